// inst_sep_v2.cu -- stream_kernel instantiations for OP_SEP, variant 2 (see sepconv_inst.cuh).
#define SEPCONV_OP OP_SEP
#define SEPCONV_VARIANT 2
#define SEPCONV_NAME stream_table_sep_v2
#include "sepconv_inst.cuh"
