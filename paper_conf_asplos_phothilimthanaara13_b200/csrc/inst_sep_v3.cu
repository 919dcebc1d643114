// inst_sep_v3.cu -- stream_kernel instantiations for OP_SEP, variant 3 (see sepconv_inst.cuh).
#define SEPCONV_OP OP_SEP
#define SEPCONV_VARIANT 3
#define SEPCONV_NAME stream_table_sep_v3
#include "sepconv_inst.cuh"
