// inst_sep_v4.cu -- stream_kernel instantiations for OP_SEP, variant 4 (see sepconv_inst.cuh).
#define SEPCONV_OP OP_SEP
#define SEPCONV_VARIANT 4
#define SEPCONV_NAME stream_table_sep_v4
#include "sepconv_inst.cuh"
