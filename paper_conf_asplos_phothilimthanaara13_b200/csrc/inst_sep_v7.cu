// inst_sep_v7.cu -- stream_kernel instantiations for OP_SEP, variant 7 (see sepconv_inst.cuh).
#define SEPCONV_OP OP_SEP
#define SEPCONV_VARIANT 7
#define SEPCONV_NAME stream_table_sep_v7
#include "sepconv_inst.cuh"
