// inst_sep_v6.cu -- stream_kernel instantiations for OP_SEP, variant 6 (see sepconv_inst.cuh).
#define SEPCONV_OP OP_SEP
#define SEPCONV_VARIANT 6
#define SEPCONV_NAME stream_table_sep_v6
#include "sepconv_inst.cuh"
