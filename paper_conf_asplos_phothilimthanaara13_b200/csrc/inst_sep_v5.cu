// inst_sep_v5.cu -- stream_kernel instantiations for OP_SEP, variant 5 (see sepconv_inst.cuh).
#define SEPCONV_OP OP_SEP
#define SEPCONV_VARIANT 5
#define SEPCONV_NAME stream_table_sep_v5
#include "sepconv_inst.cuh"
