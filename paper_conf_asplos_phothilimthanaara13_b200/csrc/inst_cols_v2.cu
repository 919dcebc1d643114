// inst_cols_v2.cu -- stream_kernel instantiations for OP_COLS, variant 2 (see sepconv_inst.cuh).
#define SEPCONV_OP OP_COLS
#define SEPCONV_VARIANT 2
#define SEPCONV_NAME stream_table_cols_v2
#include "sepconv_inst.cuh"
