// inst_cols_v1.cu -- stream_kernel instantiations for OP_COLS, variant 1 (see sepconv_inst.cuh).
#define SEPCONV_OP OP_COLS
#define SEPCONV_VARIANT 1
#define SEPCONV_NAME stream_table_cols_v1
#include "sepconv_inst.cuh"
