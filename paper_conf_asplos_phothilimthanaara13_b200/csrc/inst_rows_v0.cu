// inst_rows_v0.cu -- stream_kernel instantiations for OP_ROWS, variant 0 (see sepconv_inst.cuh).
#define SEPCONV_OP OP_ROWS
#define SEPCONV_VARIANT 0
#define SEPCONV_NAME stream_table_rows_v0
#include "sepconv_inst.cuh"
