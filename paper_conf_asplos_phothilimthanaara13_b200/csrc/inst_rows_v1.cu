// inst_rows_v1.cu -- stream_kernel instantiations for OP_ROWS, variant 1 (see sepconv_inst.cuh).
#define SEPCONV_OP OP_ROWS
#define SEPCONV_VARIANT 1
#define SEPCONV_NAME stream_table_rows_v1
#include "sepconv_inst.cuh"
