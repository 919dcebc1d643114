// inst_rows_v2.cu -- stream_kernel instantiations for OP_ROWS, variant 2 (see sepconv_inst.cuh).
#define SEPCONV_OP OP_ROWS
#define SEPCONV_VARIANT 2
#define SEPCONV_NAME stream_table_rows_v2
#include "sepconv_inst.cuh"
