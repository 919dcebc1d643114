// sepconv_dispatch.cpp -- (op, variant, K, store mode) -> kernel info / launcher, over the
// per-(op, variant) instantiation units inst_*.cu.
#include "sepconv_launch.h"

namespace sepconv {
const StreamEntry *stream_table_rows_v0();
const StreamEntry *stream_table_rows_v1();
const StreamEntry *stream_table_rows_v2();
const StreamEntry *stream_table_cols_v0();
const StreamEntry *stream_table_cols_v1();
const StreamEntry *stream_table_cols_v2();
const StreamEntry *stream_table_sep_v0();
const StreamEntry *stream_table_sep_v1();
const StreamEntry *stream_table_sep_v2();
const StreamEntry *stream_table_sep_v3();
const StreamEntry *stream_table_sep_v4();
const StreamEntry *stream_table_sep_v5();
const StreamEntry *stream_table_sep_v6();
const StreamEntry *stream_table_sep_v7();

static const StreamEntry *table(int op, int variant) {
    switch (op) {
        case OP_ROWS:
            switch (variant) {
                case 0: return stream_table_rows_v0();
                case 1: return stream_table_rows_v1();
                case 2: return stream_table_rows_v2();
            }
            break;
        case OP_COLS:
            switch (variant) {
                case 0: return stream_table_cols_v0();
                case 1: return stream_table_cols_v1();
                case 2: return stream_table_cols_v2();
            }
            break;
        case OP_SEP:
            switch (variant) {
                case 0: return stream_table_sep_v0();
                case 1: return stream_table_sep_v1();
                case 2: return stream_table_sep_v2();
                case 3: return stream_table_sep_v3();
                case 4: return stream_table_sep_v4();
                case 5: return stream_table_sep_v5();
                case 6: return stream_table_sep_v6();
                case 7: return stream_table_sep_v7();
            }
            break;
    }
    return nullptr;
}

KernelInfo stream_info(int op, int variant, int K, int smode) {
    const StreamEntry *t = table(op, variant);
    return t[K - 1].info[smode == 2 ? 1 : smode == 3 ? 2 : smode == 4 ? 3 : 0]();
}
cudaError_t stream_launch(int op, int variant, int K, int smode, const StreamParams &p, int grid, cudaStream_t st) {
    const StreamEntry *t = table(op, variant);
    return t[K - 1].launch[smode == 2 ? 1 : smode == 3 ? 2 : smode == 4 ? 3 : 0](p, grid, st);
}
}  // namespace sepconv
