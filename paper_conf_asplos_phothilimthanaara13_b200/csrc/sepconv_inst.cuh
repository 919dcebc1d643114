// sepconv_inst.cuh -- instantiation unit body: include with SEPCONV_OP (OP_ROWS/OP_COLS/OP_SEP),
// SEPCONV_VARIANT (stream_geom variant) and SEPCONV_NAME (a token) defined.  One
// translation unit per (op, variant) keeps the parallel build short.
#include "sepconv_kernels.cuh"
#include "sepconv_launch.h"

namespace sepconv {
namespace {
template <int K, int SM>
KernelInfo info_one() {
    using I = StreamInst<K, SEPCONV_OP, SEPCONV_VARIANT, SM>;
    return {reinterpret_cast<const void *>(I::kernel), I::smem, I::threads, I::G.sr, I::G.cps};
}
template <int K, int SM>
cudaError_t launch_one(const StreamParams &p, int grid, cudaStream_t st) {
    using I = StreamInst<K, SEPCONV_OP, SEPCONV_VARIANT, SM>;
    I::kernel<<<grid, I::threads, I::smem, st>>>(p);
    return cudaGetLastError();
}
// store modes: [0] 8-byte rows, [1] 16-byte rows, [2] 8-byte rows with even-width edge warps on
// the fast path -- compiled for the fused kernel at K >= 13 only (elsewhere the [0] kernel)
#define SEPCONV_E(K) ((SEPCONV_OP == OP_SEP && (K) >= 13) ? 3 : 1)
// [3] two 8-byte stores per lane (store path 2): the fused TMA configurations only
#define SEPCONV_V (SEPCONV_OP == OP_SEP && SEPCONV_VARIANT >= 2 ? 4 : 1)
const StreamEntry kTable[kMaxK] = {
    {{info_one<1, 1>, info_one<1, 2>, info_one<1, SEPCONV_E(1)>, info_one<1, SEPCONV_V>}, {launch_one<1, 1>, launch_one<1, 2>, launch_one<1, SEPCONV_E(1)>, launch_one<1, SEPCONV_V>}},
    {{info_one<2, 1>, info_one<2, 2>, info_one<2, SEPCONV_E(2)>, info_one<2, SEPCONV_V>}, {launch_one<2, 1>, launch_one<2, 2>, launch_one<2, SEPCONV_E(2)>, launch_one<2, SEPCONV_V>}},
    {{info_one<3, 1>, info_one<3, 2>, info_one<3, SEPCONV_E(3)>, info_one<3, SEPCONV_V>}, {launch_one<3, 1>, launch_one<3, 2>, launch_one<3, SEPCONV_E(3)>, launch_one<3, SEPCONV_V>}},
    {{info_one<4, 1>, info_one<4, 2>, info_one<4, SEPCONV_E(4)>, info_one<4, SEPCONV_V>}, {launch_one<4, 1>, launch_one<4, 2>, launch_one<4, SEPCONV_E(4)>, launch_one<4, SEPCONV_V>}},
    {{info_one<5, 1>, info_one<5, 2>, info_one<5, SEPCONV_E(5)>, info_one<5, SEPCONV_V>}, {launch_one<5, 1>, launch_one<5, 2>, launch_one<5, SEPCONV_E(5)>, launch_one<5, SEPCONV_V>}},
    {{info_one<6, 1>, info_one<6, 2>, info_one<6, SEPCONV_E(6)>, info_one<6, SEPCONV_V>}, {launch_one<6, 1>, launch_one<6, 2>, launch_one<6, SEPCONV_E(6)>, launch_one<6, SEPCONV_V>}},
    {{info_one<7, 1>, info_one<7, 2>, info_one<7, SEPCONV_E(7)>, info_one<7, SEPCONV_V>}, {launch_one<7, 1>, launch_one<7, 2>, launch_one<7, SEPCONV_E(7)>, launch_one<7, SEPCONV_V>}},
    {{info_one<8, 1>, info_one<8, 2>, info_one<8, SEPCONV_E(8)>, info_one<8, SEPCONV_V>}, {launch_one<8, 1>, launch_one<8, 2>, launch_one<8, SEPCONV_E(8)>, launch_one<8, SEPCONV_V>}},
    {{info_one<9, 1>, info_one<9, 2>, info_one<9, SEPCONV_E(9)>, info_one<9, SEPCONV_V>}, {launch_one<9, 1>, launch_one<9, 2>, launch_one<9, SEPCONV_E(9)>, launch_one<9, SEPCONV_V>}},
    {{info_one<10, 1>, info_one<10, 2>, info_one<10, SEPCONV_E(10)>, info_one<10, SEPCONV_V>}, {launch_one<10, 1>, launch_one<10, 2>, launch_one<10, SEPCONV_E(10)>, launch_one<10, SEPCONV_V>}},
    {{info_one<11, 1>, info_one<11, 2>, info_one<11, SEPCONV_E(11)>, info_one<11, SEPCONV_V>}, {launch_one<11, 1>, launch_one<11, 2>, launch_one<11, SEPCONV_E(11)>, launch_one<11, SEPCONV_V>}},
    {{info_one<12, 1>, info_one<12, 2>, info_one<12, SEPCONV_E(12)>, info_one<12, SEPCONV_V>}, {launch_one<12, 1>, launch_one<12, 2>, launch_one<12, SEPCONV_E(12)>, launch_one<12, SEPCONV_V>}},
    {{info_one<13, 1>, info_one<13, 2>, info_one<13, SEPCONV_E(13)>, info_one<13, SEPCONV_V>}, {launch_one<13, 1>, launch_one<13, 2>, launch_one<13, SEPCONV_E(13)>, launch_one<13, SEPCONV_V>}},
    {{info_one<14, 1>, info_one<14, 2>, info_one<14, SEPCONV_E(14)>, info_one<14, SEPCONV_V>}, {launch_one<14, 1>, launch_one<14, 2>, launch_one<14, SEPCONV_E(14)>, launch_one<14, SEPCONV_V>}},
    {{info_one<15, 1>, info_one<15, 2>, info_one<15, SEPCONV_E(15)>, info_one<15, SEPCONV_V>}, {launch_one<15, 1>, launch_one<15, 2>, launch_one<15, SEPCONV_E(15)>, launch_one<15, SEPCONV_V>}},
    {{info_one<16, 1>, info_one<16, 2>, info_one<16, SEPCONV_E(16)>, info_one<16, SEPCONV_V>}, {launch_one<16, 1>, launch_one<16, 2>, launch_one<16, SEPCONV_E(16)>, launch_one<16, SEPCONV_V>}},
    {{info_one<17, 1>, info_one<17, 2>, info_one<17, SEPCONV_E(17)>, info_one<17, SEPCONV_V>}, {launch_one<17, 1>, launch_one<17, 2>, launch_one<17, SEPCONV_E(17)>, launch_one<17, SEPCONV_V>}},
};
#undef SEPCONV_E
#undef SEPCONV_V
}  // namespace

const StreamEntry *SEPCONV_NAME() { return kTable; }
}  // namespace sepconv
