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
#define SEPCONV_ROW(K) {{info_one<K, 1>, info_one<K, 2>}}
const StreamEntry kTable[kMaxK] = {
    {{info_one<1, 1>, info_one<1, 2>}, {launch_one<1, 1>, launch_one<1, 2>}},
    {{info_one<2, 1>, info_one<2, 2>}, {launch_one<2, 1>, launch_one<2, 2>}},
    {{info_one<3, 1>, info_one<3, 2>}, {launch_one<3, 1>, launch_one<3, 2>}},
    {{info_one<4, 1>, info_one<4, 2>}, {launch_one<4, 1>, launch_one<4, 2>}},
    {{info_one<5, 1>, info_one<5, 2>}, {launch_one<5, 1>, launch_one<5, 2>}},
    {{info_one<6, 1>, info_one<6, 2>}, {launch_one<6, 1>, launch_one<6, 2>}},
    {{info_one<7, 1>, info_one<7, 2>}, {launch_one<7, 1>, launch_one<7, 2>}},
    {{info_one<8, 1>, info_one<8, 2>}, {launch_one<8, 1>, launch_one<8, 2>}},
    {{info_one<9, 1>, info_one<9, 2>}, {launch_one<9, 1>, launch_one<9, 2>}},
    {{info_one<10, 1>, info_one<10, 2>}, {launch_one<10, 1>, launch_one<10, 2>}},
    {{info_one<11, 1>, info_one<11, 2>}, {launch_one<11, 1>, launch_one<11, 2>}},
    {{info_one<12, 1>, info_one<12, 2>}, {launch_one<12, 1>, launch_one<12, 2>}},
    {{info_one<13, 1>, info_one<13, 2>}, {launch_one<13, 1>, launch_one<13, 2>}},
    {{info_one<14, 1>, info_one<14, 2>}, {launch_one<14, 1>, launch_one<14, 2>}},
    {{info_one<15, 1>, info_one<15, 2>}, {launch_one<15, 1>, launch_one<15, 2>}},
    {{info_one<16, 1>, info_one<16, 2>}, {launch_one<16, 1>, launch_one<16, 2>}},
    {{info_one<17, 1>, info_one<17, 2>}, {launch_one<17, 1>, launch_one<17, 2>}},
};
#undef SEPCONV_ROW
}  // namespace

const StreamEntry *SEPCONV_NAME() { return kTable; }
}  // namespace sepconv
