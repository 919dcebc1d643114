// sepconv_2d.cu -- instantiations of conv2d_kernel<K, MAP, kNW> for K = 1..17 and the three mappings.
#include "sepconv_kernels.cuh"
#include "sepconv_launch.h"

namespace sepconv {
namespace {
template <int K, int MAP>
KernelInfo info_one() {
    return {reinterpret_cast<const void *>(&conv2d_kernel<K, MAP, kNW>), conv2d_smem_bytes<K, MAP, kNW>(),
            kNW * 32, Conv2DCfg<K>::SR, 0};
}
template <int K, int MAP>
cudaError_t launch_one(const Conv2DParams &p, int grid, cudaStream_t st) {
    conv2d_kernel<K, MAP, kNW><<<grid, kNW * 32, conv2d_smem_bytes<K, MAP, kNW>(), st>>>(p);
    return cudaGetLastError();
}
using InfoFn = KernelInfo (*)();
using LaunchFn = cudaError_t (*)(const Conv2DParams &, int, cudaStream_t);
#define SEPCONV_ROW(K) {info_one<K, MAP_DIRECT>, info_one<K, MAP_DIRECT_VEC>, info_one<K, MAP_TMA>}
const InfoFn kInfo[kMaxK][3] = {
    SEPCONV_ROW(1),
    SEPCONV_ROW(2),
    SEPCONV_ROW(3),
    SEPCONV_ROW(4),
    SEPCONV_ROW(5),
    SEPCONV_ROW(6),
    SEPCONV_ROW(7),
    SEPCONV_ROW(8),
    SEPCONV_ROW(9),
    SEPCONV_ROW(10),
    SEPCONV_ROW(11),
    SEPCONV_ROW(12),
    SEPCONV_ROW(13),
    SEPCONV_ROW(14),
    SEPCONV_ROW(15),
    SEPCONV_ROW(16),
    SEPCONV_ROW(17)};
#undef SEPCONV_ROW
#define SEPCONV_ROW(K) {launch_one<K, MAP_DIRECT>, launch_one<K, MAP_DIRECT_VEC>, launch_one<K, MAP_TMA>}
const LaunchFn kLaunch[kMaxK][3] = {
    SEPCONV_ROW(1),
    SEPCONV_ROW(2),
    SEPCONV_ROW(3),
    SEPCONV_ROW(4),
    SEPCONV_ROW(5),
    SEPCONV_ROW(6),
    SEPCONV_ROW(7),
    SEPCONV_ROW(8),
    SEPCONV_ROW(9),
    SEPCONV_ROW(10),
    SEPCONV_ROW(11),
    SEPCONV_ROW(12),
    SEPCONV_ROW(13),
    SEPCONV_ROW(14),
    SEPCONV_ROW(15),
    SEPCONV_ROW(16),
    SEPCONV_ROW(17)};
#undef SEPCONV_ROW
}  // namespace

KernelInfo conv2d_info(int map, int K) { return kInfo[K - 1][map](); }
cudaError_t conv2d_launch(int map, int K, const Conv2DParams &p, int grid, cudaStream_t st) {
    return kLaunch[K - 1][map](p, grid, st);
}
}  // namespace sepconv
