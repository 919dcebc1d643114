// sepconv_sep.cu -- instantiations of stream_kernel for OP_SEP, K = 1..17, every mapping
// variant of stream_geom (sepconv_params.h).
#include "sepconv_kernels.cuh"
#include "sepconv_launch.h"

namespace sepconv {
namespace {
constexpr int NV = stream_variants(OP_SEP);
template <int K, int V_>
KernelInfo info_one() {
    using I = StreamInst<K, OP_SEP, V_>;
    return {reinterpret_cast<const void *>(I::kernel), I::smem, I::threads, I::G.sr, I::G.cps};
}
template <int K, int V_>
cudaError_t launch_one(const StreamParams &p, int grid, cudaStream_t st) {
    using I = StreamInst<K, OP_SEP, V_>;
    I::kernel<<<grid, I::threads, I::smem, st>>>(p);
    return cudaGetLastError();
}
template <int K, int... Vs>
struct Row {
    static constexpr KernelInfo (*info[sizeof...(Vs)])() = {info_one<K, Vs>...};
    static constexpr cudaError_t (*launch[sizeof...(Vs)])(const StreamParams &, int, cudaStream_t) = {launch_one<K, Vs>...};
};
template <int K, int... Vs>
KernelInfo info_dispatch(int v, std::integer_sequence<int, Vs...>) {
    return Row<K, Vs...>::info[v]();
}
template <int K, int... Vs>
cudaError_t launch_dispatch(int v, const StreamParams &p, int grid, cudaStream_t st, std::integer_sequence<int, Vs...>) {
    return Row<K, Vs...>::launch[v](p, grid, st);
}
using Seq = std::make_integer_sequence<int, NV>;
using InfoFn = KernelInfo (*)(int);
using LaunchFn = cudaError_t (*)(int, const StreamParams &, int, cudaStream_t);
template <int K>
KernelInfo info_k(int v) { return info_dispatch<K>(v, Seq{}); }
template <int K>
cudaError_t launch_k(int v, const StreamParams &p, int grid, cudaStream_t st) { return launch_dispatch<K>(v, p, grid, st, Seq{}); }
#define SEPCONV_ROW(K) info_k<K>
const InfoFn kInfo[kMaxK] = {
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
#define SEPCONV_ROW(K) launch_k<K>
const LaunchFn kLaunch[kMaxK] = {
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

KernelInfo stream_sep_info(int variant, int K) { return kInfo[K - 1](variant); }
cudaError_t stream_sep_launch(int variant, int K, const StreamParams &p, int grid, cudaStream_t st) {
    return kLaunch[K - 1](variant, p, grid, st);
}
}  // namespace sepconv
