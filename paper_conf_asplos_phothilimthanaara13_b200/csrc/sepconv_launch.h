// sepconv_launch.h -- host-side entry points into the kernel translation units.
#pragma once
#include <cuda_runtime.h>

#include <utility>

#include "sepconv_params.h"

namespace sepconv {

constexpr int kNW = 8;   // compute warps per CTA (each owns a 128-column strip)

struct KernelInfo {
    const void *func;    // the __global__ function (for attributes / occupancy)
    size_t smem;         // dynamic shared memory bytes
    int threads;
    int stage_rows;      // TMA box height (streaming kernels)
    int cps;             // CTAs per SM to size the grid for (0 = occupancy limit)
};

// streaming kernels: op = OP_ROWS / OP_COLS / OP_SEP; variant = 0 direct, 1 direct 16-byte,
// 2.. TMA configurations (stream_geom in sepconv_params.h); smode = 2 if every output row is
// 16-byte aligned (the 16-byte store path), else 1, or 3 (the 8-byte path with even-width
// right-edge warps on it; a distinct kernel only for the fused kernel at K >= 13), or 4 (two
// 8-byte stores per lane: store path 2 of the fused TMA configurations).
// conv2d: map = MAP_DIRECT / _VEC / MAP_TMA.  K in [1, 17].
struct StreamEntry {
    KernelInfo (*info[4])();
    cudaError_t (*launch[4])(const StreamParams &, int, cudaStream_t);
};
KernelInfo stream_info(int op, int variant, int K, int smode);
cudaError_t stream_launch(int op, int variant, int K, int smode, const StreamParams &p, int grid, cudaStream_t st);
KernelInfo conv2d_info(int map, int K);
cudaError_t conv2d_launch(int map, int K, const Conv2DParams &p, int grid, cudaStream_t st);

// utility kernels (sepconv_util.cu)
cudaError_t launch_fill_pattern(float *dst, long long n, unsigned seed, cudaStream_t st);
cudaError_t launch_l2_flush(float *scratch, long long n, cudaStream_t st);
// read a second buffer of >= 2 x L2 (zero-filled by the caller) after launch_l2_flush: L2 ends clean
cudaError_t launch_l2_clean(const float *src, long long n, float *sink, cudaStream_t st);

}  // namespace sepconv
