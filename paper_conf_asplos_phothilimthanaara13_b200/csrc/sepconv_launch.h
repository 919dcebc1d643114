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

// streaming kernels: variant = 0 direct, 1 direct 16-byte, 2.. TMA configurations
// (stream_geom in sepconv_params.h); conv2d: map = MAP_DIRECT / MAP_DIRECT_VEC / MAP_TMA.
// K in [1, 17]
KernelInfo stream_rows_info(int map, int K);
KernelInfo stream_cols_info(int map, int K);
KernelInfo stream_sep_info(int map, int K);
KernelInfo conv2d_info(int map, int K);
cudaError_t stream_rows_launch(int map, int K, const StreamParams &p, int grid, cudaStream_t st);
cudaError_t stream_cols_launch(int map, int K, const StreamParams &p, int grid, cudaStream_t st);
cudaError_t stream_sep_launch(int map, int K, const StreamParams &p, int grid, cudaStream_t st);
cudaError_t conv2d_launch(int map, int K, const Conv2DParams &p, int grid, cudaStream_t st);

// utility kernels (sepconv_util.cu)
cudaError_t launch_fill_pattern(float *dst, long long n, unsigned seed, cudaStream_t st);
cudaError_t launch_l2_flush(float *scratch, long long n, cudaStream_t st);

}  // namespace sepconv
