// sepconv_params.h -- launch parameter blocks and tile constants shared by the host
// launcher (plain C++) and the kernels (CUDA).  No device code here.
#pragma once
#include <cuda.h>
#include <stdint.h>

#ifdef __CUDACC__
#define SEPCONV_HD __host__ __device__
#else
#define SEPCONV_HD
#endif

namespace sepconv {

constexpr int kMaxK = 17;
constexpr int V = 4;                        // output columns per thread
constexpr int kWarpCols = 32 * V;           // output columns per warp strip

enum Op { OP_ROWS = 0, OP_COLS = 1, OP_SEP = 2 };

// Parameters of one launch.  Passed as a __grid_constant__ so the weights are
// read as constant-bank / uniform-register FFMA operands (2 register reads per
// FFMA: ~124 FMA/clk/SM measured on B200 vs ~88 with a register weight,
// profiles/r01_ubench_ffma.txt).
struct alignas(64) StreamParams {
    CUtensorMap tmap;            // 3-D map over the input: {cols, rows, images}
    const float *in;
    float *out;
    long long in_img_stride;     // floats between images of the input
    long long out_img_stride;
    long long ld_in, ld_out;     // row pitches (floats)
    int in_rows;                 // rows of one input image
    int in_cols;                 // valid input columns
    int out_cols;                // valid output columns
    int row_begin;               // first output row (and first input row) of this launch
    int rows;                    // output rows per image in this launch
    int nimg;
    int nstrips;                 // CTA strips = ceil(out_cols / (warps*128))
    int pad0;
    long long total;             // nimg * nstrips * rows (work units)
    float k[kMaxK];
};

struct alignas(64) Conv2DParams {
    CUtensorMap tmap;
    const float *in;
    float *out;
    long long in_img_stride, out_img_stride;
    long long ld_in, ld_out;
    int in_rows, in_cols, out_cols;
    int row_begin, rows, nimg, nstrips, pad0;
    long long total;
    float w[kMaxK * kMaxK];      // w[j*K + i] = fl(k_i * k_j)
};

// ---- per-K tile configuration -------------------------------------------------
template <int K> struct StreamCfg {
    static constexpr int HALO4 = ((K - 1) + 3) & ~3;            // halo columns, rounded to 16 B
    static constexpr int M = (20 / K) > 0 ? (20 / K) : 1;
    static constexpr int SR = K * M;                           // rows per stage: a multiple of K
    static constexpr int NS = 2;                               // stages per warp
};

template <int K> struct Conv2DCfg {
    static constexpr int SR = 8;
    static constexpr int NS = (K - 1 + SR - 1) / SR + 2;
};

SEPCONV_HD constexpr int box_width(int K, bool halo) {
    return kWarpCols + (halo ? (((K - 1) + 3) & ~3) : 0);
}

enum Map { MAP_DIRECT = 0, MAP_DIRECT_VEC = 1, MAP_TMA = 2 };

}  // namespace sepconv
