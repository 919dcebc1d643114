// sepconv_params.h -- launch parameter blocks and tile constants shared by the host
// launcher (plain C++) and the kernels (CUDA).  No device code here.
#pragma once
#include <cuda.h>
#include <cuda_runtime.h>
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
    int parts;                   // >0: row partitions per (image, strip), strided schedule; 0: contiguous;
                                 // <0: -q full-width windows + extra CTAs (SegmentIter)
    int store8;                  // 2: every output row 16-byte aligned, 1: 8-byte aligned, 0: neither
    long long total;             // nimg * nstrips * rows (work units)
    int win_rows;                // parts < 0: rows of each of the q main windows
    int extra;                   // parts < 0: CTAs sharing the last (short) window
    int steal;                   // work stealing between warps (strided schedule): a warp out of work
                                 // takes half of another's unclaimed stages when at least this many
                                 // remain (0 = off)
    unsigned epoch;              // launch id the claim words are tagged with
    unsigned long long *claims;  // claim word per (segment item, warp) (plan-owned)
    float k[kMaxK];
    float2 k2[kMaxK];            // {k_i, k_i}: the same weights as packed-FP32 operands
#ifdef SEPCONV_CTA_TRACE
    unsigned long long *trace;   // exploration builds only (tools/explore_mid.cu): per CTA
                                 // {start ns, end ns, SM id, segments}
#endif
};

struct alignas(64) Conv2DParams {
    CUtensorMap tmap;
    const float *in;
    float *out;
    long long in_img_stride, out_img_stride;
    long long ld_in, ld_out;
    int in_rows, in_cols, out_cols;
    int row_begin, rows, nimg, nstrips, parts, store8;
    long long total;
    int win_rows, extra;         // as StreamParams
    float w[kMaxK * kMaxK];      // w[j*K + i] = fl(k_i * k_j)
};

// ---- per-K tile configuration -------------------------------------------------
// Geometry of the streaming kernels (measured on B200 with tools/explore.cu, see
// profiles/r01_explore_*.txt and DESIGN.md section 6).  Each warp owns a ring of NS
// stages of SR rows x BW columns in shared memory.  RING ops need SR to be a multiple
// of K so the register ring's slot indices are compile-time.
//
// `variant` selects the mapping: 0 direct (4-byte loads), 1 direct (16-byte loads),
// 2.. the TMA configurations.  The unfused passes have one TMA configuration; the
// fused kernel has kSepTmaConfigs, all tuner candidates, because the best one moves
// with K in ways no simple model predicts:
//   cfg 0  8 warps, SR ~ 6 rows (a multiple of K), 2 stages, CTA lockstep   (shallow)
//   cfg 1  8 warps, SR ~ 8 rows, up to 3 stages, CTA lockstep               (medium)
//   cfg 2  8 warps, SR ~ 6 rows, 2 stages, warps free-running                (free)
//   cfg 3  16 warps, SR ~ 6 rows, as many stages as fit (<= 4), free-running (wide)
//   cfg 4  cfg 2 with the row pass in packed FP32 too (FFMA2 for both passes; the odd taps'
//          shifted pairs cost a few MOVs): fewer issue slots, FMA-pipe-bound at K = 15-17
//          (-2.6% at 16384^2 / K=17, tools/explore_mid.cu, profiles/r02_explore_mid.txt)
//   cfg 5  4 warps (512-column CTA strips), SR ~ 6, 2 stages, free-running, 2 CTAs per SM:
//          finer strips for widths that are not a multiple of 1024 columns (3520^2: -8%
//          at K = 3 and 9)
// "Lockstep" = a CTA barrier after every stage, so the 8 warps of a CTA read the same
// rows (4 KB of each) together: measured +13% at K=9 and +4% at K=1 on 16384^2, because
// DRAM sees whole row segments instead of 512-byte pieces at drifting times.  At K=17
// (FMA-bound) the barrier costs a little, hence cfg 2; and there 16 warps (cfg 3, 128
// registers, a few spilled) beat 8 warps with 2 stages by 10%.
constexpr int kSepTmaConfigs = 6;
constexpr int kSmemPerCta = 232448 - 1024;     // opt-in limit minus headroom

SEPCONV_HD constexpr int stream_bw(int K, int op) { return 32 * 4 + (op != OP_COLS ? (((K - 1) + 3) & ~3) : 0); }
SEPCONV_HD constexpr int stage_floats(int sr, int bw) { return (sr * bw + 31) & ~31; }   // 128-byte aligned
SEPCONV_HD constexpr int ns_fit(int nw, int sr, int bw) { return kSmemPerCta / (nw * (stage_floats(sr, bw) * 4 + 8)); }
SEPCONV_HD constexpr int clampi(int v, int lo, int hi) { return v < lo ? lo : (v > hi ? hi : v); }

struct StreamGeom {
    int nw, sr, ns, f2;
    int cps;       // CTAs per SM the grid is sized for (0 = as many as fit)
    int lock;      // 1: CTA barrier after every stage (TMA only)
};

SEPCONV_HD constexpr int sep_sr_shallow(int K) { return K >= 6 ? K : K * ((6 + K / 2) / K); }
SEPCONV_HD constexpr int sep_sr_medium(int K) { return K >= 8 ? K : K * ((8 + K - 1) / K); }

SEPCONV_HD constexpr StreamGeom stream_geom(int K, int op, int variant) {
    // packed FP32 for the column pass: halves its issue slots (FFMA2 peak is ~8% below FFMA's)
    return op == OP_SEP
               ? (variant < 2 ? StreamGeom{8, K >= 8 ? K : K * ((8 + K - 1) / K), 1, K >= 2 ? 1 : 0, 0, 0}
                  : variant == 2 ? StreamGeom{8, sep_sr_shallow(K), 2, K >= 2 ? 1 : 0, 1, 1}
                  : variant == 3 ? StreamGeom{8, sep_sr_medium(K),
                                              clampi(ns_fit(8, sep_sr_medium(K), stream_bw(K, op)), 1, 3), K >= 2 ? 1 : 0,
                                              1, 1}
                  : variant == 4 ? StreamGeom{8, sep_sr_shallow(K), 2, K >= 2 ? 1 : 0, 1, 0}
                  : variant == 5 ? StreamGeom{16, sep_sr_shallow(K),
                                              clampi(ns_fit(16, sep_sr_shallow(K), stream_bw(K, op)), 1, 4),
                                              K >= 2 ? 1 : 0, 1, 0}
                  : variant == 6 ? StreamGeom{8, sep_sr_shallow(K), 2, K >= 2 ? 2 : 0, 1, 0}
                                 : StreamGeom{4, sep_sr_shallow(K), 2, K >= 2 ? 1 : 0, 2, 0})
               : op == OP_ROWS ? StreamGeom{8, 8, clampi(ns_fit(8, 8, stream_bw(K, op)), 1, 8), 0, 0, 0}
                               : StreamGeom{8, K * ((8 + K - 1) / K),
                                            clampi(ns_fit(8, K * ((8 + K - 1) / K), stream_bw(K, op)), 1, 8),
                                            K >= 2 ? 1 : 0, 0, 0};
}
SEPCONV_HD constexpr int stream_variants(int op) { return op == OP_SEP ? 2 + kSepTmaConfigs : 3; }

template <int K> struct Conv2DCfg {
    static constexpr int SR = 8;
    static constexpr int NS = (K - 1 + SR - 1) / SR + 2;
};

SEPCONV_HD constexpr int box_width(int K, bool halo) {
    return kWarpCols + (halo ? (((K - 1) + 3) & ~3) : 0);
}

enum Map { MAP_DIRECT = 0, MAP_DIRECT_VEC = 1, MAP_TMA = 2 };

}  // namespace sepconv
