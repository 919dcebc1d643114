// sor.cu -- Poisson2D red-black SOR on sm_100a (include/sor.h; PAPER.md P:1294-1308,
// SURVEY.md 8(f) NEXT-3).
//
// Layout (reading P5): the plan splits x and b into red / black buffers, [N][ldh] each,
// red[i][k] = x[i][2k + (i & 1)], black[i][k] = x[i][2k + 1 - (i & 1)].  In split
// coordinates a cell (i, k) of colour c sits at grid column j = 2k + s, s = (i + c) & 1,
// and its four neighbours are all of the other colour:
//     N = other[i-1][k], S = other[i+1][k], W = other[i][k+s-1], E = other[i][k+s].
//
// Arithmetic (reading P6), identical in every kernel, bitwise equal to the fixed-order
// float32 oracle:  t = (((N + S) + W) + E) + b;  u' = fma(w/4, t, (1-w) * u).
//
// Kernels:
//   rb_split_kernel / rb_merge_kernel   P5 and its inverse (HBM-bound copies)
//   sor_half_kernel<COLOR>              one half-sweep in place (SOR_HALF: 2 launches
//                                       per iteration, 16 B of HBM traffic per cell)
//   sor_wave_kernel<T>                  T iterations in one pass (SOR_WAVE): each warp
//       owns a strip of 4*(32-2*HL) split columns (HL halo lanes per side, HL =
//       ceil(2T/4): the dependency cone widens by one split column per half-sweep) and
//       walks down its rows.  Rows arrive in a per-warp shared-memory ring by 3-D TMA
//       (cp.async.bulk.tensor + mbarrier; one box = the red and black row of a buffer
//       pair) PF rows ahead.  At step r the warp takes row
//       r (level 0) and computes red_t(r-2t+1), black_t(r-2t) for t = 1..T from 3-row
//       register windows of the previous level, so u and b are read once and u written
//       once per T iterations (12 B per cell per pass), out of place into the plan's
//       second buffer pair.
#include <cuda_runtime.h>

#include <algorithm>
#include <cmath>
#include <cstdlib>
#include <cstring>
#include <new>
#include <vector>

#include "../../include/sor.h"
#include "sepconv_internal.h"

namespace sor {

constexpr int kMaxDepth = 8;
constexpr int kWaveWarps = 4;            // warps per CTA of the wave kernel
constexpr int kThreads = 256;            // split / merge / half kernels

struct alignas(64) SorParams {
    CUtensorMap tmap;                    // WAVE: 3-D map {ldh, n, 6} over the plan's six split buffers
    int zu;                              // WAVE: buffer index (0 or 2) of the pair the pass reads
    const float *ur, *ub;                // iterate read by the pass (split buffers)
    float *ur_out, *ub_out;              // iterate written (HALF: the same buffers)
    const float *br, *bb;                // right-hand side, split
    long long ldh;                       // split row pitch (floats, multiple of 4)
    int n, m;                            // grid rows, columns
    float w4, om1;                       // w/4 and 1-w, formed in float32 on the host (P6)
    int nstrips, seg_rows;               // wave schedule: items = nstrips * nsegs
    long long items;
};

// interior columns of split quad k0..k0+3 for s = 0 (j = 2k) and s = 1 (j = 2k+1): bit e set
// when 1 <= j <= m-2 (reading P2: the frame is never written)
__device__ __forceinline__ unsigned col_mask(int k0, int s, int m, long long ldh) {
    unsigned msk = 0;
#pragma unroll
    for (int e = 0; e < 4; ++e) {
        const int k = k0 + e;
        const int j = 2 * k + s;
        if (k >= 0 && k < ldh && j >= 1 && j <= m - 2) msk |= 1u << e;
    }
    return msk;
}

__device__ __forceinline__ float relax1(float n, float s, float w, float e, float b, float u, float w4, float om1) {
    float t = __fadd_rn(n, s);
    t = __fadd_rn(t, w);
    t = __fadd_rn(t, e);
    t = __fadd_rn(t, b);
    // operands ordered so the uniform w/4 and 1-w sit in the constant-operand slot
    // (FMUL/FFMA R, R, c[]); multiplication commutes exactly, so P6 is unchanged
    return __fmaf_rn(t, w4, __fmul_rn(u, om1));
}

// One quad of cells: u (own colour), N/S/C the other colour's rows i-1, i+1, i at the same
// k, left = other[i][k0-1], right = other[i][k0+4]; s = row/colour parity, msk = interior
// bits.  Cells outside the interior keep u.
__device__ __forceinline__ float4 relax4(const float4 &u, const float4 &N, const float4 &S, const float4 &C,
                                         float left, float right, const float4 &b, int s, unsigned msk, float w4,
                                         float om1) {
    const float W0 = s ? C.x : left, W1 = s ? C.y : C.x, W2 = s ? C.z : C.y, W3 = s ? C.w : C.z;
    const float E0 = s ? C.y : C.x, E1 = s ? C.z : C.y, E2 = s ? C.w : C.z, E3 = s ? right : C.w;
    float4 o;
    o.x = (msk & 1u) ? relax1(N.x, S.x, W0, E0, b.x, u.x, w4, om1) : u.x;
    o.y = (msk & 2u) ? relax1(N.y, S.y, W1, E1, b.y, u.y, w4, om1) : u.y;
    o.z = (msk & 4u) ? relax1(N.z, S.z, W2, E2, b.z, u.z, w4, om1) : u.z;
    o.w = (msk & 8u) ? relax1(N.w, S.w, W3, E3, b.w, u.w, w4, om1) : u.w;
    return o;
}

__device__ __forceinline__ float4 ld4(const float *p) { return *reinterpret_cast<const float4 *>(p); }
__device__ __forceinline__ float4 ldg4(const float *p) { return __ldg(reinterpret_cast<const float4 *>(p)); }
__device__ __forceinline__ void st4(float *p, const float4 &v) { *reinterpret_cast<float4 *>(p) = v; }
// predicated 16-byte store: a branch-free body keeps ptxas from unswitching the hot loop
__device__ __forceinline__ void st4_if(float *p, const float4 &v, bool ok) {
    asm volatile(
        "{\n\t.reg .pred q;\n\tsetp.ne.u32 q, %5, 0;\n\t"
        "@q st.global.v4.f32 [%0], {%1, %2, %3, %4};\n\t}" ::"l"(p),
        "f"(v.x), "f"(v.y), "f"(v.z), "f"(v.w), "r"(static_cast<unsigned>(ok))
        : "memory");
}

// ---- P5: split and merge ------------------------------------------------------------------
// one thread per (row i, split quad k0..k0+3): grid columns 2k0 .. 2k0+7 of row i
__global__ void rb_split_kernel(const float *__restrict__ x, long long ldx, int n, int m, float *__restrict__ red,
                                float *__restrict__ black, long long ldh) {
    const long long nq = ldh / 4;
    for (long long idx = blockIdx.x * static_cast<long long>(blockDim.x) + threadIdx.x; idx < n * nq;
         idx += static_cast<long long>(gridDim.x) * blockDim.x) {
        const int i = static_cast<int>(idx / nq);
        const int k0 = static_cast<int>(idx - static_cast<long long>(i) * nq) * 4;
        const float *row = x + i * ldx;
        float v[8];
#pragma unroll
        for (int e = 0; e < 8; ++e) {
            const int j = 2 * k0 + e;
            v[e] = j < m ? row[j] : 0.f;
        }
        // row parity: red holds the even columns of even rows and the odd columns of odd rows
        const int p = i & 1;
        st4(red + i * ldh + k0, make_float4(v[p], v[2 + p], v[4 + p], v[6 + p]));
        st4(black + i * ldh + k0, make_float4(v[1 - p], v[3 - p], v[5 - p], v[7 - p]));
    }
}

__global__ void rb_merge_kernel(const float *__restrict__ red, const float *__restrict__ black, long long ldh, int n,
                                int m, float *__restrict__ x, long long ldx) {
    const long long nq = ldh / 4;
    for (long long idx = blockIdx.x * static_cast<long long>(blockDim.x) + threadIdx.x; idx < n * nq;
         idx += static_cast<long long>(gridDim.x) * blockDim.x) {
        const int i = static_cast<int>(idx / nq);
        const int k0 = static_cast<int>(idx - static_cast<long long>(i) * nq) * 4;
        const float4 r = ld4(red + i * ldh + k0), b = ld4(black + i * ldh + k0);
        const int p = i & 1;
        const float ev[4] = {p ? b.x : r.x, p ? b.y : r.y, p ? b.z : r.z, p ? b.w : r.w};   // even columns
        const float od[4] = {p ? r.x : b.x, p ? r.y : b.y, p ? r.z : b.z, p ? r.w : b.w};   // odd columns
        float *row = x + i * ldx;
#pragma unroll
        for (int e = 0; e < 4; ++e) {
            const int j = 2 * (k0 + e);
            if (j < m) row[j] = ev[e];
            if (j + 1 < m) row[j + 1] = od[e];
        }
    }
}

// ---- SOR_HALF: one colour, in place -------------------------------------------------------
template <int COLOR>
__global__ void __launch_bounds__(kThreads) sor_half_kernel(const SorParams p) {
    const long long nq = p.ldh / 4;
    const long long rows = p.n - 2;
    float *self = COLOR == 0 ? p.ur_out : p.ub_out;
    const float *__restrict__ other = COLOR == 0 ? p.ub : p.ur;
    const float *__restrict__ bs = COLOR == 0 ? p.br : p.bb;
    for (long long idx = blockIdx.x * static_cast<long long>(blockDim.x) + threadIdx.x; idx < rows * nq;
         idx += static_cast<long long>(gridDim.x) * blockDim.x) {
        const int i = 1 + static_cast<int>(idx / nq);
        const int k0 = static_cast<int>(idx - static_cast<long long>(i - 1) * nq) * 4;
        const int s = (i + COLOR) & 1;
        const long long o = i * p.ldh + k0;
        const float4 u = ld4(self + o);
        const float4 b = ldg4(bs + o);
        const float4 N = ldg4(other + o - p.ldh), S = ldg4(other + o + p.ldh), C = ldg4(other + o);
        const float left = (s == 0 && k0 > 0) ? __ldg(other + o - 1) : 0.f;
        const float right = (s == 1 && k0 + 4 < p.ldh) ? __ldg(other + o + 4) : 0.f;
        st4(self + o, relax4(u, N, S, C, left, right, b, s, col_mask(k0, s, p.m, p.ldh), p.w4, p.om1));
    }
}

// ---- SOR_WAVE: T iterations per pass ------------------------------------------------------
template <int T>
struct Wave {
    static constexpr int HL = (2 * T + 3) / 4;       // halo lanes per side
    static constexpr int OUT_LANES = 32 - 2 * HL;
    static constexpr int WOUT = 4 * OUT_LANES;       // split columns written per strip
    static constexpr int PF = 3;                     // rows prefetched ahead of the wavefront
    static constexpr int RDU = 4;                    // u ring rows (>= PF + 1), one mbarrier each
    // b ring rows: row r - 2T (black_T at step r) must survive until row r + PF lands;
    // 12 rows (T <= 4) keep a 4-warp CTA at 64 KB: 3 CTAs (12 warps) per SM
    static constexpr int RDB = (2 * T + PF + 1 <= 12) ? 12 : (2 * T + PF + 1 <= 16 ? 16 : 32);
    static constexpr int WARP_FLOATS = 128 * (2 * RDU + 2 * RDB);
    static constexpr size_t SMEM = static_cast<size_t>(kWaveWarps) * (WARP_FLOATS * 4 + RDU * 8);
    static_assert(2 * T + PF + 1 <= RDB, "b ring too shallow");
};

__device__ __forceinline__ uint32_t smem_addr(const void *p) {
    return static_cast<uint32_t>(__cvta_generic_to_shared(p));
}

// One step's refill issued by the whole (converged) warp: the operands are warp-uniform values
// computed outside any lane-divergent branch, and one elected lane runs the fence, the
// expect_tx and the two TMA boxes (u pair, b pair) under a predicate -- no `if (lane == 0)`
// region whose operands ptxas would move into uniform registers lane by lane.
__device__ __forceinline__ void refill_elected(bool go, uint32_t bar, uint32_t dst_u, uint32_t dst_b,
                                               const CUtensorMap *map, int col, int row, int zu) {
    asm volatile(
        "{\n\t.reg .pred e, g, q;\n\t"
        "elect.sync _|e, 0xffffffff;\n\t"
        "setp.ne.u32 g, %0, 0;\n\t"
        "and.pred q, e, g;\n\t"
        "@q fence.proxy.async.shared::cta;\n\t"
        "@q mbarrier.arrive.expect_tx.shared::cta.b64 _, [%1], 2048;\n\t"
        "@q cp.async.bulk.tensor.3d.shared::cluster.global.tile.mbarrier::complete_tx::bytes "
        "[%2], [%4, {%5, %6, %7}], [%1];\n\t"
        "@q cp.async.bulk.tensor.3d.shared::cluster.global.tile.mbarrier::complete_tx::bytes "
        "[%3], [%4, {%5, %6, 4}], [%1];\n\t}" ::"r"(static_cast<uint32_t>(go)),
        "r"(bar), "r"(dst_u), "r"(dst_b), "l"(reinterpret_cast<uint64_t>(map)), "r"(col), "r"(row), "r"(zu)
        : "memory");
}

// one TMA box {128 split columns, 1 row, 2 buffers}: the red and the black row of one
// buffer pair, 1 KB, columns outside [0, ldh) and rows outside [0, n) zero-filled (those cells
// are never written and only feed cells that are not)
__device__ __forceinline__ void tma_row_pair(void *dst, const CUtensorMap *map, uint64_t *bar, int col, int row,
                                             int z) {
    asm volatile(
        "cp.async.bulk.tensor.3d.shared::cluster.global.tile.mbarrier::complete_tx::bytes "
        "[%0], [%1, {%3, %4, %5}], [%2];" ::"r"(smem_addr(dst)),
        "l"(reinterpret_cast<uint64_t>(map)), "r"(smem_addr(bar)), "r"(col), "r"(row), "r"(z)
        : "memory");
}

__device__ __forceinline__ void bar_expect(uint64_t *bar, uint32_t bytes) {
    asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(smem_addr(bar)), "r"(bytes) : "memory");
}

__device__ __forceinline__ void bar_wait(uint64_t *bar, uint32_t parity) {
    uint32_t done, spins = 0;
    do {
        if (++spins == (1u << 26)) __trap();          // a lost transaction: fail loudly, never hang
        asm volatile(
            "{\n\t.reg .pred q;\n\t"
            "mbarrier.try_wait.parity.shared::cta.b64 q, [%1], %2;\n\t"
            "selp.u32 %0, 1, 0, q;\n\t}"
            : "=r"(done)
            : "r"(smem_addr(bar)), "r"(parity)
            : "memory");
    } while (!done);
}

// relax4 with the parity a compile-time constant (the 6-step unroll fixes it).  All four
// cells are evaluated and the frame / out-of-range cells then select their old value: a
// select per cell instead of a predicated FADD/FFMA chain plus a move (same bits: the
// arithmetic of every written cell is unchanged, P6)
template <int S>
__device__ __forceinline__ float4 relax4s(const float4 &u, const float4 &N, const float4 &Sv, const float4 &C,
                                          float left, float right, const float4 &b, unsigned msk, float w4,
                                          float om1) {
    float4 o;
    if constexpr (S == 0) {
        o.x = relax1(N.x, Sv.x, left, C.x, b.x, u.x, w4, om1);
        o.y = relax1(N.y, Sv.y, C.x, C.y, b.y, u.y, w4, om1);
        o.z = relax1(N.z, Sv.z, C.y, C.z, b.z, u.z, w4, om1);
        o.w = relax1(N.w, Sv.w, C.z, C.w, b.w, u.w, w4, om1);
    } else {
        o.x = relax1(N.x, Sv.x, C.x, C.y, b.x, u.x, w4, om1);
        o.y = relax1(N.y, Sv.y, C.y, C.z, b.y, u.y, w4, om1);
        o.z = relax1(N.z, Sv.z, C.z, C.w, b.z, u.z, w4, om1);
        o.w = relax1(N.w, Sv.w, C.w, right, b.w, u.w, w4, om1);
    }
    o.x = (msk & 1u) ? o.x : u.x;
    o.y = (msk & 2u) ? o.y : u.y;
    o.z = (msk & 4u) ? o.z : u.z;
    o.w = (msk & 8u) ? o.w : u.w;
    return o;
}

// Rows reach shared memory through a per-warp ring filled by TMA (lane 0, PF rows ahead, one
// mbarrier per u-ring slot covering the row's two boxes: u red + black, b red + black --
// 1 KB each, one 3-D tensor map over the six split buffers); the b ring is deeper because the deepest level
// still needs b of row r - 2T.  The step loop is unrolled 6 ways from a row that is a
// multiple of 6, so the 3-row window slots (row % 3) and the row parities (which
// neighbour column a cell needs, hence which single shuffle) are compile-time constants.
// (Measured alternatives: waiting once per 6-row block lets steps
// overlap but needs 36 KB of ring per warp -- 4 warps/SM -- and ran 20% slower.)
template <int T>
// (an explicit minimum of one CTA per SM lets ptxas spend registers freely -- 168 at T=4 instead
// of 134 -- while shared memory still holds three CTAs per SM: +5% at T=4, profiles/r01_sor_perf.txt)
__global__ void __launch_bounds__(kWaveWarps * 32, 1) sor_wave_kernel(const __grid_constant__ SorParams p) {
    using WV = Wave<T>;
    constexpr int HL = WV::HL, WOUT = WV::WOUT, PF = WV::PF, RDU = WV::RDU, RDB = WV::RDB;
    extern __shared__ __align__(128) float wsmem[];
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    float *ring = wsmem + warp * WV::WARP_FLOATS;
    float *ringU = ring;                                                 // [RDU][red, black][128] of u
    float *ringB = ring + 256 * RDU;                                     // [RDB][red, black][128] of b
    uint64_t *bars = reinterpret_cast<uint64_t *>(wsmem + kWaveWarps * WV::WARP_FLOATS) + warp * RDU;
    if (lane == 0) {
#pragma unroll
        for (int i = 0; i < RDU; ++i)
            asm volatile("mbarrier.init.shared::cta.b64 [%0], 1;" ::"r"(smem_addr(&bars[i])) : "memory");
        asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
    }
    __syncwarp();

    const long long gw = (blockIdx.x * static_cast<long long>(blockDim.x) + threadIdx.x) >> 5;
    const long long nw = (static_cast<long long>(gridDim.x) * blockDim.x) >> 5;
    const int n = p.n;
    const long long ldh = p.ldh;
    const unsigned nm2 = static_cast<unsigned>(n - 2);                  // row rho is interior iff rho-1 < n-2
    // row counter of this warp's rings.  The first steps of a segment read b slots of rows
    // above the segment (counter c - 2T .. c - 1; their values only feed rows that are never
    // written), so the counter starts past 2T: with RDB not a power of two a wrapped unsigned
    // counter would alias a slot the prologue is filling.  A multiple of 2 RDU keeps the
    // mbarrier phase parity (counter / RDU) & 1 at 0 for each barrier's first phase.
    uint32_t c = 2 * RDU * ((2 * T + 2 * RDU) / (2 * RDU));

    for (long long item = gw; item < p.items; item += nw) {
        const int strip = static_cast<int>(item % p.nstrips);
        const int seg = static_cast<int>(item / p.nstrips);
        const int q0 = seg * p.seg_rows;
        const int q1 = min(n, q0 + p.seg_rows);
        const int kbase = strip * WOUT - 4 * HL;                          // lane 0's first split column
        const int k0 = kbase + 4 * lane;
        const bool writer = lane >= HL && lane < 32 - HL && k0 < ldh;
        const unsigned m0 = col_mask(k0, 0, p.m, ldh), m1 = col_mask(k0, 1, p.m, ldh);
        int r0 = max(0, q0 - 2 * T);
        r0 -= r0 % 6;
        const int nsteps = ((q1 - 1 + 2 * T) - r0) / 6 * 6 + 6;           // whole 6-step blocks
        const uint32_t c0 = c;
        float *outR = p.ur_out + k0, *outB = p.ub_out + k0;

        auto issue = [&](int j) {                                        // step j = row r0 + j
            const uint32_t cc = c0 + j;
            uint64_t *bar = &bars[cc % RDU];
            bar_expect(bar, 2 * 1024);                                   // full boxes, OOB included
            tma_row_pair(ringU + (cc % RDU) * 256, &p.tmap, bar, kbase, r0 + j, p.zu);
            tma_row_pair(ringB + (cc % RDB) * 256, &p.tmap, bar, kbase, r0 + j, 4);
        };
        __syncwarp();                                                    // every lane is past the last segment
        if (lane == 0) {
            asm volatile("fence.proxy.async.shared::cta;" ::: "memory");
            for (int j = 0; j < min(PF, nsteps); ++j) issue(j);
        }

        float4 R[T + 1][3], B[T + 1][3];
#pragma unroll
        for (int t = 0; t <= T; ++t)
#pragma unroll
            for (int z = 0; z < 3; ++z) R[t][z] = B[t][z] = make_float4(0.f, 0.f, 0.f, 0.f);

        const float *ringBl = ringB + 4 * lane;                           // this lane's column of the b ring
#pragma unroll 1
        for (int jb = 0; jb < nsteps; jb += 6) {
            // b-ring slot of step jb; slots of the unrolled steps and levels are compile-time
            // offsets from it with one conditional wrap (no division by RDB per load)
            const int hb = static_cast<int>((c0 + jb) % RDB);
            auto bslot = [&](int off) -> const float * {                 // slot of counter c0 + jb + off
                int v = hb + off;
                if (off < 0) v += (hb < -off) ? RDB : 0;
                if (off > 0) v -= (hb >= RDB - off) ? RDB : 0;
                return ringBl + v * 256;
            };
#pragma unroll
            for (int u = 0; u < 6; ++u) {
                const int j = jb + u;
                const int r = r0 + j;                                     // r % 6 == u
                const uint32_t cc = c0 + j;
                // refill: the slot row j+PF reuses was last read at step j-2 (u) / j-2 (b, row
                // r+PF-RDB <= r-2T-1); all lanes are past step j-1 here
                __syncwarp();
                {
                    const uint32_t cn = cc + PF;                              // counter of row j + PF
                    refill_elected(j + PF < nsteps, smem_addr(&bars[cn % RDU]), smem_addr(ringU + (cn % RDU) * 256),
                                   smem_addr(ringB + (cn % RDB) * 256), &p.tmap, kbase, r + PF, p.zu);
                }
                bar_wait(&bars[cc % RDU], (cc / RDU) & 1);
                __syncwarp();
                R[0][u % 3] = *reinterpret_cast<const float4 *>(ringU + (cc % RDU) * 256 + 4 * lane);
                B[0][u % 3] = *reinterpret_cast<const float4 *>(ringU + (cc % RDU) * 256 + 128 + 4 * lane);
#pragma unroll
                for (int t = 1; t <= T; ++t) {
                    {   // red_t at rho = r - 2t + 1 (parity of u + 1)
                        const int sc = ((u - 2 * t + 1) % 3 + 3) % 3, sm = (sc + 2) % 3, sp = (sc + 1) % 3;
                        const float4 C = B[t - 1][sc];
                        const bool row_in = static_cast<unsigned>(r - 2 * t) < nm2;   // rho - 1 < n - 2
                        const float4 b = *reinterpret_cast<const float4 *>(
                            bslot(u - (2 * t - 1)));
                        if ((u + 1) % 2 == 0) {                             // rho even: red at even columns
                            const float left = __shfl_up_sync(0xffffffffu, C.w, 1);
                            R[t][sc] = relax4s<0>(R[t - 1][sc], B[t - 1][sm], B[t - 1][sp], C, left, 0.f, b,
                                                  row_in ? m0 : 0u, p.w4, p.om1);
                        } else {
                            const float right = __shfl_down_sync(0xffffffffu, C.x, 1);
                            R[t][sc] = relax4s<1>(R[t - 1][sc], B[t - 1][sm], B[t - 1][sp], C, 0.f, right, b,
                                                  row_in ? m1 : 0u, p.w4, p.om1);
                        }
                    }
                    {   // black_t at beta = r - 2t: black of row beta sits at column parity (beta+1)&1
                        const int sc = ((u - 2 * t) % 3 + 3) % 3, sm = (sc + 2) % 3, sp = (sc + 1) % 3;
                        const float4 C = R[t][sc];
                        const bool row_in = static_cast<unsigned>(r - 2 * t - 1) < nm2;
                        const float4 b = *reinterpret_cast<const float4 *>(
                            bslot(u - 2 * t) + 128);
                        if ((u + 1) % 2 == 0) {
                            const float left = __shfl_up_sync(0xffffffffu, C.w, 1);
                            B[t][sc] = relax4s<0>(B[t - 1][sc], R[t][sm], R[t][sp], C, left, 0.f, b,
                                                  row_in ? m0 : 0u, p.w4, p.om1);
                        } else {
                            const float right = __shfl_down_sync(0xffffffffu, C.x, 1);
                            B[t][sc] = relax4s<1>(B[t - 1][sc], R[t][sm], R[t][sp], C, 0.f, right, b,
                                                  row_in ? m1 : 0u, p.w4, p.om1);
                        }
                    }
                }
                const int rr = r - 2 * T + 1, bt = r - 2 * T;
                st4_if(outR + static_cast<long long>(rr) * ldh, R[T][((u - 2 * T + 1) % 3 + 3) % 3],
                       writer && rr >= q0 && rr < q1);
                st4_if(outB + static_cast<long long>(bt) * ldh, B[T][((u - 2 * T) % 3 + 3) % 3],
                       writer && bt >= q0 && bt < q1);
            }
        }
        c = c0 + nsteps;
    }
}

template <int T>
cudaError_t launch_wave(const SorParams &p, int grid, cudaStream_t st) {
    sor_wave_kernel<T><<<grid, kWaveWarps * 32, Wave<T>::SMEM, st>>>(p);
    return cudaGetLastError();
}

using WaveLaunch = cudaError_t (*)(const SorParams &, int, cudaStream_t);
static const WaveLaunch kWave[kMaxDepth + 1] = {nullptr,         launch_wave<1>, launch_wave<2>,
                                                launch_wave<3>,  launch_wave<4>, launch_wave<5>,
                                                launch_wave<6>,  launch_wave<7>, launch_wave<8>};
static const int kWout[kMaxDepth + 1] = {0,           Wave<1>::WOUT, Wave<2>::WOUT, Wave<3>::WOUT, Wave<4>::WOUT,
                                         Wave<5>::WOUT, Wave<6>::WOUT, Wave<7>::WOUT, Wave<8>::WOUT};

}  // namespace sor

using sepconv::cuda_fail;
using sepconv::fail;

struct sor_plan_s {
    int device = -1;
    int sms = 0;
    int64_t n = 0, m = 0, ldh = 0;
    float *buf = nullptr;            // one allocation: 6 buffers of n * ldh floats
    float *u[2][2] = {};             // [pair][colour]
    float *b[2] = {};
    int cur = 0;                     // pair holding the current iterate
    int variant = -1, depth = 0;     // tuned (variant < 0: untuned)
    int seg_div = 1;                 // wave schedule: row segments = (resident warps / strips) / seg_div (tuned)
    int forced_depth = 0;
    int wave_occ[sor::kMaxDepth + 1] = {};
    CUtensorMap tmap;                // {ldh, n, 6} over buf (the wave kernel's TMA source)
    // row bands (sor_comm_init): this plan holds rows [row0 - h_top, row1 + h_bot) of the grid
    bool band = false, band_external = false;
    void *comm = nullptr;
    int nranks = 1, rank = 0, halo = 0, h_top = 0, h_bot = 0;
    // sor_iterate's multi-launch sequences, captured once and replayed as CUDA graphs (keyed by
    // everything the launches bake in: omega, iterations, variant, depth, schedule, start pair)
    struct Graph {
        uint32_t omega_bits;
        int iters, variant, depth, seg_div, cur, cur_after;
        cudaGraphExec_t exec;
    };
    std::vector<Graph> graphs;
    cudaStream_t cap = nullptr;      // capture stream (the caller's may be the legacy default stream)
};

namespace {

constexpr int kDefaultDepth = 3;      // measured best at 16384^2 (profiles/r01_sor_perf.txt)

// SOR_GRAPHS=0 turns the graph replay of sor_iterate off (A/B checks)
bool graphs_enabled() {
    static const bool on = [] {
        const char *e = std::getenv("SOR_GRAPHS");
        return !(e && e[0] == '0');
    }();
    return on;
}

sepconv_status_t check_plan(sor_plan_t plan) {
    if (!plan) return fail(SEPCONV_E_INVALID, "sor plan is NULL");
    return SEPCONV_OK;
}

int grid_for(long long work, int threads, int sms) {
    const long long blocks = (work + threads - 1) / threads;
    return static_cast<int>(std::max<long long>(1, std::min<long long>(blocks, static_cast<long long>(sms) * 8)));
}

bool aligned16(const void *p) { return (reinterpret_cast<uintptr_t>(p) & 15u) == 0; }

sor::SorParams base_params(sor_plan_t plan, float omega) {
    sor::SorParams p;
    std::memset(&p, 0, sizeof p);
    p.br = plan->b[0];
    p.bb = plan->b[1];
    p.ldh = plan->ldh;
    p.n = static_cast<int>(plan->n);
    p.m = static_cast<int>(plan->m);
    p.w4 = omega * 0.25f;                      // exact (power-of-two scaling)
    p.om1 = 1.0f - omega;                      // rounded once in float32 (P6)
    return p;
}

sepconv_status_t half_iterations(sor_plan_t plan, float omega, int iters, cudaStream_t st) {
    if (plan->n < 3 || plan->m < 3) return SEPCONV_OK;         // no interior
    sor::SorParams p = base_params(plan, omega);
    p.ur = p.ur_out = plan->u[plan->cur][0];
    p.ub = p.ub_out = plan->u[plan->cur][1];
    const int grid = grid_for((plan->n - 2) * (plan->ldh / 4), sor::kThreads, plan->sms);
    for (int it = 0; it < iters; ++it) {
        sor::sor_half_kernel<0><<<grid, sor::kThreads, 0, st>>>(p);
        sor::sor_half_kernel<1><<<grid, sor::kThreads, 0, st>>>(p);
        cudaError_t e = cudaGetLastError();
        if (e != cudaSuccess) return cuda_fail(e, "sor_half_kernel launch");
        sepconv::g_launches.fetch_add(2, std::memory_order_relaxed);
    }
    return SEPCONV_OK;
}

sepconv_status_t wave_pass(sor_plan_t plan, float omega, int T, cudaStream_t st) {
    sor::SorParams p = base_params(plan, omega);
    const int src = plan->cur, dst = 1 - plan->cur;
    p.ur = plan->u[src][0];
    p.ub = plan->u[src][1];
    p.ur_out = plan->u[dst][0];
    p.ub_out = plan->u[dst][1];
    p.tmap = plan->tmap;
    p.zu = 2 * src;
    int &occ = plan->wave_occ[T];
    if (occ == 0) {
        static const void *funcs[sor::kMaxDepth + 1] = {
            nullptr,
            reinterpret_cast<const void *>(sor::sor_wave_kernel<1>),
            reinterpret_cast<const void *>(sor::sor_wave_kernel<2>),
            reinterpret_cast<const void *>(sor::sor_wave_kernel<3>),
            reinterpret_cast<const void *>(sor::sor_wave_kernel<4>),
            reinterpret_cast<const void *>(sor::sor_wave_kernel<5>),
            reinterpret_cast<const void *>(sor::sor_wave_kernel<6>),
            reinterpret_cast<const void *>(sor::sor_wave_kernel<7>),
            reinterpret_cast<const void *>(sor::sor_wave_kernel<8>)};
        static const size_t smem[sor::kMaxDepth + 1] = {0,
                                                        sor::Wave<1>::SMEM, sor::Wave<2>::SMEM, sor::Wave<3>::SMEM,
                                                        sor::Wave<4>::SMEM, sor::Wave<5>::SMEM, sor::Wave<6>::SMEM,
                                                        sor::Wave<7>::SMEM, sor::Wave<8>::SMEM};
        cudaError_t e = cudaFuncSetAttribute(funcs[T], cudaFuncAttributeMaxDynamicSharedMemorySize,
                                             static_cast<int>(smem[T]));
        if (e != cudaSuccess) return cuda_fail(e, "sor wave smem attribute");
        e = cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, funcs[T], sor::kWaveWarps * 32, smem[T]);
        if (e != cudaSuccess) return cuda_fail(e, "sor wave occupancy");
        occ = std::max(occ, 1);
    }
    // items = strips x row segments, about one per resident warp (/ seg_div, which sor_tune
    // sets: fewer, longer segments trade idle warps for less warm-up, and fewer warps per SM
    // each issue faster).  Each segment pays ~4T warm-up/drain steps, but idle warps cost more:
    // on the paper's 2048^2 a floor of 16T rows per segment left three quarters of the warps
    // idle (372 G vs 565 G cell-it/s at T=3, profiles/r01_sor_perf.txt), so segments only keep
    // >= 2T rows.  Segment rows are a multiple
    // of the 6-step unroll, so every segment starts on a block boundary and no steps are wasted
    // aligning its first block.
    p.nstrips = static_cast<int>((plan->ldh + sor::kWout[T] - 1) / sor::kWout[T]);
    const long long warps = static_cast<long long>(plan->sms) * occ * sor::kWaveWarps;
    long long nsegs = std::max<long long>(1, warps / p.nstrips / std::max(1, plan->seg_div));
    nsegs = std::min<long long>(nsegs, std::max<long long>(1, plan->n / (2 * T)));
    p.seg_rows = static_cast<int>(((plan->n + nsegs - 1) / nsegs + 5) / 6 * 6);
    nsegs = (plan->n + p.seg_rows - 1) / p.seg_rows;
    p.items = nsegs * p.nstrips;
    const long long blocks = (p.items + sor::kWaveWarps - 1) / sor::kWaveWarps;
    const int grid = static_cast<int>(std::min<long long>(blocks, static_cast<long long>(plan->sms) * occ));
    cudaError_t e = sor::kWave[T](p, grid, st);
    if (e != cudaSuccess) return cuda_fail(e, "sor_wave_kernel launch");
    sepconv::g_launches.fetch_add(1, std::memory_order_relaxed);
    plan->cur = dst;
    return SEPCONV_OK;
}

sepconv_status_t wave_iterations(sor_plan_t plan, float omega, int iters, int depth, cudaStream_t st) {
    if (plan->n < 3 || plan->m < 3) return SEPCONV_OK;
    while (iters > 0) {
        const int T = std::min(iters, depth);
        sepconv_status_t s = wave_pass(plan, omega, T, st);
        if (s != SEPCONV_OK) return s;
        iters -= T;
    }
    return SEPCONV_OK;
}

}  // namespace

extern "C" {

sepconv_status_t sor_plan(int64_t n, int64_t m, sor_plan_t *out) {
    if (!out) return fail(SEPCONV_E_INVALID, "plan output pointer is NULL");
    *out = nullptr;
    if (n < 1 || m < 1 || n > (1LL << 30) || m > (1LL << 30))
        return fail(SEPCONV_E_INVALID, "grid %lld x %lld: need 1 <= N, M <= 2^30", (long long)n, (long long)m);
    int dev = 0, count = 0;
    cudaError_t e = cudaGetDeviceCount(&count);
    if (e != cudaSuccess || count == 0) return fail(SEPCONV_E_UNSUPPORTED, "no CUDA device");
    SC_CUDA(cudaGetDevice(&dev));
    cudaDeviceProp prop;
    SC_CUDA(cudaGetDeviceProperties(&prop, dev));
    if (prop.major != 10) return fail(SEPCONV_E_UNSUPPORTED, "device is sm_%d%d; built for sm_100a", prop.major, prop.minor);
    sor_plan_t p = new (std::nothrow) sor_plan_s;
    if (!p) return fail(SEPCONV_E_NOMEM, "host allocation");
    p->device = dev;
    p->sms = prop.multiProcessorCount;
    p->n = n;
    p->m = m;
    p->ldh = (((m + 1) / 2) + 3) & ~3LL;
    const size_t one = static_cast<size_t>(n) * static_cast<size_t>(p->ldh);
    e = cudaMalloc(&p->buf, 6 * one * sizeof(float));
    if (e != cudaSuccess) {
        delete p;
        return cuda_fail(e, "sor_plan workspace");
    }
    p->u[0][0] = p->buf;
    p->u[0][1] = p->buf + one;
    p->u[1][0] = p->buf + 2 * one;
    p->u[1][1] = p->buf + 3 * one;
    p->b[0] = p->buf + 4 * one;
    p->b[1] = p->buf + 5 * one;
    {
        const uint64_t dims[3] = {static_cast<uint64_t>(p->ldh), static_cast<uint64_t>(n), 6};
        const uint64_t strides[2] = {static_cast<uint64_t>(p->ldh) * 4, one * 4};
        const uint32_t box[3] = {128, 1, 2};
        sepconv_status_t st = sepconv::encode_tmap_f32_3d(&p->tmap, p->buf, dims, strides, box);
        if (st != SEPCONV_OK) {
            cudaFree(p->buf);
            delete p;
            return st;
        }
    }
    e = cudaMemset(p->buf, 0, 6 * one * sizeof(float));
    if (e != cudaSuccess) {
        cudaFree(p->buf);
        delete p;
        return cuda_fail(e, "sor_plan memset");
    }
    *out = p;
    return SEPCONV_OK;
}

void sor_destroy(sor_plan_t plan) {
    if (!plan) return;
    cudaDeviceSynchronize();
    for (auto &g : plan->graphs) cudaGraphExecDestroy(g.exec);
    if (plan->cap) cudaStreamDestroy(plan->cap);
    if (plan->comm) sepconv::comm_release(plan->comm);
    cudaFree(plan->buf);
    delete plan;
}

static bool overlaps(const void *a, size_t abytes, const void *b, size_t bbytes) {
    const uintptr_t x = reinterpret_cast<uintptr_t>(a), y = reinterpret_cast<uintptr_t>(b);
    return x < y + bbytes && y < x + abytes;
}

sepconv_status_t sor_load(sor_plan_t plan, const float *x, int64_t ld_x, const float *b, int64_t ld_b,
                          sepconv_stream_t stream) {
    if (sepconv_status_t s = check_plan(plan)) return s;
    if (!x || !b) return fail(SEPCONV_E_INVALID, "x or b is NULL");
    ld_x = ld_x ? ld_x : plan->m;
    ld_b = ld_b ? ld_b : plan->m;
    if (ld_x < plan->m || ld_b < plan->m) return fail(SEPCONV_E_INVALID, "row pitch smaller than M");
    if ((reinterpret_cast<uintptr_t>(x) | reinterpret_cast<uintptr_t>(b)) & 3u)
        return fail(SEPCONV_E_ALIGN, "x and b must be 4-byte aligned");
    const size_t ws = 6 * static_cast<size_t>(plan->n * plan->ldh) * sizeof(float);
    if (overlaps(x, static_cast<size_t>(plan->n * ld_x) * 4, plan->buf, ws) ||
        overlaps(b, static_cast<size_t>(plan->n * ld_b) * 4, plan->buf, ws))
        return fail(SEPCONV_E_ALIAS, "x or b overlaps the plan's workspace");
    cudaStream_t st = static_cast<cudaStream_t>(stream);
    const int grid = grid_for(plan->n * (plan->ldh / 4), sor::kThreads, plan->sms);
    plan->cur = 0;
    sor::rb_split_kernel<<<grid, sor::kThreads, 0, st>>>(x, ld_x, (int)plan->n, (int)plan->m, plan->u[0][0],
                                                         plan->u[0][1], plan->ldh);
    sor::rb_split_kernel<<<grid, sor::kThreads, 0, st>>>(b, ld_b, (int)plan->n, (int)plan->m, plan->b[0], plan->b[1],
                                                         plan->ldh);
    cudaError_t e = cudaGetLastError();
    if (e != cudaSuccess) return cuda_fail(e, "rb_split_kernel launch");
    sepconv::g_launches.fetch_add(2, std::memory_order_relaxed);
    return SEPCONV_OK;
}

sepconv_status_t sor_iterate(sor_plan_t plan, float omega, int iters, sor_variant_t variant,
                             sepconv_stream_t stream) {
    if (sepconv_status_t s = check_plan(plan)) return s;
    if (!(omega > 0.f && omega < 2.f)) return fail(SEPCONV_E_INVALID, "omega %g outside (0, 2)", (double)omega);
    if (iters < 0) return fail(SEPCONV_E_INVALID, "iters %d < 0", iters);
    if (variant < SOR_HALF || variant > SOR_AUTO) return fail(SEPCONV_E_INVALID, "unknown variant %d", (int)variant);
    cudaStream_t st = static_cast<cudaStream_t>(stream);
    int v = variant, depth = plan->forced_depth;
    if (v == SOR_AUTO) v = plan->variant >= 0 ? plan->variant : SOR_WAVE;
    if (depth == 0) depth = plan->depth > 0 ? plan->depth : kDefaultDepth;
    auto direct = [&](cudaStream_t s) {
        return v == SOR_HALF ? half_iterations(plan, omega, iters, s) : wave_iterations(plan, omega, iters, depth, s);
    };
    const long long launches = (plan->n < 3 || plan->m < 3) ? 0
                               : v == SOR_HALF ? 2LL * iters : (iters + depth - 1) / depth;
    if (launches < 2 || !graphs_enabled()) return direct(st);
    cudaStreamCaptureStatus cs = cudaStreamCaptureStatusNone;
    if (cudaStreamIsCapturing(st, &cs) != cudaSuccess || cs != cudaStreamCaptureStatusNone) {
        cudaGetLastError();
        return direct(st);                                     // the caller is capturing: no nesting
    }
    // a multi-launch call replays a CUDA graph of its launch sequence: measured -2.3% per 24
    // iterations of the tuned wavefront on 2048^2 and -1.2 us per launch for half-sweeps
    // (tools/graph_probe.py, profiles/r02_graph_probe.txt); the first call of a key runs directly
    // and records the graph for the next one
    uint32_t ob;
    std::memcpy(&ob, &omega, 4);
    for (const auto &g : plan->graphs) {
        if (g.omega_bits == ob && g.iters == iters && g.variant == v && g.depth == depth && g.seg_div == plan->seg_div &&
            g.cur == plan->cur) {
            cudaError_t e = cudaGraphLaunch(g.exec, st);
            if (e != cudaSuccess) return cuda_fail(e, "sor graph launch");
            plan->cur = g.cur_after;
            sepconv::g_launches.fetch_add(static_cast<uint64_t>(launches), std::memory_order_relaxed);
            return SEPCONV_OK;
        }
    }
    const int cur0 = plan->cur;
    if (sepconv_status_t s = direct(st)) return s;
    const int cur1 = plan->cur;
    // record (nothing executes during capture); the launch counter counts executed launches only
    if (!plan->cap && cudaStreamCreateWithFlags(&plan->cap, cudaStreamNonBlocking) != cudaSuccess) {
        plan->cap = nullptr;
        cudaGetLastError();
        return SEPCONV_OK;
    }
    const uint64_t counted = sepconv::g_launches.load(std::memory_order_relaxed);
    plan->cur = cur0;
    cudaGraph_t graph = nullptr;
    cudaGraphExec_t exec = nullptr;
    bool ok = cudaStreamBeginCapture(plan->cap, cudaStreamCaptureModeThreadLocal) == cudaSuccess;
    if (ok) {
        const sepconv_status_t rs = direct(plan->cap);
        ok = cudaStreamEndCapture(plan->cap, &graph) == cudaSuccess && rs == SEPCONV_OK && plan->cur == cur1;
    }
    if (ok) ok = cudaGraphInstantiate(&exec, graph, 0) == cudaSuccess;
    if (graph) cudaGraphDestroy(graph);
    cudaGetLastError();                                        // a failed capture leaves the direct path
    sepconv::g_launches.store(counted, std::memory_order_relaxed);
    plan->cur = cur1;
    if (ok) {
        if (plan->graphs.size() >= 8) {
            cudaGraphExecDestroy(plan->graphs.front().exec);
            plan->graphs.erase(plan->graphs.begin());
        }
        plan->graphs.push_back({ob, iters, v, depth, plan->seg_div, cur0, cur1, exec});
    }
    return SEPCONV_OK;
}

sepconv_status_t sor_store(sor_plan_t plan, float *u, int64_t ld_u, sepconv_stream_t stream) {
    if (sepconv_status_t s = check_plan(plan)) return s;
    if (!u) return fail(SEPCONV_E_INVALID, "u is NULL");
    ld_u = ld_u ? ld_u : plan->m;
    if (ld_u < plan->m) return fail(SEPCONV_E_INVALID, "row pitch smaller than M");
    if (reinterpret_cast<uintptr_t>(u) & 3u) return fail(SEPCONV_E_ALIGN, "u must be 4-byte aligned");
    const size_t ws = 6 * static_cast<size_t>(plan->n * plan->ldh) * sizeof(float);
    if (overlaps(u, static_cast<size_t>(plan->n * ld_u) * 4, plan->buf, ws))
        return fail(SEPCONV_E_ALIAS, "u overlaps the plan's workspace");
    cudaStream_t st = static_cast<cudaStream_t>(stream);
    const int grid = grid_for(plan->n * (plan->ldh / 4), sor::kThreads, plan->sms);
    sor::rb_merge_kernel<<<grid, sor::kThreads, 0, st>>>(plan->u[plan->cur][0], plan->u[plan->cur][1], plan->ldh,
                                                         (int)plan->n, (int)plan->m, u, ld_u);
    cudaError_t e = cudaGetLastError();
    if (e != cudaSuccess) return cuda_fail(e, "rb_merge_kernel launch");
    sepconv::g_launches.fetch_add(1, std::memory_order_relaxed);
    return SEPCONV_OK;
}

sepconv_status_t sor_solve(sor_plan_t plan, const float *x, const float *b, float *u, float omega, int iters,
                           sor_variant_t variant, sepconv_stream_t stream) {
    if (sepconv_status_t s = sor_load(plan, x, 0, b, 0, stream)) return s;
    if (sepconv_status_t s = sor_iterate(plan, omega, iters, variant, stream)) return s;
    return sor_store(plan, u, 0, stream);
}

sepconv_status_t sor_solve_host(sor_plan_t plan, const float *x, const float *b, float *u, float omega, int iters,
                                sor_variant_t variant, sepconv_stream_t stream) {
    if (sepconv_status_t s = check_plan(plan)) return s;
    if (!x || !b || !u) return fail(SEPCONV_E_INVALID, "x, b or u is NULL");
    cudaStream_t st = static_cast<cudaStream_t>(stream);
    const size_t bytes = static_cast<size_t>(plan->n * plan->m) * sizeof(float);
    // staging: the second iterate pair (2 * N * ldh >= N * M floats, contiguous) is free
    // before the first iteration -- x goes there and is split into pair 0, then b goes
    // there and is split into the b buffers (stream order serialises the reuse)
    float *stage = plan->u[1][0];
    if (static_cast<size_t>(2 * plan->n * plan->ldh) * sizeof(float) < bytes)
        return fail(SEPCONV_E_INVALID, "internal: staging too small");
    const int grid = grid_for(plan->n * (plan->ldh / 4), sor::kThreads, plan->sms);
    plan->cur = 0;
    SC_CUDA(cudaMemcpyAsync(stage, x, bytes, cudaMemcpyHostToDevice, st));
    sor::rb_split_kernel<<<grid, sor::kThreads, 0, st>>>(stage, plan->m, (int)plan->n, (int)plan->m, plan->u[0][0],
                                                         plan->u[0][1], plan->ldh);
    SC_CUDA(cudaGetLastError());
    SC_CUDA(cudaMemcpyAsync(stage, b, bytes, cudaMemcpyHostToDevice, st));
    sor::rb_split_kernel<<<grid, sor::kThreads, 0, st>>>(stage, plan->m, (int)plan->n, (int)plan->m, plan->b[0],
                                                         plan->b[1], plan->ldh);
    SC_CUDA(cudaGetLastError());
    sepconv::g_launches.fetch_add(2, std::memory_order_relaxed);
    if (sepconv_status_t s = sor_iterate(plan, omega, iters, variant, stream)) return s;
    // merge into whichever pair is not current, then copy out
    float *du = plan->u[1 - plan->cur][0];
    sor::rb_merge_kernel<<<grid, sor::kThreads, 0, st>>>(plan->u[plan->cur][0], plan->u[plan->cur][1], plan->ldh,
                                                         (int)plan->n, (int)plan->m, du, plan->m);
    SC_CUDA(cudaGetLastError());
    sepconv::g_launches.fetch_add(1, std::memory_order_relaxed);
    SC_CUDA(cudaMemcpyAsync(u, du, bytes, cudaMemcpyDeviceToHost, st));
    SC_CUDA(cudaStreamSynchronize(st));
    return SEPCONV_OK;
}

sepconv_status_t sor_buffers(sor_plan_t plan, float **u_red, float **u_black, float **b_red, float **b_black,
                             int64_t *ldh) {
    if (sepconv_status_t s = check_plan(plan)) return s;
    if (u_red) *u_red = plan->u[plan->cur][0];
    if (u_black) *u_black = plan->u[plan->cur][1];
    if (b_red) *b_red = plan->b[0];
    if (b_black) *b_black = plan->b[1];
    if (ldh) *ldh = plan->ldh;
    return SEPCONV_OK;
}

sepconv_status_t sor_set_depth(sor_plan_t plan, int depth) {
    if (sepconv_status_t s = check_plan(plan)) return s;
    if (depth < 0 || depth > sor::kMaxDepth) return fail(SEPCONV_E_INVALID, "depth %d outside 0..%d", depth, sor::kMaxDepth);
    plan->forced_depth = depth;
    return SEPCONV_OK;
}

// ---- row bands across GPUs -------------------------------------------------------------
// Owned rows of band g: [r_g, r_{g+1}) with r_g = 2 floor(g N / 2G) (even, so every band's
// first local row has an even global index and the red/black colouring of P3 is the same in
// local and global coordinates); r_G = N.  A band plan holds its owned rows plus `halo` ghost
// rows on each side that has a neighbour.  A pass of depth T leaves the owned rows exact when
// halo >= 2T: the ghost rows are treated as fixed, and the error that introduces moves one
// row inward per half-sweep.
sepconv_status_t sor_band(int64_t n, int nbands, int g, int halo, int64_t *row0, int64_t *rows, int64_t *alloc_row0,
                          int64_t *alloc_rows) {
    if (n < 1 || nbands < 1 || g < 0 || g >= nbands) return fail(SEPCONV_E_INVALID, "band %d of %d", g, nbands);
    if (halo < 0 || (halo & 1)) return fail(SEPCONV_E_INVALID, "halo %d must be even and >= 0", halo);
    const int64_t r0 = 2 * ((static_cast<int64_t>(g) * n) / (2LL * nbands));
    const int64_t r1 = g + 1 == nbands ? n : 2 * ((static_cast<int64_t>(g + 1) * n) / (2LL * nbands));
    if (nbands > 1 && (r1 - r0) < std::max(halo, 1))
        return fail(SEPCONV_E_INVALID, "band %d has %lld rows, fewer than the %d-row halo", g, (long long)(r1 - r0), halo);
    const int64_t a0 = g > 0 ? r0 - halo : r0;
    const int64_t a1 = g + 1 < nbands ? r1 + halo : r1;
    if (a0 < 0 || a1 > n) return fail(SEPCONV_E_INVALID, "halo %d larger than the neighbouring band", halo);
    if (row0) *row0 = r0;
    if (rows) *rows = r1 - r0;
    if (alloc_row0) *alloc_row0 = a0;
    if (alloc_rows) *alloc_rows = a1 - a0;
    return SEPCONV_OK;
}

sepconv_status_t sor_comm_init(sor_plan_t plan, const unsigned char *id, int nranks, int rank, int halo) {
    if (sepconv_status_t s = check_plan(plan)) return s;
    if (nranks < 1 || rank < 0 || rank >= nranks) return fail(SEPCONV_E_INVALID, "rank %d of %d", rank, nranks);
    if (halo < 2 || (halo & 1)) return fail(SEPCONV_E_INVALID, "halo %d must be even and >= 2", halo);
    const int h_top = rank > 0 ? halo : 0, h_bot = rank + 1 < nranks ? halo : 0;
    if (plan->n - h_top - h_bot < halo && nranks > 1)
        return fail(SEPCONV_E_INVALID, "band of %lld rows cannot hold %d owned rows plus its ghost rows",
                    (long long)plan->n, halo);
    if (plan->comm) {
        sepconv::comm_release(plan->comm);
        plan->comm = nullptr;
    }
    plan->band = true;
    plan->band_external = id == nullptr;
    plan->nranks = nranks;
    plan->rank = rank;
    plan->halo = halo;
    plan->h_top = h_top;
    plan->h_bot = h_bot;
    if (id && nranks > 1) return sepconv::comm_acquire(id, nranks, rank, plan->device, &plan->comm);
    return SEPCONV_OK;
}

// refresh the ghost rows of the current iterate from the neighbours' owned rows (both colours)
static sepconv_status_t band_exchange(sor_plan_t plan, cudaStream_t st) {
    if (plan->band_external || plan->nranks == 1 || !plan->comm) return SEPCONV_OK;
    sepconv::NcclApi &a = sepconv::nccl();
    const size_t cnt = static_cast<size_t>(plan->halo) * plan->ldh;
    const int64_t n = plan->n, ldh = plan->ldh;
    sepconv::nccl_comm_t comm = plan->comm;
    sepconv::nccl_result_t r = a.GroupStart();
    for (int c = 0; c < 2 && r == 0; ++c) {
        float *buf = plan->u[plan->cur][c];
        if (plan->rank > 0) {               // first owned rows up, top ghost rows from above
            if (r == 0) r = a.Send(buf + plan->h_top * ldh, cnt, sepconv::kNcclFloat32, plan->rank - 1, comm, st);
            if (r == 0) r = a.Recv(buf, cnt, sepconv::kNcclFloat32, plan->rank - 1, comm, st);
        }
        if (plan->rank + 1 < plan->nranks) {  // last owned rows down, bottom ghost rows from below
            if (r == 0) r = a.Send(buf + (n - plan->h_bot - plan->halo) * ldh, cnt, sepconv::kNcclFloat32, plan->rank + 1,
                                   comm, st);
            if (r == 0) r = a.Recv(buf + (n - plan->halo) * ldh, cnt, sepconv::kNcclFloat32, plan->rank + 1, comm, st);
        }
    }
    sepconv::nccl_result_t r2 = a.GroupEnd();
    if (r != 0) return sepconv::nccl_fail(r, "ncclSend/ncclRecv (SOR ghost rows)");
    if (r2 != 0) return sepconv::nccl_fail(r2, "ncclGroupEnd");
    return SEPCONV_OK;
}

sepconv_status_t sor_band_iterate(sor_plan_t plan, float omega, int iters, sor_variant_t variant,
                                  sepconv_stream_t stream) {
    if (sepconv_status_t s = check_plan(plan)) return s;
    if (!plan->band) return fail(SEPCONV_E_INVALID, "sor_comm_init has not been called on this plan");
    if (!(omega > 0.f && omega < 2.f)) return fail(SEPCONV_E_INVALID, "omega %g outside (0, 2)", (double)omega);
    if (iters < 0) return fail(SEPCONV_E_INVALID, "iters %d < 0", iters);
    if (variant < SOR_HALF || variant > SOR_AUTO) return fail(SEPCONV_E_INVALID, "unknown variant %d", (int)variant);
    cudaStream_t st = static_cast<cudaStream_t>(stream);
    int v = variant, depth = plan->forced_depth;
    if (v == SOR_AUTO) v = plan->variant >= 0 ? plan->variant : SOR_WAVE;
    if (depth == 0) depth = plan->depth > 0 ? plan->depth : kDefaultDepth;
    depth = std::max(1, std::min(depth, plan->halo / 2));           // owned rows exact after each pass
    while (iters > 0) {
        const int T = v == SOR_HALF ? 1 : std::min(iters, depth);
        sepconv_status_t s = v == SOR_HALF ? half_iterations(plan, omega, 1, st) : wave_iterations(plan, omega, T, T, st);
        if (s != SEPCONV_OK) return s;
        s = band_exchange(plan, st);
        if (s != SEPCONV_OK) return s;
        iters -= T;
    }
    return SEPCONV_OK;
}

sepconv_status_t sor_tune(sor_plan_t plan, int iters_hint, int reps, int *variant_out, int *depth_out) {
    if (sepconv_status_t s = check_plan(plan)) return s;
    if (iters_hint < 1) iters_hint = 24;
    if (reps < 1) reps = 5;
    // time on the plan's own buffers (their contents are replaced by the caller's next load)
    cudaStream_t st = nullptr;
    cudaEvent_t e0, e1;
    SC_CUDA(cudaEventCreate(&e0));
    SC_CUDA(cudaEventCreate(&e1));
    const int depths[] = {0, 1, 2, 3, 4, 5, 6, 8};       // 0 = SOR_HALF
    const int divs[] = {1, 2, 3};                         // wave segments per resident warp: 1, 1/2, 1/3
    float best = 1e30f;
    int best_v = SOR_WAVE, best_d = kDefaultDepth, best_div = 1;
    const float omega = 1.5f;
    sepconv_status_t status = SEPCONV_OK;
    for (int cand = 0; cand < 8 * 3 && status == SEPCONV_OK; ++cand) {
        const int d = depths[cand / 3], div = divs[cand % 3];
        if (d == 0 && div != 1) continue;
        plan->seg_div = div;
        float times[64];
        const int R = std::min(reps, 64);
        for (int r = -1; r < R && status == SEPCONV_OK; ++r) {
            cudaEventRecord(e0, st);
            status = d == 0 ? half_iterations(plan, omega, iters_hint, st)
                            : wave_iterations(plan, omega, iters_hint, d, st);
            cudaEventRecord(e1, st);
            if (cudaEventSynchronize(e1) != cudaSuccess) status = cuda_fail(cudaGetLastError(), "sor_tune");
            float ms = 0.f;
            cudaEventElapsedTime(&ms, e0, e1);
            if (r >= 0) times[r] = ms;
        }
        if (status != SEPCONV_OK) break;
        std::sort(times, times + R);
        const float med = times[R / 2];
        if (const char *log = std::getenv("SEPCONV_TUNE_LOG"))    // diagnostics: every candidate's time
            if (FILE *f = std::fopen(log, "a")) {
                std::fprintf(f, "sor %lldx%lld depth %d seg_div %d: %.4f ms\n", (long long)plan->n, (long long)plan->m,
                             d, div, med);
                std::fclose(f);
            }
        if (med < best * 0.99f) {
            best = med;
            best_v = d == 0 ? SOR_HALF : SOR_WAVE;
            best_d = d == 0 ? kDefaultDepth : d;
            best_div = div;
        }
    }
    cudaEventDestroy(e0);
    cudaEventDestroy(e1);
    plan->seg_div = best_div;
    if (status != SEPCONV_OK) return status;
    plan->variant = best_v;
    plan->depth = best_d;
    if (variant_out) *variant_out = best_v;
    if (depth_out) *depth_out = best_d;
    return SEPCONV_OK;
}

}  // extern "C"
