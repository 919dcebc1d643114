// sepconv_kernels.cuh -- sm_100a kernels for SeparableConvolution (Fig. 1,
// P:354-408).  Included only by the per-op kernel translation units.
//
// Kernel family:
//   stream_kernel<K, OP, MAP>  column-strip streaming kernels.  Each warp owns a
//       strip of 32*V output columns (V = 4 per thread) and walks down the rows
//       of its CTA's row range.  OP selects what a warp does with each input row:
//         OP_ROWS  ConvolveRows: buf[r][c] = sum_i k_i In[r][c+i]
//         OP_COLS  ConvolveColumns over buf rows held in a K-slot
//                  register ring: out[q][c] = sum_j k_j buf[q+j][c]
//         OP_SEP   both, fused: the row pass result goes straight into the ring
//                  (the paper's `buffer`, never touches HBM)
//       MAP_TMA stages SR-row x (32V + K-1)-column boxes of In (halo included)
//       into a per-warp shared-memory ring by cp.async.bulk.tensor + mbarrier;
//       MAP_DIRECT(_VEC) reads each thread's window straight from global memory
//       through L1 (4- or 16-byte loads).
//   conv2d_kernel<K, MAP>  Convolve2D: each output row is the sum over
//       j of K-tap dot products of input row q+j with weight row w_j = fl(k_j k_i).
//
// Arithmetic order (R6, fixed for every mapping, tile and GPU count):
//   ROWS/SEP:  b = k_0*x_0; b = fma(k_i, x_i, b) for i = 1..K-1
//   COLS/SEP:  a = k_0*b_q; a = fma(k_j, b_{q+j}, a) for j = 1..K-1
//   2D:        p_j = w_j0*x_0; p_j = fma(w_ji, x_i, p_j); a = p_0; a = a + p_j
// so fused and unfused separable are bitwise identical.
#pragma once
#include <cuda.h>
#include <cuda_runtime.h>
#include <stdint.h>

#include <type_traits>

#include "sepconv_params.h"

// cache operator of the output stores ("" = default write-back)
#ifndef SEPCONV_ST_HINT
#define SEPCONV_ST_HINT ""
#endif

namespace sepconv {

// ---- PTX helpers ----------------------------------------------------------------
__device__ __forceinline__ uint32_t smem_u32(const void *p) {
    return static_cast<uint32_t>(__cvta_generic_to_shared(p));
}

__device__ __forceinline__ void mbar_init(uint64_t *bar, uint32_t count) {
    asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(smem_u32(bar)), "r"(count) : "memory");
}

__device__ __forceinline__ void fence_barrier_init() {
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
    asm volatile("fence.proxy.async.shared::cta;" ::: "memory");
}

__device__ __forceinline__ void mbar_arrive_expect_tx(uint64_t *bar, uint32_t bytes) {
    asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(smem_u32(bar)), "r"(bytes)
                 : "memory");
}

__device__ __forceinline__ void mbar_wait(uint64_t *bar, uint32_t parity) {
    const uint32_t addr = smem_u32(bar);
    uint32_t done, spins = 0;
    do {
        // a lost transaction would otherwise hang the GPU: fail loudly instead
        if (++spins == (1u << 26)) __trap();
        asm volatile(
            "{\n\t.reg .pred p;\n\t"
            "mbarrier.try_wait.parity.shared::cta.b64 p, [%1], %2;\n\t"
            "selp.u32 %0, 1, 0, p;\n\t}"
            : "=r"(done)
            : "r"(addr), "r"(parity)
            : "memory");
    } while (!done);
}

// Orders this warp's earlier generic-proxy shared-memory reads before a following
// TMA (async-proxy) write into the same stage.
__device__ __forceinline__ void fence_proxy_async_smem() {
    asm volatile("fence.proxy.async.shared::cta;" ::: "memory");
}

__device__ __forceinline__ void tma_load_3d(void *dst, const CUtensorMap *map, uint64_t *bar, int c0, int c1,
                                            int c2) {
    asm volatile(
        "cp.async.bulk.tensor.3d.shared::cluster.global.tile.mbarrier::complete_tx::bytes "
        "[%0], [%1, {%3, %4, %5}], [%2];" ::"r"(smem_u32(dst)),
        "l"(reinterpret_cast<uint64_t>(map)), "r"(smem_u32(bar)), "r"(c0), "r"(c1), "r"(c2)
        : "memory");
}

// Stage refill issued by the converged warp: one elected lane runs the proxy fence, the
// expect_tx and the box load under a predicate (no lane-0 branch; see sor.cu refill_elected).
__device__ __forceinline__ void tma_refill_elected(bool go, void *dst, const CUtensorMap *map, uint64_t *bar,
                                                   uint32_t bytes, int c0, int c1, int c2) {
    asm volatile(
        "{\n\t.reg .pred e, g, q;\n\t"
        "elect.sync _|e, 0xffffffff;\n\t"
        "setp.ne.u32 g, %6, 0;\n\t"
        "and.pred q, e, g;\n\t"
        "@q fence.proxy.async.shared::cta;\n\t"
        "@q mbarrier.arrive.expect_tx.shared::cta.b64 _, [%2], %7;\n\t"
        "@q cp.async.bulk.tensor.3d.shared::cluster.global.tile.mbarrier::complete_tx::bytes "
        "[%0], [%1, {%3, %4, %5}], [%2];\n\t}" ::"r"(smem_u32(dst)),
        "l"(reinterpret_cast<uint64_t>(map)), "r"(smem_u32(bar)), "r"(c0), "r"(c1), "r"(c2),
        "r"(static_cast<uint32_t>(go)), "r"(bytes)
        : "memory");
}

__device__ __forceinline__ void prefetch_tmap(const CUtensorMap *map) {
    asm volatile("prefetch.tensormap [%0];" ::"l"(reinterpret_cast<uint64_t>(map)) : "memory");
}

// Packed FP32 (FFMA2 / FMUL2 on sm_100): two independent IEEE RN operations per
// instruction -- bitwise the same as two fmaf / two multiplies.
__device__ __forceinline__ float2 ffma2(float2 a, float2 b, float2 c) {
    unsigned long long ra = *reinterpret_cast<unsigned long long *>(&a);
    unsigned long long rb = *reinterpret_cast<unsigned long long *>(&b);
    unsigned long long rc = *reinterpret_cast<unsigned long long *>(&c), rd;
    asm("fma.rn.f32x2 %0, %1, %2, %3;" : "=l"(rd) : "l"(ra), "l"(rb), "l"(rc));
    return *reinterpret_cast<float2 *>(&rd);
}
__device__ __forceinline__ float2 fmul2(float2 a, float2 b) {
    unsigned long long ra = *reinterpret_cast<unsigned long long *>(&a);
    unsigned long long rb = *reinterpret_cast<unsigned long long *>(&b), rd;
    asm("mul.rn.f32x2 %0, %1, %2;" : "=l"(rd) : "l"(ra), "l"(rb));
    return *reinterpret_cast<float2 *>(&rd);
}

__device__ __forceinline__ float4 ld_shared4(const float *p) {
    return *reinterpret_cast<const float4 *>(p);
}

// Output cursor: this thread's 4-column slot of one output row, advanced one row
// per step.  Stores are branch-free -- every case is a predicated st.global --
// because a branch inside the unrolled step body makes ptxas move the weights from
// uniform registers into vector registers, and FFMA R,R,R,R issues ~30% slower than
// FFMA R,R,UR,R on B200 (profiles/r01_ubench_ffma.txt).  16-byte stores when the
// row address is 16-byte aligned (c is a multiple of 4, so the alignment is
// warp-uniform), 2 x 8-byte when it is 8-byte aligned, 4 x 4-byte otherwise and at
// the ragged right edge (per-element guards computed once per segment).
struct OutCursor {
    float *ptr;              // &out[row][c] of the row the next store() writes
    long long ld;            // row pitch (floats)
    bool full;               // all 4 columns of this thread are inside the image
    bool e1, e2, e3, e0;     // column c+e is inside the image
    bool last4;              // this thread's 4 columns end the row exactly
    __device__ __forceinline__ void init(float *rowp, long long ld_, int c, int out_cols) {
        ptr = rowp + c;
        ld = ld_;
        full = c + V <= out_cols;
        last4 = c + V == out_cols;
        e0 = c < out_cols;
        e1 = c + 1 < out_cols;
        e2 = c + 2 < out_cols;
        e3 = c + 3 < out_cols;
    }
    // Fast path: every row start is 8-byte aligned (checked by the host).  A 16-byte aligned row
    // is one STG.128 per lane.  An 8-byte aligned row is re-cut into 16-byte aligned chunks with
    // two shuffles -- lane l stores (lane l-1's v2, v3, its own v0, v1) -- plus one 8-byte store
    // at each end of the warp's span, so every sector is written once and whole instead of twice
    // in halves.  EDGE: the warp may be a right-edge warp of an even output width (each lane has
    // 4, 2 or 0 columns inside): a lane with 2 stores 8 bytes, the last lane with 4 closes the
    // span; the extra predicates cost a few instructions per row, so only the widths whose hot
    // loop is large enough for a second copy of it to hurt (K >= 13) compile them
    template <bool EDGE>
    __device__ __forceinline__ void store_fast(const float (&v)[V], bool ok, int lane) {
        const unsigned a8 = static_cast<unsigned>(reinterpret_cast<uintptr_t>(ptr)) & 8u;
        const float u2 = __shfl_up_sync(0xffffffffu, v[2], 1);
        const float u3 = __shfl_up_sync(0xffffffffu, v[3], 1);
        if constexpr (EDGE) {
            const bool in2 = e1;                               // columns c, c+1 inside
            const unsigned p16 = ok && a8 == 0 && full;
            const unsigned ph = ok && a8 == 0 && !full && in2;
            const unsigned pm = ok && a8 != 0 && lane != 0 && in2;
            const unsigned p0 = ok && a8 != 0 && lane == 0 && in2;
            const unsigned p31 = ok && a8 != 0 && full && (lane == 31 || last4);
            asm volatile(
                "{\n\t.reg .pred q16, qh, qm, q0, q31;\n\t"
                "setp.ne.u32 q16, %7, 0;\n\t"
                "setp.ne.u32 qm, %8, 0;\n\t"
                "setp.ne.u32 q0, %9, 0;\n\t"
                "setp.ne.u32 q31, %10, 0;\n\t"
                "setp.ne.u32 qh, %11, 0;\n\t"
                "@q16 st.global" SEPCONV_ST_HINT ".v4.f32 [%0], {%1, %2, %3, %4};\n\t"
                "@qh st.global" SEPCONV_ST_HINT ".v2.f32 [%0], {%1, %2};\n\t"
                "@qm st.global" SEPCONV_ST_HINT ".v4.f32 [%0+-8], {%5, %6, %1, %2};\n\t"
                "@q0 st.global" SEPCONV_ST_HINT ".v2.f32 [%0], {%1, %2};\n\t"
                "@q31 st.global" SEPCONV_ST_HINT ".v2.f32 [%0+8], {%3, %4};\n\t}"
                ::"l"(ptr), "f"(v[0]), "f"(v[1]), "f"(v[2]), "f"(v[3]), "f"(u2), "f"(u3), "r"(p16), "r"(pm), "r"(p0),
                "r"(p31), "r"(ph)
                : "memory");
        } else {
            const unsigned p16 = ok && a8 == 0;
            const unsigned pm = ok && a8 != 0 && lane != 0;
            const unsigned p0 = ok && a8 != 0 && lane == 0;
            const unsigned p31 = ok && a8 != 0 && lane == 31;
            asm volatile(
                "{\n\t.reg .pred q16, qm, q0, q31;\n\t"
                "setp.ne.u32 q16, %7, 0;\n\t"
                "setp.ne.u32 qm, %8, 0;\n\t"
                "setp.ne.u32 q0, %9, 0;\n\t"
                "setp.ne.u32 q31, %10, 0;\n\t"
                "@q16 st.global" SEPCONV_ST_HINT ".v4.f32 [%0], {%1, %2, %3, %4};\n\t"
                "@qm st.global" SEPCONV_ST_HINT ".v4.f32 [%0+-8], {%5, %6, %1, %2};\n\t"
                "@q0 st.global" SEPCONV_ST_HINT ".v2.f32 [%0], {%1, %2};\n\t"
                "@q31 st.global" SEPCONV_ST_HINT ".v2.f32 [%0+8], {%3, %4};\n\t}"
                ::"l"(ptr), "f"(v[0]), "f"(v[1]), "f"(v[2]), "f"(v[3]), "f"(u2), "f"(u3), "r"(p16), "r"(pm), "r"(p0),
                "r"(p31)
                : "memory");
        }
        ptr += ld;
    }
    // Fastest path: every row start is 16-byte aligned (out base, ld_out and image
    // stride multiples of 4 floats): one predicated STG.128, nothing else.  `full` also
    // admits the right-edge warp when the output width is a multiple of 4 (each lane's four
    // columns are then all inside or all outside), so every warp of the pass runs this one
    // loop body (see the dispatch in stream_kernel).
    __device__ __forceinline__ void store_fast16(const float (&v)[V], bool ok) {
        const unsigned p16 = ok && full;
        asm volatile(
            "{\n\t.reg .pred q16;\n\t"
            "setp.ne.u32 q16, %5, 0;\n\t"
            "@q16 st.global" SEPCONV_ST_HINT ".v4.f32 [%0], {%1, %2, %3, %4};\n\t}"
            ::"l"(ptr), "f"(v[0]), "f"(v[1]), "f"(v[2]), "f"(v[3]), "r"(p16)
            : "memory");
        ptr += ld;
    }
    // Ragged right edge / 4-byte aligned rows of the streaming kernels: per-element
    // predicated 4-byte stores only (cheap in registers: this body is compiled next to the
    // hot one and the kernel's register budget is the larger of the two).
    __device__ __forceinline__ void store_scalar(const float (&v)[V], bool ok) {
        const unsigned q0 = ok && e0, q1 = ok && e1, q2 = ok && e2, q3 = ok && e3;
        asm volatile(
            "{\n\t.reg .pred q0, q1, q2, q3;\n\t"
            "setp.ne.u32 q0, %5, 0;\n\t"
            "setp.ne.u32 q1, %6, 0;\n\t"
            "setp.ne.u32 q2, %7, 0;\n\t"
            "setp.ne.u32 q3, %8, 0;\n\t"
            "@q0 st.global.f32 [%0], %1;\n\t"
            "@q1 st.global.f32 [%0+4], %2;\n\t"
            "@q2 st.global.f32 [%0+8], %3;\n\t"
            "@q3 st.global.f32 [%0+12], %4;\n\t}"
            ::"l"(ptr), "f"(v[0]), "f"(v[1]), "f"(v[2]), "f"(v[3]), "r"(q0), "r"(q1), "r"(q2), "r"(q3)
            : "memory");
        ptr += ld;
    }
    // 8-byte rows without shuffles: two predicated 8-byte stores per lane (each 32-byte sector
    // is written in two halves by the two instructions); fewer live registers than store_fast
    // (EDGE: a right-edge warp of an even output width; each lane stores the pairs that are inside)
    template <bool EDGE>
    __device__ __forceinline__ void store_v2x2(const float (&v)[V], bool ok) {
        const unsigned qa = ok && (!EDGE || e1), qb = ok && (!EDGE || full);
        asm volatile(
            "{\n\t.reg .pred qa, qb;\n\t"
            "setp.ne.u32 qa, %5, 0;\n\t"
            "setp.ne.u32 qb, %6, 0;\n\t"
            "@qa st.global" SEPCONV_ST_HINT ".v2.f32 [%0], {%1, %2};\n\t"
            "@qb st.global" SEPCONV_ST_HINT ".v2.f32 [%0+8], {%3, %4};\n\t}"
            ::"l"(ptr), "f"(v[0]), "f"(v[1]), "f"(v[2]), "f"(v[3]), "r"(qa), "r"(qb)
            : "memory");
        ptr += ld;
    }
    // MODE 2: 16-byte rows, 1: 8-byte rows (shuffled into 16-byte chunks), 3: 8-byte rows as
    // two 8-byte stores, 0: ragged edge / 4-byte rows
    template <int MODE, bool EDGE = false>
    __device__ __forceinline__ void put(const float (&v)[V], bool ok, int lane) {
        if constexpr (MODE == 2) store_fast16(v, ok);
        else if constexpr (MODE == 1) store_fast<EDGE>(v, ok, lane);
        else if constexpr (MODE == 3) store_v2x2<EDGE>(v, ok);
        else store_scalar(v, ok);
    }
    // write v to the cursor row if ok, then move to the next row
    __device__ __forceinline__ void store(const float (&v)[V], bool ok) {
        const unsigned a = static_cast<unsigned>(reinterpret_cast<uintptr_t>(ptr)) & 15u;
        const bool fast = full && (a & 7u) == 0;
        const unsigned p16 = ok && fast && a == 0;
        const unsigned p8 = ok && fast && a == 8;
        const bool ps = ok && !fast;
        const unsigned q0 = ps && e0, q1 = ps && e1, q2 = ps && e2, q3 = ps && e3;
        asm volatile(
            "{\n\t.reg .pred q16, q8, q0, q1, q2, q3;\n\t"
            "setp.ne.u32 q16, %5, 0;\n\t"
            "setp.ne.u32 q8, %6, 0;\n\t"
            "setp.ne.u32 q0, %7, 0;\n\t"
            "setp.ne.u32 q1, %8, 0;\n\t"
            "setp.ne.u32 q2, %9, 0;\n\t"
            "setp.ne.u32 q3, %10, 0;\n\t"
            "@q16 st.global" SEPCONV_ST_HINT ".v4.f32 [%0], {%1, %2, %3, %4};\n\t"
            "@q8 st.global.v2.f32 [%0], {%1, %2};\n\t"
            "@q8 st.global.v2.f32 [%0+8], {%3, %4};\n\t"
            "@q0 st.global.f32 [%0], %1;\n\t"
            "@q1 st.global.f32 [%0+4], %2;\n\t"
            "@q2 st.global.f32 [%0+8], %3;\n\t"
            "@q3 st.global.f32 [%0+12], %4;\n\t}"
            ::"l"(ptr), "f"(v[0]), "f"(v[1]), "f"(v[2]), "f"(v[3]), "r"(p16), "r"(p8), "r"(q0), "r"(q1), "r"(q2),
            "r"(q3)
            : "memory");
        ptr += ld;
    }
};

// Direct mapping: this thread's window of XW floats of one input row, read
// through L1 (neighbouring lanes overlap, so most of it hits).  Branch-free (see
// store_out4): the row and the columns are clamped into the image instead of
// guarded.  A clamped row or column only ever feeds an output cell that is not
// stored (a valid output column c' < in_cols-K+1 reads columns <= in_cols-1; a
// step past the segment's last input row completes no stored row), so the
// duplicated values are harmless and every load stays inside the allocation.
template <int XW, bool VEC>
__device__ __forceinline__ void load_window_global(float (&x)[(XW + 3) & ~3], const float *__restrict__ img,
                                                   int r, int c, int in_rows, int in_cols, long long ld_in) {
    constexpr int XV = (XW + 3) / 4;
    const float *__restrict__ rowp = img + static_cast<long long>(min(r, in_rows - 1)) * ld_in;
    if constexpr (VEC) {
        const int cmax = (in_cols - 1) & ~3;
#pragma unroll
        for (int v = 0; v < XV; ++v) {
            const float4 t = __ldg(reinterpret_cast<const float4 *>(rowp + min(c + 4 * v, cmax)));
            x[4 * v + 0] = t.x; x[4 * v + 1] = t.y; x[4 * v + 2] = t.z; x[4 * v + 3] = t.w;
        }
    } else {
#pragma unroll
        for (int e = 0; e < XV * 4; ++e) x[e] = __ldg(rowp + min(c + e, in_cols - 1));
    }
}

// ---- work decomposition ------------------------------------------------------------------
// A segment = (image n, CTA strip s, output rows [q0, q0+nrows)); each segment costs K-1
// warm-up rows.  Two schedules (chosen by the host):
//   parts > 0: items (n, part j, strip s) with the strip index fastest, CTA b takes items
//     b, b+grid, ...; part j = rows [j*rows/parts, (j+1)*rows/parts).  Consecutive CTAs walk
//     the same rows of neighbouring strips, so the CTAs in flight touch a few row windows
//     (TLB- and L2-friendly: halo columns of neighbouring strips are read at the same time).
//   parts = 0: CTA b takes the contiguous range [b*total/grid, (b+1)*total/grid) of the
//     (image, strip, row) space -- exactly balanced, used when items would not divide evenly.
//   parts = -q: every slot busy when the S = nimg*nstrips strips do not divide the slots:
//     CTAs b < q*S take one segment each, rows [j*P, (j+1)*P) of strip b % S with
//     j = b / S (q full-width windows of P = win_rows rows, strip-fastest as above); the
//     e = extra remaining CTAs split the last window, rows [q*P, rows), CTA x taking the
//     strips x, x+e, ...  The host sizes P so both kinds finish together.
struct SegmentIter {
    long long total, u, u_end, item, items;
    int rows, nstrips, parts, win_rows, extra;
    __device__ SegmentIter(long long total_, int rows_, int nstrips_, int parts_, int nimg, int win_rows_ = 0,
                           int extra_ = 0)
        : total(total_), rows(rows_), nstrips(nstrips_), parts(parts_), win_rows(win_rows_), extra(extra_) {
        u = total * blockIdx.x / gridDim.x;
        u_end = total * (blockIdx.x + 1) / gridDim.x;
        item = blockIdx.x;
        items = static_cast<long long>(nimg) * nstrips * (parts > 0 ? parts : 1);
    }
    __device__ bool next(int &n, int &s, int &q0, int &nrows) {
        if (parts < 0) {
            const long long S = items;                         // nimg * nstrips
            const long long nmain = static_cast<long long>(-parts) * S;
            long long sidx;
            if (item < nmain) {                                // main CTA: one segment
                sidx = item % S;
                q0 = static_cast<int>((item / S) * win_rows);
                nrows = win_rows;
                item = nmain + S * extra;                      // done (never < nmain again)
            } else {
                // extra CTA x = blockIdx.x - nmain: item walks x, x + e, ... (offset by nmain)
                if (item >= nmain + S * extra) return false;
                const long long x = item - nmain;              // x + t*e on the t-th call
                if (x >= S) return false;
                sidx = x;
                q0 = -parts * win_rows;
                nrows = rows - q0;
                if (nrows <= 0) return false;
                item += extra;
            }
            n = static_cast<int>(sidx / nstrips);
            s = static_cast<int>(sidx - static_cast<long long>(n) * nstrips);
            return true;
        }
        if (parts > 0) {
            if (item >= items) return false;
            s = static_cast<int>(item % nstrips);
            const long long t = item / nstrips;
            const int j = static_cast<int>(t % parts);
            n = static_cast<int>(t / parts);
            q0 = static_cast<int>(static_cast<long long>(rows) * j / parts);
            nrows = static_cast<int>(static_cast<long long>(rows) * (j + 1) / parts) - q0;
            item += gridDim.x;
            return true;
        }
        if (u >= u_end) return false;
        const long long sidx = u / rows;                       // (image, strip) index
        q0 = static_cast<int>(u - sidx * rows);
        const long long seg_end = min(u_end, (sidx + 1) * static_cast<long long>(rows));
        nrows = static_cast<int>(seg_end - u);
        u = seg_end;
        n = static_cast<int>(sidx / nstrips);
        s = static_cast<int>(sidx - static_cast<long long>(n) * nstrips);
        return true;
    }
};

// ---- work stealing between warps ---------------------------------------------------------
// With p.steal > 0 (strided schedule), warp w of segment item d owns the claim word
// claims[d * NW + w] = epoch:32 | front:16 | end:16, in TMA stages ("chunks") of that warp's
// column strip.  The owner claims its stages one at a time from the front (an atomic add one
// stage ahead of use, so the latency hides behind a stage of arithmetic); a warp that has run
// out of work takes half of the largest unclaimed remainder from the back by compare-and-swap
// and computes it as an ordinary segment (K-1 warm-up rows).  A thief always leaves the owner
// its next stage, so the owner stops exactly where the thief starts: every output row is
// computed by one warp, with the same arithmetic as any other schedule.  Words of an earlier
// launch carry an older epoch and are ignored.
__device__ __forceinline__ unsigned long long claim_word(unsigned epoch, int front, int end) {
    return (static_cast<unsigned long long>(epoch) << 32) | (static_cast<unsigned long long>(front) << 16) |
           static_cast<unsigned long long>(end);
}

// segment of item d under the strided schedule (SegmentIter, parts > 0)
__device__ __forceinline__ void strided_item(long long d, int rows, int nstrips, int parts, int &n, int &s, int &q0,
                                             int &nrows) {
    s = static_cast<int>(d % nstrips);
    const long long t = d / nstrips;
    const int j = static_cast<int>(t % parts);
    n = static_cast<int>(t / parts);
    q0 = static_cast<int>(static_cast<long long>(rows) * j / parts);
    nrows = static_cast<int>(static_cast<long long>(rows) * (j + 1) / parts) - q0;
}

// Called by all 32 lanes of a warp with no work left: steals half of the largest unclaimed
// remainder (at least p.steal stages) of any warp of this launch.  Returns the stolen rows as a
// segment of warp slot wslot, or false when nothing is worth stealing.
template <int K, int SR, int NW>
__device__ bool steal_stages(const StreamParams &p, int lane, int &n, int &s, int &wslot, int &q0, int &nrows) {
    const long long nwords = static_cast<long long>(p.nimg) * p.nstrips * p.parts * NW;
    for (int attempt = 0; attempt < 64; ++attempt) {
        int best_rem = 0;
        long long best_v = -1;
        unsigned long long best_w = 0;
        for (long long v = lane; v < nwords; v += 32) {
            const unsigned long long w = *reinterpret_cast<volatile unsigned long long *>(p.claims + v);
            if (static_cast<unsigned>(w >> 32) != p.epoch) continue;
            const int rem = static_cast<int>(w & 0xffff) - static_cast<int>((w >> 16) & 0xffff);
            if (rem > best_rem) {
                best_rem = rem;
                best_v = v;
                best_w = w;
            }
        }
#pragma unroll
        for (int o = 16; o; o >>= 1) {                          // warp argmax (ties: lower index)
            const int r2 = __shfl_xor_sync(0xffffffffu, best_rem, o);
            const long long v2 = __shfl_xor_sync(0xffffffffu, best_v, o);
            const unsigned long long w2 = __shfl_xor_sync(0xffffffffu, best_w, o);
            if (r2 > best_rem || (r2 == best_rem && v2 < best_v)) {
                best_rem = r2;
                best_v = v2;
                best_w = w2;
            }
        }
        if (best_rem < p.steal || best_rem < 2) return false;
        const int f = static_cast<int>((best_w >> 16) & 0xffff), e = static_cast<int>(best_w & 0xffff);
        const int e_new = e - (e - f) / 2;                       // >= f + 1: the owner keeps its next stage
        int won = 0;
        if (lane == 0)
            won = atomicCAS(p.claims + best_v, best_w, (best_w & ~0xffffull) | static_cast<unsigned>(e_new)) == best_w;
        if (!__shfl_sync(0xffffffffu, won, 0)) continue;        // the word moved: look again
        wslot = static_cast<int>(best_v % NW);
        strided_item(best_v / NW, p.rows, p.nstrips, p.parts, n, s, q0, nrows);
        const int r0 = e_new * SR - (K - 1);                      // output rows of stages [e_new, e)
        const int r1 = min(e * SR - (K - 1), nrows);
        q0 += r0;
        nrows = r1 - r0;
        return true;
    }
    return false;
}

// ---- the streaming kernel -----------------------------------------------------------
// One CTA = NW independent warps over NW adjacent 128-column strips; the CTA's
// share of the (image, CTA-strip, row) space is contiguous, split evenly over
// the grid so the row granularity is 1 and no CTA idles at the end.
template <int K, int OP, int MAP, int NW, int SR_, int NS_, int F2, int SM = 1, int LOCK = 0>
__global__ void __launch_bounds__(NW * 32, MAP == MAP_TMA ? 1 : 2) stream_kernel(const __grid_constant__ StreamParams p) {
    constexpr bool TMA = MAP == MAP_TMA;
    constexpr bool HALO = OP != OP_COLS;
    constexpr bool ROWCONV = OP != OP_COLS;
    constexpr bool RING = OP != OP_ROWS;
    constexpr int XW = HALO ? V + K - 1 : V;
    constexpr int XV = (XW + 3) / 4;
    constexpr int BW = stream_bw(K, OP);
    constexpr int SR = SR_;  // rows per stage
    constexpr int NS = NS_;
    constexpr int BOX_BYTES = SR * BW * 4;                     // bytes one TMA box delivers
    constexpr int STAGE = (SR * BW + 31) & ~31;                // floats per stage (128-byte TMA alignment)
    constexpr int RK = RING ? K : 1;                           // ring slots
    static_assert(BW <= 256, "TMA box width");
    static_assert(BW == box_width(K, HALO), "box width");
    static_assert(!RING || SR % K == 0, "ring period must divide the stage");
    static_assert(!TMA || NW * NS * (STAGE * 4 + 8) <= kSmemPerCta, "shared memory per CTA");

    extern __shared__ __align__(128) float smem[];
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    float *wsm = smem + (TMA ? warp * NS * STAGE : 0);
    uint64_t *wbar = reinterpret_cast<uint64_t *>(smem + NW * NS * STAGE) + warp * NS;

    if constexpr (TMA) {
        if (lane == 0) {
            if (warp == 0) prefetch_tmap(&p.tmap);
#pragma unroll
            for (int s = 0; s < NS; ++s) mbar_init(&wbar[s], 1);
            fence_barrier_init();
        }
        __syncwarp();
    }

    SegmentIter seg(p.total, p.rows, p.nstrips, p.parts, p.nimg, p.win_rows, p.extra);
    uint32_t kc = 0;                                           // chunks consumed by this warp
#ifdef SEPCONV_CTA_TRACE
    unsigned long long t_start = 0, nseg = 0;
    if (threadIdx.x == 0) asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t_start));
#endif

    // work stealing between warps: free-running warps only (lockstep CTAs share barriers; the
    // 16-warp CTAs' 128-register budget has no room for the claim state)
    constexpr bool STEAL = TMA && RING && !LOCK && NW <= 8;
    // SM = 3: the 8-byte store path with even-width right-edge warps on it too (the host picks it
    // for K >= 13 on images up to 8192 columns; see the store-path dispatch below)
    // store path 2 (SM = 4) carries its right-edge warp from K = 13 up as mode 3 does: two
    // predicated 8-byte stores per lane instead of a second copy of the loop (2048^2 / K=15 19.2 ->
    // 14.3 us, 3520^2 / 4096^2 -10%; mixed below K = 13, profiles/r02_explore_v2edge.txt)
    constexpr bool EDGE8 = SM == 3 || SM == 5 || (SM == 4 && K >= 13);
    constexpr int SMS = (SM >= 3) ? 1 : SM;                    // the store path proper
    // SM = 4 (store path 2): 8-byte rows as two 8-byte stores per lane at any warp count -- no
    // shuffles, a smaller loop body; faster at 2048^2-3520^2 (K = 7-15: -4-14%), slower at 16384^2
    // (each 32-byte sector written in two halves: +3-13%), so a tuner candidate
    // (tools/explore_mid.cu EXPLORE_V2X2, profiles/r02_explore_v2x2.txt).  SM = 5 (exploration
    // only): store path 2 with even-width right-edge warps on it (store_v2x2<EDGE>)
    const bool steal_on = STEAL && p.steal > 0 && p.parts > 0;
    bool thief = false;
    int n, s, q0, nrows;
    for (;;) {
        int wslot = warp;                                      // column slot (a thief takes its victim's)
        unsigned long long *word = nullptr;                    // this warp-segment's claim word (owner)
        if (!thief) {
            if (seg.next(n, s, q0, nrows)) {
                if (steal_on) word = p.claims + (seg.item - gridDim.x) * NW + warp;
            } else if (steal_on) {
                thief = true;
            } else {
                break;
            }
        }
        if (thief && !steal_stages<K, SR, NW>(p, lane, n, s, wslot, q0, nrows)) break;
#ifdef SEPCONV_CTA_TRACE
        ++nseg;
#endif
        if constexpr (TMA && LOCK) {
            // the lockstep barrier's thread count depends on the strip: a warp must not reach
            // the next segment's barriers while another still uses this one's (a CTA whose
            // segments span a full strip and a narrow right-edge strip of a batch or of a
            // window schedule would otherwise mix counts on barrier 1)
            __syncthreads();
        }
        const int wcol = s * (NW * kWarpCols) + wslot * kWarpCols;  // warp's first column
        if (wcol >= p.out_cols) continue;
        // warps of this strip that have columns (named-barrier thread count for LOCK)
        const int lock_threads = 32 * min(NW, (p.out_cols - s * (NW * kWarpCols) + kWarpCols - 1) / kWarpCols);
        (void)lock_threads;
        const int c = wcol + lane * V;                         // this thread's first column
        const int in_row0 = p.row_begin + q0;
        const int steps = nrows + (RING ? K - 1 : 0);
        const int nchunks = (steps + SR - 1) / SR;
        const float *__restrict__ in_img = p.in + n * p.in_img_stride;
        float *out_rows = p.out + n * p.out_img_stride + static_cast<long long>(in_row0) * p.ld_out;
        // the cursor starts at the row step 0 completes: q = -(K-1) for RING ops
        OutCursor oc;
        oc.init(out_rows - (RING ? static_cast<long long>(K - 1) * p.ld_out : 0LL), p.ld_out, c, p.out_cols);

        if constexpr (TMA) {
            __syncwarp();                                      // every lane is past the previous segment's reads
            if (lane == 0) {
                fence_proxy_async_smem();                      // ... which precede these async-proxy writes
                const int npro = nchunks < NS ? nchunks : NS;
                if (word) atomicExch(word, claim_word(p.epoch, npro, nchunks));   // open for thieves
                for (int ch = 0; ch < npro; ++ch) {
                    const int st = (kc + ch) % NS;
                    mbar_arrive_expect_tx(&wbar[st], BOX_BYTES);
                    tma_load_3d(wsm + st * STAGE, &p.tmap, &wbar[st], wcol, in_row0 + ch * SR, n);
                }
            }
        }

        // two copies of the hot loop: the fast store path SM and the general one, which
        // only runs at the ragged right edge (or for rows that are not 8-byte aligned)
        auto run_chunks = [&](auto mode_tag) {
        constexpr int SMODE = decltype(mode_tag)::value;
        float acc[RK][V];
#pragma unroll
        for (int a = 0; a < RK; ++a)
#pragma unroll
            for (int e = 0; e < V; ++e) acc[a][e] = 0.f;

        // stealing: stages [0, limit) are this warp's; the claim of stage `next` is issued one
        // refill ahead of its use (pend, lane 0)
        int limit = nchunks;
        unsigned long long pend = 0;
        if (STEAL && word != nullptr && lane == 0 && NS < nchunks) pend = atomicAdd(word, 1ull << 16);
        for (int ch = 0; ch < limit; ++ch, ++kc) {
            const int st = kc % NS;
            const float *stage = wsm + st * STAGE;
            if constexpr (TMA) mbar_wait(&wbar[st], (kc / NS) & 1);
#pragma unroll
            for (int pr = 0; pr < SR; ++pr) {
                const int t = ch * SR + pr;                    // step = input row - in_row0
                float x[XV * 4];
                if constexpr (TMA) {
#pragma unroll
                    for (int v = 0; v < XV; ++v) {
                        const float4 tt = ld_shared4(stage + pr * BW + lane * V + 4 * v);
                        x[4 * v + 0] = tt.x; x[4 * v + 1] = tt.y; x[4 * v + 2] = tt.z; x[4 * v + 3] = tt.w;
                    }
                } else {
                    load_window_global<XW, MAP == MAP_DIRECT_VEC>(x, in_img, in_row0 + t, c, p.in_rows,
                                                                 p.in_cols, p.ld_in);
                }
                float b[V];
                if constexpr (ROWCONV) {
                    if constexpr (F2 == 2) {
                        // same per-element order as the scalar path, two columns per instruction:
                        // xp[m] = (x_2m, x_2m+1) are the loaded pairs, xs[m] = (x_2m+1, x_2m+2) the
                        // shifted pairs odd taps need (built once per step, shared by both column pairs)
                        constexpr int NP = (XW + 1) / 2;
                        float2 xp[NP], xs[NP];
#pragma unroll
                        for (int m = 0; m < NP; ++m) xp[m] = make_float2(x[2 * m], x[2 * m + 1]);
#pragma unroll
                        for (int m = 0; m + 1 < NP; ++m) xs[m] = make_float2(x[2 * m + 1], x[2 * m + 2]);
#pragma unroll
                        for (int e = 0; e < V; e += 2) {
                            float2 bb = fmul2(p.k2[0], xp[e / 2]);
#pragma unroll
                            for (int i = 1; i < K; ++i)
                                bb = ffma2(p.k2[i], ((e + i) & 1) ? xs[(e + i) / 2] : xp[(e + i) / 2], bb);
                            b[e] = bb.x;
                            b[e + 1] = bb.y;
                        }
                    } else if constexpr (F2 == 3 && K >= 2) {
                        // exploration only (tools/explore_mid.cu; no product configuration uses
                        // it: it changes the summation order R6): two independent chains over
                        // even / odd taps, halving the row pass's dependent-FMA depth
#pragma unroll
                        for (int e = 0; e < V; ++e) {
                            float b0 = p.k[0] * x[e], b1 = p.k[1] * x[e + 1];
#pragma unroll
                            for (int i = 2; i < K; ++i) {
                                if (i & 1) b1 = fmaf(p.k[i], x[e + i], b1);
                                else b0 = fmaf(p.k[i], x[e + i], b0);
                            }
                            b[e] = b0 + b1;
                        }
                    } else {
#pragma unroll
                        for (int e = 0; e < V; ++e) {
                            b[e] = p.k[0] * x[e];
#pragma unroll
                            for (int i = 1; i < K; ++i) b[e] = fmaf(p.k[i], x[e + i], b[e]);
                        }
                    }
                } else {
#pragma unroll
                    for (int e = 0; e < V; ++e) b[e] = x[e];
                }
                if constexpr (RING) {
#pragma unroll
                    for (int j = 0; j < K; ++j) {
                        const int slot = ((pr - j) % K + K) % K;
                        if constexpr (F2 >= 1) {
#pragma unroll
                            for (int e = 0; e < V; e += 2) {
                                const float2 bb = make_float2(b[e], b[e + 1]);
                                float2 aa = (j == 0) ? fmul2(p.k2[0], bb)
                                                     : ffma2(p.k2[j], bb, make_float2(acc[slot][e], acc[slot][e + 1]));
                                acc[slot][e] = aa.x;
                                acc[slot][e + 1] = aa.y;
                            }
                        } else {
#pragma unroll
                            for (int e = 0; e < V; ++e)
                                acc[slot][e] = (j == 0) ? p.k[0] * b[e] : fmaf(p.k[j], b[e], acc[slot][e]);
                        }
                    }
                    const int q = t - (K - 1);                 // output row completed by this step
                    oc.put<SMODE, EDGE8>(acc[(pr + 1) % K], static_cast<unsigned>(q) < static_cast<unsigned>(nrows), lane);
                } else {
                    oc.put<SMODE, EDGE8>(b, t < nrows, lane);
                }
            }
            if constexpr (TMA) {
                if constexpr (LOCK) {
                    // CTA lockstep: the active warps of this strip finish the stage together.
                    // Non-.aligned barrier: the edge warp of a strip runs the other copy of this
                    // loop (scalar stores), i.e. a different barrier instruction with the same id
                    asm volatile("barrier.sync 1, %0;" ::"r"(lock_threads) : "memory");
                } else {
                    __syncwarp();
                }
                bool go = ch + NS < limit;
                if (STEAL && word != nullptr && go) {          // warp-uniform
                    const unsigned long long r = __shfl_sync(0xffffffffu, pend, 0);
                    if (((r >> 16) & 0xffff) < (r & 0xffff)) {  // stage ch + NS is ours
                        if (lane == 0 && ch + NS + 1 < nchunks) pend = atomicAdd(word, 1ull << 16);
                    } else {                                   // a thief has the rest
                        limit = ch + NS;
                        go = false;
                    }
                }
                tma_refill_elected(go, wsm + st * STAGE, &p.tmap, &wbar[st], BOX_BYTES, wcol,
                                   in_row0 + (ch + NS) * SR, n);
            }
        }
        };
        // SM (a template parameter) is the store path of warps wholly inside the image; the
        // host instantiates SM = 2 when every row start is 16-byte aligned, else SM = 1 (or 3)
        // (16-warp configurations take the 8-byte rows as two 8-byte stores: the shuffled form
        // spills at their 128-register budget)
        constexpr int SMF = (SM == 4 || SM == 5 || (SMS == 1 && NW >= 16)) ? 3 : SMS;
        // The right-edge warp of a ragged width joins the 16-byte path when the width is a
        // multiple of 4 (store_fast16 masks its outside lanes): a second copy of the ~38 KB
        // K=17 loop running on some SMs slowed those CTAs and their TPC neighbours by 6-12%
        // at 16384^2 (the last two CTA strips; profiles/r02_cta_strips.txt)
        // The same holds for the 8-byte store paths (SM = 3) when the output width is even: each
        // lane then has 4, 2 or 0 columns inside and store_fast<EDGE8> / store_v2x2<EDGE8>
        // predicate the pairs.  Measured (profiles/r02x_edge8_ab.txt): 2048^2 / K = 13-17
        // -11-19%, 3520^2 -4-9%, but +2-6% at 16384^2 (the predicates cost every warp a few
        // instructions per row, and there the edge warp is 1 of 128), and up to +10% for K = 7 at
        // mid sizes -- hence the host's choice of SM = 3 only for K >= 13 and widths <= 8192
        const bool edge_ok = SMF == 2 ? (p.out_cols & 3) == 0 : (EDGE8 && (p.out_cols & 1) == 0);
        const bool fast = (wcol + kWarpCols <= p.out_cols || edge_ok) && p.store8 >= SMS;
        if (fast) run_chunks(std::integral_constant<int, SMF>{});
        else run_chunks(std::integral_constant<int, 0>{});
    }
#ifdef SEPCONV_CTA_TRACE
    __syncthreads();
    if (threadIdx.x == 0) {
        unsigned long long t_end;
        unsigned smid;
        asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t_end));
        asm volatile("mov.u32 %0, %%smid;" : "=r"(smid));
        p.trace[4 * blockIdx.x + 0] = t_start;
        p.trace[4 * blockIdx.x + 1] = t_end;
        p.trace[4 * blockIdx.x + 2] = smid;
        p.trace[4 * blockIdx.x + 3] = nseg;
    }
#endif
}

template <int K, int OP, int MAP, int NW, int SR, int NS, int F2>
constexpr size_t stream_smem_bytes() {
    return MAP == MAP_TMA ? static_cast<size_t>(NW) * NS * ((SR * stream_bw(K, OP) + 31) & ~31) * 4 + NW * NS * 8
                          : 0;
}

// The kernel for (K, OP, variant) with the geometry of stream_geom (sepconv_params.h).
template <int K, int OP, int VARIANT, int SM>
struct StreamInst {
    static constexpr StreamGeom G = stream_geom(K, OP, VARIANT);
    static constexpr int MAP = VARIANT >= 2 ? MAP_TMA : VARIANT;
    static constexpr auto kernel = &stream_kernel<K, OP, MAP, G.nw, G.sr, G.ns, G.f2, SM, G.lock>;
    static constexpr size_t smem = stream_smem_bytes<K, OP, MAP, G.nw, G.sr, G.ns, G.f2>();
    static constexpr int threads = G.nw * 32;
};

// ---- Convolve2D ------------------------------------------------------------------------
// Per output row q: a = sum_j (sum_i w_ji x_{q+j, c+i}).  TMA mapping keeps a
// per-warp ring of NS stages of SR rows; rows [q, q+K-1] must be resident, a
// stage is refilled once q has passed it.
template <int K, int MAP, int NW>
__global__ void __launch_bounds__(NW * 32, 1) conv2d_kernel(const __grid_constant__ Conv2DParams p) {
    constexpr bool TMA = MAP == MAP_TMA;
    constexpr int XW = V + K - 1;
    constexpr int XV = (XW + 3) / 4;
    constexpr int BW = box_width(K, true);
    constexpr int SR = Conv2DCfg<K>::SR;
    constexpr int NS = Conv2DCfg<K>::NS;
    constexpr int STAGE = SR * BW;
    static_assert((STAGE * 4) % 128 == 0, "TMA destinations must be 128-byte aligned");
    constexpr int RING_ROWS = NS * SR;

    extern __shared__ __align__(128) float smem[];
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    float *wsm = smem + (TMA ? warp * NS * STAGE : 0);
    uint64_t *wbar = reinterpret_cast<uint64_t *>(smem + NW * NS * STAGE) + warp * NS;
    if constexpr (TMA) {
        if (lane == 0) {
            if (warp == 0) prefetch_tmap(&p.tmap);
#pragma unroll
            for (int s = 0; s < NS; ++s) mbar_init(&wbar[s], 1);
            fence_barrier_init();
        }
        __syncwarp();
    }

    SegmentIter seg(p.total, p.rows, p.nstrips, p.parts, p.nimg, p.win_rows, p.extra);
    uint32_t kc = 0;

    int n, s, q0, nrows;
    while (seg.next(n, s, q0, nrows)) {
        const int wcol = s * (NW * kWarpCols) + warp * kWarpCols;
        if (wcol >= p.out_cols) continue;
        const int c = wcol + lane * V;
        const int in_row0 = p.row_begin + q0;
        const int nchunks = (nrows + K - 1 + SR - 1) / SR;
        const float *__restrict__ in_img = p.in + n * p.in_img_stride;
        float *out_rows = p.out + n * p.out_img_stride + static_cast<long long>(in_row0) * p.ld_out;
        const uint32_t kc0 = kc;
        int waited = 0;
        OutCursor oc;
        oc.init(out_rows, p.ld_out, c, p.out_cols);

        if constexpr (TMA) {
            __syncwarp();                                      // every lane is past the previous segment's reads
            if (lane == 0) {
                fence_proxy_async_smem();                      // ... which precede these async-proxy writes
                const int npro = nchunks < NS ? nchunks : NS;
                for (int ch = 0; ch < npro; ++ch) {
                    const int st = (kc0 + ch) % NS;
                    mbar_arrive_expect_tx(&wbar[st], STAGE * 4);
                    tma_load_3d(wsm + st * STAGE, &p.tmap, &wbar[st], wcol, in_row0 + ch * SR, n);
                }
            }
        }
        const int ring_base = static_cast<int>(kc0 % NS) * SR;     // ring row of segment row 0

        for (int q = 0; q < nrows; ++q) {
            if constexpr (TMA) {
                const int need = (q + K - 1) / SR;
                while (waited <= need) {
                    const uint32_t g = kc0 + waited;
                    mbar_wait(&wbar[g % NS], (g / NS) & 1);
                    ++waited;
                }
            }
            float a[V];
            int rr = ring_base + q;
            if (rr >= RING_ROWS) rr -= RING_ROWS * (rr / RING_ROWS);
#pragma unroll
            for (int j = 0; j < K; ++j) {
                float x[XV * 4];
                if constexpr (TMA) {
                    const float *rowp = wsm + rr * BW + lane * V;
#pragma unroll
                    for (int v = 0; v < XV; ++v) {
                        const float4 tt = ld_shared4(rowp + 4 * v);
                        x[4 * v + 0] = tt.x; x[4 * v + 1] = tt.y; x[4 * v + 2] = tt.z; x[4 * v + 3] = tt.w;
                    }
                    rr = (rr + 1 == RING_ROWS) ? 0 : rr + 1;
                } else {
                    load_window_global<XW, MAP == MAP_DIRECT_VEC>(x, in_img, in_row0 + q + j, c, p.in_rows,
                                                                 p.in_cols, p.ld_in);
                }
#pragma unroll
                for (int e = 0; e < V; ++e) {
                    float pj = p.w[j * K] * x[e];
#pragma unroll
                    for (int i = 1; i < K; ++i) pj = fmaf(p.w[j * K + i], x[e + i], pj);
                    a[e] = (j == 0) ? pj : a[e] + pj;
                }
            }
            oc.store(a, true);
            if constexpr (TMA) {
                // rows < q+1 are dead; a stage is free once q+1 crosses its end
                if ((q + 1) % SR == 0) {
                    const int done_chunk = (q + 1) / SR - 1;
                    const int next = done_chunk + NS;
                    __syncwarp();
                    if (lane == 0 && next < nchunks) {
                        const int st = (kc0 + done_chunk) % NS;
                        fence_proxy_async_smem();
                        mbar_arrive_expect_tx(&wbar[st], STAGE * 4);
                        tma_load_3d(wsm + st * STAGE, &p.tmap, &wbar[st], wcol, in_row0 + next * SR, n);
                    }
                }
            }
        }
        if constexpr (TMA) {
            // consume (wait on) any chunk issued but not needed by the last row
            const int issued = nchunks;
            while (waited < issued) {
                const uint32_t g = kc0 + waited;
                mbar_wait(&wbar[g % NS], (g / NS) & 1);
                ++waited;
            }
        }
        kc = kc0 + nchunks;
    }
}

template <int K, int MAP, int NW>
constexpr size_t conv2d_smem_bytes() {
    return MAP == MAP_TMA ? static_cast<size_t>(NW) * Conv2DCfg<K>::NS * Conv2DCfg<K>::SR * box_width(K, true) * 4 +
                     NW * Conv2DCfg<K>::NS * 8
               : 0;
}

}  // namespace sepconv
