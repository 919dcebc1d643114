// explore_mid.cu -- design-space exploration of the fused kernel on mid-size images (not the
// product).  For each stream_kernel instantiation below and each image side, the marginal
// pass time after a clean L2 flush (write 2 x L2 + read 2 x L2): event time of n x [flush,
// pass] minus n x [flush], so the ~2 us event granularity averages out; 16384^2 times
// back-to-back passes.  Also sweeps the strided schedule's part count around the default.
//   nvcc -std=c++17 -O3 -gencode arch=compute_100a,code=sm_100a -I../paper_conf_asplos_phothilimthanaara13_b200/csrc \
//        explore_mid.cu -o explore_mid -lcuda
//   ./explore_mid [sizes...]
#include <cuda.h>
#include <cuda_runtime.h>

#include <algorithm>
#include <cstdio>
#include <cstring>
#include <vector>

#include "sepconv_kernels.cuh"

using namespace sepconv;

typedef CUresult (*EncodeTiledFn)(CUtensorMap *, CUtensorMapDataType, cuuint32_t, void *, const cuuint64_t *,
                                  const cuuint64_t *, const cuuint32_t *, const cuuint32_t *, CUtensorMapInterleave,
                                  CUtensorMapSwizzle, CUtensorMapL2promotion, CUtensorMapFloatOOBfill);
static EncodeTiledFn enc;
static int SMS = 148;
static float *din, *dout, *wfl, *rfl, *sink;
static long long fl_n4;
static cudaEvent_t e0, e1;

__global__ void fill_k(float4 *p, long long n) {
    for (long long i = blockIdx.x * (long long)blockDim.x + threadIdx.x; i < n; i += (long long)gridDim.x * blockDim.x)
        p[i] = make_float4(1.f, 1.f, 1.f, 1.f);
}
__global__ void read_k(const float4 *p, long long n, float *s) {
    float a = 0.f;
    for (long long i = blockIdx.x * (long long)blockDim.x + threadIdx.x; i < n; i += (long long)gridDim.x * blockDim.x)
        a += p[i].x;
    if (a < 0.f) *s = a;
}
static void flush() {
    fill_k<<<148 * 8, 256>>>((float4 *)wfl, fl_n4);
    read_k<<<148 * 8, 256>>>((const float4 *)rfl, fl_n4, sink);
}
template <typename F>
static float batch(F f, int n) {
    f();
    cudaDeviceSynchronize();
    cudaEventRecord(e0);
    for (int i = 0; i < n; ++i) f();
    cudaEventRecord(e1);
    cudaEventSynchronize(e1);
    float ms;
    cudaEventElapsedTime(&ms, e0, e1);
    return ms * 1000.f / n;
}
template <typename F>
static float pass_time(F f, bool cold) {
    float t[3];
    for (int b = 0; b < 3; ++b) {
        if (cold) {
            const float tf = batch(flush, 60);
            t[b] = batch([&] { flush(); f(); }, 60) - tf;
        } else {
            t[b] = batch(f, 20);
        }
    }
    std::sort(t, t + 3);
    return t[1];
}

template <int K, int NW, int SR, int NS, int F2, int SM = 2, int LOCK = 0>
static void run_cfg(int H, const char *tag, int cps_want = 1) {
    const int W = H;
    auto kern = stream_kernel<K, OP_SEP, MAP_TMA, NW, SR, NS, F2, SM, LOCK>;
    size_t smem = stream_smem_bytes<K, OP_SEP, MAP_TMA, NW, SR, NS, F2>();
    if (smem > 232448) { printf("skip (smem %zu)\n", smem); return; }
    cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
    int occ = 0;
    cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, kern, NW * 32, smem);
    const int cps = std::min(cps_want, occ);
    StreamParams p;
    memset(&p, 0, sizeof p);
    p.in = din; p.out = dout;
    p.ld_in = W; p.ld_out = W - K + 1;
    p.in_img_stride = (long long)H * W; p.out_img_stride = (long long)(H - K + 1) * (W - K + 1);
    p.in_rows = H; p.in_cols = W; p.out_cols = W - K + 1;
    p.row_begin = 0; p.rows = H - K + 1; p.nimg = 1;
    p.nstrips = (p.out_cols + NW * 128 - 1) / (NW * 128);
    p.total = (long long)p.nstrips * p.rows;
    for (int i = 0; i < K; ++i) { p.k[i] = 1.0f / K; p.k2[i] = make_float2(p.k[i], p.k[i]); }
    p.store8 = ((W - K + 1) % 4 == 0) ? 2 : (((W - K + 1) % 2 == 0) ? 1 : 0);
    if (SM == 2 && p.store8 != 2) { printf("skip SM2 (rows not 16-byte aligned)\n"); return; }
    if ((SM == 1 || SM >= 3) && p.store8 < 1) { printf("skip SM%d (rows not 8-byte aligned)\n", SM); return; }
    cuuint64_t dims[3] = {(cuuint64_t)W, (cuuint64_t)H, 1};
    cuuint64_t str[2] = {(cuuint64_t)W * 4, (cuuint64_t)H * W * 4};
    cuuint32_t box[3] = {(cuuint32_t)stream_bw(K, OP_SEP), (cuuint32_t)SR, 1}, es[3] = {1, 1, 1};
    CUresult r = enc(&p.tmap, CU_TENSOR_MAP_DATA_TYPE_FLOAT32, 3, din, dims, str, box, es, CU_TENSOR_MAP_INTERLEAVE_NONE,
                     CU_TENSOR_MAP_SWIZZLE_NONE, CU_TENSOR_MAP_L2_PROMOTION_L2_256B, CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
    if (r) { printf("encode failed %d\n", (int)r); return; }
    const int slots = SMS * cps;
    const bool cold = H <= 4096;
    const double bytes = 4.0 * ((double)H * W + (double)(H - K + 1) * (W - K + 1));
    // default: one round of items (parts = slots / strips), then a few alternatives
    const int p0 = std::max(1, slots / p.nstrips);
    float best = 1e30f;
    int best_parts = 0;
    for (int parts : {p0, std::max(1, p0 / 2), p0 * 2, std::max(1, (2 * p0) / 3), (3 * p0) / 2}) {
        p.parts = parts;
        const int grid = std::min<long long>(slots, (long long)p.nstrips * parts);
        const float us = pass_time([&] { kern<<<grid, NW * 32, smem>>>(p); }, cold);
        if (us < best) { best = us; best_parts = parts; }
    }
    cudaError_t e = cudaGetLastError();
    printf("H=%5d K=%2d %-10s NW=%2d SR=%2d NS=%d F2=%d L=%d cps=%d/%d smem=%3zuKB strips=%d parts=%4d: %7.2f us %6.0f GB/s %s\n",
           H, K, tag, NW, SR, NS, F2, LOCK, cps, occ, smem / 1024, p.nstrips, best_parts, best, bytes / best / 1e3,
           e ? cudaGetErrorString(e) : "");
    fflush(stdout);
}

int main(int argc, char **argv) {
    std::vector<int> sizes;
    for (int i = 1; i < argc; ++i) sizes.push_back(atoi(argv[i]));
    if (sizes.empty()) sizes = {2048, 4096, 16384};
    void *fp = nullptr;
    cudaDriverEntryPointQueryResult q;
    cudaGetDriverEntryPoint("cuTensorMapEncodeTiled", &fp, cudaEnableDefault, &q);
    enc = (EncodeTiledFn)fp;
    cudaDeviceProp prop;
    cudaGetDeviceProperties(&prop, 0);
    SMS = prop.multiProcessorCount;
    const size_t big = (size_t)16384 * 16384 * 4;
    cudaMalloc(&din, big);
    cudaMalloc(&dout, big);
    cudaMemset(din, 0, big);
    fl_n4 = 2LL * prop.l2CacheSize / 16;
    cudaMalloc(&wfl, fl_n4 * 16);
    cudaMalloc(&rfl, fl_n4 * 16);
    cudaMalloc(&sink, 16);
    cudaMemset(rfl, 0, fl_n4 * 16);
    cudaEventCreate(&e0);
    cudaEventCreate(&e1);
    // (EXPLORE_CS, CTA-shared stages: measured and rejected in round 2, the kernel code reverted;
    //  profiles/r02_explore_cta_stage.txt)
    // (EXPLORE_IWARM, a dry pass over the hot loop before the first segment to pull its code into the
    //  instruction caches while the prologue loads fly: 2-12% slower at 2048-4096^2, reverted;
    //  profiles/r02_explore_iwarm.txt)
    if (getenv("EXPLORE_HINT")) {                  // store cache hint (compile with -DSEPCONV_ST_HINT='".cs"')
        for (int H : sizes) {
            run_cfg<17, 8, 17, 2, 2>(H, "tma4");
            run_cfg<17, 8, 17, 2, 1>(H, "tma2");
            run_cfg<9, 8, 9, 2, 1, 2, 1>(H, "tma0");
            run_cfg<9, 4, 9, 2, 1, 2>(H, "tma5", 2);
            run_cfg<3, 8, 6, 2, 1, 1>(H, "tma2");
            run_cfg<5, 8, 5, 2, 1, 2>(H, "tma2");
        }
        return 0;
    }
    if (getenv("EXPLORE_V2EDGE")) {                // store path 2 with / without the right-edge warp on it
        for (int rep = 0; rep < 3; ++rep)
            for (int H : sizes) {
                run_cfg<3, 8, 9, 3, 1, 4, 1>(H, "tma1v2");
                run_cfg<3, 8, 9, 3, 1, 5, 1>(H, "tma1v2e");
                run_cfg<7, 8, 7, 2, 1, 4>(H, "tma2v2");
                run_cfg<7, 8, 7, 2, 1, 5>(H, "tma2v2e");
                run_cfg<7, 4, 7, 2, 1, 4>(H, "tma5v2", 2);
                run_cfg<7, 4, 7, 2, 1, 5>(H, "tma5v2e", 2);
                run_cfg<11, 8, 11, 2, 1, 4>(H, "tma2v2");
                run_cfg<11, 8, 11, 2, 1, 5>(H, "tma2v2e");
                run_cfg<15, 8, 15, 2, 1, 4>(H, "tma2v2");
                run_cfg<15, 8, 15, 2, 1, 5>(H, "tma2v2e");
            }
        return 0;
    }
    if (getenv("EXPLORE_V2X2")) {                  // 8-byte rows: shuffled 16-byte chunks (SM 1) vs two 8-byte stores (SM 4)
        for (int rep = 0; rep < 3; ++rep)
            for (int H : sizes) {
                run_cfg<3, 8, 9, 3, 1, 1, 1>(H, "tma1");
                run_cfg<3, 8, 9, 3, 1, 4, 1>(H, "tma1-v2x2");
                run_cfg<7, 8, 7, 2, 1, 1>(H, "tma2");
                run_cfg<7, 8, 7, 2, 1, 4>(H, "tma2-v2x2");
                run_cfg<11, 8, 11, 3, 1, 1, 1>(H, "tma1");
                run_cfg<11, 8, 11, 3, 1, 4, 1>(H, "tma1-v2x2");
                run_cfg<15, 8, 15, 2, 1, 1>(H, "tma2");
                run_cfg<15, 8, 15, 2, 1, 4>(H, "tma2-v2x2");
            }
        return 0;
    }
    if (getenv("EXPLORE_EDGE8")) {                 // 8-byte store paths with an even-width right edge
        for (int H : sizes) {
            run_cfg<15, 8, 15, 2, 1, 1>(H, "tma2");
            run_cfg<15, 8, 15, 2, 1, 1, 1>(H, "tma0");
            run_cfg<17, 8, 17, 2, 1, 1>(H, "tma2s8");
            run_cfg<17, 8, 17, 2, 2, 1>(H, "tma4s8");
            run_cfg<13, 8, 13, 3, 1, 1, 1>(H, "tma1s8");
            run_cfg<11, 8, 11, 3, 1, 1, 1>(H, "tma1");
            run_cfg<7, 8, 7, 2, 1, 1>(H, "tma2");
        }
        return 0;
    }
    if (getenv("EXPLORE_DEEPLOCK")) {              // deeper lockstep rings for the HBM-bound small widths
        for (int rep = 0; rep < 2; ++rep)
            for (int H : sizes) {
                run_cfg<3, 8, 6, 2, 1, 1, 1>(H, "tma0");
                run_cfg<3, 8, 9, 3, 1, 1, 1>(H, "tma1");
                run_cfg<3, 8, 6, 2, 1, 1>(H, "tma2");
                run_cfg<3, 8, 6, 4, 1, 1, 1>(H, "8w4s-lock");
                run_cfg<3, 8, 6, 6, 1, 1, 1>(H, "8w6s-lock");
                run_cfg<3, 8, 9, 5, 1, 1, 1>(H, "8w5sx9-lock");
                run_cfg<5, 8, 5, 2, 1, 2, 1>(H, "tma0");
                run_cfg<5, 8, 10, 3, 1, 2, 1>(H, "tma1");
                run_cfg<5, 8, 5, 2, 1, 2>(H, "tma2");
                run_cfg<5, 8, 5, 6, 1, 2, 1>(H, "8w6s-lock");
                run_cfg<5, 8, 10, 5, 1, 2, 1>(H, "8w5sx10-lock");
                run_cfg<7, 8, 7, 2, 1, 1, 1>(H, "tma0");
                run_cfg<7, 8, 7, 2, 1, 1>(H, "tma2");
                run_cfg<7, 8, 7, 5, 1, 1, 1>(H, "8w5s-lock");
                run_cfg<7, 8, 14, 3, 1, 1, 1>(H, "8w3sx14-lock");
            }
        return 0;
    }
    if (getenv("EXPLORE_DEEP")) {                  // deeper free-running rings for short segments
        for (int H : sizes) {
            run_cfg<3, 8, 6, 2, 1, 1>(H, "tma2");
            run_cfg<3, 8, 6, 9, 1, 1>(H, "8w9s");
            run_cfg<3, 8, 6, 6, 1, 1>(H, "8w6s");
            run_cfg<3, 8, 6, 4, 1, 1>(H, "8w4s");
            run_cfg<3, 8, 6, 6, 1, 1, 1>(H, "8w6s-lock");
            run_cfg<3, 4, 6, 4, 1, 1>(H, "4w4s-x2", 2);
            run_cfg<5, 8, 5, 2, 1, 2>(H, "tma2");
            run_cfg<5, 8, 5, 8, 1, 2>(H, "8w8s");
            run_cfg<7, 8, 7, 2, 1, 1>(H, "tma2");
            run_cfg<7, 8, 7, 6, 1, 1>(H, "8w6s");
            run_cfg<7, 4, 7, 2, 1, 1>(H, "tma5", 2);
            run_cfg<7, 4, 7, 4, 1, 1>(H, "4w4s-x2", 2);
            run_cfg<9, 8, 9, 2, 1, 2>(H, "tma2");
            run_cfg<9, 8, 9, 5, 1, 2>(H, "8w5s");
            run_cfg<9, 4, 9, 2, 1, 2>(H, "tma5", 2);
            run_cfg<11, 8, 11, 2, 1, 1>(H, "tma2");
            run_cfg<11, 8, 11, 4, 1, 1>(H, "8w4s");
            run_cfg<13, 8, 13, 2, 1, 2>(H, "tma2");
            run_cfg<13, 8, 13, 3, 1, 2>(H, "8w3s");
        }
        return 0;
    }
    if (getenv("EXPLORE_K17")) {                   // round-2 follow-up: packed-FP32 row pass variants at K=17
        for (int H : sizes) {
            run_cfg<17, 8, 17, 2, 2>(H, "rowffma2");
            run_cfg<17, 8, 17, 2, 2, 2, 1>(H, "rowf2-lock");
            run_cfg<17, 16, 17, 1, 2>(H, "16w-rowf2");
            run_cfg<17, 16, 17, 1, 1>(H, "16w1s");
            run_cfg<15, 8, 15, 2, 2, 1>(H, "k15rowf2");
            run_cfg<15, 8, 15, 2, 1, 1>(H, "k15base");
            run_cfg<13, 8, 13, 2, 2, 2>(H, "k13rowf2");
            run_cfg<13, 8, 13, 2, 1, 2, 1>(H, "k13lock");
        }
        return 0;
    }
    for (int H : sizes) {
        // K = 17: the product's tma2 (8 warps, 2 stages, FFMA2 column pass), its FFMA2 row pass,
        // split row chains, fewer warps with deeper rings, 4-warp CTAs x2 per SM
        run_cfg<17, 8, 17, 2, 1>(H, "base");
        run_cfg<17, 8, 17, 2, 2>(H, "rowffma2");
        run_cfg<17, 8, 17, 2, 3>(H, "split");
        run_cfg<17, 6, 17, 3, 1>(H, "6w3s");
        run_cfg<17, 6, 17, 3, 3>(H, "6w3s-spl");
        run_cfg<17, 4, 17, 2, 1>(H, "4w2s-x2", 2);
        run_cfg<17, 4, 17, 2, 3>(H, "4w2s-x2sp", 2);
        run_cfg<17, 4, 17, 3, 1>(H, "4w3s");
        run_cfg<17, 16, 17, 1, 1>(H, "16w1s");
        // K = 9 and 3
        run_cfg<9, 8, 9, 2, 1, 1>(H, "base");
        run_cfg<9, 8, 9, 2, 3, 1>(H, "split");
        run_cfg<9, 4, 9, 2, 1, 1>(H, "4w2s-x2", 2);
        run_cfg<9, 8, 9, 4, 1, 1>(H, "8w4s");
        run_cfg<3, 8, 6, 2, 1, 1>(H, "base");
        run_cfg<3, 8, 6, 6, 1, 1>(H, "8w6s");
        run_cfg<3, 4, 6, 2, 1, 1>(H, "4w2s-x2", 2);
    }
    return 0;
}
