// cta_trace.cu -- where does a pass's time go across SMs? (not the product)  Runs fused
// configurations once after a clean L2 flush with a per-CTA trace (globaltimer at CTA start and
// end, SM id, segments; compiled in only under SEPCONV_CTA_TRACE) and prints the start skew, the
// spread of CTA durations and the slowest SMs, for the mid-size imbalance of DESIGN.md section 6.
//   nvcc -std=c++17 -O3 -DSEPCONV_CTA_TRACE -gencode arch=compute_100a,code=sm_100a \
//        -I../paper_conf_asplos_phothilimthanaara13_b200/csrc cta_trace.cu -o cta_trace -lcuda
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
static float *din, *dout, *wfl, *rfl, *sink;
static unsigned long long *dtrace;
static long long fl_n4;

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

template <int K, int NW, int SR, int NS, int F2, int SM = 2, int LOCK = 0>
static void trace_cfg(int H, const char *tag, int parts_mult = 1, int Win = 0) {
    const int W = Win ? Win : H;
    auto kern = stream_kernel<K, OP_SEP, MAP_TMA, NW, SR, NS, F2, SM, LOCK>;
    const size_t smem = stream_smem_bytes<K, OP_SEP, MAP_TMA, NW, SR, NS, F2>();
    cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
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
    p.trace = dtrace;
    cuuint64_t dims[3] = {(cuuint64_t)W, (cuuint64_t)H, 1};
    cuuint64_t str[2] = {(cuuint64_t)W * 4, (cuuint64_t)H * W * 4};
    cuuint32_t box[3] = {(cuuint32_t)stream_bw(K, OP_SEP), (cuuint32_t)SR, 1}, es[3] = {1, 1, 1};
    enc(&p.tmap, CU_TENSOR_MAP_DATA_TYPE_FLOAT32, 3, din, dims, str, box, es, CU_TENSOR_MAP_INTERLEAVE_NONE,
        CU_TENSOR_MAP_SWIZZLE_NONE, CU_TENSOR_MAP_L2_PROMOTION_L2_256B, CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
    const int slots = 148;
    p.parts = std::max(1, slots / p.nstrips) * parts_mult;
    const int grid = std::min<long long>(slots, (long long)p.nstrips * p.parts);
    for (int rep = 0; rep < 3; ++rep) {                 // the last repetition is reported
        fill_k<<<148 * 8, 256>>>((float4 *)wfl, fl_n4);
        read_k<<<148 * 8, 256>>>((const float4 *)rfl, fl_n4, sink);
        kern<<<grid, NW * 32, smem>>>(p);
        cudaDeviceSynchronize();
    }
    std::vector<unsigned long long> t(4 * grid);
    cudaMemcpy(t.data(), dtrace, t.size() * 8, cudaMemcpyDeviceToHost);
    unsigned long long s0 = ~0ull, s1 = 0, e0 = ~0ull, e1 = 0;
    std::vector<double> dur(grid);
    for (int b = 0; b < grid; ++b) {
        s0 = std::min(s0, t[4 * b]); s1 = std::max(s1, t[4 * b]);
        e0 = std::min(e0, t[4 * b + 1]); e1 = std::max(e1, t[4 * b + 1]);
        dur[b] = (t[4 * b + 1] - t[4 * b]) * 1e-3;
    }
    std::vector<int> order(grid);
    for (int b = 0; b < grid; ++b) order[b] = b;
    std::sort(order.begin(), order.end(), [&](int a, int c) { return dur[a] > dur[c]; });
    double avg = 0;
    for (double d : dur) avg += d;
    avg /= grid;
    printf("H=%5d K=%2d %-8s grid=%d parts=%d: start skew %.2f us, CTA duration min %.2f avg %.2f max %.2f us, "
           "first end %.2f, last end %.2f us after first start\n", H, K, tag, grid, p.parts, (s1 - s0) * 1e-3,
           dur[order.back()], avg, dur[order[0]], (e0 - s0) * 1e-3, (e1 - s0) * 1e-3);
    printf("    slowest CTAs (block: SM, us, segments):");
    for (int i = 0; i < 6; ++i) {
        const int b = order[i];
        printf(" %d:%llu,%.1f,%llu", b, t[4 * b + 2], dur[b], t[4 * b + 3]);
    }
    printf("\n    fastest CTAs:");
    for (int i = 0; i < 4; ++i) {
        const int b = order[grid - 1 - i];
        printf(" %d:%llu,%.1f,%llu", b, t[4 * b + 2], dur[b], t[4 * b + 3]);
    }
    printf("\n");
    if (getenv("CTA_TRACE_STRIPS")) {                    // mean CTA duration per CTA strip
        printf("    W=%d strips=%d by strip:", W, p.nstrips);
        for (int q = 0; q < p.nstrips; ++q) {
            double sum = 0;
            int cnt = 0;
            for (int b = q; b < grid; b += p.nstrips) sum += dur[b], ++cnt;
            printf(" %.1f", cnt ? sum / cnt : 0.0);
        }
        printf("\n");
    }
    if (getenv("CTA_TRACE_DUMP")) {                      // per-SM duration, for stability checks
        printf("    dump %s H=%d K=%d:", tag, H, K);
        for (int b = 0; b < grid; ++b) printf(" %llu:%.2f", t[4 * b + 2], dur[b]);
        printf("\n");
    }
    fflush(stdout);
}

int main(int argc, char **argv) {
    void *fp = nullptr;
    cudaDriverEntryPointQueryResult q;
    cudaGetDriverEntryPoint("cuTensorMapEncodeTiled", &fp, cudaEnableDefault, &q);
    enc = (EncodeTiledFn)fp;
    cudaDeviceProp prop;
    cudaGetDeviceProperties(&prop, 0);
    const size_t big = (size_t)16384 * 17440 * 4;
    cudaMalloc(&din, big);
    cudaMalloc(&dout, big);
    cudaMemset(din, 0, big);
    fl_n4 = 2LL * prop.l2CacheSize / 16;
    cudaMalloc(&wfl, fl_n4 * 16);
    cudaMalloc(&rfl, fl_n4 * 16);
    cudaMalloc(&sink, 16);
    cudaMalloc(&dtrace, 4 * 4096 * 8);
    cudaMemset(rfl, 0, fl_n4 * 16);
    if (argc > 1 && !strcmp(argv[1], "strips")) {         // which strips are slow, and why
        for (int W : {16384, 16400, 16128, 15376, 17424}) trace_cfg<17, 8, 17, 2, 2>(16384, "tma4", 1, W);
        for (int W : {16384, 16400}) trace_cfg<9, 8, 9, 2, 1, 2, 1>(16384, "tma0", 1, W);
        return 0;
    }
    if (argc > 1 && !strcmp(argv[1], "mid")) {            // mid sizes after the right-edge change
        for (int rep = 0; rep < 2; ++rep)
            for (int H : {2048, 4096}) {
                trace_cfg<17, 8, 17, 2, 2>(H, "tma4");
                trace_cfg<17, 8, 17, 2, 1>(H, "tma2");
                trace_cfg<17, 16, 17, 1, 1>(H, "tma3");
                trace_cfg<9, 8, 9, 2, 1, 2, 1>(H, "tma0");
            }
        return 0;
    }
    if (argc > 1 && !strcmp(argv[1], "stability")) {      // the same launches repeated
        for (int rep = 0; rep < 3; ++rep) {
            trace_cfg<17, 8, 17, 2, 2>(16384, "tma4");
            trace_cfg<17, 8, 17, 2, 1>(16384, "tma2");
            trace_cfg<9, 8, 9, 2, 1, 2, 1>(16384, "tma0");
            trace_cfg<17, 8, 17, 2, 2>(4096, "tma4");
        }
        return 0;
    }
    for (int H : {2048, 4096, 16384}) {
        trace_cfg<17, 8, 17, 2, 2>(H, "tma4");
        trace_cfg<17, 8, 17, 2, 1>(H, "tma2");
        trace_cfg<17, 16, 17, 1, 1>(H, "tma3");
        trace_cfg<9, 8, 9, 2, 1, 2, 1>(H, "tma0");
        trace_cfg<3, 8, 6, 2, 1, 1>(H, "tma2");
    }
    trace_cfg<17, 8, 17, 2, 2>(16384, "tma4x3", 3);
    return 0;
}
