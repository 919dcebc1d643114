// explore.cu -- design-space exploration for the streaming kernels on one B200 (not the
// product; the product's configurations live in sepconv_params.h).  Times stream_kernel
// instantiations with different warps/CTA, stage rows, stage counts, grid sizes and TMA
// L2 promotion on a 16384^2 image, next to a plain float4 copy of the same bytes.
//   nvcc -std=c++17 -O3 -gencode arch=compute_100a,code=sm_100a -I../paper_conf_asplos_phothilimthanaara13_b200/csrc explore.cu -o explore
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
static int H = 16384, W = 16384, SMS = 148;
static float *din, *dout;
static cudaEvent_t e0, e1;

__global__ void copy_kernel(const float4 *__restrict__ a, float4 *__restrict__ b, long long n) {
    for (long long i = blockIdx.x * (long long)blockDim.x + threadIdx.x; i < n; i += (long long)gridDim.x * blockDim.x)
        b[i] = a[i];
}

static int g_reps = 10, g_onlyK = 0;
template <typename F>
static float time_it_(F f, int reps);
template <typename F>
static float time_it(F f, int reps = -1) { return time_it_(f, reps < 0 ? g_reps : reps); }
template <typename F>
static float time_it_(F f, int reps) {
    std::vector<float> t;
    for (int r = 0; r < reps + 2; ++r) {
        cudaEventRecord(e0);
        f();
        cudaEventRecord(e1);
        cudaEventSynchronize(e1);
        float ms;
        cudaEventElapsedTime(&ms, e0, e1);
        if (r >= 2) t.push_back(ms * 1000.f);
    }
    std::sort(t.begin(), t.end());
    return t[t.size() / 2];
}

template <int K, int OP, int MAP, int NW, int SR, int NS, int F2 = 0, int SM = 1, int LOCK = 0>
static void run_cfg(int ctas_per_sm, CUtensorMapL2promotion prom, const char *tag, int parts = 0) {
    if (g_onlyK && g_onlyK != K) return;
    auto kern = stream_kernel<K, OP, MAP, NW, SR, NS, F2, SM, LOCK>;
    size_t smem = stream_smem_bytes<K, OP, MAP, NW, SR, NS, F2>();
    if (MAP == MAP_TMA && NW * NS * (((SR * stream_bw(K, OP) + 31) & ~31) * 4 + 8) > kSmemPerCta) { printf("skip\n"); return; }
    if (smem > 232448) { printf("skip (smem %zu)\n", smem); return; }
    cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
    int occ = 0;
    cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, kern, NW * 32, smem);
    int cps = std::min(ctas_per_sm, occ);
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
    if (MAP == MAP_TMA) {
        cuuint64_t dims[3] = {(cuuint64_t)W, (cuuint64_t)H, 1};
        cuuint64_t str[2] = {(cuuint64_t)W * 4, (cuuint64_t)H * W * 4};
        cuuint32_t box[3] = {(cuuint32_t)stream_bw(K, OP), (cuuint32_t)SR, 1}, es[3] = {1, 1, 1};
        CUresult r = enc(&p.tmap, CU_TENSOR_MAP_DATA_TYPE_FLOAT32, 3, din, dims, str, box, es, CU_TENSOR_MAP_INTERLEAVE_NONE,
                         CU_TENSOR_MAP_SWIZZLE_NONE, prom, CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
        if (r) { printf("encode failed %d\n", (int)r); return; }
    }
    int grid = SMS * cps;
    if (parts < 0) {   // auto: as many row parts as fit the grid
        parts = std::max(1, grid / p.nstrips);
        grid = std::min<long long>(grid, (long long)p.nstrips * parts);
    }
    p.parts = parts;
    float us = time_it([&] { kern<<<grid, NW * 32, smem>>>(p); });
    cudaError_t e = cudaGetLastError();
    double bytes = 4.0 * ((double)H * W + (double)(H - K + 1) * (W - K + 1));
    printf("K=%2d L=%d SM=%d F2=%d %-6s map=%d NW=%2d SR=%2d NS=%d cps=%d/%d prom=%d parts=%d grid=%d smem=%3zuKB : %7.1f us  %6.0f GB/s %s\n", K, LOCK, SM, F2, tag, MAP, NW,
           SR, NS, cps, occ, (int)prom, parts, grid, smem / 1024, us, bytes / us / 1e3, e ? cudaGetErrorString(e) : "");
}

int main(int argc, char **argv) {
    if (argc > 1) g_reps = atoi(argv[1]);
    if (argc > 2) g_onlyK = atoi(argv[2]);
    void *fp = nullptr;
    cudaDriverEntryPointQueryResult q;
    cudaGetDriverEntryPoint("cuTensorMapEncodeTiled", &fp, cudaEnableDefault, &q);
    enc = (EncodeTiledFn)fp;
    cudaDeviceProp prop;
    cudaGetDeviceProperties(&prop, 0);
    SMS = prop.multiProcessorCount;
    cudaMalloc(&din, (size_t)H * W * 4);
    cudaMalloc(&dout, (size_t)H * W * 4);
    cudaMemset(din, 0, (size_t)H * W * 4);
    cudaEventCreate(&e0);
    cudaEventCreate(&e1);
    long long n4 = (long long)H * W / 4;
    for (int g : {SMS * 16}) {
        float us = time_it([&] { copy_kernel<<<g, 512>>>((const float4 *)din, (float4 *)dout, n4); });
        printf("copy float4 grid=%d: %.1f us %.0f GB/s\n", g, us, 8.0 * H * W / us / 1e3);
    }
    const auto P0 = CU_TENSOR_MAP_L2_PROMOTION_NONE, P256 = CU_TENSOR_MAP_L2_PROMOTION_L2_256B,
               P128 = CU_TENSOR_MAP_L2_PROMOTION_L2_128B;
    run_cfg<17, OP_SEP, MAP_TMA, 16, 17, 1, 1, 2, 0>(1, P0, "x", -1);
    run_cfg<17, OP_SEP, MAP_TMA, 8, 17, 2, 1, 2, 0>(1, P0, "x", -1);
    run_cfg<15, OP_SEP, MAP_TMA, 16, 15, 1, 1, 1, 0>(1, P0, "x", -1);
    run_cfg<15, OP_SEP, MAP_TMA, 8, 15, 2, 1, 1, 0>(1, P0, "x", -1);
    run_cfg<13, OP_SEP, MAP_TMA, 16, 13, 1, 1, 1, 0>(1, P0, "x", -1);
    run_cfg<13, OP_SEP, MAP_TMA, 8, 13, 3, 1, 1, 0>(1, P0, "x", -1);
    run_cfg<11, OP_SEP, MAP_TMA, 16, 11, 1, 1, 1, 0>(1, P0, "x", -1);
    run_cfg<11, OP_SEP, MAP_TMA, 8, 11, 2, 1, 1, 1>(1, P0, "x", -1);
    run_cfg<9, OP_SEP, MAP_TMA, 8, 9, 2, 1, 2, 1>(1, P0, "x", -1);
    run_cfg<3, OP_SEP, MAP_TMA, 8, 6, 2, 1, 1, 0>(1, P0, "x", -1);
    run_cfg<5, OP_SEP, MAP_TMA, 8, 5, 2, 1, 2, 0>(1, P0, "x", -1);
    run_cfg<7, OP_SEP, MAP_TMA, 8, 7, 2, 1, 1, 0>(1, P0, "x", -1);
    return 0;
}
