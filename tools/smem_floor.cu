// smem_floor.cu -- does a kernel that needs ~200 KB of dynamic shared memory pay an L1/shared
// carveout change after the clean flush (whose kernels use no shared memory)?  Marginal time of an
// empty 148-CTA kernel after the flush, with 0 and with 200 KB of dynamic shared memory, and the
// same with the flush kernels' preferred carveout set to the maximum shared-memory split.
//   nvcc -std=c++17 -O3 -gencode arch=compute_100a,code=sm_100a smem_floor.cu -o smem_floor
#include <cuda_runtime.h>

#include <algorithm>
#include <cstdio>

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
__global__ void empty_k(float *s, int use) {
    extern __shared__ float sm[];
    if (use && threadIdx.x == 1023) s[0] = sm[0];
}

static float *wfl, *rfl, *sink;
static long long fl_n4;
static cudaEvent_t e0, e1;
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
static float marginal(F f) {
    float t[5];
    for (int b = 0; b < 5; ++b) {
        const float tf = batch(flush, 60);
        t[b] = batch([&] { flush(); f(); }, 60) - tf;
    }
    std::sort(t, t + 5);
    return t[2];
}

int main() {
    cudaDeviceProp prop;
    cudaGetDeviceProperties(&prop, 0);
    fl_n4 = 2LL * prop.l2CacheSize / 16;
    cudaMalloc(&wfl, fl_n4 * 16);
    cudaMalloc(&rfl, fl_n4 * 16);
    cudaMalloc(&sink, 16);
    cudaMemset(rfl, 0, fl_n4 * 16);
    cudaEventCreate(&e0);
    cudaEventCreate(&e1);
    const int big = 200 * 1024;
    cudaFuncSetAttribute(empty_k, cudaFuncAttributeMaxDynamicSharedMemorySize, big);
    for (int carve = 0; carve < 2; ++carve) {
        if (carve) {
            cudaFuncSetAttribute(fill_k, cudaFuncAttributePreferredSharedMemoryCarveout, 100);
            cudaFuncSetAttribute(read_k, cudaFuncAttributePreferredSharedMemoryCarveout, 100);
        }
        for (int smem : {0, 48 * 1024, big}) {
            for (int threads : {256, 1024}) {
                const float us = marginal([&] { empty_k<<<148, threads, smem>>>(sink, smem > 0); });
                printf("flush carveout %-8s empty kernel 148 x %4d threads, %6d B dynamic smem: %6.2f us marginal\n",
                       carve ? "max-smem" : "default", threads, smem, us);
            }
        }
        const float tf = batch(flush, 60);
        printf("flush carveout %-8s flush alone %.2f us\n", carve ? "max-smem" : "default", tf);
    }
    printf("%s\n", cudaGetErrorString(cudaGetLastError()));
    return 0;
}
