// latency_probe.cu -- what a CUDA-event pair around ONE kernel measures on this B200 when
// the kernel follows an L2 flush (not the product; evidence for DESIGN.md section 9).
//   nvcc -std=c++17 -O3 -gencode arch=compute_100a,code=sm_100a latency_probe.cu -o latency_probe
// Prints, for an empty kernel and for a kernel that only touches 200 KB of dynamic shared
// memory, the median event time around the kernel after (a) a flush by kernels that use no
// shared memory and (b) the same flush kernels set to the max-shared carveout, plus the
// marginal cost of the kernel inside a batch of [flush, kernel] pairs.
#include <cuda_runtime.h>

#include <algorithm>
#include <cstdio>
#include <vector>

__global__ void fill_k(float4 *p, long long n) {
    for (long long i = blockIdx.x * (long long)blockDim.x + threadIdx.x; i < n; i += (long long)gridDim.x * blockDim.x)
        p[i] = make_float4(1.f, 1.f, 1.f, 1.f);
}
__global__ void read_k(const float4 *p, long long n, float *sink) {
    float a = 0.f;
    for (long long i = blockIdx.x * (long long)blockDim.x + threadIdx.x; i < n; i += (long long)gridDim.x * blockDim.x)
        a += p[i].x;
    if (a < 0.f) *sink = a;
}
__global__ void empty_k() {}
__global__ void smem_k(float *sink) {
    extern __shared__ float s[];
    s[threadIdx.x] = threadIdx.x;
    __syncthreads();
    if (s[(threadIdx.x + 1) % blockDim.x] < 0.f) *sink = 1.f;
}

int main() {
    int l2 = 0;
    cudaDeviceGetAttribute(&l2, cudaDevAttrL2CacheSize, 0);
    const long long n4 = 2LL * l2 / 16;
    float4 *w, *r;
    float *sink;
    cudaMalloc(&w, n4 * 16);
    cudaMalloc(&r, n4 * 16);
    cudaMalloc(&sink, 16);
    cudaMemset(r, 0, n4 * 16);
    const int smem = 200 * 1024;
    cudaFuncSetAttribute(smem_k, cudaFuncAttributeMaxDynamicSharedMemorySize, smem);
    cudaEvent_t e0, e1;
    cudaEventCreate(&e0);
    cudaEventCreate(&e1);
    auto flush = [&]() {
        fill_k<<<148 * 8, 256>>>(w, n4);
        read_k<<<148 * 8, 256>>>(r, n4, sink);
    };
    auto single = [&](auto kern, const char *name) {
        std::vector<float> t;
        for (int i = 0; i < 60; ++i) {
            flush();
            cudaEventRecord(e0);
            kern();
            cudaEventRecord(e1);
            cudaEventSynchronize(e1);
            float ms;
            cudaEventElapsedTime(&ms, e0, e1);
            if (i >= 10) t.push_back(ms * 1000.f);
        }
        std::sort(t.begin(), t.end());
        float mean = 0;
        for (float x : t) mean += x;
        printf("%-44s single-event median %6.2f us  mean %6.2f us  min %6.2f\n", name, t[t.size() / 2], mean / t.size(),
               t[0]);
    };
    auto batch = [&](auto body, int n) {
        body();
        cudaDeviceSynchronize();
        cudaEventRecord(e0);
        for (int i = 0; i < n; ++i) body();
        cudaEventRecord(e1);
        cudaEventSynchronize(e1);
        float ms;
        cudaEventElapsedTime(&ms, e0, e1);
        return ms * 1000.f / n;
    };
    auto empty = [&]() { empty_k<<<148, 256>>>(); };
    auto sm = [&]() { smem_k<<<148, 256, smem>>>(sink); };
    for (int carve = 0; carve < 2; ++carve) {
        if (carve) {
            cudaFuncSetAttribute(fill_k, cudaFuncAttributePreferredSharedMemoryCarveout, 100);
            cudaFuncSetAttribute(read_k, cudaFuncAttributePreferredSharedMemoryCarveout, 100);
        }
        printf("-- flush kernels carveout: %s\n", carve ? "max shared" : "default");
        single(empty, "empty kernel 148x256");
        single(sm, "200 KB smem kernel 148x256");
        const float tf = batch(flush, 200);
        printf("%-44s marginal in [flush, kernel] x200: %6.2f us\n", "empty kernel",
               batch([&]() { flush(); empty(); }, 200) - tf);
        printf("%-44s marginal in [flush, kernel] x200: %6.2f us\n", "200 KB smem kernel",
               batch([&]() { flush(); sm(); }, 200) - tf);
        printf("%-44s back-to-back x1000: %6.2f us\n", "empty kernel", batch(empty, 1000));
        printf("%-44s back-to-back x1000: %6.2f us\n", "200 KB smem kernel", batch(sm, 1000));
    }
    return 0;
}
