// bs_small.cu -- Black-Scholes at the paper's 500 000 options: grid / vector-width
// variants of the product kernels, marginal time after the clean flush (write 2 x L2, read 2 x L2;
// event time of n x [flush, pass] minus n x [flush]).  Exploration only.
//   nvcc -std=c++17 -O3 -gencode arch=compute_100a,code=sm_100a -I../paper_conf_asplos_phothilimthanaara13_b200/csrc \
//        bs_small.cu -o bs_small
#include <cuda_runtime.h>

#include <algorithm>
#include <cstdio>
#include <cstdlib>
#include <vector>

#include "bs_kernels.cuh"

using namespace bs;

// two options per thread from 8-byte loads
__global__ void bs_kernel_f2(const float2 *__restrict__ s, const float2 *__restrict__ x, const float2 *__restrict__ t,
                             long long n2, float r, float v, float inv_v, float2 *__restrict__ call,
                             float2 *__restrict__ put) {
    for (long long i = blockIdx.x * (long long)blockDim.x + threadIdx.x; i < n2; i += (long long)gridDim.x * blockDim.x) {
        const float2 S = __ldcs(s + i), X = __ldcs(x + i), T = __ldcs(t + i);
        float2 c, p;
        price1(S.x, X.x, T.x, r, v, inv_v, c.x, p.x);
        price1(S.y, X.y, T.y, r, v, inv_v, c.y, p.y);
        __stcs(call + i, c);
        __stcs(put + i, p);
    }
}

static float *wfl, *rfl, *sink;
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
static float marginal(F f) {
    float t[5];
    for (int b = 0; b < 5; ++b) {
        const float tf = batch(flush, 60);
        t[b] = batch([&] { flush(); f(); }, 60) - tf;
    }
    std::sort(t, t + 5);
    return t[2];
}

__global__ void init_k(float *s, float *x, float *t, long long n) {
    for (long long i = blockIdx.x * (long long)blockDim.x + threadIdx.x; i < n; i += (long long)gridDim.x * blockDim.x) {
        const unsigned h = (unsigned)(i * 2654435761u);
        s[i] = 5.f + 25.f * (h & 0xffff) / 65536.f;
        x[i] = 1.f + 99.f * (h >> 16) / 65536.f;
        t[i] = 0.25f + 9.75f * ((h * 7u) & 0xffff) / 65536.f;
    }
}

int main(int argc, char **argv) {
    std::vector<long long> sizes;
    for (int i = 1; i < argc; ++i) sizes.push_back(atoll(argv[i]));
    if (sizes.empty()) sizes = {500000, 1 << 20, 1 << 22};
    cudaDeviceProp prop;
    cudaGetDeviceProperties(&prop, 0);
    const int sms = prop.multiProcessorCount;
    fl_n4 = 2LL * prop.l2CacheSize / 16;
    cudaMalloc(&wfl, fl_n4 * 16);
    cudaMalloc(&rfl, fl_n4 * 16);
    cudaMalloc(&sink, 16);
    cudaMemset(rfl, 0, fl_n4 * 16);
    cudaEventCreate(&e0);
    cudaEventCreate(&e1);
    const long long nmax = *std::max_element(sizes.begin(), sizes.end());
    float *s, *x, *t, *c, *p;
    for (float **a : {&s, &x, &t, &c, &p}) cudaMalloc(a, nmax * 4);
    init_k<<<1024, 256>>>(s, x, t, nmax);
    const float r = 0.02f, v = 0.30f, iv = 1.0f / v;
    const float empty_us = marginal([&] { fill_k<<<sms, 256>>>((float4 *)c, 0); });
    printf("empty %d-CTA kernel: %.2f us marginal\n", sms, empty_us);
    for (long long n : sizes) {
        const long long n4 = n / 4, n2 = n / 2;
        const double bytes = 20.0 * n;
        auto rep = [&](const char *tag, float us) {
            printf("n=%9lld %-34s %7.2f us  %7.1f G opt/s  %6.0f GB/s\n", n, tag, us, n / us / 1e3, bytes / us / 1e3);
        };
        auto vec = [&](auto kern, int threads, long long cap, const char *tag) {
            const long long blocks = std::min<long long>((n4 + threads - 1) / threads, cap);
            rep(tag, marginal([&] {
                    kern<<<(int)blocks, threads>>>((const float4 *)s, (const float4 *)x, (const float4 *)t, n4, r, v, iv,
                                                   (float4 *)c, (float4 *)p);
                }));
        };
        vec(bs_kernel_vec<2>, 256, 4LL * sms, "product vec<2> 256t <=4/SM");
        vec(bs_kernel_vec<1>, 256, 1LL << 30, "vec<1> 256t one group/thread");
        vec(bs_kernel_vec<1>, 128, 1LL << 30, "vec<1> 128t one group/thread");
        vec(bs_kernel_vec<1>, 64, 1LL << 30, "vec<1> 64t one group/thread");
        for (int th : {128, 256}) {
            const long long blocks = (n2 + th - 1) / th;
            char tag[64];
            snprintf(tag, sizeof tag, "f2 %dt one pair/thread", th);
            rep(tag, marginal([&] {
                    bs_kernel_f2<<<(int)blocks, th>>>((const float2 *)s, (const float2 *)x, (const float2 *)t, n2, r, v,
                                                      iv, (float2 *)c, (float2 *)p);
                }));
        }
        for (int th : {128, 256}) {
            const long long blocks = (n + th - 1) / th;
            char tag[64];
            snprintf(tag, sizeof tag, "scalar %dt one option/thread", th);
            rep(tag, marginal([&] { bs_kernel_scalar<<<(int)blocks, th>>>(s, x, t, n, r, v, iv, c, p); }));
        }
    }
    printf("%s\n", cudaGetErrorString(cudaGetLastError()));
    return 0;
}
