// bs.cu -- Black-Scholes European option pricing on sm_100a (include/bs.h; PAPER.md
// P:1270-1276).
//
// One option per entry (reading B1), the textbook formula (B2) in float32 with the
// SFU lg2 / ex2 / rcp / rsqrt (B3) and a Chebyshev erfc (B5).  Purely elementwise: 12 B read and
// 8 B written per option; each thread prices 4 options from 16-byte loads (the scalar
// path takes unaligned pointers and the ragged tail).  The host variant streams chunks
// through a two-slot device workspace on two streams so the copy engines overlap.
#include <cuda_runtime.h>

#include <algorithm>
#include <cstdint>
#include <map>
#include <mutex>

#include "../../include/bs.h"
#include "sepconv_internal.h"

#include "bs_kernels.cuh"

namespace bs {

static int sms_of_current() {
    static std::mutex mu;
    static std::map<int, int> cache;
    int dev = 0;
    cudaGetDevice(&dev);
    std::lock_guard<std::mutex> lock(mu);
    auto it = cache.find(dev);
    if (it != cache.end()) return it->second;
    int sms = 0;
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev);
    cache[dev] = sms > 0 ? sms : 148;
    return cache[dev];
}

static cudaError_t launch(const float *s, const float *x, const float *t, long long n, float r, float v, float *call,
                          float *put, cudaStream_t st) {
    if (n <= 0) return cudaSuccess;
    const int sms = sms_of_current();
    const uintptr_t all = reinterpret_cast<uintptr_t>(s) | reinterpret_cast<uintptr_t>(x) |
                          reinterpret_cast<uintptr_t>(t) | reinterpret_cast<uintptr_t>(call) |
                          reinterpret_cast<uintptr_t>(put);
    long long done = 0;
    if ((all & 15u) == 0 && n >= 4) {
        const long long n4 = n / 4;
        // one float4 group (4 options) per thread, one thread per group: a plain (not persistent)
        // grid, so the hardware block scheduler keeps every SM full to the end.  Round 1 picked a
        // persistent grid of 4 CTAs per SM with 2 groups per thread per trip (860 us on 2^28);
        // against it the plain grid is 12-14% faster from 4M options up (2^26: 195 vs 225 us,
        // 6.9 TB/s) and equal at 500 000 (tools/bs_small.cu, profiles/r02_bs_small.txt)
        const long long blocks = std::min<long long>((n4 + kThreads - 1) / kThreads, 1LL << 30);
        auto kern = bs_kernel_vec<1>;
        kern<<<static_cast<int>(blocks), kThreads, 0, st>>>(
            reinterpret_cast<const float4 *>(s), reinterpret_cast<const float4 *>(x), reinterpret_cast<const float4 *>(t),
            n4, r, v, 1.0f / v, reinterpret_cast<float4 *>(call), reinterpret_cast<float4 *>(put));
        sepconv::g_launches.fetch_add(1, std::memory_order_relaxed);
        done = n4 * 4;
    }
    if (done < n) {
        const long long rem = n - done;
        const long long blocks = std::min<long long>((rem + kThreads - 1) / kThreads, static_cast<long long>(sms) * 8);
        bs_kernel_scalar<<<static_cast<int>(blocks), kThreads, 0, st>>>(s + done, x + done, t + done, rem, r, v,
                                                                        1.0f / v, call + done, put + done);
        sepconv::g_launches.fetch_add(1, std::memory_order_relaxed);
    }
    return cudaGetLastError();
}

// host pipeline workspace, one per device
struct HostWs {
    static constexpr long long kChunk = 8LL << 20;   // options per chunk (160 MB of device buffers per slot)
    float *buf[2] = {nullptr, nullptr};               // per slot: s, x, t, call, put
    cudaStream_t st[2] = {nullptr, nullptr};
    cudaEvent_t ev[2] = {nullptr, nullptr};
};

static HostWs *host_ws(sepconv_status_t *status) {
    static std::mutex mu;
    static std::map<int, HostWs *> all;
    int dev = 0;
    cudaGetDevice(&dev);
    std::lock_guard<std::mutex> lock(mu);
    auto it = all.find(dev);
    if (it != all.end()) return it->second;
    HostWs *w = new HostWs;
    for (int i = 0; i < 2; ++i) {
        cudaError_t e = cudaMalloc(&w->buf[i], 5 * HostWs::kChunk * sizeof(float));
        if (e == cudaSuccess) e = cudaStreamCreateWithFlags(&w->st[i], cudaStreamNonBlocking);
        if (e == cudaSuccess) e = cudaEventCreateWithFlags(&w->ev[i], cudaEventDisableTiming);
        if (e != cudaSuccess) {
            *status = sepconv::cuda_fail(e, "bs_price_host workspace");
            return nullptr;
        }
    }
    all[dev] = w;
    return w;
}

}  // namespace bs

using sepconv::cuda_fail;
using sepconv::fail;

static bool bs_overlap(const void *a, const void *b, size_t bytes) {
    const uintptr_t x = reinterpret_cast<uintptr_t>(a), y = reinterpret_cast<uintptr_t>(b);
    return x < y + bytes && y < x + bytes;
}

static sepconv_status_t bs_check(const float *s, const float *x, const float *t, int64_t n, float v, float *call,
                                 float *put) {
    if (n < 0) return fail(SEPCONV_E_INVALID, "n = %lld < 0", static_cast<long long>(n));
    if (!(v > 0.f)) return fail(SEPCONV_E_INVALID, "volatility %g must be > 0", static_cast<double>(v));
    if (n == 0) return SEPCONV_OK;
    if (!s || !x || !t || !call || !put) return fail(SEPCONV_E_INVALID, "NULL pointer");
    const uintptr_t all = reinterpret_cast<uintptr_t>(s) | reinterpret_cast<uintptr_t>(x) |
                          reinterpret_cast<uintptr_t>(t) | reinterpret_cast<uintptr_t>(call) |
                          reinterpret_cast<uintptr_t>(put);
    if (all & 3u) return fail(SEPCONV_E_ALIGN, "pointers must be 4-byte aligned");
    const size_t bytes = static_cast<size_t>(n) * sizeof(float);
    const void *ins[3] = {s, x, t};
    for (const void *in : ins)
        if (bs_overlap(in, call, bytes) || bs_overlap(in, put, bytes))
            return fail(SEPCONV_E_ALIAS, "an output overlaps an input");
    if (bs_overlap(call, put, bytes)) return fail(SEPCONV_E_ALIAS, "call and put overlap");
    return SEPCONV_OK;
}

extern "C" {

sepconv_status_t bs_price(const float *s, const float *x, const float *t, int64_t n, float r, float v, float *call,
                          float *put, sepconv_stream_t stream) {
    if (sepconv_status_t st = bs_check(s, x, t, n, v, call, put)) return st;
    cudaError_t e = bs::launch(s, x, t, n, r, v, call, put, static_cast<cudaStream_t>(stream));
    if (e != cudaSuccess) return cuda_fail(e, "bs kernel launch");
    return SEPCONV_OK;
}

sepconv_status_t bs_price_host(const float *s, const float *x, const float *t, int64_t n, float r, float v,
                               float *call, float *put, sepconv_stream_t stream) {
    if (sepconv_status_t st = bs_check(s, x, t, n, v, call, put)) return st;
    if (n == 0) return SEPCONV_OK;
    sepconv_status_t status = SEPCONV_OK;
    bs::HostWs *w = bs::host_ws(&status);
    if (!w) return status;
    cudaStream_t user = static_cast<cudaStream_t>(stream);
    cudaEvent_t start;
    SC_CUDA(cudaEventCreateWithFlags(&start, cudaEventDisableTiming));
    SC_CUDA(cudaEventRecord(start, user));
    for (int i = 0; i < 2; ++i) SC_CUDA(cudaStreamWaitEvent(w->st[i], start, 0));
    const long long C = bs::HostWs::kChunk;
    long long chunk = 0;
    for (long long off = 0; off < n; off += C, ++chunk) {
        const long long m = std::min(C, n - off);
        const int slot = static_cast<int>(chunk & 1);
        cudaStream_t st = w->st[slot];
        float *d = w->buf[slot];
        float *ds = d, *dx = d + C, *dt = d + 2 * C, *dc = d + 3 * C, *dp = d + 4 * C;
        const size_t b = static_cast<size_t>(m) * sizeof(float);
        SC_CUDA(cudaMemcpyAsync(ds, s + off, b, cudaMemcpyHostToDevice, st));
        SC_CUDA(cudaMemcpyAsync(dx, x + off, b, cudaMemcpyHostToDevice, st));
        SC_CUDA(cudaMemcpyAsync(dt, t + off, b, cudaMemcpyHostToDevice, st));
        cudaError_t e = bs::launch(ds, dx, dt, m, r, v, dc, dp, st);
        if (e != cudaSuccess) return cuda_fail(e, "bs kernel launch");
        SC_CUDA(cudaMemcpyAsync(call + off, dc, b, cudaMemcpyDeviceToHost, st));
        SC_CUDA(cudaMemcpyAsync(put + off, dp, b, cudaMemcpyDeviceToHost, st));
    }
    for (int i = 0; i < 2; ++i) {
        SC_CUDA(cudaEventRecord(w->ev[i], w->st[i]));
        SC_CUDA(cudaStreamWaitEvent(user, w->ev[i], 0));
    }
    cudaEventDestroy(start);
    SC_CUDA(cudaStreamSynchronize(user));
    return SEPCONV_OK;
}

}  // extern "C"
