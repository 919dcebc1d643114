// bs.cu -- Black-Scholes European option pricing on sm_100a (include/bs.h; PAPER.md
// P:1270-1276).
//
// One option per entry (reading B1), the textbook formula (B2) in float32 with the
// accurate libdevice logf / expf / erfcf and SFU reciprocals (B3).  Purely elementwise: 12 B read and
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

namespace bs {

constexpr int kThreads = 256;

// The kernel is issue-bound (ncu: 83% issue-active at 180 instructions per option with IEEE
// division and sqrt), so the two divisions and the square root use the SFU: 1/(v sqrt T) =
// rsqrt(T) / v (1/v formed once on the host), sqrt T = T rsqrt(T), S/X = __fdividef.  Each
// adds ~2 ulp to d1 or to the quotient inside the log, inside the B4 bound.
__device__ __forceinline__ void price1(float S, float X, float T, float r, float v, float inv_v, float &call,
                                       float &put) {
    const float rs = rsqrtf(T);
    const float vs = v * (T * rs);                      // v sqrt T
    const float d1 = (logf(__fdividef(S, X)) + (r + 0.5f * v * v) * T) * (rs * inv_v);
    const float d2 = d1 - vs;
    const float disc = X * expf(-r * T);
    const float k = 0.70710678118654752f;             // 1 / sqrt 2
    const float n1 = 0.5f * erfcf(-d1 * k);            // N(d1)
    const float n2 = 0.5f * erfcf(-d2 * k);            // N(d2)
    call = S * n1 - disc * n2;
    put = disc * (1.0f - n2) - S * (1.0f - n1);        // N(-d) = 1 - N(d)
}

__global__ void __launch_bounds__(kThreads) bs_kernel_vec(const float4 *__restrict__ s, const float4 *__restrict__ x,
                                                          const float4 *__restrict__ t, long long n4, float r, float v,
                                                          float inv_v, float4 *__restrict__ call, float4 *__restrict__ put) {
    for (long long i = blockIdx.x * static_cast<long long>(blockDim.x) + threadIdx.x; i < n4;
         i += static_cast<long long>(gridDim.x) * blockDim.x) {
        const float4 S = __ldcs(s + i), X = __ldcs(x + i), T = __ldcs(t + i);    // streamed once
        float4 c, p;
        price1(S.x, X.x, T.x, r, v, inv_v, c.x, p.x);
        price1(S.y, X.y, T.y, r, v, inv_v, c.y, p.y);
        price1(S.z, X.z, T.z, r, v, inv_v, c.z, p.z);
        price1(S.w, X.w, T.w, r, v, inv_v, c.w, p.w);
        __stcs(call + i, c);
        __stcs(put + i, p);
    }
}

__global__ void __launch_bounds__(kThreads) bs_kernel_scalar(const float *__restrict__ s, const float *__restrict__ x,
                                                             const float *__restrict__ t, long long n, float r, float v,
                                                             float inv_v, float *__restrict__ call, float *__restrict__ put) {
    for (long long i = blockIdx.x * static_cast<long long>(blockDim.x) + threadIdx.x; i < n;
         i += static_cast<long long>(gridDim.x) * blockDim.x) {
        float c, p;
        price1(s[i], x[i], t[i], r, v, inv_v, c, p);
        call[i] = c;
        put[i] = p;
    }
}

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
        const long long blocks = std::min<long long>((n4 + kThreads - 1) / kThreads, static_cast<long long>(sms) * 8);
        bs_kernel_vec<<<static_cast<int>(blocks), kThreads, 0, st>>>(
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
