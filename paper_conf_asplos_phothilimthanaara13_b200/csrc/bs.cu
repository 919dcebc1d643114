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

namespace bs {

constexpr int kThreads = 256;

// SFU approximations, flush-to-zero (inputs here are never denormal: S, X, T > 0 are
// normal and 1 + z/2 >= 1; an ex2 result below 2^-126 flushes to 0, an absolute error
// below 1e-38).  One MUFU instruction each, without the denormal rescaling libdevice
// and the non-ftz intrinsics wrap around them.
__device__ __forceinline__ float rcp_ftz(float x) {
    float y;
    asm("rcp.approx.ftz.f32 %0, %1;" : "=f"(y) : "f"(x));
    return y;
}
__device__ __forceinline__ float rsqrt_ftz(float x) {
    float y;
    asm("rsqrt.approx.ftz.f32 %0, %1;" : "=f"(y) : "f"(x));
    return y;
}
__device__ __forceinline__ float ex2_ftz(float x) {
    float y;
    asm("ex2.approx.ftz.f32 %0, %1;" : "=f"(y) : "f"(x));
    return y;
}
__device__ __forceinline__ float lg2_ftz(float x) {
    float y;
    asm("lg2.approx.ftz.f32 %0, %1;" : "=f"(y) : "f"(x));
    return y;
}

constexpr float kLn2 = 0.69314718055994531f;
constexpr float kLog2e = 1.44269504088896341f;

// The kernel was issue-bound (ncu: 85% issue-active at 159 instructions per option with
// libdevice logf/expf/erfcf), so every transcendental is one SFU instruction plus FMAs
// (reading B3): 1/(v sqrt T) = rsqrt(T) / v (1/v formed once on the host), sqrt T =
// T rsqrt(T), ln(S/X) = ln2 lg2(S rcp(X)), e^{-rT} = ex2(-rT log2e).  Each adds a few
// ulp (lg2.approx: ~2^-22 absolute) to d1, to the discount or to the tail below --
// inside the B4 bound, whose d1 allowance is 16 eps (|ln S/X| + 1 + ...)/(v sqrt T).
//
// The normal CDF (reading B5): N(d) and its complement 1 - N(d) from one tail value
// e = erfc(|d|/sqrt 2)/2 -- N(d) = 1 - e, 1 - N(d) = e for d >= 0 and the other way
// round for d < 0 -- so the put's N(-d) is never formed by cancellation.  erfc on
// [0, inf) is the Chebyshev fit of Numerical Recipes (Press et al., 2nd ed., section
// 6.2, "erfcc"): erfc(z) = t exp(-z^2 + P(t)), t = 1/(1 + z/2), P of degree 9, fractional
// error < 1.2e-7 everywhere; here ~15 instructions (an SFU reciprocal, 11 FMAs, ex2)
// against ~40 for libdevice erfcf.  Float32 evaluation adds |z^2| 2^-24 relative in the
// exponent, negligible where the tail matters.
__device__ __forceinline__ float erfc_tail(float z) {   // z >= 0
    const float t = rcp_ftz(fmaf(0.5f, z, 1.0f));
    float p = 0.17087277f;
    p = fmaf(p, t, -0.82215223f);
    p = fmaf(p, t, 1.48851587f);
    p = fmaf(p, t, -1.13520398f);
    p = fmaf(p, t, 0.27886807f);
    p = fmaf(p, t, -0.18628806f);
    p = fmaf(p, t, 0.09678418f);
    p = fmaf(p, t, 0.37409196f);
    p = fmaf(p, t, 1.00002368f);
    p = fmaf(p, t, -1.26551223f);
    return t * ex2_ftz(fmaf(-z, z, p) * kLog2e);
}

__device__ __forceinline__ void price1(float S, float X, float T, float r, float v, float inv_v, float &call,
                                       float &put) {
    const float rs = rsqrt_ftz(T);
    const float vs = v * (T * rs);                      // v sqrt T
    const float d1 = fmaf(kLn2, lg2_ftz(S * rcp_ftz(X)), (r + 0.5f * v * v) * T) * (rs * inv_v);
    const float d2 = d1 - vs;
    const float disc = X * ex2_ftz((-r * kLog2e) * T);
    const float k = 0.70710678118654752f;             // 1 / sqrt 2
    const float e1 = 0.5f * erfc_tail(fabsf(d1) * k);
    const float e2 = 0.5f * erfc_tail(fabsf(d2) * k);
    const float n1 = d1 >= 0.f ? 1.0f - e1 : e1;       // N(d1)
    const float m1 = d1 >= 0.f ? e1 : 1.0f - e1;       // N(-d1)
    const float n2 = d2 >= 0.f ? 1.0f - e2 : e2;
    const float m2 = d2 >= 0.f ? e2 : 1.0f - e2;
    call = S * n1 - disc * n2;
    put = disc * m2 - S * m1;
}

// U float4 groups per thread per trip (stride apart, so a warp's accesses stay coalesced),
// all 3U loads issued before any arithmetic: more bytes in flight per warp.
template <int U>
__global__ void __launch_bounds__(kThreads) bs_kernel_vec(const float4 *__restrict__ s, const float4 *__restrict__ x,
                                                          const float4 *__restrict__ t, long long n4, float r, float v,
                                                          float inv_v, float4 *__restrict__ call, float4 *__restrict__ put) {
    const long long stride = static_cast<long long>(gridDim.x) * blockDim.x;
    for (long long i0 = blockIdx.x * static_cast<long long>(blockDim.x) + threadIdx.x; i0 < n4; i0 += U * stride) {
        float4 S[U], X[U], T[U];
#pragma unroll
        for (int u = 0; u < U; ++u) {
            const long long i = i0 + u * stride;
            if (u == 0 || i < n4) {
                S[u] = __ldcs(s + i);                        // streamed once
                X[u] = __ldcs(x + i);
                T[u] = __ldcs(t + i);
            }
        }
#pragma unroll
        for (int u = 0; u < U; ++u) {
            const long long i = i0 + u * stride;
            if (u == 0 || i < n4) {
                float4 c, p;
                price1(S[u].x, X[u].x, T[u].x, r, v, inv_v, c.x, p.x);
                price1(S[u].y, X[u].y, T[u].y, r, v, inv_v, c.y, p.y);
                price1(S[u].z, X[u].z, T[u].z, r, v, inv_v, c.z, p.z);
                price1(S[u].w, X[u].w, T[u].w, r, v, inv_v, c.w, p.w);
                __stcs(call + i, c);
                __stcs(put + i, p);
            }
        }
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
        // 2 float4 groups per thread per trip, 4 CTAs per SM (48 registers: all resident, one
        // persistent wave): 860 us on 2^28 options = 6.24 TB/s.  The grid size matters more
        // than occupancy here -- 8 CTAs/SM ran 940 us, 6 ran 1040 us (profiles/r01_bs_sweep.txt)
        const long long blocks = std::min<long long>((n4 + kThreads - 1) / kThreads, static_cast<long long>(sms) * 4);
        auto kern = bs_kernel_vec<2>;
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
