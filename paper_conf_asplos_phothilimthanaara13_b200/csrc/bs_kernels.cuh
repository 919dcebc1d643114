// bs_kernels.cuh -- the Black-Scholes device code (include/bs.h, DESIGN.md
// section 12): SFU helpers, the Chebyshev erfc tail, price1 and the two kernels.  Included by bs.cu
// (the product) and by tools/bs_small.cu (exploration); no host code here.
#pragma once
#include <cuda_runtime.h>

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

}  // namespace bs
