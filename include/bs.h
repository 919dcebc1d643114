/*
 * bs.h -- C ABI of libsepconv.so, part 3: B200-native Black-Scholes option pricing
 * (Phothilimthana et al., ASPLOS'13, /root/reference/PAPER.md
 * "Black-Scholes implements a mathematical model of a financial market to
 * solve for the price of European options.  Each entry of the output matrix can be
 * computed from the input matrix by applying the Black-Scholes formula"; test input
 * 500000 options, Fig. 8).
 *
 * Readings:
 *   B1  one option per entry: spot S, strike X, years to expiry T (float32 arrays of n);
 *       the riskless rate r and the volatility v are scalars of the call;
 *   B2  the textbook formula: d1 = (ln(S/X) + (r + v^2/2) T) / (v sqrt T), d2 = d1 - v sqrt T,
 *       call = S N(d1) - X e^{-rT} N(d2), put = X e^{-rT} N(-d2) - S N(-d1),
 *       N(x) = erfc(-x / sqrt 2) / 2;
 *   B3  float32, every transcendental one SFU instruction (ftz): ln(S/X) = ln2 lg2(S rcp X),
 *       e^{-rT} = ex2(-rT log2e), 1/(v sqrt T) = rsqrt(T)/v (a few ulp each);
 *   B5  N(d) and 1 - N(d) from one tail e = erfc(|d|/sqrt 2)/2, erfc the Chebyshev fit of
 *       Numerical Recipes 6.2 "erfcc" (fractional error < 1.2e-7);
 *   B4  tolerance vs the double definition: |g - o| <= 16 eps (S phi(d1) dd + X e^{-rT}
 *       phi(d2) dd + S + X e^{-rT}), eps = 2^-24, dd the conditioning of d1 (oracle).
 * The paper's CPU/GPU work split (25/75 on its laptop) is not built: there
 * is no CPU path; a multi-GPU run shards the options (no exchange).
 *
 * Storage: device pointers of the current device, n float32 each; outputs written in
 * full, inputs untouched.  S, X, T > 0 and v > 0 are the caller's contract (not checked
 * per element on the device).  Errors: sepconv_status_t, detail in sepconv_last_error().
 */
#ifndef BS_H
#define BS_H

#include "sepconv.h"

#ifdef __cplusplus
extern "C" {
#endif

/* Price n options on `stream` (asynchronous).  call/put must not overlap the inputs
 * or each other (E_ALIAS); all pointers 4-byte aligned (E_ALIGN); 16-byte aligned
 * pointers take the vectorised path.  n = 0 is a no-op; E_INVALID for v <= 0 or n < 0. */
sepconv_status_t bs_price(const float *s, const float *x, const float *t, int64_t n, float r, float v, float *call,
                          float *put, sepconv_stream_t stream);

/* The same with HOST buffers (pinned or pageable): copies in, prices, copies out,
 * synchronously on `stream`, in chunks through a library-owned device workspace. */
sepconv_status_t bs_price_host(const float *s, const float *x, const float *t, int64_t n, float r, float v,
                               float *call, float *put, sepconv_stream_t stream);

#ifdef __cplusplus
}
#endif
#endif /* BS_H */
