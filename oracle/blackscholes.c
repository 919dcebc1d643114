/*
 * blackscholes.c -- CPU ORACLE FOR Black-Scholes.  TEST INFRASTRUCTURE ONLY.
 *
 * Only tests/, __graft_entry__.smoke() and bench.py's cpu_baseline / --impl
 * reference legs may load this code.  The product path (libsepconv.so and the
 * Python binding) never links, imports or calls it, and shares no source,
 * header, table or helper with it.
 *
 * What it computes: "Black-Scholes
 * implements a mathematical model of a financial market to solve for the price
 * of European options.  Each entry of the output matrix can be computed from the
 * input matrix by applying the Black-Scholes formula."  Test input: 500000
 * options (Fig. 8).  The formula itself is the textbook one (Black and
 * Scholes 1973), written out in double precision with the standard normal CDF
 * N(x) = erfc(-x / sqrt 2) / 2 from libm (readings B1-B4):
 *
 *   d1 = (ln(S/X) + (r + v^2/2) T) / (v sqrt T),   d2 = d1 - v sqrt T
 *   call = S N(d1) - X e^{-rT} N(d2)
 *   put  = X e^{-rT} N(-d2) - S N(-d1)
 *
 * for each option i: spot S[i], strike X[i], years to expiry T[i]; the riskless
 * rate r and volatility v are scalars.  err_call[i] and err_put[i] (nullable)
 * receive the first-order rounding-error scales of a float32 evaluation of the
 * call and of the put (reading B4).
 *
 * Parity status: pinned by tests/test_bs_oracle.py (a textbook worked example,
 * put-call parity, the v -> 0 and T -> 0 limits, delta = N(d1) by finite
 * differences, monotonicity); not "parity unpinned".
 */
#include <math.h>
#include <stdint.h>

static double cnd(double x) { return 0.5 * erfc(-x / sqrt(2.0)); }

int oracle_black_scholes(const float *s, const float *x, const float *t, int64_t n, double r, double v,
                         double *call, double *put, double *err_call, double *err_put) {
    if (n < 0 || !(v > 0.0)) return -1;
    for (int64_t i = 0; i < n; ++i) {
        const double S = (double)s[i], X = (double)x[i], T = (double)t[i];
        if (!(S > 0.0) || !(X > 0.0) || !(T > 0.0)) return -1;
        const double sqrtT = sqrt(T);
        const double d1 = (log(S / X) + (r + 0.5 * v * v) * T) / (v * sqrtT);
        const double d2 = d1 - v * sqrtT;
        const double disc = X * exp(-r * T);
        call[i] = S * cnd(d1) - disc * cnd(d2);
        put[i] = disc * cnd(-d2) - S * cnd(-d1);
        if (err_call || err_put) {
            /* B4: a float32 evaluation perturbs d1 and d2 by a few ulps of the magnitudes
             * that form them -- |ln(S/X)| + 1 (the log of a rounded quotient), (r + v^2/2) T,
             * v sqrt T -- divided by v sqrt T, plus a few ulps of |d1| (the argument of the
             * tail's exponential grows like d^2); through N that moves each term by
             * S phi(d1) dd and disc phi(d2) dd.  Each product and CDF adds a few ulps of its
             * own term -- S N(d1) and disc N(d2) for the call, disc N(-d2) and S N(-d1) for
             * the put -- and the two terms cancel at most completely.  Results below the
             * float32 normal range flush to zero (reading B3): an absolute allowance of
             * (S + disc) 2^-100, i.e. 16 eps x that = 2^-120 (S + disc) > FLT_MIN (S + disc). */
            const double phi1 = exp(-0.5 * d1 * d1) / sqrt(2.0 * 3.14159265358979323846);
            const double phi2 = exp(-0.5 * d2 * d2) / sqrt(2.0 * 3.14159265358979323846);
            const double dd = (fabs(log(S / X)) + 1.0 + fabs(r + 0.5 * v * v) * T + v * sqrtT) / (v * sqrtT) +
                              fabs(d1) + 1.0;
            const double sens = S * phi1 * dd + disc * phi2 * dd;
            const double ftz = (S + disc) * 0x1p-100;
            if (err_call) err_call[i] = sens + S * cnd(d1) + disc * cnd(d2) + ftz;
            if (err_put) err_put[i] = sens + disc * cnd(-d2) + S * cnd(-d1) + ftz;
        }
    }
    return 0;
}
