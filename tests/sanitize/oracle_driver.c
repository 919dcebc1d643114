/* oracle_driver.c -- exercises every oracle entry point (oracle/*.c, test infrastructure) on
 * small and degenerate shapes under AddressSanitizer + UndefinedBehaviorSanitizer
 * (tests/test_sanitize_cpu.py builds it with -fsanitize=address,undefined
 * -fno-sanitize-recover=all, so any report aborts with a non-zero status).  Values are
 * checked by the pins elsewhere; here only memory and UB hygiene, plus argument rejection. */
#include <math.h>
#include <stdint.h>
#include <stdio.h>
#include <stdlib.h>

int oracle_num_cpus(void);
int oracle_convolve2d(const float *in, int64_t h, int64_t w, int64_t ld, const float *kernel, int K, double *out,
                      double *absum, int nthreads);
int oracle_convolve_rows(const float *in, int64_t h, int64_t w, int64_t ld, const float *kernel, int K, double *out);
int oracle_convolve_columns(const double *in, int64_t h, int64_t w, const float *kernel, int K, double *out);
int oracle_separable(const float *in, int64_t h, int64_t w, int64_t ld, const float *kernel, int K, double *buffer,
                     double *out);
int oracle_sor_rb(const float *x, const float *b, int64_t n, int64_t m, double w, int iters, double *u);
int oracle_sor_rb_f32(const float *x, const float *b, int64_t n, int64_t m, float w, int iters, float *u);
int oracle_rb_split(const float *x, int64_t n, int64_t m, float *red, float *black);
int oracle_rb_merge(const float *red, const float *black, int64_t n, int64_t m, float *x);
int oracle_poisson_residual(const double *u, const float *b, int64_t n, int64_t m, double *r);
int oracle_black_scholes(const float *s, const float *x, const float *t, int64_t n, double r, double v, double *call,
                         double *put, double *err_call, double *err_put);

static int failures = 0;
#define EXPECT(c)                                                         \
    do {                                                                  \
        if (!(c)) {                                                       \
            fprintf(stderr, "%s:%d: expectation failed: %s\n", __FILE__, __LINE__, #c); \
            ++failures;                                                   \
        }                                                                 \
    } while (0)

/* exact-size heap blocks so ASan sees any overrun */
static float *fbuf(int64_t n, float v) {
    float *p = (float *)malloc((size_t)(n > 0 ? n : 1) * sizeof(float));
    for (int64_t i = 0; i < n; ++i) p[i] = v + (float)(i % 13) * 0.25f;
    return p;
}
static double *dbuf(int64_t n) { return (double *)malloc((size_t)(n > 0 ? n : 1) * sizeof(double)); }

int main(void) {
    EXPECT(oracle_num_cpus() >= 1);
    /* SeparableConvolution: every K on images from K x K up, pitched input, all thread counts */
    for (int K = 1; K <= 17; K += 2)
        for (int64_t h = K; h <= K + 3; ++h)
            for (int64_t w = K; w <= K + 5; w += 2) {
                const int64_t ld = w + (K % 3), ho = h - K + 1, wo = w - K + 1;
                float *in = fbuf(h * ld, 0.5f), *k = fbuf(K, 0.125f);
                double *o = dbuf(ho * wo), *s = dbuf(ho * wo), *rows = dbuf(h * wo), *cols = dbuf(ho * wo),
                       *buf = dbuf(h * wo), *sep = dbuf(ho * wo);
                for (int nt = 0; nt <= 3; ++nt) EXPECT(oracle_convolve2d(in, h, w, ld, k, K, o, nt ? s : NULL, nt) == 0);
                EXPECT(oracle_convolve_rows(in, h, w, ld, k, K, rows) == 0);
                EXPECT(oracle_convolve_columns(rows, h, wo, k, K, cols) == 0);
                EXPECT(oracle_separable(in, h, w, ld, k, K, buf, sep) == 0);
                for (int64_t i = 0; i < ho * wo; ++i) EXPECT(fabs(sep[i] - o[i]) <= 1e-12 * (fabs(o[i]) + 1.0));
                free(in); free(k); free(o); free(s); free(rows); free(cols); free(buf); free(sep);
            }
    {   /* rejections: nothing is touched */
        float *in = fbuf(16, 1.f), *k = fbuf(5, 1.f);
        double *o = dbuf(16);
        EXPECT(oracle_convolve2d(in, 4, 4, 4, k, 5, o, NULL, 1) != 0);
        EXPECT(oracle_convolve2d(in, 4, 4, 3, k, 3, o, NULL, 1) != 0);
        EXPECT(oracle_convolve2d(NULL, 4, 4, 4, k, 3, o, NULL, 1) != 0);
        EXPECT(oracle_convolve2d(in, 4, 4, 4, k, 0, o, NULL, 1) != 0);
        EXPECT(oracle_convolve_rows(in, 4, 4, 4, k, 5, o) != 0);
        EXPECT(oracle_separable(in, 4, 4, 4, k, 3, NULL, o) != 0);
        free(in); free(k); free(o);
    }
    /* Poisson2D red-black SOR: degenerate and small grids, split/merge round trips */
    for (int64_t n = 1; n <= 7; ++n)
        for (int64_t m = 1; m <= 8; ++m) {
            float *x = fbuf(n * m, 0.1f), *b = fbuf(n * m, 0.01f), *u32 = fbuf(n * m, 0.f);
            double *u = dbuf(n * m), *r = dbuf(n * m);
            const int64_t mh = (m + 1) / 2;
            float *red = fbuf(n * mh, 0.f), *black = fbuf(n * mh, 0.f), *back = fbuf(n * m, 0.f);
            EXPECT(oracle_sor_rb(x, b, n, m, 1.5, 3, u) == 0);
            EXPECT(oracle_sor_rb_f32(x, b, n, m, 1.5f, 3, u32) == 0);
            EXPECT(oracle_rb_split(x, n, m, red, black) == 0);
            EXPECT(oracle_rb_merge(red, black, n, m, back) == 0);
            for (int64_t i = 0; i < n * m; ++i) EXPECT(back[i] == x[i]);
            EXPECT(oracle_poisson_residual(u, b, n, m, r) == 0);
            free(x); free(b); free(u32); free(u); free(r); free(red); free(black); free(back);
        }
    /* Black-Scholes: with and without the error scales; rejected inputs */
    {
        const int64_t n = 257;
        float *s = fbuf(n, 5.f), *x = fbuf(n, 1.f), *t = fbuf(n, 0.25f);
        double *c = dbuf(n), *p = dbuf(n), *ec = dbuf(n), *ep = dbuf(n);
        EXPECT(oracle_black_scholes(s, x, t, n, 0.02, 0.3, c, p, ec, ep) == 0);
        EXPECT(oracle_black_scholes(s, x, t, n, 0.02, 0.3, c, p, NULL, NULL) == 0);
        EXPECT(oracle_black_scholes(s, x, t, 0, 0.02, 0.3, c, p, ec, ep) == 0);
        EXPECT(oracle_black_scholes(s, x, t, n, 0.02, 0.0, c, p, NULL, NULL) != 0);
        x[7] = 0.f;
        EXPECT(oracle_black_scholes(s, x, t, n, 0.02, 0.3, c, p, NULL, NULL) != 0);
        free(s); free(x); free(t); free(c); free(p); free(ec); free(ep);
    }
    if (failures) {
        fprintf(stderr, "oracle_driver: %d expectation(s) failed\n", failures);
        return 1;
    }
    printf("oracle sanitize ok\n");
    return 0;
}
