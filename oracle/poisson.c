/*
 * poisson.c -- CPU ORACLE FOR Poisson2D SOR.  TEST INFRASTRUCTURE ONLY.
 *
 * Only tests/, __graft_entry__.smoke() and bench.py's cpu_baseline / --impl
 * reference legs may load this code.  The product path (libsepconv.so and the
 * Python binding) never links, imports or calls it, and shares no source,
 * header, table or helper with it.
 *
 * What it computes: "This
 * benchmark solves Poisson's equation using Red-Black Successive
 * Over-Relaxation (SOR).  Before main iteration, the algorithm splits the
 * input matrix into separate buffers of red and black cells for cache
 * efficiency."  The paper states nothing else about the method; the readings
 * below are DESIGN.md P1-P8 (section 11):
 *
 *   P1  the 5-point discretisation of -Laplace(u) = f with the grid spacing
 *       folded into the right-hand side b:
 *         4 u[i][j] - u[i-1][j] - u[i+1][j] - u[i][j-1] - u[i][j+1] = b[i][j]
 *       for every interior cell (1 <= i <= N-2, 1 <= j <= M-2);
 *   P2  Dirichlet boundary: the outer frame of the input matrix X holds the
 *       boundary values and is never written; the interior of X is the
 *       initial guess;
 *   P3  red cells have (i + j) even, black cells (i + j) odd; one iteration
 *       is a red half-sweep followed by a black half-sweep;
 *   P4  the SOR update (Young's over-relaxed Gauss-Seidel) uses the newest
 *       neighbour values:
 *         u[i][j] <- (1 - w) u[i][j] + (w / 4) (u[i-1][j] + u[i+1][j]
 *                                               + u[i][j-1] + u[i][j+1] + b[i][j])
 *   P5  split layout: row i of the red buffer holds the red cells of row i
 *       in column order, red[i][k] = X[i][2k + (i & 1)]; black[i][k] =
 *       X[i][2k + 1 - (i & 1)]; both buffers have pitch ceil(M/2).
 *
 * oracle_sor_rb() is P1-P4 written out on the unsplit matrix, in double, in
 * the textbook loop order (colour, row, column); the split is a layout, so
 * the oracle needs no split to compute the iterate.  oracle_sor_rb_f32() is
 * the same loops in float32 with one fixed evaluation order (P6):
 *   t = ((((u_N + u_S) + u_W) + u_E) + b);  u' = fmaf(w/4, t, (1 - w) * u)
 * with w/4 and 1-w formed in float -- a bitwise reference for the GPU kernels,
 * which compute every cell in that order.  oracle_rb_split/merge are P5.
 *
 * Parity status: every function is pinned by tests/test_poisson_oracle.py
 * (a direct sparse solve of P1 as the fixed point, discrete-harmonic and
 * quadratic closed forms, Young's asymptotic rate for the red-black ordering,
 * a hand-derived worked iteration, split/merge index closed forms); none is
 * "parity unpinned".
 */
#include <math.h>
#include <stdint.h>
#include <string.h>

/* ---- P1-P4 in double on the full matrix ----------------------------------- */
int oracle_sor_rb(const float *x, const float *b, int64_t n, int64_t m, double w, int iters, double *u) {
    if (n < 1 || m < 1 || iters < 0) return -1;
    for (int64_t i = 0; i < n * m; ++i) u[i] = (double)x[i];
    for (int it = 0; it < iters; ++it) {
        for (int color = 0; color < 2; ++color) {           /* P3: red (even) first, then black */
            for (int64_t i = 1; i + 1 < n; ++i) {
                for (int64_t j = 1; j + 1 < m; ++j) {
                    if (((i + j) & 1) != color) continue;
                    const double nb = u[(i - 1) * m + j] + u[(i + 1) * m + j] + u[i * m + j - 1] +
                                      u[i * m + j + 1];
                    u[i * m + j] = (1.0 - w) * u[i * m + j] + (w / 4.0) * (nb + (double)b[i * m + j]);
                }
            }
        }
    }
    return 0;
}

/* ---- the same in float32, one fixed evaluation order (P6) ------- */
int oracle_sor_rb_f32(const float *x, const float *b, int64_t n, int64_t m, float w, int iters, float *u) {
    if (n < 1 || m < 1 || iters < 0) return -1;
    const float w4 = w * 0.25f, om1 = 1.0f - w;
    memcpy(u, x, sizeof(float) * (size_t)(n * m));
    for (int it = 0; it < iters; ++it) {
        for (int color = 0; color < 2; ++color) {
            for (int64_t i = 1; i + 1 < n; ++i) {
                for (int64_t j = 1; j + 1 < m; ++j) {
                    if (((i + j) & 1) != color) continue;
                    float t = u[(i - 1) * m + j] + u[(i + 1) * m + j];
                    t = t + u[i * m + j - 1];
                    t = t + u[i * m + j + 1];
                    t = t + b[i * m + j];
                    const float v = om1 * u[i * m + j];
                    u[i * m + j] = fmaf(w4, t, v);
                }
            }
        }
    }
    return 0;
}

/* ---- P5: the red/black split and its inverse ------------------------------- */
int oracle_rb_split(const float *x, int64_t n, int64_t m, float *red, float *black) {
    if (n < 1 || m < 1) return -1;
    const int64_t mh = (m + 1) / 2;
    for (int64_t i = 0; i < n; ++i) {
        for (int64_t j = 0; j < m; ++j) {
            if (((i + j) & 1) == 0) red[i * mh + j / 2] = x[i * m + j];
            else black[i * mh + j / 2] = x[i * m + j];
        }
    }
    return 0;
}

int oracle_rb_merge(const float *red, const float *black, int64_t n, int64_t m, float *x) {
    if (n < 1 || m < 1) return -1;
    const int64_t mh = (m + 1) / 2;
    for (int64_t i = 0; i < n; ++i)
        for (int64_t j = 0; j < m; ++j)
            x[i * m + j] = (((i + j) & 1) == 0) ? red[i * mh + j / 2] : black[i * mh + j / 2];
    return 0;
}

/* ---- the residual of P1 (interior cells; 0 on the frame), double ---------- */
int oracle_poisson_residual(const double *u, const float *b, int64_t n, int64_t m, double *r) {
    if (n < 1 || m < 1) return -1;
    for (int64_t i = 0; i < n; ++i) {
        for (int64_t j = 0; j < m; ++j) {
            if (i == 0 || j == 0 || i + 1 == n || j + 1 == m) {
                r[i * m + j] = 0.0;
                continue;
            }
            r[i * m + j] = (double)b[i * m + j] - (4.0 * u[i * m + j] - u[(i - 1) * m + j] - u[(i + 1) * m + j] -
                                                   u[i * m + j - 1] - u[i * m + j + 1]);
        }
    }
    return 0;
}
