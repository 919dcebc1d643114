/*
 * sor.h -- C ABI of libsepconv.so, part 2: B200-native Poisson2D red-black SOR
 * (the second data-parallel benchmark of Phothilimthana et
 * al., ASPLOS'13).
 *
 * The paper: "This benchmark solves Poisson's equation using Red-Black Successive
 * Over-Relaxation (SOR).  Before main iteration, the algorithm splits the input
 * matrix into separate buffers of red and black cells for cache efficiency"
 * (P:1296-1299); its test input is 2048^2 (Fig. 8).  Everything else is a
 * reading:
 *   P1  4 u[i][j] - u[i-1][j] - u[i+1][j] - u[i][j-1] - u[i][j+1] = b[i][j] on the
 *       interior cells of an N x M grid (grid spacing folded into b);
 *   P2  Dirichlet boundary: the outer frame of x holds it and is never written;
 *   P3  red = (i + j) even, updated first; then black;
 *   P4  u <- (1 - w) u + (w/4) (u_N + u_S + u_W + u_E + b), newest neighbours;
 *   P5  split: red[i][k] = x[i][2k + (i & 1)], black[i][k] = x[i][2k + 1 - (i & 1)];
 *   P6  float32, every cell evaluated as t = (((u_N + u_S) + u_W) + u_E) + b,
 *       u' = fmaf(w/4, t, (1 - w) * u) with w/4 and 1-w formed in float32 -- so a
 *       result is bitwise independent of the variant, the tile and the launch split,
 *       and bitwise equal to the fixed-order float32 oracle.
 *
 * Storage: x, b and u are row-major float32 [N][ld] (ld >= M floats), device
 * memory of the plan's device.  The plan owns the split buffers: u_red, u_black,
 * b_red, b_black, each [N][ldh] with ldh = round_up(ceil(M/2), 4) (16-byte rows);
 * cells past a row's count of its colour are padding (never read as data).
 *
 * Errors: sepconv_status_t (include/sepconv.h), detail via sepconv_last_error().
 * Threading: one host thread per plan at a time.  All device work is asynchronous
 * on the caller's stream (NULL = legacy default stream).
 */
#ifndef SOR_H
#define SOR_H

#include "sepconv.h"

#ifdef __cplusplus
extern "C" {
#endif

typedef struct sor_plan_s *sor_plan_t;             /* opaque, owned by the library */

/* How one iteration is executed (all bitwise identical, P6):
 *   SOR_HALF   two launches per iteration, one per colour (the paper's structure:
 *              a red pass, then a black pass over the split buffers);
 *   SOR_WAVE   T iterations fused in one pass: each warp walks its column strip
 *              down the rows with a register-resident wavefront (red row r of
 *              iteration t, black row r-1, red row r-2 of iteration t+1, ...),
 *              reading u and b once and writing u once per T iterations
 *              (out-of-place into the plan's second buffer pair);
 *   SOR_AUTO   the tuned choice (sor_tune), else SOR_WAVE. */
typedef enum { SOR_HALF = 0, SOR_WAVE = 1, SOR_AUTO = 2 } sor_variant_t;

/* Plan an N x M grid on the current device.  N, M >= 1.  Allocates the split
 * buffers (and the second pair SOR_WAVE uses): 6 * N * ldh * 4 bytes. */
sepconv_status_t sor_plan(int64_t n, int64_t m, sor_plan_t *plan);

/* P5: split x (initial guess + boundary) and b into the plan's red/black buffers.
 * ld_x, ld_b: row pitches in floats (0 = M).  x and b must not overlap the plan. */
sepconv_status_t sor_load(sor_plan_t plan, const float *x, int64_t ld_x, const float *b, int64_t ld_b,
                          sepconv_stream_t stream);

/* P3-P4: `iters` >= 0 red-black iterations with relaxation factor 0 < omega < 2 on
 * the split buffers.  E_INVALID for omega outside (0, 2) or iters < 0.
 * A call of two or more kernel launches is recorded (on its first use) as a CUDA graph keyed by
 * omega, iters, variant, depth, schedule and the buffer pair it starts from, and replayed on
 * `stream` by later calls with the same key (env SOR_GRAPHS=0: always direct launches).  If
 * `stream` is being captured by the caller, the launches go into the caller's capture; the
 * plan's host-side state (which pair holds the iterate) advances at capture time. */
sepconv_status_t sor_iterate(sor_plan_t plan, float omega, int iters, sor_variant_t variant,
                             sepconv_stream_t stream);

/* Inverse of the split: write the current iterate to u [N][ld_u] (ld_u 0 = M).
 * Every cell is written, the boundary frame included (unchanged from x). */
sepconv_status_t sor_store(sor_plan_t plan, float *u, int64_t ld_u, sepconv_stream_t stream);

/* load + iterate + store. */
sepconv_status_t sor_solve(sor_plan_t plan, const float *x, const float *b, float *u, float omega, int iters,
                           sor_variant_t variant, sepconv_stream_t stream);

/* The same with HOST buffers (pinned or pageable, dense [N][M]): copies in, solves,
 * copies out, synchronously on `stream`.  The paper's timings include the
 * transfers. */
sepconv_status_t sor_solve_host(sor_plan_t plan, const float *x, const float *b, float *u, float omega,
                                int iters, sor_variant_t variant, sepconv_stream_t stream);

/* Device pointers of the current split iterate and right-hand side, and ldh (for
 * tests and tools; valid until the next sor_iterate / sor_destroy). */
sepconv_status_t sor_buffers(sor_plan_t plan, float **u_red, float **u_black, float **b_red, float **b_black,
                             int64_t *ldh);

/* Empirical choice between SOR_HALF and SOR_WAVE (wavefront depths 1..8, each with 1, 1/2
 * or 1/3 row segments per resident warp -- the wave schedule's size-like tunable) for this
 * grid at `iters_hint` iterations: median of `reps` event-timed runs on the legacy
 * default stream (synchronous).  It iterates the plan's own buffers, so call it
 * before sor_load (or load again afterwards).  Writes the chosen variant and depth
 * (nullable outputs); SOR_AUTO uses them from then on. */
sepconv_status_t sor_tune(sor_plan_t plan, int iters_hint, int reps, int *variant, int *depth);

/* Force the wavefront depth SOR_WAVE uses (0 = the tuned / default depth).  For
 * tests and measurements; E_INVALID outside 0..8. */
sepconv_status_t sor_set_depth(sor_plan_t plan, int depth);

/* ---- row bands across GPUs (one process per GPU) ----------------------------------
 * Band g of G owns grid rows [row0, row0 + rows), row0 = 2 floor(g N / 2G) (even: the
 * colouring P3 is the same in band and grid coordinates); it is planned as a grid of
 * alloc_rows rows starting at grid row alloc_row0: `halo` ghost rows above and below where
 * a neighbour exists.  The caller loads x and b for those alloc rows (sor_load) and stores
 * the result (sor_store: the owned rows are rows [row0 - alloc_row0, + rows)).
 * E_INVALID when a band is thinner than the halo or the halo is odd. */
sepconv_status_t sor_band(int64_t n, int nbands, int g, int halo, int64_t *row0, int64_t *rows, int64_t *alloc_row0,
                          int64_t *alloc_rows);

/* Make `plan` (planned with alloc_rows x M) band `rank` of `nranks` with `halo` ghost rows
 * (even, >= 2).  id: a sepconv_nccl_unique_id() shared by all ranks (NCCL communicator,
 * reference-counted per id), or NULL for external mode, where the caller refreshes the
 * ghost rows between calls (tests on one GPU). */
sepconv_status_t sor_comm_init(sor_plan_t plan, const unsigned char *id, int nranks, int rank, int halo);

/* `iters` iterations of the band in passes of depth T <= halo/2 (SOR_WAVE) or 1 (SOR_HALF);
 * after every pass the ghost rows of both colours are exchanged with the neighbours by
 * NCCL grouped send/recv on `stream` (skipped in external mode).  The owned rows equal the
 * single-GPU result bit for bit. */
sepconv_status_t sor_band_iterate(sor_plan_t plan, float omega, int iters, sor_variant_t variant,
                                  sepconv_stream_t stream);

void sor_destroy(sor_plan_t plan);                  /* NULL-safe; waits for the device */

#ifdef __cplusplus
}
#endif
#endif /* SOR_H */
