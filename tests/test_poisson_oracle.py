"""Pins for the Poisson2D red-black SOR oracle (oracle/poisson.c; PAPER.md P:1294-1308,
readings DESIGN.md section 11).  None re-types the oracle's update: each checks it against
a direct sparse solve of the equation (scipy, the Kronecker-sum Laplacian), closed forms
(discrete-harmonic and quadratic fixed points), Young's asymptotic convergence rates of
red-black SOR, a hand-derived worked iteration, index closed forms of the split, or an
invariance.  CPU only (-m "not gpu")."""
import math
import os

import numpy as np
import pytest
import scipy.sparse as sp
import scipy.sparse.linalg as spla

import oracle
from paper_conf_asplos_phothilimthanaara13_b200 import synth

GOLDEN = os.path.join(os.path.dirname(__file__), "golden")
EPS32 = 2.0 ** -24


def _laplacian_2d(ni, mi):
    """A of reading P1 on an ni x mi interior: the Kronecker sum of two 1-D second
    differences tridiag(-1, 2, -1) -- the textbook 5-point operator (row-major cells)."""
    def t(k):
        return sp.diags([-np.ones(k - 1), 2 * np.ones(k), -np.ones(k - 1)], [-1, 0, 1])
    return (sp.kron(sp.identity(ni), t(mi)) + sp.kron(t(ni), sp.identity(mi))).tocsc()


def _direct_solution(x, b):
    """Solve A u = b + (boundary contributions) for the interior with scipy's sparse LU."""
    n, m = x.shape
    ni, mi = n - 2, m - 2
    rhs = b[1:-1, 1:-1].astype(np.float64).copy()
    xd = x.astype(np.float64)
    rhs[0, :] += xd[0, 1:-1]
    rhs[-1, :] += xd[-1, 1:-1]
    rhs[:, 0] += xd[1:-1, 0]
    rhs[:, -1] += xd[1:-1, -1]
    u = xd.copy()
    u[1:-1, 1:-1] = spla.spsolve(_laplacian_2d(ni, mi), rhs.reshape(-1)).reshape(ni, mi)
    return u


# ---- fixed point = the direct solve of the equation (P1, P2) -----------------------------
@pytest.mark.parametrize("shape", [(12, 15), (9, 9), (20, 7)])
def test_converges_to_direct_sparse_solve(shape):
    n, m = shape
    x, b = synth.poisson_problem(n, m, seed=n * 100 + m, guess="uniform")
    b = (b * np.float32((max(n, m) - 1) ** 2)).astype(np.float32)    # O(1) source: a visible b term
    want = _direct_solution(x, b)
    u = oracle.sor_rb(x, b, synth.omega_opt(n, m), 400)
    assert np.max(np.abs(u - want)) <= 1e-10 * max(1.0, np.max(np.abs(want)))
    # the boundary frame is never written (P2)
    assert np.array_equal(u[0], x[0]) and np.array_equal(u[-1], x[-1])
    assert np.array_equal(u[:, 0], x[:, 0]) and np.array_equal(u[:, -1], x[:, -1])
    # and the residual of the direct solution vanishes (pins oracle_poisson_residual)
    assert np.max(np.abs(oracle.poisson_residual(want, b))) <= 1e-10


def test_residual_closed_form():
    """r = b - A u for u = i^2 (A u = -2 on every interior cell) and b = 1: r = 3."""
    n, m = 6, 7
    u = np.array([[float(i * i) for _ in range(m)] for i in range(n)])
    r = oracle.poisson_residual(u, np.ones((n, m), np.float32))
    assert np.all(r[1:-1, 1:-1] == 3.0)
    assert np.all(r[0] == 0) and np.all(r[:, 0] == 0)


# ---- closed-form fixed points ------------------------------------------------------------
def _harmonic(n, m):
    i, j = np.meshgrid(np.arange(n, dtype=np.float64), np.arange(m, dtype=np.float64), indexing="ij")
    return 3.0 + 2.0 * i - 5.0 * j + i * j + (i * i - j * j)      # discrete Laplacian = 0


@pytest.mark.parametrize("omega", [0.5, 1.0, 1.5, 1.9])
def test_discrete_harmonic_is_a_fixed_point(omega):
    n, m = 11, 14
    h = _harmonic(n, m).astype(np.float32)
    zero = np.zeros((n, m), np.float32)
    u = oracle.sor_rb(h, zero, omega, 5)
    assert np.max(np.abs(u - h)) <= 1e-12 * np.max(np.abs(h))
    if omega == 1.0:                      # integer data, w/4 = 1/4: exact in float32
        assert np.array_equal(oracle.sor_rb_f32(h, zero, omega, 5), h)


def test_quadratic_with_constant_source_is_a_fixed_point():
    """u = i^2 + j^2: 4u - (sum of neighbours) = -4, so b = -4 makes u the solution."""
    n, m = 10, 13
    i, j = np.meshgrid(np.arange(n), np.arange(m), indexing="ij")
    q = (i * i + j * j).astype(np.float32)
    b = np.full((n, m), -4.0, np.float32)
    for omega in (1.0, 1.7):
        assert np.max(np.abs(oracle.sor_rb(q, b, omega, 4) - q)) <= 1e-12 * q.max()
    assert np.array_equal(oracle.sor_rb_f32(q, b, 1.0, 4), q)
    # starting from a zero interior it converges there (the boundary carries the data)
    x = q.copy()
    x[1:-1, 1:-1] = 0
    assert np.max(np.abs(oracle.sor_rb(x, b, synth.omega_opt(n, m), 300) - q)) <= 1e-9 * q.max()


# ---- Young's theory: asymptotic rate of red-black SOR (pins ordering and the role of w) ----
def _rate(omega, n, iters):
    x = synth.poisson_problem(n, n, seed=5, guess="uniform")[0]
    x[0, :] = x[-1, :] = x[:, 0] = x[:, -1] = 0                    # solution 0: u is the error
    zero = np.zeros_like(x)
    u1 = oracle.sor_rb(x, zero, omega, iters)
    u2 = oracle.sor_rb(x, zero, omega, iters + 1)          # one more sweep, all in double
    return np.linalg.norm(u2) / np.linalg.norm(u1)


def test_gauss_seidel_rate_is_jacobi_rate_squared():
    """w = 1: rho(red-black GS) = mu^2, mu = cos(pi h) the Jacobi radius (Young).  Jacobi
    (old values only) would converge at mu, a black-first or lexicographic sweep differs in
    transients but a wrong stencil or neighbour changes mu itself."""
    n = 18                                                           # 16 x 16 interior
    mu = math.cos(math.pi / (n - 1))
    assert _rate(1.0, n, 150) == pytest.approx(mu * mu, rel=2e-4)


def test_sor_rate_below_optimal_omega():
    """w < w_opt: rho = ((w mu + sqrt(w^2 mu^2 - 4 (w - 1))) / 2)^2 (Young's formula)."""
    n, omega = 18, 1.4
    mu = math.cos(math.pi / (n - 1))
    rho = ((omega * mu + math.sqrt(omega * omega * mu * mu - 4 * (omega - 1))) / 2) ** 2
    assert _rate(omega, n, 200) == pytest.approx(rho, rel=2e-3)


def test_optimal_omega_beats_gauss_seidel():
    n = 34
    x = synth.poisson_problem(n, n, seed=9, guess="uniform")[0]
    x[0, :] = x[-1, :] = x[:, 0] = x[:, -1] = 0
    zero = np.zeros_like(x)
    e_gs = np.linalg.norm(oracle.sor_rb(x, zero, 1.0, 60))
    e_opt = np.linalg.norm(oracle.sor_rb(x, zero, synth.omega_opt(n, n), 60))
    assert e_opt < 1e-3 * e_gs                       # (w_opt - 1)^60 vs mu^120


# ---- hand-derived worked iterations (tests/golden/poisson_5x5_delta.txt) ------------------
def _golden_cases():
    cases, cur = [], None
    with open(os.path.join(GOLDEN, "poisson_5x5_delta.txt")) as f:
        for line in f:
            line = line.strip()
            if not line or line.startswith("#") or line.startswith("n ") or line.startswith("m "):
                continue
            if line.startswith("case"):
                kv = dict(t.split("=") for t in line.split()[1:])
                cur = (float(kv["w"]), int(kv["iters"]), [])
                cases.append(cur)
            else:
                cur[2].append([float(v) for v in line.split()])
    return cases


@pytest.mark.parametrize("case", _golden_cases(), ids=lambda c: "w%g_it%d" % (c[0], c[1]))
def test_worked_example(case):
    omega, iters, rows = case
    want = np.array(rows)
    x = np.zeros((5, 5), np.float32)
    b = np.zeros((5, 5), np.float32)
    b[2, 2] = 4.0
    assert np.array_equal(oracle.sor_rb(x, b, omega, iters), want)
    assert np.array_equal(oracle.sor_rb_f32(x, b, omega, iters), want.astype(np.float32))


# ---- split / merge (P5) --------------------------------------------------------------------
def test_split_closed_form():
    x = np.array([[10 * i + j for j in range(5)] for i in range(3)], np.float32)
    red, black = oracle.rb_split(x)
    assert np.array_equal(red, [[0, 2, 4], [11, 13, 0], [20, 22, 24]])
    assert np.array_equal(black, [[1, 3, 0], [10, 12, 14], [21, 23, 0]])


@pytest.mark.parametrize("shape", [(1, 1), (1, 6), (7, 1), (4, 4), (5, 9), (8, 3)])
def test_split_merge_roundtrip(shape):
    x = synth.uniform_image(*shape, seed=3)
    red, black = oracle.rb_split(x)
    assert red.shape == (shape[0], (shape[1] + 1) // 2)
    assert np.array_equal(oracle.rb_merge(red, black, shape[1]), x)


# ---- float32 evaluation vs the double definition (P6, P7) ----------------------
def _abs_scale_golden():
    lines = [ln for ln in open(os.path.join(GOLDEN, "sor_abs_scale_4x4.txt")) if ln.strip() and not ln.startswith("#")]
    sec, d = None, {}
    for ln in lines:
        tok = ln.split()
        if len(tok) == 1:
            sec = tok[0]
            d[sec] = []
        elif tok[0] == "iters2_cell11":
            d["cell11"] = float(tok[1])
        else:
            d[sec].append([float(v) for v in tok])
    return (np.array(d["x"], np.float32), np.array(d["b"], np.float32), np.array(d["iters1"]), d["cell11"])


def test_abs_scale_hand_derived():
    """sor_abs_scale (the magnitudes the P7 bound scales with) on a hand-derived 4x4 case at
    w = 3/2 (tests/golden/sor_abs_scale_4x4.txt): pins |1-w| (not 1-w), w/4, |b|, the
    red-then-black order with new red values, and the fixed frame.  Exact binary fractions."""
    x, b, want1, cell11 = _abs_scale_golden()
    assert np.array_equal(oracle.sor_abs_scale(x, b, 1.5, 1), want1)
    assert oracle.sor_abs_scale(x, b, 1.5, 2)[1, 1] == cell11


def _one_sweep_ratio(omega, state, b):
    """max |f32 - f64| / (8 eps A_1) over one iteration from the same float32 state."""
    u64 = oracle.sor_rb(state, b, omega, 1)
    u32 = oracle.sor_rb_f32(state, b, omega, 1)
    bound = 8 * EPS32 * oracle.sor_abs_scale(state, b, omega, 1)
    inner = bound > 0
    return np.max(np.abs(u32 - u64)[inner] / bound[inner]), np.all(np.abs(u32 - u64) <= bound)


@pytest.mark.parametrize("omega", [0.8, 1.0, 1.6, 1.95])
def test_f32_one_sweep_within_and_near_the_bound(omega):
    """The P7 bound is a per-sweep statement: one iteration of the float32 evaluation order
    (P6) from a float32 state stays within 8 eps A_1, and the bound is TIGHT -- the observed
    error reaches at least 5% of it somewhere (an inflated bound, e.g. a dropped |1-w| or a
    wrong sweep order in sor_abs_scale, would fail the lower check).  States: the initial
    guess and the float32-rounded double iterate after 5 and 20 iterations."""
    n, m = 21, 26
    x, b = synth.poisson_problem(n, m, seed=17, guess="uniform")
    for t in (0, 5, 20):
        state = oracle.sor_rb(x, b, omega, t).astype(np.float32) if t else x
        ratio, within = _one_sweep_ratio(omega, state, b)
        assert within, (t, ratio)
        assert ratio >= 0.05, (t, ratio)


@pytest.mark.parametrize("omega", [0.8, 1.0])
def test_f32_within_running_error_bound(omega):
    """Several sweeps under-relaxed / Gauss-Seidel (w <= 1, where the magnitude iteration does
    not outgrow the iterate): within 8 eps T A_T and at least 1% of it.  Over-relaxed sweeps
    are covered per sweep above (their magnitude iteration grows like (|1-w| + w)^T)."""
    n, m, iters = 21, 26, 3
    x, b = synth.poisson_problem(n, m, seed=17, guess="uniform")
    u64 = oracle.sor_rb(x, b, omega, iters)
    u32 = oracle.sor_rb_f32(x, b, omega, iters)
    bound = 8 * EPS32 * iters * oracle.sor_abs_scale(x, b, omega, iters)
    assert np.all(np.abs(u32 - u64) <= bound + 1e-30)
    inner = bound > 0
    assert np.max(np.abs(u32 - u64)[inner] / bound[inner]) >= 0.01

def test_transpose_invariance():
    """(i + j) parity is symmetric, so transposing x and b transposes the iterate."""
    x, b = synth.poisson_problem(13, 17, seed=23, guess="uniform")
    u = oracle.sor_rb(x, b, 1.3, 7)
    ut = oracle.sor_rb(np.ascontiguousarray(x.T), np.ascontiguousarray(b.T), 1.3, 7)
    assert np.max(np.abs(ut.T - u)) <= 1e-14


def test_degenerate_grids_have_no_interior():
    for n, m in ((1, 1), (2, 5), (5, 2)):
        x, b = synth.poisson_problem(n, m, seed=1, guess="uniform")
        assert np.array_equal(oracle.sor_rb(x, b, 1.5, 3), x.astype(np.float64))
        assert np.array_equal(oracle.sor_rb_f32(x, b, 1.5, 3), x)
