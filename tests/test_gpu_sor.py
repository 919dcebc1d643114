"""GPU parity for Poisson2D red-black SOR (include/sor.h)
through the C ABI, against the CPU oracle (oracle/poisson.c).

Bar: the split, the merge and every iterate are BIT-EXACT against the fixed-order float32
oracle (reading P6) for every variant and wavefront depth; the iterate is also within the
running-error bound (P7) of the double-precision definition.  Runs only on a B200 (-m gpu)."""
import numpy as np
import pytest

import oracle
from paper_conf_asplos_phothilimthanaara13_b200 import sepconv as sc, sor, synth

torch = pytest.importorskip("torch")
pytestmark = pytest.mark.gpu
EPS32 = 2.0 ** -24


def _dev(a):
    return torch.from_numpy(np.ascontiguousarray(a)).cuda()


class _Raw:
    """A raw device pointer viewed as a float32 [rows][cols] tensor (no copy)."""

    def __init__(self, ptr, rows, cols):
        self.__cuda_array_interface__ = {"data": (int(ptr), False), "shape": (rows, cols),
                                         "typestr": "<f4", "version": 2}


def _split_from_device(p, n, m):
    (ur, ub, br, bb), ldh = p.buffers()
    torch.cuda.synchronize()
    return [torch.as_tensor(_Raw(ptr, n, ldh), device="cuda").cpu().numpy()[:, :(m + 1) // 2]
            for ptr in (ur, ub, br, bb)]


def gpu_solve(x, b, omega, iters, variant="wave", depth=0, plan=None):
    n, m = x.shape
    p = plan or sor.SorPlan(n, m)
    if depth:
        p.set_depth(depth)
    u = torch.full((n, m), float("nan"), device="cuda")
    p.solve(_dev(x), _dev(b), u, omega, iters, variant)
    torch.cuda.synchronize()
    got = u.cpu().numpy()
    assert not np.any(np.isnan(got)), "a cell of u was not written"
    return got


SHAPES = [(5, 5), (3, 3), (9, 14), (67, 131), (300, 1100), (1500, 300), (257, 1031)]


def test_split_and_merge_bitwise():
    for n, m in [(1, 1), (3, 5), (8, 9), (67, 131), (300, 1100)]:
        x, b = synth.poisson_problem(n, m, seed=n + m, guess="uniform")
        p = sor.SorPlan(n, m)
        p.load(_dev(x), _dev(b))
        ur, ub, br, bb = _split_from_device(p, n, m)
        want_ur, want_ub = oracle.rb_split(x)
        want_br, want_bb = oracle.rb_split(b)
        # cells past a row's count of its colour are padding: compare the real cells only
        cnt_red = [(m + 1 - (i & 1)) // 2 for i in range(n)]
        cnt_black = [m // 2 if (i & 1) == 0 else (m + 1) // 2 for i in range(n)]
        for got, want, cnt in ((ur, want_ur, cnt_red), (ub, want_ub, cnt_black), (br, want_br, cnt_red),
                               (bb, want_bb, cnt_black)):
            for i in range(n):
                assert np.array_equal(got[i, :cnt[i]], want[i, :cnt[i]]), i
        assert np.array_equal(oracle.rb_merge(ur, ub, m), x)
        assert np.array_equal(oracle.rb_merge(br, bb, m), b)
        u = torch.full((n, m), float("nan"), device="cuda")
        p.store(u)
        torch.cuda.synchronize()
        assert np.array_equal(u.cpu().numpy(), x)                 # merge(split(x)) == x


@pytest.mark.parametrize("shape", SHAPES, ids=lambda s: "%dx%d" % s)
@pytest.mark.parametrize("variant,depth", [("half", 0), ("wave", 1), ("wave", 2), ("wave", 3), ("wave", 4),
                                           ("wave", 5), ("wave", 8)])
def test_iterates_bitwise_vs_f32_oracle(shape, variant, depth):
    n, m = shape
    x, b = synth.poisson_problem(n, m, seed=7 * n + m, guess="uniform")
    omega = synth.omega_opt(n, m)
    for iters in (1, 7):
        got = gpu_solve(x, b, omega, iters, variant, depth)
        want = oracle.sor_rb_f32(x, b, omega, iters)
        assert np.array_equal(got, want), f"iters={iters}: max diff {np.max(np.abs(got - want))}"


@pytest.mark.parametrize("variant,depth", [("half", 0), ("wave", 2), ("wave", 3)])
def test_graph_replay_bitwise_and_counted(variant, depth):
    """sor_iterate records a multi-launch call as a CUDA graph and replays it for the next call
    with the same key (omega, iterations, variant, depth, schedule, starting buffer pair): the
    replays -- from both buffer pairs -- stay bitwise equal to the oracle and count the launches
    they execute."""
    n, m = 257, 1031
    x, b = synth.poisson_problem(n, m, seed=5, guess="uniform")
    omega = synth.omega_opt(n, m)
    p = sor.SorPlan(n, m)
    if depth:
        p.set_depth(depth)
    dx, db = _dev(x), _dev(b)
    u = torch.empty((n, m), device="cuda")
    iters = 5
    launches = 2 * iters if variant == "half" else -(-iters // depth)
    want = {k: oracle.sor_rb_f32(x, b, omega, k * iters) for k in (1, 2)}
    for rep in range(3):                  # rep 0 records, later reps replay
        p.load(dx, db)
        for k in (1, 2):                  # the second call starts where the first left the pair index
            c0 = sc.launch_count()
            p.iterate(omega, iters, variant)
            torch.cuda.synchronize()
            assert sc.launch_count() - c0 == launches
            p.store(u)
            torch.cuda.synchronize()
            got = u.cpu().numpy()
            assert np.array_equal(got, want[k]), f"rep {rep} call {k}: max diff {np.max(np.abs(got - want[k]))}"


def test_graph_replay_inside_a_callers_capture():
    """A caller capturing its own stream gets the direct launches (no nested capture): the
    captured call replays bitwise equal to the oracle.  As with any stateful call under capture,
    the plan's host-side state (which buffer pair holds the iterate) advances when the call is
    captured, and the replay performs the recorded passes."""
    n, m = 130, 300
    x, b = synth.poisson_problem(n, m, seed=9, guess="uniform")
    omega = 1.5
    p = sor.SorPlan(n, m)
    p.set_depth(2)
    p.load(_dev(x), _dev(b))
    torch.cuda.synchronize()
    g = torch.cuda.CUDAGraph()
    s = torch.cuda.Stream()
    with torch.cuda.graph(g, stream=s):
        p.iterate(omega, 6, "wave", torch.cuda.current_stream())
    torch.cuda.synchronize()
    g.replay()                            # the capture executed nothing; the replay runs the passes
    torch.cuda.synchronize()
    u = torch.empty((n, m), device="cuda")
    p.store(u)
    torch.cuda.synchronize()
    assert np.array_equal(u.cpu().numpy(), oracle.sor_rb_f32(x, b, omega, 6))


@pytest.mark.parametrize("omega", [0.7, 1.0, 1.5, 1.97])
def test_within_running_error_bound_of_double(omega):
    """Reading P7 per sweep: one GPU iteration from a float32 state (the initial guess, and the
    rounded double iterate after 9 iterations) is within 8 eps A_1 of one double iteration from
    the same state, and reaches >= 5% of that bound somewhere (the bound is not vacuous).  For
    w <= 1 also 3 sweeps against 8 eps T A_T."""
    n, m = 131, 77
    x, b = synth.poisson_problem(n, m, seed=3, guess="uniform")
    for t in (0, 9):
        state = oracle.sor_rb(x, b, omega, t).astype(np.float32) if t else x
        got = gpu_solve(state, b, omega, 1, "auto")
        u64 = oracle.sor_rb(state, b, omega, 1)
        bound = 8 * EPS32 * oracle.sor_abs_scale(state, b, omega, 1)
        assert np.all(np.abs(got - u64) <= bound + 1e-30)
        inner = bound > 0
        assert np.max(np.abs(got - u64)[inner] / bound[inner]) >= 0.05
    if omega <= 1.0:
        got = gpu_solve(x, b, omega, 3, "auto")
        bound = 8 * EPS32 * 3 * oracle.sor_abs_scale(x, b, omega, 3)
        assert np.all(np.abs(got - oracle.sor_rb(x, b, omega, 3)) <= bound + 1e-30)


def test_worked_example_on_gpu():
    x = np.zeros((5, 5), np.float32)
    b = np.zeros((5, 5), np.float32)
    b[2, 2] = 4.0
    want = np.zeros((5, 5), np.float32)
    want[2, 2] = 1.25
    want[1, 2] = want[2, 1] = want[2, 3] = want[3, 2] = 0.375
    want[1, 1] = want[1, 3] = want[3, 1] = want[3, 3] = 0.125
    for variant in ("half", "wave"):
        assert np.array_equal(gpu_solve(x, b, 1.0, 2, variant), want)


def test_degenerate_grids():
    for n, m in ((1, 1), (2, 5), (5, 2), (1, 9), (3, 3)):
        x, b = synth.poisson_problem(n, m, seed=1, guess="uniform")
        for variant in ("half", "wave"):
            got = gpu_solve(x, b, 1.5, 3, variant)
            assert np.array_equal(got, oracle.sor_rb_f32(x, b, 1.5, 3))


def test_harmonic_fixed_point_large_grid_exact():
    """A discrete-harmonic integer field with b = 0 is a fixed point; at w = 1 every update
    is exact in float32, so it must come back bit for bit (any index error breaks it)."""
    n, m = 1030, 2050
    i, j = np.meshgrid(np.arange(n, dtype=np.float64), np.arange(m, dtype=np.float64), indexing="ij")
    h = (7.0 + 3.0 * i - 2.0 * j + i * j).astype(np.float32)          # |4u| < 2^24: exact
    zero = np.zeros((n, m), np.float32)
    for variant, depth in (("half", 0), ("wave", 4)):
        assert np.array_equal(gpu_solve(h, zero, 1.0, 6, variant, depth), h)


def test_solve_host_and_tune():
    n, m = 300, 1100
    x, b = synth.poisson_problem(n, m, seed=11, guess="uniform")
    omega = synth.omega_opt(n, m)
    p = sor.SorPlan(n, m)
    v, d = p.tune(iters_hint=8, reps=3)
    assert v in (sor.SOR_HALF, sor.SOR_WAVE) and 1 <= d <= sor.MAX_DEPTH
    u = np.full((n, m), np.nan, np.float32)
    p.solve_host(x, b, u, omega, 9, "auto")
    assert np.array_equal(u, oracle.sor_rb_f32(x, b, omega, 9))


def test_errors():
    p = sor.SorPlan(16, 16)
    x = torch.zeros((16, 16), device="cuda")
    for omega, iters in ((0.0, 1), (2.0, 1), (1.5, -1)):
        with pytest.raises(sor.SepconvError) as ei:
            p.solve(x, x, torch.zeros_like(x), omega, iters)
        assert ei.value.code == "E_INVALID"
    with pytest.raises(sor.SepconvError) as ei:
        p.set_depth(9)
    assert ei.value.code == "E_INVALID"


def test_sampled_blocks_at_bench_size():
    """16384^2 (the bench's large grid) after 8 iterations: cells farther than 2T = 16 from
    a crop's border depend only on the crop, so the oracle run on an even-offset crop (colour
    parity preserved) gives them exactly (bitwise, float32 order P6)."""
    n = m = 16384
    iters = 8
    x, b = synth.poisson_problem(n, m, seed=synth.BENCH_SEED_BASE + 40, guess="uniform")
    got = gpu_solve(x, b, synth.omega_opt(n, m), iters, "auto")
    margin = 2 * iters
    for (i0, j0) in ((0, 0), (8190, 4096), (n - 160, m - 200), (0, m - 200), (5000, 0)):
        h, w = 160, 200
        cx = np.ascontiguousarray(x[i0:i0 + h, j0:j0 + w])
        cb = np.ascontiguousarray(b[i0:i0 + h, j0:j0 + w])
        want = oracle.sor_rb_f32(cx, cb, synth.omega_opt(n, m), iters)
        top = 0 if i0 == 0 else margin
        left = 0 if j0 == 0 else margin
        bottom = h if i0 + h == n else h - margin
        right = w if j0 + w == m else w - margin
        assert np.array_equal(got[i0 + top:i0 + bottom, j0 + left:j0 + right], want[top:bottom, left:right]), (i0, j0)


# ---- row bands on one GPU: the band path of sor_band_iterate with the ghost-row exchange
# ---- done by the test (external mode); NCCL itself with one rank --------------------------
def _rows_view(ptr, ldh, r0, nrows):
    return torch.as_tensor(_Raw(int(ptr) + 4 * r0 * ldh, nrows, ldh), device="cuda")


@pytest.mark.parametrize("G,halo,variant", [(2, 6, "wave"), (3, 8, "wave"), (4, 2, "half"), (3, 4, "wave")])
def test_bands_external_exchange_equal_whole_grid(G, halo, variant):
    N, M, iters = 301, 517, 9
    x, b = synth.poisson_problem(N, M, seed=55, guess="uniform")
    omega = synth.omega_opt(N, M)
    want = gpu_solve(x, b, omega, iters, variant, depth=max(1, halo // 2))
    bands = []
    for g in range(G):
        r0, rows, a0, arows = sor.band(N, G, g, halo)
        p = sor.SorPlan(arows, M)
        p.set_depth(max(1, halo // 2))
        p.load(_dev(x[a0:a0 + arows]), _dev(b[a0:a0 + arows]))
        p.comm_init(None, G, g, halo)
        bands.append((p, r0, rows, a0, arows))
    T = 1 if variant == "half" else halo // 2
    left = iters
    while left > 0:
        t = min(T, left)
        for p, *_ in bands:
            p.band_iterate(omega, t, variant)
        torch.cuda.synchronize()
        # the exchange a NCCL run does: neighbours' first/last owned rows into the ghost rows
        views = []
        for p, r0, rows, a0, arows in bands:
            (ur, ub, _, _), ldh = p.buffers()
            views.append((ur, ub, ldh, r0 - a0, a0 + arows - (r0 + rows), arows))
        for g in range(G):
            ur, ub, ldh, h_top, h_bot, n = views[g]
            for c in range(2):
                mine = (ur, ub)[c]
                if g > 0:
                    pur, pub, _, ph_top, ph_bot, pn = views[g - 1]
                    _rows_view(mine, ldh, 0, halo).copy_(_rows_view((pur, pub)[c], ldh, pn - ph_bot - halo, halo))
                if g < G - 1:
                    nur, nub, _, nh_top, _, _ = views[g + 1]
                    _rows_view(mine, ldh, n - halo, halo).copy_(_rows_view((nur, nub)[c], ldh, nh_top, halo))
        torch.cuda.synchronize()
        left -= t
    got = []
    for p, r0, rows, a0, arows in bands:
        u = torch.full((arows, M), float("nan"), device="cuda")
        p.store(u)
        torch.cuda.synchronize()
        got.append(u[r0 - a0:r0 - a0 + rows].cpu().numpy())
    assert np.array_equal(np.concatenate(got, 0), want)


def test_band_nccl_single_rank_equals_plain():
    from paper_conf_asplos_phothilimthanaara13_b200 import sepconv as sc
    N, M = 130, 250
    x, b = synth.poisson_problem(N, M, seed=3, guess="uniform")
    want = gpu_solve(x, b, 1.6, 8, "wave", depth=4)
    p = sor.SorPlan(N, M)
    p.set_depth(4)
    p.load(_dev(x), _dev(b))
    p.comm_init(sc.nccl_unique_id(), 1, 0, 8)
    p.band_iterate(1.6, 8, "wave")
    u = torch.empty((N, M), device="cuda")
    p.store(u)
    torch.cuda.synchronize()
    assert np.array_equal(u.cpu().numpy(), want)
