"""Seeded random configurations through the C ABI against the oracle:
batch sizes, odd shapes (including images whose right edge leaves a narrow CTA strip, so the
window / strided schedules hand CTAs segments of different strips), pitches, misaligned
pointers, every kernel width and every tuner candidate.  Each case: within the 1e-5 metric of
the oracle, separable candidates bitwise equal to each other, nothing written outside the
valid region (NaN canaries).  -m gpu only."""
import numpy as np
import pytest

import oracle
from paper_conf_asplos_phothilimthanaara13_b200 import sepconv as sc
from paper_conf_asplos_phothilimthanaara13_b200 import synth

torch = pytest.importorskip("torch")
pytestmark = pytest.mark.gpu
TOL = 1e-5


def case(rng):
    K = int(rng.integers(1, 18))
    n = int(rng.choice([1, 1, 2, 3]))
    # widths near multiples of the 8- and 16-warp CTA strips (1024 / 2048 output columns)
    base = int(rng.choice([128, 1024, 2048, 3072, 4096]))
    w = max(K, base + int(rng.integers(-40, 60)) + K - 1)
    h = int(rng.integers(K, 260))
    ld_in = w + int(rng.choice([0, 0, 1, 3, 4, 9]))
    wo = w - K + 1
    ld_out = wo + int(rng.choice([0, 0, 2, 5, 8]))
    off_in = int(rng.choice([0, 0, 0, 1, 2]))
    off_out = int(rng.choice([0, 0, 0, 1, 3]))
    signed = bool(rng.integers(0, 2))
    return K, n, h, w, ld_in, ld_out, off_in, off_out, signed


@pytest.mark.parametrize("seed", range(64))
def test_random_configuration(seed):
    rng = np.random.default_rng(0xF0220 + seed)
    K, n, h, w, ld_in, ld_out, off_in, off_out, signed = case(rng)
    ho, wo = h - K + 1, w - K + 1
    imgs = np.stack([synth.uniform_image(h, w, seed=seed, n=i) for i in range(n)]) - np.float32(0.5 if signed else 0)
    k = synth.random_kernel(K, seed=seed, signed=signed)
    src = np.full((n, h, ld_in), np.nan, np.float32)
    src[:, :, :w] = imgs
    guard = 1024
    dev_in = torch.full((guard + off_in + src.size + guard,), float("nan"), device="cuda")
    dev_in[guard + off_in:guard + off_in + src.size] = torch.from_numpy(src.reshape(-1)).cuda()
    p = sc.Plan(h, w, K, n=n, ld_in=ld_in, ld_out=ld_out)
    in_ptr = dev_in.data_ptr() + 4 * (guard + off_in)
    want = [oracle.convolve2d(imgs[i], k, with_absum=True) for i in range(n)]
    sep_ref = None
    for c in p.candidates():
        out_len = n * ho * ld_out
        dev_out = torch.full((guard + off_out + out_len + guard,), float("nan"), device="cuda")
        p.run_choice(in_ptr, k, dev_out.data_ptr() + 4 * (guard + off_out), c)
        torch.cuda.synchronize()
        full = dev_out.cpu().numpy()
        assert np.all(np.isnan(full[:guard + off_out])) and np.all(np.isnan(full[guard + off_out + out_len:])), c.name
        got = full[guard + off_out:guard + off_out + out_len].reshape(n, ho, ld_out)
        assert np.all(np.isnan(got[:, :, wo:])), f"{c.name}: pitch padding written"
        got = got[:, :, :wo]
        for i in range(n):
            o, s = want[i]
            err = np.max(np.abs(got[i].astype(np.float64) - o) / np.where(s > 0, s, 1.0))
            assert err <= TOL, f"{c.name} K={K} n={n} {h}x{w}: error {err:.3e}"
        if c.algo == sc.SEPCONV_SEPARABLE:
            if sep_ref is None:
                sep_ref = got.copy()
            else:
                assert np.array_equal(got, sep_ref), f"{c.name} differs from the other separable candidates"


@pytest.mark.parametrize("seed", range(24))
def test_random_sor_configuration(seed):
    """Poisson2D red-black SOR: random grids, wavefront depths and
    iteration counts (segment splits, ragged strips, partial last passes) bitwise equal to the
    fixed-order float32 oracle."""
    from paper_conf_asplos_phothilimthanaara13_b200 import sor
    rng = np.random.default_rng(0x50F + seed)
    n = int(rng.integers(3, 420))
    m = int(rng.choice([int(rng.integers(3, 300)), int(rng.integers(200, 3000))]))
    depth = int(rng.integers(1, 9))
    iters = int(rng.integers(1, 10))
    omega = float(rng.choice([1.0, 1.5, 1.9]))
    x, b = synth.poisson_problem(n, m, seed=seed, guess="uniform")
    want = oracle.sor_rb_f32(x, b, omega, iters)
    with sor.SorPlan(n, m) as sp:
        for v, d in (("wave", depth), ("half", 0)):
            sp.set_depth(d)
            u = torch.full((n, m), float("nan"), device="cuda")
            sp.solve(torch.from_numpy(x).cuda(), torch.from_numpy(b).cuda(), u, omega, iters, v)
            torch.cuda.synchronize()
            assert np.array_equal(u.cpu().numpy(), want), f"{v} depth {d}: {n}x{m}, {iters} iterations"


@pytest.mark.parametrize("seed", range(16))
def test_random_black_scholes_configuration(seed):
    """Black-Scholes: random counts (vector body + ragged tail), pointer
    offsets (scalar path), rates and volatilities, within the B4 bound of the double oracle."""
    from paper_conf_asplos_phothilimthanaara13_b200 import bs
    rng = np.random.default_rng(0xB5 + seed)
    n = int(rng.choice([int(rng.integers(1, 64)), int(rng.integers(1000, 300000))]))
    off = int(rng.integers(0, 4))
    r = float(rng.uniform(-0.02, 0.1))
    v = float(rng.uniform(0.02, 1.2))
    s, x, t = synth.bs_options(n, seed=seed)
    dev = [torch.empty(n + off, dtype=torch.float32, device="cuda") for _ in range(5)]
    for d, a in zip(dev[:3], (s, x, t)):
        d[off:] = torch.from_numpy(a)
    dev[3].fill_(float("nan"))
    dev[4].fill_(float("nan"))
    bs.price(dev[0][off:], dev[1][off:], dev[2][off:], r, v, dev[3][off:], dev[4][off:], n=n)
    torch.cuda.synchronize()
    oc, op, sc_c, sc_p = oracle.black_scholes(s, x, t, r, v, with_scale=True)
    for got, want, scale in ((dev[3][off:], oc, sc_c), (dev[4][off:], op, sc_p)):
        g = got.cpu().numpy()
        assert not np.any(np.isnan(g))
        assert np.all(np.abs(g - want) <= 16 * 2.0 ** -24 * scale)
