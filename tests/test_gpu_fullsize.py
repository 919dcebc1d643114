"""Whole-output parity at the configurations bench.py times (BASELINE.json configs[1], [3], [4]).

Every output cell of the GPU result is compared with the oracle's Fig. 1 definition
(oracle.convolve2d, float64, all host cores): max |g - o| / S <= 1e-5
(R14; S = o for the non-negative benchmark data).  Plans are tuned exactly as
bench.py tunes them (Plan.tune(reps=10) on the same seeded image), so the picks checked are
the ones the bench runs on this box -- whatever they are; no test assumes a pick.

* 16384^2, K = 3, 5, ..., 17: the tuned AUTO pick; at K = 3 and 17 also every fused TMA
  configuration under both work schedules (window and strided, $SEPCONV_SCHED), i.e. every
  window and part boundary row.
* 2048^2 (C2), K = 3, 7, 11, 15, 17: the tuned pick and every candidate.
* 64 x 4096^2, K = 11 (C5): the tuned pick, images 0, 31 and 63 whole.
-m gpu only."""
import os

import numpy as np
import pytest

import oracle
from paper_conf_asplos_phothilimthanaara13_b200 import sepconv as sc
from paper_conf_asplos_phothilimthanaara13_b200 import synth
from tests.parity import TOL

torch = pytest.importorskip("torch")
pytestmark = pytest.mark.gpu
TUNE_REPS = 10                     # bench.py --tune-reps default


def _oracle_on_gpu(img, k):
    o, s = oracle.convolve2d(img, k, with_absum=True)
    return torch.from_numpy(o).cuda(), torch.from_numpy(s).cuda()


def _err(out, o, s):
    """max |g - o| / S over every cell, on the device (float64)."""
    assert not torch.isnan(out).any().item(), "an output cell was not written"
    g = out.double()
    zero = s == 0
    assert not bool(((g - o).abs() * zero).any().item()), "nonzero output where every term is zero"
    return float(((g - o).abs() / torch.where(zero, torch.ones_like(s), s)).max().item())


@pytest.fixture(scope="module")
def big():
    img = synth.uniform_image(16384, 16384, seed=synth.BENCH_SEED_BASE + 3)   # bench.py's image
    dev = torch.from_numpy(img).cuda()
    yield img, dev
    del dev
    torch.cuda.empty_cache()


def _with_sched(mode, fn):
    old = os.environ.get("SEPCONV_SCHED")
    os.environ["SEPCONV_SCHED"] = mode
    try:
        return fn()
    finally:
        if old is None:
            del os.environ["SEPCONV_SCHED"]
        else:
            os.environ["SEPCONV_SCHED"] = old


@pytest.mark.parametrize("K", [3, 5, 7, 9, 11, 13, 15, 17])
def test_16384_tuned_pick_whole_output(K, big):
    img, dev = big
    H = W = 16384
    k = synth.binomial_kernel(K)
    o, s = _oracle_on_gpu(img, k)
    p = sc.Plan(H, W, K)
    pick = p.tune(reps=TUNE_REPS)
    out = torch.empty((H - K + 1, W - K + 1), dtype=torch.float32, device="cuda")
    checked = []

    def run(choice=None):
        out.fill_(float("nan"))
        if choice is None:
            p.run(dev, k, out, "auto")
        else:
            p.run_choice(dev, k, out, choice)
        torch.cuda.synchronize()
        return _err(out, o, s)

    err = run()
    assert err <= TOL, (pick.name, err)
    checked.append((pick.name, "auto", err))
    if K in (3, 17):
        for c in p.candidates():
            if not (c.algo == sc.SEPCONV_SEPARABLE and c.fused and c.mapping == sc.MAP_TMA):
                continue
            for mode in ("win", "nowin"):
                e = _with_sched(mode, lambda: run(c))
                assert e <= TOL, (c.name, mode, e)
                checked.append((c.name, mode, e))
    print("16384^2 K=%d:" % K, checked)
    del o, s
    torch.cuda.empty_cache()


@pytest.mark.parametrize("K", [3, 7, 11, 15, 17])
def test_2048_every_candidate_and_pick_whole_output(K):
    H = W = 2048
    img = synth.uniform_image(H, W, seed=synth.BENCH_SEED_BASE + 1)
    dev = torch.from_numpy(img).cuda()
    k = synth.binomial_kernel(K)
    o, s = _oracle_on_gpu(img, k)
    p = sc.Plan(H, W, K)
    pick = p.tune(reps=TUNE_REPS)
    out = torch.empty((H - K + 1, W - K + 1), dtype=torch.float32, device="cuda")
    for c in [None] + p.candidates():
        out.fill_(float("nan"))
        if c is None:
            p.run(dev, k, out, "auto")
        else:
            p.run_choice(dev, k, out, c)
        torch.cuda.synchronize()
        e = _err(out, o, s)
        assert e <= TOL, (c.name if c else "auto=" + pick.name, e)


def test_batch_64x4096_k11_tuned_images_0_31_63():
    N, H, W, K = 64, 4096, 4096, 11
    seed = synth.BENCH_SEED_BASE + 4                      # bench.py's batch seed
    k = synth.binomial_kernel(K)
    dev = torch.rand((N, H, W), dtype=torch.float32, device="cuda")
    picks = (0, 31, 63)
    imgs = {n: synth.uniform_image(H, W, seed, n=n) for n in picks}
    for n in picks:
        dev[n].copy_(torch.from_numpy(imgs[n]))
    p = sc.Plan(H, W, K, n=N)
    p.tune(reps=TUNE_REPS)
    out = torch.full((N, H - K + 1, W - K + 1), float("nan"), dtype=torch.float32, device="cuda")
    p.run(dev, k, out, "auto")
    torch.cuda.synchronize()
    assert not torch.isnan(out).any().item()
    for n in picks:
        o, s = _oracle_on_gpu(imgs[n], k)
        assert _err(out[n], o, s) <= TOL, n
