"""The achievable floor at mid sizes: a device-to-device copy of the same bytes as one pass
(read H*W floats, write (H-K+1)*(W-K+1) ~ H*W floats) timed exactly as bench.py times a pass
(clean L2 flush before every pass, marginal batch difference), next to the tuned fused pass.
    python tools/copy_floor.py [--sizes 2048,3520,4096] [--widths 3,17] [--n 100]"""
import argparse
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

from paper_conf_asplos_phothilimthanaara13_b200 import sepconv as sc, synth  # noqa: E402

ap = argparse.ArgumentParser()
ap.add_argument("--sizes", default="2048,3520,4096")
ap.add_argument("--widths", default="3,17")
ap.add_argument("--n", type=int, default=100)
a = ap.parse_args()


def batch(fn, n):
    fn()
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    for _ in range(n):
        fn()
    e1.record()
    torch.cuda.synchronize()
    return e0.elapsed_time(e1) * 1e3 / n


def cold(fn):
    for _ in range(20):
        sc.l2_flush()
    ts = []
    for _ in range(3):
        f0 = batch(sc.l2_flush, a.n)
        fp = batch(lambda: (sc.l2_flush(), fn()), a.n)
        f1 = batch(sc.l2_flush, a.n)
        ts.append(fp - 0.5 * (f0 + f1))
    return sorted(ts)[1]


empty = torch.empty(1, device="cuda")
print("empty kernel (fill_ of 4 bytes) after a flush: %.2f us" % cold(lambda: empty.fill_(0.0)), flush=True)
for H in [int(s) for s in a.sizes.split(",")]:
    x = torch.from_numpy(synth.uniform_image(H, H, seed=synth.BENCH_SEED_BASE + 3)).cuda()
    y = torch.empty_like(x)
    t_copy = cold(lambda: y.copy_(x))
    mb = 8.0 * H * H / 1e6
    print("%5d^2 copy (torch) %7.2f us  %5.0f GB/s" % (H, t_copy, mb * 1e3 / t_copy), flush=True)
    for K in [int(k) for k in a.widths.split(",")]:
        p = sc.Plan(H, H, K)
        c = p.tune(reps=10, force=True)
        out = torch.empty((H - K + 1, H - K + 1), device="cuda")
        k = synth.binomial_kernel(K)
        t = cold(lambda: p.run_choice(x, k, out, c))
        print("%5d^2 K=%2d %-28s %7.2f us  = %.2f x the copy" % (H, K, c.name, t, t / t_copy), flush=True)
