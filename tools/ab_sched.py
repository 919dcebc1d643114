"""A/B of the work schedules (SEPCONV_SCHED = nowin | default) on the 16384^2 image.

    python tools/ab_sched.py [--size 16384] [--widths 3,9,15,17] [--reps 30] [--cands sep-fused-tma0,...]

For every width and fused candidate, launches alternate between the modes (the env var is
read per launch), each timed with CUDA events on the launching stream; prints the median
time and algorithmic GB/s per mode."""
import argparse
import os
import statistics
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch

from paper_conf_asplos_phothilimthanaara13_b200 import sepconv as sc, synth

ap = argparse.ArgumentParser()
ap.add_argument("--size", type=int, default=16384)
ap.add_argument("--widths", default="3,9,13,15,17")
ap.add_argument("--reps", type=int, default=30)
ap.add_argument("--modes", default="nowin,default")
ap.add_argument("--cands", default="")
a = ap.parse_args()

H = W = a.size
x = torch.rand((H, W), device="cuda")
modes = a.modes.split(",")
for K in [int(v) for v in a.widths.split(",")]:
    out = torch.empty((H - K + 1, W - K + 1), device="cuda")
    p = sc.Plan(H, W, K)
    k = synth.binomial_kernel(K)
    cands = [c for c in p.candidates() if c.algo == sc.SEPCONV_SEPARABLE and c.fused and c.mapping == sc.MAP_TMA]
    if a.cands:
        want = set(a.cands.split(","))
        cands = [c for c in cands if c.name in want]
    byts = 4.0 * (H * W + (H - K + 1) * (W - K + 1))
    for c in cands:
        times = {m: [] for m in modes}
        for r in range(a.reps + 2):
            for m in modes:
                if m == "default":
                    os.environ.pop("SEPCONV_SCHED", None)
                else:
                    os.environ["SEPCONV_SCHED"] = m
                e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                torch.cuda.synchronize()
                e0.record()
                p.run_choice(x, k, out, c)
                e1.record()
                torch.cuda.synchronize()
                if r >= 2:
                    times[m].append(e0.elapsed_time(e1) * 1e3)
        line = f"K={K:2d} {c.name:18s}"
        for m in modes:
            t = statistics.median(times[m])
            line += f"  {m}: {t:7.1f} us {byts / t / 1e3:6.0f} GB/s ({byts / t / 8e6:5.1%} of 8TB/s)"
        print(line, flush=True)
    p.close()
os.environ.pop("SEPCONV_SCHED", None)
