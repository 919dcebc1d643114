"""Median device time of every fused-separable candidate on the 16384^2 image at chosen widths,
for A/B comparisons of two builds:  python tools/ab_cands.py [--root DIR] [--widths 13,15,17]
(--root: the repo copy whose package is imported)."""
import argparse, os, statistics, sys
ap = argparse.ArgumentParser()
ap.add_argument("--root", default=os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
ap.add_argument("--widths", default="13,15,17")
ap.add_argument("--reps", type=int, default=15)
ap.add_argument("--size", type=int, default=16384)
a = ap.parse_args()
sys.path.insert(0, a.root)
import torch
from paper_conf_asplos_phothilimthanaara13_b200 import sepconv as sc, synth
print("lib", sc.LIB_PATH)
H = W = a.size
x = torch.rand((H, W), device="cuda")
for K in [int(k) for k in a.widths.split(",")]:
    out = torch.empty((H - K + 1, W - K + 1), device="cuda")
    k = synth.binomial_kernel(K)
    with sc.Plan(H, W, K) as p:
        for c in p.candidates():
            if not c.name.startswith("sep-fused-tma"):
                continue
            for _ in range(3):
                p.run_choice(x, k, out, c)
            ts = []
            for _ in range(a.reps):
                e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                e0.record(); p.run_choice(x, k, out, c); e1.record(); torch.cuda.synchronize()
                ts.append(e0.elapsed_time(e1) * 1e3)
            print(f"K={K:2d} {c.name:18s} {statistics.median(ts):8.1f} us", flush=True)
    del out
