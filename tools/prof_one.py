"""Run one candidate at one width on the 16384^2 image: warm-up launch + N profiled launches.

    python tools/prof_one.py --k 17 --cand sep-fused-tma [--n 2] [--size 16384]
Used under ncu (-s <warm-ups> -c <n>) to capture a single kernel."""
import argparse, os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch
from paper_conf_asplos_phothilimthanaara13_b200 import sepconv as sc, synth

ap = argparse.ArgumentParser()
ap.add_argument("--k", type=int, default=17)
ap.add_argument("--cand", default="sep-fused-tma")
ap.add_argument("--n", type=int, default=2)
ap.add_argument("--size", type=int, default=16384)
a = ap.parse_args()
names = {"sep-fused-tma0": (1, 1, 1, 0), "sep-fused-tma1": (1, 1, 1, 1), "sep-fused-tma2": (1, 1, 1, 2),
         "sep-fused-tma3": (1, 1, 1, 3), "sep-fused-tma0s8": (1, 1, 1, 0, 1), "sep-fused-tma1s8": (1, 1, 1, 1, 1),
         "sep-fused-tma2s8": (1, 1, 1, 2, 1), "sep-fused-tma3s8": (1, 1, 1, 3, 1),
         "sep-fused-direct": (1, 0, 1), "2d-tma": (0, 1, 0), "2d-direct": (0, 0, 0),
         "sep-unfused-tma": (1, 1, 0), "sep-unfused-direct": (1, 0, 0)}
names["sep-fused-tma"] = names["sep-fused-tma0"]
for cfg in range(8):                       # every fused TMA configuration, both store paths
    names["sep-fused-tma%d" % cfg] = (1, 1, 1, cfg)
    names["sep-fused-tma%ds8" % cfg] = (1, 1, 1, cfg, 1)
    names["sep-fused-tma%dv2" % cfg] = (1, 1, 1, cfg, 2)
H = W = a.size
x = torch.rand((H, W), device="cuda")
out = torch.empty((H - a.k + 1, W - a.k + 1), device="cuda")
p = sc.Plan(H, W, a.k)
c = sc.Choice(*names[a.cand])
k = synth.binomial_kernel(a.k)
p.run_choice(x, k, out, c)
torch.cuda.synchronize()
for _ in range(a.n):
    p.run_choice(x, k, out, c)
torch.cuda.synchronize()
print("done", a.cand, a.k)
