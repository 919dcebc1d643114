"""One SOR_WAVE pass (or HALF iteration) on an n x n grid, for ncu captures:
    ncu --set full -k regex:sor_wave -c 1 python tools/prof_sor.py --n 16384 --depth 4"""
import argparse, os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch
from paper_conf_asplos_phothilimthanaara13_b200 import sor, synth

ap = argparse.ArgumentParser()
ap.add_argument("--n", type=int, default=16384)
ap.add_argument("--depth", type=int, default=4)
ap.add_argument("--variant", default="wave")
a = ap.parse_args()
x = torch.rand((a.n, a.n), device="cuda")
b = torch.rand((a.n, a.n), device="cuda") * (1.0 / (a.n - 1) ** 2)
p = sor.SorPlan(a.n, a.n)
p.load(x, b)
p.set_depth(a.depth)
it = a.depth if a.variant == "wave" else 1
p.iterate(synth.omega_opt(a.n, a.n), it, a.variant)      # warm-up pass
p.iterate(synth.omega_opt(a.n, a.n), it, a.variant)      # profiled pass
torch.cuda.synchronize()
print("done")
