"""One SOR call on n^2 for ncu (not the product): python tools/sor_prof_one.py <n> <variant> [iters]"""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

from paper_conf_asplos_phothilimthanaara13_b200 import sor, synth  # noqa: E402

n = int(sys.argv[1])
variant = sys.argv[2]
iters = int(sys.argv[3]) if len(sys.argv) > 3 else 24
x, b = synth.poisson_problem(n, n, seed=3, guess="uniform")
p = sor.SorPlan(n, n)
p.load(torch.from_numpy(x).cuda(), torch.from_numpy(b).cuda())
p.iterate(1.9, iters, variant)
torch.cuda.synchronize()
p.iterate(1.9, iters, variant)
torch.cuda.synchronize()
