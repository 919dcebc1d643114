"""One Black-Scholes launch on 2^28 options, for ncu captures (-k regex:bs_kernel -s 1 -c 1)."""
import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch
from paper_conf_asplos_phothilimthanaara13_b200 import bs, synth
n = 1 << 28
s, x, t = (torch.from_numpy(a).cuda() for a in synth.bs_options(n, seed=1))
c, p = torch.empty_like(s), torch.empty_like(s)
for _ in range(2):
    bs.price(s, x, t, synth.BS_RATE, synth.BS_VOL, c, p)
torch.cuda.synchronize()
print("done")
