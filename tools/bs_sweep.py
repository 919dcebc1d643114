"""Time bs_price on 2^28 device-resident options (median of 20, CUDA events).
    python tools/bs_sweep.py
(profiles/r01_bs_sweep.txt was taken with temporary BS_U / BS_CPS environment switches for the
unroll and the grid size; the kernel now hard-codes the winner: U = 2, 4 CTAs per SM.)"""
import os, sys, statistics
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch
from paper_conf_asplos_phothilimthanaara13_b200 import bs, synth
n = 1 << 28
g = torch.Generator(device="cuda").manual_seed(1)
s = 5 + 25 * torch.rand(n, device="cuda", generator=g)
x = 1 + 99 * torch.rand(n, device="cuda", generator=g)
t = 0.25 + 9.75 * torch.rand(n, device="cuda", generator=g)
c, p = torch.empty_like(s), torch.empty_like(s)
ts = []
for it in range(25):
    a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    a.record(); bs.price(s, x, t, synth.BS_RATE, synth.BS_VOL, c, p); b.record(); torch.cuda.synchronize()
    if it >= 5: ts.append(a.elapsed_time(b))
m = statistics.median(ts)
print(f"bs_kernel_vec<2>, 4 CTAs/SM: {m*1e3:.1f} us  {n/m/1e6:.0f} G opt/s  {20*n/m/1e6:.0f} GB/s")
