"""Small-shape runs of the NEXT-3/4 kernels for compute-sanitizer: the SOR split/merge,
half-sweep and every wavefront depth (including the band path), and Black-Scholes on
aligned and unaligned buffers.  Usage: python tools/sanitize_next.py"""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np  # noqa: E402
import torch  # noqa: E402

from paper_conf_asplos_phothilimthanaara13_b200 import bs, sor, synth  # noqa: E402

for n, m in ((37, 53), (130, 600)):
    x, b = synth.poisson_problem(n, m, seed=2, guess="uniform")
    dx, db = torch.from_numpy(x).cuda(), torch.from_numpy(b).cuda()
    u = torch.empty((n, m), device="cuda")
    p = sor.SorPlan(n, m)
    for v, d in [("half", 0)] + [("wave", d) for d in range(1, 9)]:
        p.set_depth(d)
        p.solve(dx, db, u, 1.5, 7, v)
        torch.cuda.synchronize()
        print("ok sor", n, m, v, d, flush=True)
    p.close()
    r0, rows, a0, arows = sor.band(n, 2, 1, 4)
    q = sor.SorPlan(arows, m)
    q.load(dx[a0:a0 + arows].contiguous(), db[a0:a0 + arows].contiguous())
    q.comm_init(None, 2, 1, 4)
    q.band_iterate(1.5, 5, "wave")
    torch.cuda.synchronize()
    print("ok sor band", n, m, flush=True)
for n, off in ((1003, 0), (1003, 1), (4, 0)):
    s, xx, t = (torch.from_numpy(a).cuda() for a in synth.bs_options(n + off, seed=4))
    c = torch.empty(n + off, device="cuda")
    pp = torch.empty(n + off, device="cuda")
    bs.price(s[off:], xx[off:], t[off:], synth.BS_RATE, synth.BS_VOL, c[off:], pp[off:], n=n)
    torch.cuda.synchronize()
    print("ok bs", n, off, flush=True)
