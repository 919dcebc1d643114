"""Small-shape run of every tuner candidate through the C ABI, for compute-sanitizer
(memcheck / racecheck / synccheck).  Usage: python tools/sanitize.py [K,K,...]"""
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch  # noqa: E402

from paper_conf_asplos_phothilimthanaara13_b200 import sepconv as sc  # noqa: E402
from paper_conf_asplos_phothilimthanaara13_b200 import synth  # noqa: E402

Ks = [int(x) for x in sys.argv[1].split(",")] if len(sys.argv) > 1 else [3, 17]
# (1200, 700) and (300, 4200): many short segments, several per CTA (the schedule allows 8-row segments)
for (h, w) in ((40, 1100), (67, 131), (1200, 700), (300, 4200)):
    img = torch.from_numpy(synth.uniform_image(h, w, seed=1)).cuda()
    for K in Ks:
        if K > min(h, w):
            continue
        p = sc.Plan(h, w, K)
        out = torch.empty((h - K + 1, w - K + 1), device="cuda")
        for c in p.candidates():
            p.run_choice(img, synth.binomial_kernel(K), out, c)
            torch.cuda.synchronize()
            print("ok", h, w, K, c.name, flush=True)
