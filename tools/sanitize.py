"""Small-shape run of every candidate and width through the C ABI, for compute-sanitizer."""
import sys, os
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np, torch
from paper_conf_asplos_phothilimthanaara13_b200 import sepconv as sc, synth
cands = [sc.Choice(1, 1, 1), sc.Choice(1, 0, 1), sc.Choice(0, 1, 0), sc.Choice(0, 0, 0), sc.Choice(1, 1, 0), sc.Choice(1, 0, 0)]
Ks = [int(x) for x in sys.argv[1].split(",")] if len(sys.argv) > 1 else [1, 3, 8, 17]
for (h, w) in ((67, 131), (40, 1100)):
    img = torch.from_numpy(synth.uniform_image(h, w, seed=1)).cuda()
    for K in Ks:
        if K > min(h, w):
            continue
        p = sc.Plan(h, w, K)
        out = torch.empty((h - K + 1, w - K + 1), device="cuda")
        for c in cands:
            p.run_choice(img, synth.binomial_kernel(K), out, c)
            torch.cuda.synchronize()
            print("ok", h, w, K, c.name, flush=True)
