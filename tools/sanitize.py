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

# the host pipeline (banded copy-in / kernel / copy-out) and row bands in external-halo mode
h, w, K = 700, 2100, 5
img = synth.uniform_image(h, w, seed=2)
src = torch.from_numpy(img).pin_memory()
dst = torch.empty((h - K + 1, w - K + 1)).pin_memory()
p = sc.Plan(h, w, K)
for v in ("separable", "2d"):
    p.run_host(src, synth.binomial_kernel(K), dst, v)
    print("ok run_host", v, flush=True)
dev = torch.from_numpy(img).cuda()
for g in range(2):
    r0, rows, owned, alloc = sc.band(h, K, 2, g)
    band = dev[r0:r0 + alloc].contiguous()
    q = sc.Plan(alloc, w, K)
    q.comm_init(None, 2, g)
    out = torch.empty((rows, w - K + 1), device="cuda")
    q.run_band(band, synth.binomial_kernel(K), out, "auto")
    torch.cuda.synchronize()
    print("ok run_band", g, flush=True)

# round 2: schedule overrides (the mutation search's tunables), the replay fast path and the
# clean L2 flush
h, w, K = 1200, 2300, 13
img = torch.from_numpy(synth.uniform_image(h, w, seed=3)).cuda()
out = torch.empty((h - K + 1, w - K + 1), device="cuda")
p = sc.Plan(h, w, K)
for cfg in range(6):
    for parts, grid in ((1, 1), (7, 20), (300, 0)):
        p.run_choice(img, synth.binomial_kernel(K), out,
                     sc.Choice(sc.SEPCONV_SEPARABLE, sc.MAP_TMA, 1, cfg, sched_parts=parts, sched_grid=grid))
        torch.cuda.synchronize()
    print("ok overrides cfg", cfg, flush=True)
# work stealing between warps (claim words, the owners' stage claims, the thieves' scan and
# compare-and-swap): one segment per CTA, several per CTA, and few long ones
for cfg in (2, 4, 5):
    for parts, grid in ((49, 0), (300, 0), (4, 9)):
        for steal in (2, 8):
            p.run_choice(img, synth.binomial_kernel(K), out,
                         sc.Choice(sc.SEPCONV_SEPARABLE, sc.MAP_TMA, 1, cfg, sched_parts=parts, sched_grid=grid,
                                   sched_steal=steal))
            torch.cuda.synchronize()
    print("ok work stealing cfg", cfg, flush=True)
run = p.bind(img, synth.binomial_kernel(K), out, "separable")
for _ in range(3):
    run()
sc.l2_flush()
torch.cuda.synchronize()
print("ok replay + l2_flush", flush=True)
