"""Per-call cost of sepconv_run on small images: host wall time per call (1000 back-to-back
calls, no sync between) and device time per call (CUDA events around the same loop).
    python tools/small_latency.py"""
import os, sys, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch
from paper_conf_asplos_phothilimthanaara13_b200 import sepconv as sc, synth
for (h, K) in [(64, 3), (2048, 3), (2048, 17), (4096, 17)]:
    x = torch.rand((h, h), device="cuda")
    out = torch.empty((h - K + 1, h - K + 1), device="cuda")
    k = synth.binomial_kernel(K)
    with sc.Plan(h, h, K) as p:
        p.tune(reps=10)
        lib, h_, xp, op_, kb = sc.lib(), p.handle, x.data_ptr(), out.data_ptr(), sc._kernel_buf(k, K)
        kp, st = kb.ctypes.data, sc._stream(None)
        raw = lambda: lib.sepconv_run(h_, xp, kp, op_, 2, st)
        cands = [("auto", None), ("auto-raw-ctypes", raw), ("auto-bind", p.bind(x, k, out, "auto"))] + \
            [(c.name, c) for c in p.candidates()]
        if os.environ.get("AUTO_ONLY"):
            cands = cands[:3]
        for name, c in cands:
            run = (lambda: p.run(x, k, out, "auto")) if c is None else (c if callable(c) else (lambda c=c: p.run_choice(x, k, out, c)))
            for _ in range(20):
                run()
            torch.cuda.synchronize()
            n = 500
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            t0 = time.perf_counter()
            e0.record()
            for _ in range(n):
                run()
            e1.record()
            t1 = time.perf_counter()
            torch.cuda.synchronize()
            print(f"{h}^2 K={K} {name:20s} host {1e6 * (t1 - t0) / n:7.2f} us/call  device {1e3 * e0.elapsed_time(e1) / n:7.2f} us/call", flush=True)
