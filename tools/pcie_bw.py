"""Host<->device copy ceiling of the box (the roof of every `e2e` number).

    python tools/pcie_bw.py [--mb 1024] [--chunk-mb 64]

Pinned host buffers, CUDA events: H2D alone, D2H alone, and both directions at once on two
streams (the duplex ceiling a banded copy-in / kernel / copy-out pipeline can reach).
"""
import argparse
import json

import torch

ap = argparse.ArgumentParser()
ap.add_argument("--mb", type=int, default=1024)
ap.add_argument("--chunk-mb", type=int, default=64)
ap.add_argument("--reps", type=int, default=5)
a = ap.parse_args()
n = a.mb << 18
h_in = torch.empty(n, dtype=torch.float32).pin_memory()
h_out = torch.empty(n, dtype=torch.float32).pin_memory()
d_a = torch.empty(n, dtype=torch.float32, device="cuda")
d_b = torch.empty(n, dtype=torch.float32, device="cuda")
s1, s2 = torch.cuda.Stream(), torch.cuda.Stream()
chunk = a.chunk_mb << 18


def timed(fn):
    best = 1e30
    for _ in range(a.reps):
        torch.cuda.synchronize()
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record()
        fn()
        torch.cuda.synchronize()
        e1.record()
        torch.cuda.synchronize()
        best = min(best, e0.elapsed_time(e1))
    return best


def h2d():
    with torch.cuda.stream(s1):
        for o in range(0, n, chunk):
            d_a[o:o + chunk].copy_(h_in[o:o + chunk], non_blocking=True)


def d2h():
    with torch.cuda.stream(s2):
        for o in range(0, n, chunk):
            h_out[o:o + chunk].copy_(d_b[o:o + chunk], non_blocking=True)


def both():
    h2d()
    d2h()


nbytes = n * 4
t1, t2, t3 = timed(h2d), timed(d2h), timed(both)
res = {"bytes": nbytes, "chunk_bytes": chunk * 4,
       "h2d_gbs": nbytes / t1 / 1e6, "d2h_gbs": nbytes / t2 / 1e6,
       "duplex_each_gbs": nbytes / t3 / 1e6, "duplex_total_gbs": 2 * nbytes / t3 / 1e6}
print(json.dumps(res))
