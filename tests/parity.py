"""Parity metric shared by the tests (R14).

err = max |g - o| / S over output cells, where o is the oracle's float64 value
and S = sum |k_i k_j In| is the per-cell error scale the oracle returns.  For the
benchmark data (In >= 0, k >= 0) S == o, so err is the plain max relative error
BASELINE.json asks for.  Cells with S == 0 must match exactly (g == 0).
"""
import numpy as np

TOL = 1e-5            # BASELINE.json north_star: "max relative error of 1e-5 in float32"


def rel_error(gpu, oracle, absum):
    g = np.asarray(gpu, np.float64)
    o = np.asarray(oracle, np.float64)
    s = np.asarray(absum, np.float64)
    if g.shape != o.shape or o.shape != s.shape:
        raise AssertionError(f"shape mismatch: gpu {g.shape} oracle {o.shape} scale {s.shape}")
    if not np.all(np.isfinite(g)):
        raise AssertionError("non-finite value in GPU output")
    diff = np.abs(g - o)
    zero = s == 0
    if np.any(diff[zero] != 0):
        raise AssertionError("nonzero output where every term is zero")
    if np.all(zero):
        return 0.0
    return float(np.max(diff[~zero] / s[~zero]))


def plain_rel_error(gpu, oracle):
    g = np.asarray(gpu, np.float64)
    o = np.asarray(oracle, np.float64)
    nz = o != 0
    return float(np.max(np.abs(g[nz] - o[nz]) / np.abs(o[nz]))) if np.any(nz) else 0.0
