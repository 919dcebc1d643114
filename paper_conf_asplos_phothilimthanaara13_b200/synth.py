"""Seeded synthetic inputs shared by the tests, bench.py and the oracle checks.

This module holds NONE of the method's arithmetic: it only draws images and
kernels.  Both the CUDA path and the CPU oracle receive the bytes it returns.

Images are counter-based (splitmix64 of a per-pixel counter), so any row band
of a large image can be regenerated on its own and every value is reproducible
from (seed, n, r, c):

    z = splitmix64(seed * 2^32 + n * H * W + r * W + c)
    uniform image:  In = (z >> 40) * 2^-24            exact float32 in [0, 1)
    integer image:  In = (z >> 32) mod 31 - 15        in {-15..15}

The benchmark kernel is the normalised binomial k_i = C(K-1, i) / 2^(K-1)
(DESIGN.md "Input recipe"): positive, sum 1, exact in float32 for K <= 17.
"""
from __future__ import annotations

import math

import numpy as np

_GOLDEN = np.uint64(0x9E3779B97F4A7C15)
_M1 = np.uint64(0xBF58476D1CE4E5B9)
_M2 = np.uint64(0x94D049BB133111EB)

BENCH_SEED_BASE = 0x5EC0000


def _splitmix64(x: np.ndarray) -> np.ndarray:
    with np.errstate(over="ignore"):
        z = x + _GOLDEN
        z = (z ^ (z >> np.uint64(30))) * _M1
        z = (z ^ (z >> np.uint64(27))) * _M2
        return z ^ (z >> np.uint64(31))


def _counters(seed: int, n: int, h: int, w: int, r0: int, r1: int) -> np.ndarray:
    base = (np.uint64(seed & 0xFFFFFFFF) << np.uint64(32)) + np.uint64(n * h * w)
    rows = np.arange(r0, r1, dtype=np.uint64)[:, None] * np.uint64(w)
    cols = np.arange(w, dtype=np.uint64)[None, :]
    with np.errstate(over="ignore"):
        return base + rows + cols


def uniform_image(h: int, w: int, seed: int, n: int = 0, rows=None,
                  chunk_rows: int = 1024) -> np.ndarray:
    """float32 [rows][w] with exact 24-bit values in [0,1); rows defaults to all h."""
    r0, r1 = (0, h) if rows is None else rows
    out = np.empty((r1 - r0, w), np.float32)
    for a in range(r0, r1, chunk_rows):
        b = min(r1, a + chunk_rows)
        z = _splitmix64(_counters(seed, n, h, w, a, b))
        out[a - r0:b - r0] = (z >> np.uint64(40)).astype(np.float32) * np.float32(2.0 ** -24)
    return out


def integer_image(h: int, w: int, seed: int, n: int = 0) -> np.ndarray:
    """float32 [h][w] with integer values in {-15..15} (exact in any order, pin P5)."""
    z = _splitmix64(_counters(seed, n, h, w, 0, h))
    return (((z >> np.uint64(32)) % np.uint64(31)).astype(np.int64) - 15).astype(np.float32)


def uniform_batch(nimg: int, h: int, w: int, seed: int) -> np.ndarray:
    return np.stack([uniform_image(h, w, seed, n) for n in range(nimg)])


def binomial_kernel(K: int) -> np.ndarray:
    """k_i = C(K-1, i) / 2^(K-1): the benchmark (Gaussian-blur) kernel."""
    return np.array([math.comb(K - 1, i) / 2.0 ** (K - 1) for i in range(K)], np.float32)


def random_kernel(K: int, seed: int, signed: bool = False) -> np.ndarray:
    rng = np.random.default_rng(seed)
    if signed:
        return rng.uniform(-1.0, 1.0, K).astype(np.float32)
    k = rng.uniform(0.0, 1.0, K)
    return (k / k.sum()).astype(np.float32)


def integer_kernel(K: int, seed: int) -> np.ndarray:
    rng = np.random.default_rng(seed)
    return rng.integers(-3, 4, K).astype(np.float32)


def delta_kernel(K: int, m: int) -> np.ndarray:
    k = np.zeros(K, np.float32)
    k[m] = 1.0
    return k


def box_kernel(K: int, normalized: bool = False) -> np.ndarray:
    return np.full(K, (1.0 / K) if normalized else 1.0, np.float32)


# ---- Poisson2D SOR inputs (input recipe) ------------------------------
def poisson_problem(n: int, m: int, seed: int, guess: str = "zero"):
    """(x, b) for an [n][m] grid: x carries the Dirichlet boundary (uniform [0,1) on the outer
    frame) and the initial guess of the interior (0, or uniform [0,1) with guess="uniform");
    b = f / (max(n, m) - 1)^2 with f uniform [0,1): the right-hand side with the grid spacing
    h = 1/(max(n,m)-1) folded in (reading P1), so the solution is O(1)."""
    u = uniform_image(n, m, seed, n=0)
    x = np.zeros((n, m), np.float32)
    x[0, :], x[-1, :], x[:, 0], x[:, -1] = u[0, :], u[-1, :], u[:, 0], u[:, -1]
    if guess == "uniform" and n > 2 and m > 2:
        x[1:-1, 1:-1] = u[1:-1, 1:-1]
    h2 = float(max(n, m) - 1) ** 2 if max(n, m) > 1 else 1.0
    b = (uniform_image(n, m, seed, n=1) / np.float32(h2)).astype(np.float32)
    return x, b


def omega_opt(n: int, m: int) -> float:
    """Young's optimal relaxation factor for the model problem on the larger side,
    2 / (1 + sin(pi / (max(n, m) - 1))) -- the bench's default w (an input, not a result)."""
    s = max(n, m) - 1
    return 2.0 / (1.0 + math.sin(math.pi / s)) if s > 1 else 1.0


# ---- Black-Scholes inputs (input recipe) ------------------------------
BS_RATE, BS_VOL = 0.02, 0.30


def bs_options(n: int, seed: int):
    """(spot, strike, years) float32 arrays of n options from the counter generator:
    S uniform [5, 30), X uniform [1, 100), T uniform [0.25, 10) -- the ranges of the
    classic GPU Black-Scholes benchmark; r = BS_RATE, v = BS_VOL are scalars."""
    u = uniform_image(3, n, seed)
    s = (np.float32(5.0) + np.float32(25.0) * u[0]).astype(np.float32)
    x = (np.float32(1.0) + np.float32(99.0) * u[1]).astype(np.float32)
    t = (np.float32(0.25) + np.float32(9.75) * u[2]).astype(np.float32)
    return s, x, t
