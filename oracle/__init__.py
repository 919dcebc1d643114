"""CPU oracles for SeparableConvolution and Poisson2D SOR -- TEST INFRASTRUCTURE ONLY.

Only ``tests/``, ``__graft_entry__.smoke()`` and ``bench.py``'s
``cpu_baseline`` / ``--impl reference`` legs may import this package.  The
product path (``libsepconv.so`` and ``paper_conf_asplos_phothilimthanaara13_b200``)
never imports, links or calls it, and the two share no code.

The arithmetic lives in ``oracle.c`` (plain C, double precision, the paper's
Fig. 1 loops written out; P:354-408 of /root/reference/PAPER.md).  This module
only compiles it with gcc and marshals numpy arrays through ctypes.  The one
piece of Python logic here, :func:`band_rows`, is the row-band partition
reading of DESIGN.md R18 written out independently of the product's C code.

``poisson.c`` is the Poisson2D red-black SOR oracle (readings
DESIGN.md section 11), wrapped by the ``sor_*`` / ``rb_*`` functions below;
``blackscholes.c`` the Black-Scholes oracle,
wrapped by :func:`black_scholes`.

Parity status: every function is pinned by ``tests/test_oracle_pins.py`` and
``tests/test_poisson_oracle.py`` and ``tests/test_bs_oracle.py``.
"""
from __future__ import annotations

import ctypes
import os
import subprocess
import threading

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "oracle.c")
_SRCS = [_SRC, os.path.join(_HERE, "poisson.c"), os.path.join(_HERE, "blackscholes.c")]
_LIB = os.path.join(_HERE, "liboracle.so")
_lock = threading.Lock()
_lib = None


def build(force: bool = False) -> str:
    """Compile oracle.c, poisson.c and blackscholes.c into liboracle.so (gcc -O2, no fast-math)."""
    if force or not os.path.exists(_LIB) or any(os.path.getmtime(_LIB) < os.path.getmtime(s) for s in _SRCS):
        tmp = _LIB + ".tmp.%d" % os.getpid()
        subprocess.check_call(["gcc", "-O2", "-std=c11", "-fPIC", "-shared", "-pthread",
                               "-fno-fast-math", "-ffp-contract=off", "-o", tmp, *_SRCS, "-lm"])
        os.replace(tmp, _LIB)
    return _LIB


def _load():
    global _lib
    with _lock:
        if _lib is None:
            lib = ctypes.CDLL(build())
            f32p = np.ctypeslib.ndpointer(np.float32, flags="C_CONTIGUOUS")
            f64p = np.ctypeslib.ndpointer(np.float64, flags="C_CONTIGUOUS")
            i64, i32 = ctypes.c_int64, ctypes.c_int
            lib.oracle_convolve2d.argtypes = [f32p, i64, i64, i64, f32p, i32, f64p,
                                              ctypes.c_void_p, i32]
            lib.oracle_convolve_rows.argtypes = [f32p, i64, i64, i64, f32p, i32, f64p]
            lib.oracle_convolve_columns.argtypes = [f64p, i64, i64, f32p, i32, f64p]
            lib.oracle_separable.argtypes = [f32p, i64, i64, i64, f32p, i32, f64p, f64p]
            lib.oracle_num_cpus.argtypes = []
            lib.oracle_sor_rb.argtypes = [f32p, f32p, i64, i64, ctypes.c_double, i32, f64p]
            lib.oracle_sor_rb_f32.argtypes = [f32p, f32p, i64, i64, ctypes.c_float, i32, f32p]
            lib.oracle_rb_split.argtypes = [f32p, i64, i64, f32p, f32p]
            lib.oracle_rb_merge.argtypes = [f32p, f32p, i64, i64, f32p]
            lib.oracle_poisson_residual.argtypes = [f64p, f32p, i64, i64, f64p]
            lib.oracle_black_scholes.argtypes = [f32p, f32p, f32p, i64, ctypes.c_double, ctypes.c_double,
                                                 f64p, f64p, ctypes.c_void_p, ctypes.c_void_p]
            for fn in (lib.oracle_convolve2d, lib.oracle_convolve_rows,
                       lib.oracle_convolve_columns, lib.oracle_separable, lib.oracle_num_cpus,
                       lib.oracle_sor_rb, lib.oracle_sor_rb_f32, lib.oracle_rb_split,
                       lib.oracle_rb_merge, lib.oracle_poisson_residual, lib.oracle_black_scholes):
                fn.restype = ctypes.c_int
            _lib = lib
    return _lib


def num_cpus() -> int:
    return int(_load().oracle_num_cpus())


def _image(x):
    x = np.asarray(x)
    if x.dtype != np.float32 or x.ndim != 2:
        raise TypeError("oracle expects a 2-D float32 image")
    return np.ascontiguousarray(x)


def _kernel(k):
    k = np.ascontiguousarray(np.asarray(k, dtype=np.float32).reshape(-1))
    if k.size < 1:
        raise ValueError("empty kernel")
    return k


def convolve2d(image, kernel, with_absum: bool = False, nthreads: int = 0):
    """Choice 1 / Convolve2D in double.

    Returns Out [H-K+1][W-K+1] float64 and, if ``with_absum``, the per-cell
    sum of |term| used as the error scale (R14)."""
    img, k = _image(image), _kernel(kernel)
    h, w = img.shape
    K = k.size
    if h < K or w < K:
        raise ValueError("image smaller than kernel")
    out = np.empty((h - K + 1, w - K + 1), np.float64)
    absum = np.empty_like(out) if with_absum else None
    rc = _load().oracle_convolve2d(img, h, w, w, k, K, out,
                                   absum.ctypes.data if with_absum else None, int(nthreads))
    if rc != 0:
        raise ValueError("oracle_convolve2d rejected its arguments")
    return (out, absum) if with_absum else out


def convolve_rows(image, kernel):
    """ConvolveRows: [H][W] -> [H][W-K+1], double."""
    img, k = _image(image), _kernel(kernel)
    h, w = img.shape
    out = np.empty((h, w - k.size + 1), np.float64)
    if _load().oracle_convolve_rows(img, h, w, w, k, k.size, out) != 0:
        raise ValueError("oracle_convolve_rows rejected its arguments")
    return out


def convolve_columns(buffer, kernel):
    """ConvolveColumns: [H][Wb] double -> [H-K+1][Wb], double."""
    buf = np.ascontiguousarray(np.asarray(buffer, dtype=np.float64))
    k = _kernel(kernel)
    h, w = buf.shape
    out = np.empty((h - k.size + 1, w), np.float64)
    if _load().oracle_convolve_columns(buf, h, w, k, k.size, out) != 0:
        raise ValueError("oracle_convolve_columns rejected its arguments")
    return out


def separable(image, kernel):
    """Choice 2: ConvolveRows into buffer, then ConvolveColumns."""
    img, k = _image(image), _kernel(kernel)
    h, w = img.shape
    K = k.size
    if h < K or w < K:
        raise ValueError("image smaller than kernel")
    buf = np.empty((h, w - K + 1), np.float64)
    out = np.empty((h - K + 1, w - K + 1), np.float64)
    if _load().oracle_separable(img, h, w, w, k, K, buf, out) != 0:
        raise ValueError("oracle_separable rejected its arguments")
    return out


def convolve2d_batch(images, kernel, with_absum: bool = False, nthreads: int = 0):
    """Convolve2D applied to each image of an [N][H][W] batch independently."""
    outs = [convolve2d(np.asarray(im), kernel, with_absum, nthreads) for im in images]
    if with_absum:
        return np.stack([o for o, _ in outs]), np.stack([a for _, a in outs])
    return np.stack(outs)


def band_rows(ho: int, nbands: int, g: int):
    """Row-band partition of the output (R18).

    Band g owns output rows [floor(g*Ho/G), floor((g+1)*Ho/G)); computing them
    needs input rows [row0, row1 + K - 1)."""
    return (ho * g) // nbands, (ho * (g + 1)) // nbands


def convolve2d_bands(image, kernel, nbands: int):
    """Each band convolved on its own from its input rows (owned + K-1 halo rows
    from the successor band, P:374 windows extend to +y), then concatenated."""
    img, k = _image(image), _kernel(kernel)
    K = k.size
    ho = img.shape[0] - K + 1
    parts = []
    for g in range(nbands):
        r0, r1 = band_rows(ho, nbands, g)
        if r1 > r0:
            parts.append(convolve2d(np.ascontiguousarray(img[r0:r1 + K - 1]), k))
    return np.concatenate(parts, axis=0)


# ---- Poisson2D red-black SOR (poisson.c) ----------------
def _grid(x, name):
    x = np.asarray(x)
    if x.dtype != np.float32 or x.ndim != 2:
        raise TypeError("%s must be a 2-D float32 matrix" % name)
    return np.ascontiguousarray(x)


def sor_rb(x, b, omega: float, iters: int):
    """Red-black SOR (readings P1-P4) in double from the initial guess / boundary x and the
    right-hand side b (both [N][M] float32); returns the iterate [N][M] float64."""
    x, b = _grid(x, "x"), _grid(b, "b")
    if x.shape != b.shape:
        raise ValueError("x and b differ in shape")
    u = np.empty(x.shape, np.float64)
    if _load().oracle_sor_rb(x, b, x.shape[0], x.shape[1], float(omega), int(iters), u) != 0:
        raise ValueError("oracle_sor_rb rejected its arguments")
    return u


def sor_rb_f32(x, b, omega: float, iters: int):
    """The same iteration in float32 with the fixed evaluation order of DESIGN.md P6."""
    x, b = _grid(x, "x"), _grid(b, "b")
    if x.shape != b.shape:
        raise ValueError("x and b differ in shape")
    u = np.empty(x.shape, np.float32)
    if _load().oracle_sor_rb_f32(x, b, x.shape[0], x.shape[1], float(np.float32(omega)), int(iters), u) != 0:
        raise ValueError("oracle_sor_rb_f32 rejected its arguments")
    return u


def rb_split(x):
    """Reading P5: red[i][k] = x[i][2k + (i & 1)], black[i][k] = x[i][2k + 1 - (i & 1)];
    both [N][ceil(M/2)] (cells past the row's end are left 0)."""
    x = _grid(x, "x")
    n, m = x.shape
    red = np.zeros((n, (m + 1) // 2), np.float32)
    black = np.zeros_like(red)
    if _load().oracle_rb_split(x, n, m, red, black) != 0:
        raise ValueError("oracle_rb_split rejected its arguments")
    return red, black


def rb_merge(red, black, m: int):
    red, black = _grid(red, "red"), _grid(black, "black")
    n = red.shape[0]
    x = np.empty((n, m), np.float32)
    if _load().oracle_rb_merge(red, black, n, m, x) != 0:
        raise ValueError("oracle_rb_merge rejected its arguments")
    return x


def poisson_residual(u, b):
    """r = b - A u on interior cells (reading P1), 0 on the boundary frame; double."""
    u = np.ascontiguousarray(np.asarray(u, np.float64))
    b = _grid(b, "b")
    r = np.empty(u.shape, np.float64)
    if _load().oracle_poisson_residual(u, b, u.shape[0], u.shape[1], r) != 0:
        raise ValueError("oracle_poisson_residual rejected its arguments")
    return r


def sor_abs_scale(x, b, omega: float, iters: int):
    """The absolute-value iteration A_{t+1} = |1-w| A_t + (w/4) (sum |neighbours| + |b|),
    A_0 = |x| (frame fixed): a per-cell bound on the magnitudes every float32 evaluation of
    P4 combines, used to scale the rounding-error bound (P7): the red-black sweep
    order of oracle_sor_rb with the coefficients |1-w| and w/4 applied to magnitudes."""
    a = np.abs(_grid(x, "x")).astype(np.float64)
    bb = np.abs(_grid(b, "b")).astype(np.float64)
    n, m = a.shape
    c0, c1 = abs(1.0 - omega), omega / 4.0
    ii, jj = np.meshgrid(np.arange(n), np.arange(m), indexing="ij")
    interior = (ii > 0) & (ii < n - 1) & (jj > 0) & (jj < m - 1)
    masks = [interior & ((ii + jj) % 2 == c) for c in (0, 1)]
    for _ in range(int(iters)):
        for mask in masks:
            nb = np.zeros_like(a)
            nb[1:-1, 1:-1] = a[:-2, 1:-1] + a[2:, 1:-1] + a[1:-1, :-2] + a[1:-1, 2:]
            a = np.where(mask, c0 * a + c1 * (nb + bb), a)
    return a


# ---- Black-Scholes (blackscholes.c) -----------------------
def black_scholes(s, x, t, r: float, v: float, with_scale: bool = False):
    """European call and put prices in double for float32 spot s, strike x, expiry t (years)
    and scalar rate r, volatility v.  With ``with_scale`` also the float32 error scales of the
    call and of the put (reading B4): returns (call, put, scale_call, scale_put)."""
    s, x, t = (np.ascontiguousarray(np.asarray(a, np.float32).reshape(-1)) for a in (s, x, t))
    if not (s.size == x.size == t.size):
        raise ValueError("s, x, t differ in length")
    call = np.empty(s.size, np.float64)
    put = np.empty(s.size, np.float64)
    sc = np.empty(s.size, np.float64) if with_scale else None
    sp = np.empty(s.size, np.float64) if with_scale else None
    rc = _load().oracle_black_scholes(s, x, t, s.size, float(r), float(v), call, put,
                                      sc.ctypes.data if with_scale else None,
                                      sp.ctypes.data if with_scale else None)
    if rc != 0:
        raise ValueError("oracle_black_scholes rejected its arguments")
    return (call, put, sc, sp) if with_scale else (call, put)
