"""CPU oracle for SeparableConvolution -- TEST INFRASTRUCTURE ONLY.

Only ``tests/``, ``__graft_entry__.smoke()`` and ``bench.py``'s
``cpu_baseline`` / ``--impl reference`` legs may import this package.  The
product path (``libsepconv.so`` and ``paper_conf_asplos_phothilimthanaara13_b200``)
never imports, links or calls it, and the two share no code.

The arithmetic lives in ``oracle.c`` (plain C, double precision, the paper's
Fig. 1 loops written out; P:354-408 of /root/reference/PAPER.md).  This module
only compiles it with gcc and marshals numpy arrays through ctypes.  The one
piece of Python logic here, :func:`band_rows`, is the row-band partition
reading of DESIGN.md R18 written out independently of the product's C code.

Parity status: every function is pinned by ``tests/test_oracle_pins.py``.
"""
from __future__ import annotations

import ctypes
import os
import subprocess
import threading

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "oracle.c")
_LIB = os.path.join(_HERE, "liboracle.so")
_lock = threading.Lock()
_lib = None


def build(force: bool = False) -> str:
    """Compile oracle.c into liboracle.so with plain gcc (-O2, no fast-math)."""
    if force or not os.path.exists(_LIB) or os.path.getmtime(_LIB) < os.path.getmtime(_SRC):
        tmp = _LIB + ".tmp.%d" % os.getpid()
        subprocess.check_call(["gcc", "-O2", "-std=c11", "-fPIC", "-shared", "-pthread",
                               "-fno-fast-math", "-ffp-contract=off", "-o", tmp, _SRC, "-lm"])
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
            for fn in (lib.oracle_convolve2d, lib.oracle_convolve_rows,
                       lib.oracle_convolve_columns, lib.oracle_separable, lib.oracle_num_cpus):
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
