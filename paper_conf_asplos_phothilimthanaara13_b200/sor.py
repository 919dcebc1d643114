"""ctypes binding of include/sor.h (Poisson2D red-black SOR) -- argument
marshalling only: every step runs in libsepconv.so's CUDA kernels, and loading fails
loudly if the library is missing (no CPU fallback)."""
from __future__ import annotations

import ctypes

from .sepconv import SepconvError, _check, _ptr, _stream, lib as _sepconv_lib

SOR_HALF, SOR_WAVE, SOR_AUTO = 0, 1, 2
VARIANTS = {"half": SOR_HALF, "wave": SOR_WAVE, "auto": SOR_AUTO}
MAX_DEPTH = 8

_SIG_DONE = False


def lib() -> ctypes.CDLL:
    global _SIG_DONE
    L = _sepconv_lib()
    if not _SIG_DONE:
        P, I, I64, F = ctypes.c_void_p, ctypes.c_int, ctypes.c_int64, ctypes.c_float
        pP, pI, pI64 = ctypes.POINTER(P), ctypes.POINTER(I), ctypes.POINTER(I64)
        sig = {
            "sor_plan": (I, [I64, I64, pP]),
            "sor_load": (I, [P, P, I64, P, I64, P]),
            "sor_iterate": (I, [P, F, I, I, P]),
            "sor_store": (I, [P, P, I64, P]),
            "sor_solve": (I, [P, P, P, P, F, I, I, P]),
            "sor_solve_host": (I, [P, P, P, P, F, I, I, P]),
            "sor_buffers": (I, [P, pP, pP, pP, pP, pI64]),
            "sor_tune": (I, [P, I, I, pI, pI]),
            "sor_set_depth": (I, [P, I]),
            "sor_band": (I, [I64, I, I, I, pI64, pI64, pI64, pI64]),
            "sor_comm_init": (I, [P, ctypes.c_char_p, I, I, I]),
            "sor_band_iterate": (I, [P, F, I, I, P]),
            "sor_destroy": (None, [P]),
        }
        for name, (res, args) in sig.items():
            fn = getattr(L, name)
            fn.restype = res
            fn.argtypes = args
        _SIG_DONE = True
    return L


def exported_symbols():
    return ["sor_plan", "sor_load", "sor_iterate", "sor_store", "sor_solve", "sor_solve_host", "sor_buffers",
            "sor_tune", "sor_set_depth", "sor_band", "sor_comm_init", "sor_band_iterate", "sor_destroy"]


def band(n: int, nbands: int, g: int, halo: int):
    """sor_band: (row0, rows, alloc_row0, alloc_rows) of band g of nbands."""
    vals = [ctypes.c_int64() for _ in range(4)]
    _check(lib().sor_band(int(n), int(nbands), int(g), int(halo), *[ctypes.byref(v) for v in vals]), "sor_band")
    return tuple(int(v.value) for v in vals)


def _variant(v) -> int:
    return VARIANTS[v.lower()] if isinstance(v, str) else int(v)


class SorPlan:
    """Owns a sor_plan_t for an n x m grid on the current device.  x, b, u: float32 [n][ld]."""

    def __init__(self, n: int, m: int):
        self.n, self.m = int(n), int(m)
        self._h = ctypes.c_void_p()
        _check(lib().sor_plan(self.n, self.m, ctypes.byref(self._h)), "sor_plan")

    def close(self):
        if self._h and self._h.value:
            lib().sor_destroy(self._h)
            self._h = ctypes.c_void_p()

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass

    def __enter__(self):
        return self

    def __exit__(self, *exc):
        self.close()

    def load(self, x, b, ld_x: int = 0, ld_b: int = 0, stream=None):
        _check(lib().sor_load(self._h, _ptr(x), int(ld_x), _ptr(b), int(ld_b), _stream(stream)), "sor_load")

    def iterate(self, omega: float, iters: int, variant="auto", stream=None):
        _check(lib().sor_iterate(self._h, float(omega), int(iters), _variant(variant), _stream(stream)),
               "sor_iterate")

    def store(self, u, ld_u: int = 0, stream=None):
        _check(lib().sor_store(self._h, _ptr(u), int(ld_u), _stream(stream)), "sor_store")
        return u

    def solve(self, x, b, u, omega: float, iters: int, variant="auto", stream=None):
        _check(lib().sor_solve(self._h, _ptr(x), _ptr(b), _ptr(u), float(omega), int(iters), _variant(variant),
                               _stream(stream)), "sor_solve")
        return u

    def solve_host(self, x, b, u, omega: float, iters: int, variant="auto", stream=None):
        """HOST buffers (numpy / pinned torch CPU tensors), dense [n][m]; synchronous."""
        _check(lib().sor_solve_host(self._h, _ptr(x), _ptr(b), _ptr(u), float(omega), int(iters),
                                    _variant(variant), _stream(stream)), "sor_solve_host")
        return u

    def buffers(self):
        """(u_red, u_black, b_red, b_black) device pointers and ldh."""
        ptrs = [ctypes.c_void_p() for _ in range(4)]
        ldh = ctypes.c_int64()
        _check(lib().sor_buffers(self._h, *[ctypes.byref(p) for p in ptrs], ctypes.byref(ldh)), "sor_buffers")
        return tuple(int(p.value or 0) for p in ptrs), int(ldh.value)

    def tune(self, iters_hint: int = 24, reps: int = 5):
        v, d = ctypes.c_int(), ctypes.c_int()
        _check(lib().sor_tune(self._h, int(iters_hint), int(reps), ctypes.byref(v), ctypes.byref(d)), "sor_tune")
        return int(v.value), int(d.value)

    def set_depth(self, depth: int):
        _check(lib().sor_set_depth(self._h, int(depth)), "sor_set_depth")

    def comm_init(self, unique_id: bytes | None, nranks: int, rank: int, halo: int):
        """Band `rank` of `nranks` with `halo` ghost rows; unique_id=None = external mode."""
        _check(lib().sor_comm_init(self._h, unique_id, int(nranks), int(rank), int(halo)), "sor_comm_init")

    def band_iterate(self, omega: float, iters: int, variant="auto", stream=None):
        _check(lib().sor_band_iterate(self._h, float(omega), int(iters), _variant(variant), _stream(stream)),
               "sor_band_iterate")


__all__ = ["SorPlan", "SOR_HALF", "SOR_WAVE", "SOR_AUTO", "SepconvError", "exported_symbols", "lib"]
