"""ctypes binding of include/bs.h (Black-Scholes) -- argument marshalling only:
the pricing runs in libsepconv.so's CUDA kernels; loading fails loudly if the library is
missing (no CPU fallback)."""
from __future__ import annotations

import ctypes

from .sepconv import SepconvError, _check, _ptr, _stream, lib as _sepconv_lib

_SIG_DONE = False


def lib() -> ctypes.CDLL:
    global _SIG_DONE
    L = _sepconv_lib()
    if not _SIG_DONE:
        P, I64, F = ctypes.c_void_p, ctypes.c_int64, ctypes.c_float
        for name in ("bs_price", "bs_price_host"):
            fn = getattr(L, name)
            fn.restype = ctypes.c_int
            fn.argtypes = [P, P, P, I64, F, F, P, P, P]
        _SIG_DONE = True
    return L


def exported_symbols():
    return ["bs_price", "bs_price_host"]


def price(s, x, t, r: float, v: float, call, put, n: int | None = None, stream=None):
    """bs_price on device buffers (torch CUDA float32 tensors or raw pointers), async."""
    n = int(n if n is not None else s.numel())
    _check(lib().bs_price(_ptr(s), _ptr(x), _ptr(t), n, float(r), float(v), _ptr(call), _ptr(put),
                          _stream(stream)), "bs_price")
    return call, put


def price_host(s, x, t, r: float, v: float, call, put, n: int | None = None, stream=None):
    """bs_price_host on HOST buffers (numpy arrays or pinned torch CPU tensors); synchronous."""
    if n is None:
        n = s.numel() if hasattr(s, "numel") else s.size
    _check(lib().bs_price_host(_ptr(s), _ptr(x), _ptr(t), int(n), float(r), float(v), _ptr(call), _ptr(put),
                               _stream(stream)), "bs_price_host")
    return call, put


__all__ = ["price", "price_host", "exported_symbols", "lib", "SepconvError"]
