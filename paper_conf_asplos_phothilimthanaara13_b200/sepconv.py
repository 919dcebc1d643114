"""Thin Python binding of libsepconv.so (include/sepconv.h) -- argument marshalling only.

Every step of SeparableConvolution runs in the library's sm_100a kernels; this
module converts Python/torch arguments to the C ABI's plain pointers and sizes
and turns status codes into exceptions.  There is no fallback: if the library
is missing or cannot be loaded, :func:`lib` raises.

The names follow the C ABI (``sepconv_plan`` -> :func:`plan`, ``sepconv_run`` ->
:meth:`Plan.run`, ``sepconv_tune`` -> :meth:`Plan.tune`, ...).
"""
from __future__ import annotations

import ctypes
import os
import threading
from dataclasses import dataclass

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
LIB_PATH = os.path.join(_HERE, "libsepconv.so")

SEPCONV_2D, SEPCONV_SEPARABLE, SEPCONV_AUTO = 0, 1, 2
MAP_DIRECT, MAP_TMA = 0, 1
TUNE_FORCE, TUNE_NO_L2_FLUSH = 1, 2
SRC_DEFAULT, SRC_TUNED, SRC_SELECTOR, SRC_EXPLICIT = 0, 1, 2, 3
SELECTOR_LEVELS = 12
MAX_K = 17
NCCL_ID_BYTES = 128
VARIANTS = {"2d": SEPCONV_2D, "separable": SEPCONV_SEPARABLE, "auto": SEPCONV_AUTO}

STATUS = {0: "OK", -1: "E_INVALID", -2: "E_ALIGN", -3: "E_ALIAS", -4: "E_UNSUPPORTED",
          -5: "E_NOMEM", -6: "E_CUDA", -7: "E_NCCL"}


class SepconvError(RuntimeError):
    def __init__(self, status: int, where: str, detail: str):
        self.status = status
        self.code = STATUS.get(status, str(status))
        super().__init__(f"{where}: {self.code}: {detail}")


class _Desc(ctypes.Structure):
    _fields_ = [("n", ctypes.c_int64), ("h", ctypes.c_int64), ("w", ctypes.c_int64), ("k", ctypes.c_int),
                ("ld_in", ctypes.c_int64), ("ld_out", ctypes.c_int64), ("device", ctypes.c_int)]


class _Choice(ctypes.Structure):
    _fields_ = [("algo", ctypes.c_int), ("mapping", ctypes.c_int), ("fused", ctypes.c_int),
                ("config", ctypes.c_int), ("store_path", ctypes.c_int), ("warps", ctypes.c_int),
                ("ctas_per_sm", ctypes.c_int),
                ("median_us", ctypes.c_float), ("sched_parts", ctypes.c_int), ("sched_grid", ctypes.c_int),
                ("sched_steal", ctypes.c_int), ("source", ctypes.c_int)]


class _TuneOpts(ctypes.Structure):
    _fields_ = [("reps", ctypes.c_int), ("cache_path", ctypes.c_char_p), ("flags", ctypes.c_int),
                ("mutations", ctypes.c_int), ("seed", ctypes.c_uint32)]


class _Selector(ctypes.Structure):
    _fields_ = [("k", ctypes.c_int), ("m", ctypes.c_int), ("cutoffs", ctypes.c_int64 * (SELECTOR_LEVELS - 1)),
                ("algos", _Choice * SELECTOR_LEVELS)]


@dataclass(frozen=True)
class Choice:
    algo: int
    mapping: int
    fused: int
    config: int = 0
    store_path: int = 0
    warps: int = 8
    ctas_per_sm: int = 1
    median_us: float = 0.0
    sched_parts: int = 0          # tuned work-schedule override (0 = the library's model)
    sched_grid: int = 0
    source: int = SRC_EXPLICIT    # SRC_DEFAULT / SRC_TUNED / SRC_SELECTOR / SRC_EXPLICIT
    sched_steal: int = 0          # work-stealing threshold in stages (0 = off); strided overrides only

    @property
    def base_name(self) -> str:
        """The candidate's name without a schedule override."""
        a = "2d" if self.algo == SEPCONV_2D else ("sep-fused" if self.fused else "sep-unfused")
        m = ("-tma" if self.mapping == MAP_TMA else "-direct")
        if self.algo == SEPCONV_SEPARABLE and self.fused and self.mapping == MAP_TMA:
            m += "%d" % self.config + ("", "s8", "v2")[self.store_path]
        return a + m

    @property
    def name(self) -> str:
        s = ("@p%dg%d" % (self.sched_parts, self.sched_grid)) if self.sched_parts else ""
        return self.base_name + s + ("st%d" % self.sched_steal if self.sched_parts and self.sched_steal else "")

    def key(self):
        return (self.algo, self.mapping, self.fused, self.config, self.store_path, self.sched_parts, self.sched_grid,
                self.sched_steal)

    def _c(self) -> _Choice:
        return _Choice(self.algo, self.mapping, self.fused, self.config, self.store_path, self.warps, self.ctas_per_sm,
                       self.median_us, self.sched_parts, self.sched_grid, self.sched_steal, self.source)

    @staticmethod
    def _from(c: _Choice) -> "Choice":
        return Choice(c.algo, c.mapping, c.fused, c.config, c.store_path, c.warps, c.ctas_per_sm, float(c.median_us),
                      c.sched_parts, c.sched_grid, c.source, c.sched_steal)


@dataclass(frozen=True)
class Selector:
    """sepconv_selector_t: SELECT(input, s) = algos[i] with cutoffs[i] > n*h*w >= cutoffs[i-1]
    (P:820-829)."""
    k: int
    cutoffs: tuple
    algos: tuple

    def _c(self) -> _Selector:
        s = _Selector()
        s.k, s.m = self.k, len(self.algos)
        for i, c in enumerate(self.cutoffs):
            s.cutoffs[i] = int(c)
        for i, a in enumerate(self.algos):
            s.algos[i] = a._c()
        return s

    @staticmethod
    def _from(s: _Selector) -> "Selector":
        return Selector(s.k, tuple(int(s.cutoffs[i]) for i in range(s.m - 1)),
                        tuple(Choice._from(s.algos[i]) for i in range(s.m)))

    def select(self, size: int) -> Choice:
        """sepconv_select (host arithmetic in the library)."""
        out = _Choice()
        c = self._c()
        _check(lib().sepconv_select(ctypes.byref(c), int(size), ctypes.byref(out)), "sepconv_select")
        return Choice._from(out)


_lib = None
_lock = threading.Lock()


def lib() -> ctypes.CDLL:
    """Load libsepconv.so (RuntimeError if it is absent: there is no CPU fallback)."""
    global _lib
    with _lock:
        if _lib is not None:
            return _lib
        if not os.path.exists(LIB_PATH):
            raise RuntimeError(f"{LIB_PATH} is missing: build it with "
                               "`python -m paper_conf_asplos_phothilimthanaara13_b200.build`")
        L = ctypes.CDLL(LIB_PATH)
        P, I, I64, F = ctypes.c_void_p, ctypes.c_int, ctypes.c_int64, ctypes.c_float
        pI64 = ctypes.POINTER(ctypes.c_int64)
        sig = {
            "sepconv_plan": (I, [I64, I64, I, ctypes.POINTER(P)]),
            "sepconv_plan_ex": (I, [ctypes.POINTER(_Desc), ctypes.POINTER(P)]),
            "sepconv_destroy": (None, [P]),
            "sepconv_out_shape": (I, [P, pI64, pI64]),
            "sepconv_run": (I, [P, P, P, P, I, P]),
            "sepconv_run_choice": (I, [P, P, P, P, ctypes.POINTER(_Choice), P]),
            "sepconv_run_host": (I, [P, P, P, P, I, P]),
            "sepconv_tune": (I, [P, ctypes.POINTER(_TuneOpts), ctypes.POINTER(_Choice)]),
            "sepconv_tune_selector": (I, [I, I, ctypes.POINTER(ctypes.c_int64), I, ctypes.POINTER(_TuneOpts),
                                          ctypes.POINTER(_Selector)]),
            "sepconv_select": (I, [ctypes.POINTER(_Selector), I64, ctypes.POINTER(_Choice)]),
            "sepconv_get_choice": (I, [P, I, ctypes.POINTER(_Choice)]),
            "sepconv_set_choice": (I, [P, I, ctypes.POINTER(_Choice)]),
            "sepconv_num_candidates": (I, [P]),
            "sepconv_get_candidate": (I, [P, I, ctypes.POINTER(_Choice)]),
            "sepconv_band": (I, [I64, I, I, I, pI64, pI64, pI64, pI64]),
            "sepconv_nccl_unique_id": (I, [ctypes.c_char_p]),
            "sepconv_comm_init": (I, [P, ctypes.c_char_p, I, I]),
            "sepconv_run_band": (I, [P, P, P, P, I, P]),
            "sepconv_band_trace": (I, [P, I]),
            "sepconv_band_timeline": (I, [P, ctypes.POINTER(ctypes.c_float)]),
            "sepconv_status_str": (ctypes.c_char_p, [I]),
            "sepconv_last_error": (ctypes.c_char_p, []),
            "sepconv_version": (ctypes.c_char_p, []),
            "sepconv_launch_count": (ctypes.c_uint64, []),
            "sepconv_l2_flush": (I, [P]),
        }
        for name, (res, args) in sig.items():
            fn = getattr(L, name)
            fn.restype = res
            fn.argtypes = args
        _ = F
        _lib = L
        return L


def _check(st: int, where: str):
    if st != 0:
        raise SepconvError(st, where, (lib().sepconv_last_error() or b"").decode())


def l2_flush(stream=None):
    """sepconv_l2_flush: the clean L2 flush the tuner and bench.py time passes after."""
    _check(lib().sepconv_l2_flush(_stream(stream)), "sepconv_l2_flush")


def version() -> str:
    return lib().sepconv_version().decode()


def launch_count() -> int:
    """Kernels this library has launched in this process."""
    return int(lib().sepconv_launch_count())


def exported_symbols():
    return ["sepconv_plan", "sepconv_plan_ex", "sepconv_destroy", "sepconv_out_shape", "sepconv_run",
            "sepconv_run_choice", "sepconv_run_host", "sepconv_tune", "sepconv_tune_selector", "sepconv_select",
            "sepconv_get_choice", "sepconv_set_choice",
            "sepconv_num_candidates", "sepconv_get_candidate", "sepconv_band", "sepconv_nccl_unique_id",
            "sepconv_comm_init", "sepconv_run_band", "sepconv_band_trace", "sepconv_band_timeline",
            "sepconv_status_str", "sepconv_last_error",
            "sepconv_version", "sepconv_launch_count", "sepconv_l2_flush"]


def _variant(v) -> int:
    if isinstance(v, str):
        return VARIANTS[v.lower()]
    return int(v)


def _kernel_buf(kernel, K: int):
    k = np.ascontiguousarray(np.asarray(kernel, dtype=np.float32).reshape(-1))
    if k.size != K:
        raise ValueError(f"kernel has {k.size} taps, plan expects K={K}")
    return k


def _ptr(x) -> int:
    """Raw pointer from an int, a torch tensor (device or host) or a numpy array."""
    if x is None:
        return 0
    if isinstance(x, int):
        return x
    if hasattr(x, "data_ptr"):
        return int(x.data_ptr())
    if isinstance(x, np.ndarray):
        return int(x.ctypes.data)
    raise TypeError(f"cannot take a pointer of {type(x)!r}")


def _stream(stream) -> int:
    if stream is None:
        import torch
        try:          # the raw handle without building a torch.cuda.Stream object (~µs per call)
            return int(torch._C._cuda_getCurrentRawStream(torch._C._cuda_getDevice()))
        except AttributeError:
            return int(torch.cuda.current_stream().cuda_stream)
    if isinstance(stream, int):
        return stream
    return int(stream.cuda_stream)


def band(H: int, K: int, G: int, g: int):
    """sepconv_band: (out_row0, out_rows, in_rows_owned, in_rows_alloc) of band g of G."""
    vals = [ctypes.c_int64() for _ in range(4)]
    _check(lib().sepconv_band(H, K, G, g, *[ctypes.byref(v) for v in vals]), "sepconv_band")
    return tuple(int(v.value) for v in vals)


def nccl_unique_id() -> bytes:
    buf = ctypes.create_string_buffer(NCCL_ID_BYTES)
    _check(lib().sepconv_nccl_unique_id(buf), "sepconv_nccl_unique_id")
    return buf.raw


class Plan:
    """Owns a sepconv_plan_t.  Shapes: in [n][h][ld_in], out [n][h-k+1][ld_out], float32."""

    def __init__(self, h: int, w: int, k: int, n: int = 1, ld_in: int = 0, ld_out: int = 0, device: int = -1):
        self.n, self.h, self.w, self.k = int(n), int(h), int(w), int(k)
        self.ld_in = int(ld_in) or self.w
        self.ld_out = int(ld_out) or (self.w - self.k + 1)
        self._h = ctypes.c_void_p()
        d = _Desc(self.n, self.h, self.w, self.k, int(ld_in), int(ld_out), int(device))
        _check(lib().sepconv_plan_ex(ctypes.byref(d), ctypes.byref(self._h)), "sepconv_plan_ex")

    # -- lifecycle --
    def close(self):
        if self._h and self._h.value:
            lib().sepconv_destroy(self._h)
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

    @property
    def handle(self):
        return self._h

    def out_shape(self):
        ho, wo = ctypes.c_int64(), ctypes.c_int64()
        _check(lib().sepconv_out_shape(self._h, ctypes.byref(ho), ctypes.byref(wo)), "sepconv_out_shape")
        return int(ho.value), int(wo.value)

    # -- running --
    def run(self, inp, kernel, out, variant="auto", stream=None):
        """sepconv_run on device buffers (torch CUDA tensors or raw pointers), async on `stream`."""
        k = _kernel_buf(kernel, self.k)
        _check(lib().sepconv_run(self._h, _ptr(inp), k.ctypes.data, _ptr(out), _variant(variant),
                                 _stream(stream)), "sepconv_run")
        return out

    def bind(self, inp, kernel, out, variant="auto", stream=None):
        """A prepared sepconv_run for a hot loop: the arguments are marshalled once (pointers,
        kernel buffer, variant, raw stream handle) and the returned callable only makes the C
        call and checks its status -- no per-call numpy or torch work."""
        k = _kernel_buf(kernel, self.k)
        fn = lib().sepconv_run
        args = (self._h, ctypes.c_void_p(_ptr(inp)), ctypes.c_void_p(k.ctypes.data), ctypes.c_void_p(_ptr(out)),
                ctypes.c_int(_variant(variant)), ctypes.c_void_p(_stream(stream)))

        def call(_fn=fn, _args=args, _keep=k):
            st = _fn(*_args)
            if st:
                _check(st, "sepconv_run")
        return call

    def run_choice(self, inp, kernel, out, choice: Choice, stream=None):
        k = _kernel_buf(kernel, self.k)
        c = choice._c()
        _check(lib().sepconv_run_choice(self._h, _ptr(inp), k.ctypes.data, _ptr(out), ctypes.byref(c),
                                        _stream(stream)), "sepconv_run_choice")
        return out

    def run_host(self, inp, kernel, out, variant="auto", stream=None):
        """sepconv_run_host on HOST buffers (numpy arrays or pinned torch CPU tensors); synchronous."""
        k = _kernel_buf(kernel, self.k)
        _check(lib().sepconv_run_host(self._h, _ptr(inp), k.ctypes.data, _ptr(out), _variant(variant),
                                      _stream(stream)), "sepconv_run_host")
        return out

    # -- tuning --
    def tune(self, reps: int = 20, cache_path: str | None = None, force: bool = False,
             no_l2_flush: bool = False, mutations: int = 0, seed: int = 0) -> Choice:
        """sepconv_tune: exhaustive pass + `mutations` schedule mutations (0 = 12, < 0 = none)."""
        flags = (TUNE_FORCE if force else 0) | (TUNE_NO_L2_FLUSH if no_l2_flush else 0)
        opts = _TuneOpts(int(reps), cache_path.encode() if cache_path else None, flags, int(mutations), int(seed))
        out = _Choice()
        _check(lib().sepconv_tune(self._h, ctypes.byref(opts), ctypes.byref(out)), "sepconv_tune")
        return Choice._from(out)

    def get_choice(self, variant="auto") -> Choice:
        out = _Choice()
        _check(lib().sepconv_get_choice(self._h, _variant(variant), ctypes.byref(out)), "sepconv_get_choice")
        return Choice._from(out)

    def set_choice(self, choice: Choice, variant="auto"):
        """sepconv_set_choice: `variant` resolves to `choice` on this plan from now on."""
        c = choice._c()
        _check(lib().sepconv_set_choice(self._h, _variant(variant), ctypes.byref(c)), "sepconv_set_choice")

    def candidates(self):
        res = []
        for i in range(lib().sepconv_num_candidates(self._h)):
            c = _Choice()
            _check(lib().sepconv_get_candidate(self._h, i, ctypes.byref(c)), "sepconv_get_candidate")
            res.append(Choice._from(c))
        return res

    # -- row bands --
    def comm_init(self, unique_id: bytes | None, nranks: int, rank: int):
        """NCCL communicator for row bands; unique_id=None = external-halo mode (caller moves halos)."""
        if unique_id is not None and len(unique_id) != NCCL_ID_BYTES:
            raise ValueError("NCCL unique id must be 128 bytes")
        _check(lib().sepconv_comm_init(self._h, unique_id, int(nranks), int(rank)), "sepconv_comm_init")

    def band_trace(self, enable: bool = True):
        """sepconv_band_trace: record the phase timeline of later run_band calls."""
        _check(lib().sepconv_band_trace(self._h, int(bool(enable))), "sepconv_band_trace")

    def band_timeline(self):
        """sepconv_band_timeline: {interior, exchange, tail: (start_ms, end_ms)} of the last run_band."""
        ms = (ctypes.c_float * 6)()
        _check(lib().sepconv_band_timeline(self._h, ms), "sepconv_band_timeline")
        return {"interior": (ms[0], ms[1]), "exchange": (ms[2], ms[3]), "tail": (ms[4], ms[5])}

    def run_band(self, in_band, kernel, out_band, variant="auto", stream=None):
        k = _kernel_buf(kernel, self.k)
        _check(lib().sepconv_run_band(self._h, _ptr(in_band), k.ctypes.data, _ptr(out_band), _variant(variant),
                                      _stream(stream)), "sepconv_run_band")
        return out_band


def tune_selector(K: int, sides=None, reps: int = 10, cache_path: str | None = None, device: int = -1,
                  no_l2_flush: bool = False) -> Selector:
    """sepconv_tune_selector: the size selector for width K (12 square levels by default)."""
    arr = None
    n = 0
    if sides is not None:
        n = len(sides)
        arr = (ctypes.c_int64 * n)(*[int(x) for x in sides])
    opts = _TuneOpts(int(reps), cache_path.encode() if cache_path else None,
                     TUNE_NO_L2_FLUSH if no_l2_flush else 0, -1, 0)
    out = _Selector()
    _check(lib().sepconv_tune_selector(int(K), int(device), arr, n, ctypes.byref(opts), ctypes.byref(out)),
           "sepconv_tune_selector")
    return Selector._from(out)


def plan(H: int, W: int, K: int) -> Plan:
    """sepconv_plan: one dense H x W image, width-K kernel, current device."""
    return Plan(H, W, K)


def plan_ex(n: int, h: int, w: int, k: int, ld_in: int = 0, ld_out: int = 0, device: int = -1) -> Plan:
    return Plan(h, w, k, n=n, ld_in=ld_in, ld_out=ld_out, device=device)


def convolve(inp, kernel, variant="auto", out=None, plan_obj: Plan | None = None, stream=None):
    """Convenience: torch CUDA float32 [h][w] or [n][h][w] in -> new (or given) out tensor."""
    import torch
    if not (inp.is_cuda and inp.dtype == torch.float32):
        raise TypeError("convolve expects a CUDA float32 tensor")
    x = inp if inp.dim() == 3 else inp.unsqueeze(0)
    n, h, w = x.shape
    if x.stride(-1) != 1 or x.stride(0) != h * x.stride(1):
        raise ValueError("rows must be contiguous and images packed back to back")
    K = int(np.asarray(kernel).size)
    p = plan_obj or Plan(h, w, K, n=n, ld_in=x.stride(1), device=x.device.index)
    if out is None:
        out = torch.empty((n, h - K + 1, w - K + 1), dtype=torch.float32, device=x.device)
    p.run(x, kernel, out, variant, stream)
    return out if inp.dim() == 3 else out[0]
