"""B200 GPU sample sort -- thin Python binding over libgss.so (include/gss.h).

Every step of the sort runs in the CUDA kernels of ``libgss.so`` (built for
sm_100a from ``csrc/``); this module only marshals arguments: it takes torch
tensors for device memory and streams, allocates the scratch buffer the C ABI
asks for, and raises ``RuntimeError`` on a non-zero status.  There is no CPU
fallback: without the built library every call raises.

Method: Leischner, Osipov & Sanders, "GPU Sample Sort" (IPDPS 2010),
PAPER.md Algorithm 1 and sections 4-5.
"""
from __future__ import annotations

import ctypes
import os
from dataclasses import dataclass

import torch

from . import _build

__all__ = ["sort", "sort_host", "Sorter", "HostSorter", "HostPipeline", "partition", "partition_by", "sample", "Profiler", "Stats", "temp_bytes",
           "library_path", "KERNEL_KINDS"]

KERNEL_KINDS = ["init", "sample", "classify", "scan", "scatter", "plan", "small_sort", "copy", "overflow", "h2d",
                "d2h", "other"]
FLAG_RECOMPUTE_IDS = 1
FLAG_TREE_CLASSIFY = 512

_u32, _u64, _vp, _sz = ctypes.c_uint32, ctypes.c_uint64, ctypes.c_void_p, ctypes.c_size_t


class _Stats(ctypes.Structure):
    _fields_ = [("levels", _u32), ("launches", _u32), ("levels_launched", _u32), ("error_flags", _u32),
                ("split_elems", _u64 * 16), ("split_buckets", _u64 * 16), ("small_buckets", _u64),
                ("small_elems", _u64), ("max_small", _u64), ("eq_buckets", _u64), ("eq_elems", _u64),
                ("overflow_buckets", _u64), ("overflow_elems", _u64), ("cluster_buckets", _u64)]


class _Params(ctypes.Structure):
    _fields_ = [("k", _u32), ("oversample", _u32), ("small_threshold", _u64), ("tile", _u32),
                ("max_levels", _u32), ("k_policy", _u32), ("fill_div", _u32), ("seed", _u64), ("flags", _u32),
                ("cls_arrays", _u32), ("stats", ctypes.POINTER(_Stats)), ("profiler", _vp), ("error_out", _vp)]


@dataclass
class Stats:
    levels: int
    launches: int
    levels_launched: int
    error_flags: int
    split_elems: list
    split_buckets: list
    small_buckets: int
    small_elems: int
    max_small: int
    eq_buckets: int
    eq_elems: int
    overflow_buckets: int
    overflow_elems: int
    cluster_buckets: int = 0

    @staticmethod
    def _from(s: _Stats) -> "Stats":
        L = 16
        return Stats(s.levels, s.launches, s.levels_launched, s.error_flags, list(s.split_elems[:L]),
                     list(s.split_buckets[:L]), s.small_buckets, s.small_elems, s.max_small, s.eq_buckets,
                     s.eq_elems, s.overflow_buckets, s.overflow_elems, s.cluster_buckets)


_LIB = None
_STATUS = {0: "GSS_SUCCESS", 1: "GSS_ERROR_INVALID_VALUE", 2: "GSS_ERROR_TEMP_TOO_SMALL",
           3: "GSS_ERROR_NOT_SUPPORTED", 4: "GSS_ERROR_CUDA", 5: "GSS_ERROR_NCCL", 6: "GSS_ERROR_CAPACITY"}


def library_path() -> str:
    return _build.LIB


def _lib():
    """Load libgss.so; raise loudly if it was not built (no fallback path)."""
    global _LIB
    if _LIB is None:
        if not os.path.exists(_build.LIB):
            raise RuntimeError(f"libgss.so is not built ({_build.LIB}); run "
                               "`python -m paper_conf_ipps_leischneros10_b200._build` (or __graft_entry__.build())")
        lib = ctypes.CDLL(_build.LIB)
        P = ctypes.POINTER(_Params)
        szp = ctypes.POINTER(_sz)
        for name in ("gss_sort_u32", "gss_sort_u64", "gss_sort_u64_descending", "gss_sort_u32_descending",
                     "gss_sort_f32", "gss_sort_f64", "gss_sort_host_u32", "gss_sort_host_u64"):
            f = getattr(lib, name)
            f.restype = ctypes.c_int
            f.argtypes = [_vp, _vp, _sz, _vp, szp, _vp, P]
        for name in ("gss_sort_pairs_u32", "gss_sort_pairs_u64", "gss_sort_host_pairs_u32",
                     "gss_sort_host_pairs_u64", "gss_sort_pairs_u32_descending", "gss_sort_pairs_u64_descending"):
            f = getattr(lib, name)
            f.restype = ctypes.c_int
            f.argtypes = [_vp, _vp, _vp, _vp, _sz, _vp, szp, _vp, P]
        for name in ("gss_partition_u32", "gss_partition_u64"):
            f = getattr(lib, name)
            f.restype = ctypes.c_int
            f.argtypes = [_vp, _vp, _vp, _vp, _sz, _vp, _vp, _vp, _vp, szp, _vp, P]
        for name in ("gss_partition_by_u32", "gss_partition_by_u64", "gss_partition_by_eq_u32",
                     "gss_partition_by_eq_u64"):
            f = getattr(lib, name)
            f.restype = ctypes.c_int
            f.argtypes = [_vp, _vp, _vp, _vp, _sz, _vp, _u32, _vp, _vp, szp, _vp]
        for name in ("gss_sample_u32", "gss_sample_u64"):
            f = getattr(lib, name)
            f.restype = ctypes.c_int
            f.argtypes = [_vp, _sz, _u64, _u32, _u64, _vp, _sz, _vp]
        lib.gss_host_pipeline_create.restype = ctypes.c_int
        lib.gss_host_pipeline_create.argtypes = [ctypes.POINTER(_vp), _u32, _u32, _sz, P, _vp, szp]
        lib.gss_host_pipeline_run.restype = ctypes.c_int
        lib.gss_host_pipeline_run.argtypes = [_vp, _vp, _vp, _vp, _vp, _vp]
        lib.gss_host_pipeline_flush.restype = ctypes.c_int
        lib.gss_host_pipeline_flush.argtypes = [_vp, _vp]
        lib.gss_host_pipeline_destroy.restype = ctypes.c_int
        lib.gss_host_pipeline_destroy.argtypes = [_vp]
        lib.gss_status_string.restype = ctypes.c_char_p
        lib.gss_status_string.argtypes = [ctypes.c_int]
        lib.gss_version.restype = _u32
        lib.gss_default_params.restype = ctypes.c_int
        lib.gss_default_params.argtypes = [_u32, _u32, P]
        lib.gss_profiler_create.restype = ctypes.c_int
        lib.gss_profiler_create.argtypes = [ctypes.POINTER(_vp)]
        lib.gss_profiler_destroy.restype = ctypes.c_int
        lib.gss_profiler_destroy.argtypes = [_vp]
        lib.gss_profiler_reset.restype = ctypes.c_int
        lib.gss_profiler_reset.argtypes = [_vp]
        lib.gss_profiler_read.restype = ctypes.c_int
        lib.gss_profiler_read.argtypes = [_vp, ctypes.POINTER(ctypes.c_double), ctypes.POINTER(_u64)]
        _LIB = lib
    return _LIB


def _check(rc: int, what: str):
    if rc != 0:
        raise RuntimeError(f"{what}: {_STATUS.get(rc, rc)}")


class Profiler:
    """CUDA-event time of every kernel a call launches (per kernel kind)."""

    def __init__(self):
        h = _vp()
        _check(_lib().gss_profiler_create(ctypes.byref(h)), "gss_profiler_create")
        self._h = h

    def reset(self):
        _check(_lib().gss_profiler_reset(self._h), "gss_profiler_reset")

    def read(self) -> dict:
        """{kind: (ms, launches)} accumulated since the last reset (synchronises the events)."""
        ms = (ctypes.c_double * len(KERNEL_KINDS))()
        ln = (_u64 * len(KERNEL_KINDS))()
        _check(_lib().gss_profiler_read(self._h, ms, ln), "gss_profiler_read")
        return {k: (ms[i], int(ln[i])) for i, k in enumerate(KERNEL_KINDS)}

    def __del__(self):
        try:
            if self._h and _LIB is not None:
                _LIB.gss_profiler_destroy(self._h)
        except Exception:
            pass


def _params(k=None, M=None, a=None, tile=None, seed=None, k_policy=None, fill_div=None, max_levels=None,
            flags=0, stats=None, profiler=None, cls_arrays=None, error_out=None):
    p = _Params()
    p.k = k or 0
    p.small_threshold = M or 0
    p.oversample = a or 0
    p.tile = tile or 0
    p.seed = seed or 0
    p.k_policy = {None: 0, "adaptive": 1, "fixed": 2}[k_policy] if not isinstance(k_policy, int) else k_policy
    p.fill_div = fill_div or 0
    p.max_levels = max_levels or 0
    p.flags = flags
    p.cls_arrays = cls_arrays or 0
    if error_out is not None:
        if not (error_out.is_cuda and error_out.dtype in (torch.int32, torch.uint32) and error_out.numel() >= 1):
            raise ValueError("error_out must be a CUDA int32/uint32 tensor")
        p.error_out = error_out.data_ptr()
    if stats is not None:
        p.stats = ctypes.pointer(stats)
    if profiler is not None:
        p.profiler = profiler._h
    return p


def _kind(t: torch.Tensor) -> str:
    if t.dtype == torch.uint32:
        return "u32"
    if t.dtype == torch.uint64:
        return "u64"
    if t.dtype == torch.float32:
        return "f32"
    if t.dtype == torch.float64:
        return "f64"
    raise TypeError(f"keys must be torch.uint32, uint64, float32 or float64, got {t.dtype}")


def _stream(t: torch.Tensor, stream):
    if stream is not None:
        return stream.cuda_stream if hasattr(stream, "cuda_stream") else int(stream)
    return torch.cuda.current_stream(t.device).cuda_stream


def _ptr(t):
    return None if t is None else ctypes.c_void_p(t.data_ptr())


def _temp(fn, args_before_temp, stream_and_params, device, stream=None):
    """Scratch of the size the C ABI asks for.  When the call runs on a stream
    other than the current one, the scratch is recorded on that stream so the
    caching allocator does not hand it out while the call's kernels run."""
    tb = _sz(0)
    _check(fn(*args_before_temp, None, ctypes.byref(tb), *stream_and_params), fn.__name__ + " (temp query)")
    temp = torch.empty(max(tb.value, 1), dtype=torch.uint8, device=device)
    if isinstance(stream, torch.cuda.Stream):
        temp.record_stream(stream)
    return temp, tb


def _check_out(t: torch.Tensor | None, like: torch.Tensor, what: str):
    """An output buffer must match its input in dtype, length and device and be contiguous."""
    if t is None:
        return
    if t.dtype != like.dtype or t.numel() != like.numel() or t.device != like.device or not t.is_contiguous():
        raise ValueError(f"{what} must be a contiguous {like.dtype} tensor of {like.numel()} elements on "
                         f"{like.device}, got {t.dtype} x {t.numel()} on {t.device}")


def sort(keys: torch.Tensor, values: torch.Tensor | None = None, *, out: torch.Tensor | None = None,
         values_out: torch.Tensor | None = None, descending: bool = False, stats: bool = False,
         profiler: Profiler | None = None, stream=None, **params):
    """Sort device keys (torch.uint32 / torch.uint64, CUDA) and optional values;
    float32 / float64 keys (keys only) sort in IEEE-754 totalOrder.

    Returns (keys_out, values_out) or, with stats=True, (keys_out, values_out, Stats).
    params: k, M, a, tile, seed, k_policy ('adaptive'|'fixed'), fill_div, max_levels, flags."""
    lib = _lib()
    if not keys.is_cuda:
        raise ValueError("sort() takes CUDA tensors; use sort_host() for host buffers")
    with torch.cuda.device(keys.device):
        return _sort(lib, keys, values, out, values_out, descending, stats, profiler, stream, params)


def _sort(lib, keys, values, out, values_out, descending, stats, profiler, stream, params):
    keys = keys.contiguous()
    kind = _kind(keys)
    n = keys.numel()
    _check_out(out, keys, "out")
    out = torch.empty_like(keys) if out is None else out
    st = _Stats() if stats else None
    p = _params(stats=st, profiler=profiler, **params)
    s = _stream(keys, stream)
    if values is not None:
        if kind in ("f32", "f64"):
            raise NotImplementedError("float keys are exported keys-only")
        values = values.contiguous()
        if values.dtype != keys.dtype or values.numel() != n or values.device != keys.device:
            raise TypeError("values must have the key dtype, length and device")
        _check_out(values_out, values, "values_out")
        vout = torch.empty_like(values) if values_out is None else values_out
        fn = getattr(lib, f"gss_sort_pairs_{kind}{'_descending' if descending else ''}")
        head = (_ptr(keys), _ptr(values), _ptr(out), _ptr(vout), n)
    else:
        vout = None
        if descending:
            if kind not in ("u32", "u64"):
                raise NotImplementedError("descending order is exported for u32 / u64 keys")
            fn = getattr(lib, f"gss_sort_{kind}_descending")
        else:
            fn = getattr(lib, f"gss_sort_{kind}")
        head = (_ptr(keys), _ptr(out), n)
    temp, tb = _temp(fn, head, (s, ctypes.byref(p)), keys.device, stream)
    _check(fn(*head, _ptr(temp), ctypes.byref(tb), s, ctypes.byref(p)), fn.__name__)
    if stats:
        return out, vout, Stats._from(st)
    return out, vout


def temp_bytes(kind: str, n: int, pairs: bool = False, host: bool = False, **params) -> int:
    """Scratch bytes the C ABI asks for (host-only computation, no GPU access)."""
    lib = _lib()
    p = _params(**params)
    tb = _sz(0)
    pre = "gss_sort_host_" if host else "gss_sort_"
    if pairs:
        fn = getattr(lib, f"{pre}pairs_{kind}")
        rc = fn(None, None, None, None, n, None, ctypes.byref(tb), None, ctypes.byref(p))
    else:
        fn = getattr(lib, f"{pre}{kind}")
        rc = fn(None, None, n, None, ctypes.byref(tb), None, ctypes.byref(p))
    _check(rc, fn.__name__)
    return tb.value


class Sorter:
    """Repeated device sorts of n keys (and values) with a persistent scratch
    buffer: the call a benchmark or a serving loop makes."""

    def __init__(self, kind: str, n: int, pairs: bool = False, device=None, descending: bool = False, **params):
        self.lib = _lib()
        self.kind, self.n, self.pairs = kind, n, pairs
        self.device = torch.device(device or "cuda")
        self.params = params
        self.temp = torch.empty(max(temp_bytes(kind, n, pairs, **params), 1), dtype=torch.uint8, device=self.device)
        if descending:
            if kind not in ("u32", "u64"):
                raise NotImplementedError("descending order is exported for u32 / u64 keys")
            self.fn = getattr(self.lib, f"gss_sort_{'pairs_' if pairs else ''}{kind}_descending")
        else:
            self.fn = getattr(self.lib, f"gss_sort_{'pairs_' if pairs else ''}{kind}")

    def __call__(self, keys, out, vals=None, vals_out=None, stream=None, profiler=None, stats=False):
        st = _Stats() if stats else None
        p = _params(stats=st, profiler=profiler, **self.params)
        s = stream.cuda_stream if stream is not None else torch.cuda.current_stream(self.device).cuda_stream
        tb = _sz(self.temp.numel())
        if self.pairs:
            rc = self.fn(_ptr(keys), _ptr(vals), _ptr(out), _ptr(vals_out), self.n, _ptr(self.temp),
                         ctypes.byref(tb), s, ctypes.byref(p))
        else:
            rc = self.fn(_ptr(keys), _ptr(out), self.n, _ptr(self.temp), ctypes.byref(tb), s, ctypes.byref(p))
        _check(rc, self.fn.__name__)
        return Stats._from(st) if stats else None


class HostSorter:
    """End-to-end sort of HOST buffers through gss_sort_host_*: the call
    enqueues host->device copy, sort and device->host copy.  Keeps its
    device scratch between calls."""

    def __init__(self, kind: str, n: int, pairs: bool = False, device=None, **params):
        self.lib = _lib()
        self.kind, self.n, self.pairs = kind, n, pairs
        self.device = torch.device(device or "cuda")
        self.params = params
        self.temp = torch.empty(max(temp_bytes(kind, n, pairs, host=True, **params), 1), dtype=torch.uint8,
                                device=self.device)
        self.fn = getattr(self.lib, f"gss_sort_host_{'pairs_' if pairs else ''}{kind}")

    def __call__(self, h_keys, h_out, h_vals=None, h_vals_out=None, stream=None, profiler=None, stats=False):
        st = _Stats() if stats else None
        p = _params(stats=st, profiler=profiler, **self.params)
        s = stream.cuda_stream if stream is not None else torch.cuda.current_stream(self.device).cuda_stream
        tb = _sz(self.temp.numel())
        if self.pairs:
            rc = self.fn(_ptr(h_keys), _ptr(h_vals), _ptr(h_out), _ptr(h_vals_out), self.n, _ptr(self.temp),
                         ctypes.byref(tb), s, ctypes.byref(p))
        else:
            rc = self.fn(_ptr(h_keys), _ptr(h_out), self.n, _ptr(self.temp), ctypes.byref(tb), s, ctypes.byref(p))
        _check(rc, self.fn.__name__)
        return Stats._from(st) if stats else None


class HostPipeline:
    """Pipelined end-to-end sorts of host (pinned) arrays through gss_host_pipeline_*:
    consecutive calls overlap host->device copy, sort and device->host copy."""

    def __init__(self, kind: str, n: int, pairs: bool = False, device=None, **params):
        self.lib = _lib()
        self.n = n
        self.device = torch.device(device or "cuda")
        kb = 4 if kind == "u32" else 8
        self._p = _params(**params)
        tb = _sz(0)
        _check(self.lib.gss_host_pipeline_create(None, kb, kb if pairs else 0, n, ctypes.byref(self._p), None,
                                                 ctypes.byref(tb)), "gss_host_pipeline_create (query)")
        self.temp = torch.empty(max(tb.value, 1), dtype=torch.uint8, device=self.device)
        h = _vp()
        _check(self.lib.gss_host_pipeline_create(ctypes.byref(h), kb, kb if pairs else 0, n, ctypes.byref(self._p),
                                                 _ptr(self.temp), ctypes.byref(tb)), "gss_host_pipeline_create")
        self._h = h

    def __call__(self, h_keys, h_out, h_vals=None, h_vals_out=None, stream=None):
        s = stream.cuda_stream if stream is not None else torch.cuda.current_stream(self.device).cuda_stream
        _check(self.lib.gss_host_pipeline_run(self._h, _ptr(h_keys), _ptr(h_vals), _ptr(h_out), _ptr(h_vals_out), s),
               "gss_host_pipeline_run")

    def flush(self, stream=None):
        """Make `stream` wait for the last run's output (then synchronise it)."""
        s = stream.cuda_stream if stream is not None else torch.cuda.current_stream(self.device).cuda_stream
        _check(self.lib.gss_host_pipeline_flush(self._h, s), "gss_host_pipeline_flush")

    def __del__(self):
        try:
            if getattr(self, "_h", None) and _LIB is not None:
                _LIB.gss_host_pipeline_destroy(self._h)
        except Exception:
            pass


def sort_host(h_keys: torch.Tensor, h_values: torch.Tensor | None = None, **params):
    """Sort host (pinned) tensors end to end; returns host tensors (synchronises)."""
    kind = _kind(h_keys)
    hs = HostSorter(kind, h_keys.numel(), h_values is not None, **params)
    out = torch.empty_like(h_keys, pin_memory=True)
    vout = torch.empty_like(h_values, pin_memory=True) if h_values is not None else None
    hs(h_keys, out, h_values, vout)
    torch.cuda.current_stream(hs.device).synchronize()
    return out, vout


def partition(keys: torch.Tensor, values: torch.Tensor | None = None, *, stream=None, **params):
    """One k-way distribution step (Phases 1-4) over the whole input.

    Returns (keys_out, values_out, splitters, offsets, info) where info is
    (k_b, k_s, eq, K), splitters holds k_s-1 keys and offsets K+1 boundaries."""
    lib = _lib()
    kind = _kind(keys)
    keys = keys.contiguous()
    if values is not None:
        values = values.contiguous()
        if values.dtype != keys.dtype or values.numel() != keys.numel() or values.device != keys.device:
            raise TypeError("values must have the key dtype, length and device")
    n = keys.numel()
    out = torch.empty_like(keys)
    vout = torch.empty_like(values) if values is not None else None
    # k_b may exceed params['k'] only up to the ABI maximum: the default k is
    # resolved from n inside the library (256 .. 1024), so size for 1024
    kcap = 1024
    spl = torch.empty(kcap, dtype=keys.dtype, device=keys.device)
    off = torch.zeros(2 * kcap + 1, dtype=torch.uint64, device=keys.device)
    info = torch.zeros(4, dtype=torch.uint32, device=keys.device)
    p = _params(**params)
    with torch.cuda.device(keys.device):
        s = _stream(keys, stream)
        fn = getattr(lib, f"gss_partition_{kind}")
        head = (_ptr(keys), _ptr(values), _ptr(out), _ptr(vout), n, _ptr(spl), _ptr(off), _ptr(info))
        temp, tb = _temp(fn, head, (s, ctypes.byref(p)), keys.device, stream)
        _check(fn(*head, _ptr(temp), ctypes.byref(tb), s, ctypes.byref(p)), fn.__name__)
        if isinstance(stream, torch.cuda.Stream):
            stream.synchronize()
        inf = [int(x) for x in info.cpu().tolist()]
    kb, ks, eq, K = inf
    return out, vout, spl[: max(ks - 1, 0)], off[: K + 1], tuple(inf)


def partition_by(keys: torch.Tensor, values: torch.Tensor | None, splitters: torch.Tensor, *, stream=None,
                 eq: bool = False):
    """Stable partition of keys into len(splitters)+1 buckets by given sorted
    splitters (ties go left).  Returns (keys_out, values_out, counts[u64]).
    eq=True: equality mode (R4), 2*len(splitters)+1 buckets (gss_partition_by_eq)."""
    lib = _lib()
    kind = _kind(keys)
    keys = keys.contiguous()
    if values is not None:
        values = values.contiguous()
        if values.dtype != keys.dtype or values.numel() != keys.numel() or values.device != keys.device:
            raise TypeError("values must have the key dtype, length and device")
    if splitters.dtype != keys.dtype or splitters.device != keys.device:
        raise TypeError("splitters must have the key dtype and device")
    spl = splitters.contiguous()          # kept alive until the call returns (and recorded on `stream`)
    n = keys.numel()
    out = torch.empty_like(keys)
    vout = torch.empty_like(values) if values is not None else None
    nspl = spl.numel()
    counts = torch.zeros(2 * nspl + 1 if eq else nspl + 1, dtype=torch.uint64, device=keys.device)
    with torch.cuda.device(keys.device):
        s = _stream(keys, stream)
        fn = getattr(lib, f"gss_partition_by_{'eq_' if eq else ''}{kind}")
        head = (_ptr(keys), _ptr(values), _ptr(out), _ptr(vout), n, _ptr(spl), nspl, _ptr(counts))
        tb = _sz(0)
        _check(fn(*head, None, ctypes.byref(tb), s), fn.__name__)
        temp = torch.empty(max(tb.value, 1), dtype=torch.uint8, device=keys.device)
        if isinstance(stream, torch.cuda.Stream):
            temp.record_stream(stream)
            spl.record_stream(stream)
        _check(fn(*head, _ptr(temp), ctypes.byref(tb), s), fn.__name__)
    return out, vout, counts


def sample(keys: torch.Tensor, s: int, lo_global: int = 0, level_tag: int = 255, seed: int = 5489, *, stream=None):
    """s keys at positions mulhi64(H(seed, level_tag, lo_global, j), n) (R2)."""
    lib = _lib()
    kind = _kind(keys)
    out = torch.empty(s, dtype=keys.dtype, device=keys.device)
    fn = getattr(lib, f"gss_sample_{kind}")
    _check(fn(_ptr(keys), keys.numel(), lo_global, level_tag, seed, _ptr(out), s, _stream(keys, stream)), fn.__name__)
    return out
