"""Distributed sample sort across GPUs -- thin binding over gss_dist_* (include/gss.h).

The method is the paper's sample sort (Algorithm 1) applied
across ranks, the setting the paper names as sample sort's home (P:24-25,
P:195-196): large random samples give splitters that balance the ranks
(P:228-233).  Everything runs inside libgss.so on the caller's stream: the
global sample, its all-gather and sort, the splitter choice, the
equality-mode partition, the count all-gather, the exchange plan, the NCCL
all-to-all-v and the local sort.  This module only shares the NCCL unique id
(through the torch.distributed process group), allocates buffers and
marshals arguments.  ``plan`` exposes the host-side exchange plan
(gss_dist_plan) so its logic is testable without a GPU.
"""
from __future__ import annotations

import ctypes

import numpy as np
import torch
import torch.distributed as dist

from . import _check, _lib, _params, _ptr, _kind

__all__ = ["DistSorter", "plan"]

_u32, _u64, _vp, _sz = ctypes.c_uint32, ctypes.c_uint64, ctypes.c_void_p, ctypes.c_size_t


def _bind(lib):
    if getattr(lib, "_gss_dist_bound", False):
        return lib
    P = ctypes.c_void_p
    lib.gss_dist_unique_id.restype = ctypes.c_int
    lib.gss_dist_unique_id.argtypes = [ctypes.c_char_p]
    lib.gss_dist_create.restype = ctypes.c_int
    lib.gss_dist_create.argtypes = [ctypes.POINTER(_vp), ctypes.c_char_p, ctypes.c_int, ctypes.c_int, ctypes.c_int]
    lib.gss_dist_destroy.restype = ctypes.c_int
    lib.gss_dist_destroy.argtypes = [_vp]
    szp = ctypes.POINTER(_sz)
    for w in ("u32", "u64"):
        f = getattr(lib, f"gss_dist_sort_{w}")
        f.restype = ctypes.c_int
        f.argtypes = [_vp, _vp, _sz, _vp, _sz, szp, _vp, szp, _vp, P]
        f = getattr(lib, f"gss_dist_sort_pairs_{w}")
        f.restype = ctypes.c_int
        f.argtypes = [_vp, _vp, _vp, _sz, _vp, _vp, _sz, szp, _vp, szp, _vp, P]
    lib.gss_dist_last_exchange.restype = ctypes.c_int
    lib.gss_dist_last_exchange.argtypes = [_vp, _vp, _vp, _vp]
    lib.gss_dist_plan.restype = ctypes.c_int
    lib.gss_dist_plan.argtypes = [_u32, _u32, _u32, _vp, _vp, _vp, _vp, _vp]
    lib._gss_dist_bound = True
    return lib


def plan(P: int, me: int, counts: np.ndarray):
    """gss_dist_plan (host only): counts is the P x (2P-1) matrix of every rank's
    global-level bucket sizes.  Returns (cuts[P+1], send_off[P], send_cnt[P], recv_cnt[P])."""
    lib = _bind(_lib())
    c = np.ascontiguousarray(counts, dtype=np.uint64)
    K = 2 * P - 1
    assert c.shape == (P, K)
    cuts = np.zeros(P + 1, dtype=np.uint64)
    so, sc, rc = (np.zeros(P, dtype=np.uint64) for _ in range(3))
    p = lambda a: a.ctypes.data_as(ctypes.c_void_p)  # noqa: E731
    _check(lib.gss_dist_plan(P, me, K, p(c), p(cuts), p(so), p(sc), p(rc)), "gss_dist_plan")
    return cuts, so, sc, rc


class DistSorter:
    """Sorts a global array spread over the ranks of a torch.distributed
    process group (one process per GPU): each call passes this rank's shard
    and returns this rank's contiguous range of the global sorted order."""

    def __init__(self, kind: str, n_local: int, pairs: bool = False, device=None, group=None,
                 capacity: int | None = None, **params):
        self.lib = _bind(_lib())
        self.kind, self.n_local, self.pairs = kind, n_local, pairs
        self.device = torch.device(device) if device is not None else torch.device("cuda", torch.cuda.current_device())
        self.group = group
        self.rank = dist.get_rank(group)
        self.world = dist.get_world_size(group)
        self.params = params
        # receive capacity: the plan balances to about n/P (+-2 % at 16 Ki samples per rank)
        self.capacity = capacity if capacity is not None else n_local + n_local // 4 + 65536
        uid = ctypes.create_string_buffer(128)
        if self.rank == 0:
            _check(self.lib.gss_dist_unique_id(uid), "gss_dist_unique_id")
        obj = [bytes(uid.raw) if self.rank == 0 else None]
        dist.broadcast_object_list(obj, src=dist.get_global_rank(group, 0) if group is not None else 0, group=group)
        h = _vp()
        with torch.cuda.device(self.device):
            _check(self.lib.gss_dist_create(ctypes.byref(h), obj[0], self.rank, self.world, self.device.index),
                   "gss_dist_create")
        self._h = h
        dt = torch.uint32 if kind == "u32" else torch.uint64
        self.kout = torch.empty(self.capacity, dtype=dt, device=self.device)
        self.vout = torch.empty(self.capacity, dtype=dt, device=self.device) if pairs else None
        self.fn = getattr(self.lib, f"gss_dist_sort_{'pairs_' if pairs else ''}{kind}")
        tb = _sz(0)
        p = _params(**params)
        self._call(None, None, None, tb, p)
        self.temp = torch.empty(max(tb.value, 1), dtype=torch.uint8, device=self.device)
        self.n_out = 0

    def _call(self, keys, vals, temp, tb, p, stream=None):
        n_out = _sz(0)
        s = stream.cuda_stream if stream is not None else torch.cuda.current_stream(self.device).cuda_stream
        if self.pairs:
            rc = self.fn(self._h, _ptr(keys), _ptr(vals), self.n_local, _ptr(self.kout), _ptr(self.vout),
                         self.capacity, ctypes.byref(n_out), _ptr(temp), ctypes.byref(tb), s, ctypes.byref(p))
        else:
            rc = self.fn(self._h, _ptr(keys), self.n_local, _ptr(self.kout), self.capacity, ctypes.byref(n_out),
                         _ptr(temp), ctypes.byref(tb), s, ctypes.byref(p))
        _check(rc, self.fn.__name__)
        return int(n_out.value)

    def __call__(self, keys: torch.Tensor, vals: torch.Tensor | None = None, stream=None, profiler=None,
                 stats: bool = False):
        """Returns (sorted local range of keys, values or None, received count)."""
        if _kind(keys) != self.kind or keys.numel() != self.n_local or keys.device != self.device:
            raise ValueError(f"keys must be {self.kind} x {self.n_local} on {self.device}")
        if self.pairs and (vals is None or vals.dtype != keys.dtype or vals.numel() != self.n_local):
            raise ValueError("values must have the key dtype and length")
        from . import _Stats, Stats
        st = _Stats() if stats else None
        p = _params(stats=st, profiler=profiler, **self.params)
        tb = _sz(self.temp.numel())
        with torch.cuda.device(self.device):
            self.n_out = self._call(keys.contiguous(), vals.contiguous() if self.pairs else None, self.temp, tb, p,
                                    stream)
        k = self.kout[: self.n_out]
        v = self.vout[: self.n_out] if self.pairs else None
        if stats:
            return k, v, self.n_out, Stats._from(st)
        return k, v, self.n_out

    def last_exchange(self):
        """(send counts, receive counts, cuts) of the last call on this rank."""
        P = self.world
        s, r, c = np.zeros(P, dtype=np.uint64), np.zeros(P, dtype=np.uint64), np.zeros(P + 1, dtype=np.uint64)
        p = lambda a: a.ctypes.data_as(ctypes.c_void_p)  # noqa: E731
        _check(self.lib.gss_dist_last_exchange(self._h, p(s), p(r), p(c)), "gss_dist_last_exchange")
        return [int(x) for x in s], [int(x) for x in r], [int(x) for x in c]

    def __del__(self):
        try:
            if getattr(self, "_h", None):
                self.lib.gss_dist_destroy(self._h)
                self._h = None
        except Exception:
            pass

    # ------------------------------------------------------------------
    def verify(self, x_local_input, v_local_input=None) -> bool:
        """Global checks of the last result (not timed): every range sorted, ranges
        ordered across ranks, total count and an order-independent fingerprint of
        the keys -- of the (key, value) pairs when values are given -- preserved."""
        y = self.kout[: self.n_out].cpu().numpy()
        good = bool(np.all(y[1:] >= y[:-1])) if y.size > 1 else True
        first = int(y[0]) if y.size else None
        last = int(y[-1]) if y.size else None
        objs = [None] * self.world
        dist.all_gather_object(objs, (first, last, int(y.size)), group=self.group)
        prev = None
        for f, l, cnt in objs:
            if cnt == 0:
                continue
            if prev is not None and f < prev:
                good = False
            prev = l

        def fp(a, b=None):
            z = a.astype(np.uint64) * np.uint64(0x9E3779B97F4A7C15)
            if b is not None:
                z = z ^ (b.astype(np.uint64) * np.uint64(0xBF58476D1CE4E5B9))
            v = int(np.bitwise_xor.reduce(z ^ (z >> np.uint64(29)))) if a.size else 0
            return v - (1 << 64) if v >= (1 << 63) else v          # as a signed 64-bit value
        yv = self.vout[: self.n_out].cpu().numpy() if (self.pairs and v_local_input is not None) else None
        xin = np.asarray(x_local_input)
        vin = np.asarray(v_local_input) if yv is not None else None
        mine = [fp(xin, vin), fp(y, yv), len(xin), y.size]
        allv = [None] * self.world
        dist.all_gather_object(allv, mine, group=self.group)
        fin = fout = nin = nout = 0
        for t in allv:
            fin ^= t[0]; fout ^= t[1]; nin += t[2]; nout += t[3]
        return good and fin == fout and nin == nout
