"""CPU oracle for GPU sample sort -- TEST INFRASTRUCTURE ONLY.

A ctypes wrapper over ``oracle/liboracle.so`` (built from ``oracle/oracle.c``,
a plain sequential C implementation of Algorithm 1 of Leischner, Osipov &
Sanders, "GPU Sample Sort", with the Section 5 details
P:279-352 and the readings listed in DESIGN.md).

Only ``tests/``, ``__graft_entry__.smoke()`` and ``bench.py`` (the
``cpu_baseline`` leg and ``--impl reference``) may import this package.  The
product package ``paper_conf_ipps_leischneros10_b200`` never imports it and
shares no code with it.
"""
from __future__ import annotations

import ctypes
import os
import subprocess
from dataclasses import dataclass, field

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "oracle.c")
_REF = os.path.join(_HERE, "libref.cc")
_LIB = os.path.join(_HERE, "liboracle.so")


def build(force: bool = False) -> str:
    """Compile oracle.c with gcc (plain -O2, no vectorisation tricks; OpenMP only
    for the thread-parallel timing mode) plus the library-sort references."""
    newest = max(os.path.getmtime(_SRC), os.path.getmtime(_REF), os.path.getmtime(__file__))
    if force or not os.path.exists(_LIB) or os.path.getmtime(_LIB) < newest:
        tmp = _LIB + f".{os.getpid()}.tmp"
        o1, o2 = tmp + ".oracle.o", tmp + ".libref.o"
        subprocess.check_call(["gcc", "-O2", "-Wall", "-fopenmp", "-fPIC", "-c", "-o", o1, _SRC])
        subprocess.check_call(["g++", "-O2", "-Wall", "-fopenmp", "-fPIC", "-c", "-o", o2, _REF])
        subprocess.check_call(["g++", "-shared", "-fopenmp", "-o", tmp, o1, o2])
        os.replace(tmp, _LIB)
        for o in (o1, o2):
            os.remove(o)
    return _LIB


class _Params(ctypes.Structure):
    _fields_ = [
        ("k", ctypes.c_uint32),
        ("a", ctypes.c_uint32),
        ("M", ctypes.c_uint64),
        ("k_policy", ctypes.c_uint32),
        ("fill_div", ctypes.c_uint32),
        ("sample_cap", ctypes.c_uint32),
        ("threads", ctypes.c_uint32),
        ("seed", ctypes.c_uint64),
    ]


_lib = None


def _load():
    global _lib
    if _lib is None:
        lib = ctypes.CDLL(build())
        u64, u32, vp = ctypes.c_uint64, ctypes.c_uint32, ctypes.c_void_p
        pp = ctypes.POINTER(_Params)
        lib.oracle_splitmix64.restype = u64
        lib.oracle_splitmix64.argtypes = [u64]
        lib.oracle_sample_hash.restype = u64
        lib.oracle_sample_hash.argtypes = [u64, u32, u64, u64]
        lib.oracle_choose_kb.restype = u32
        lib.oracle_choose_kb.argtypes = [pp, u64]
        lib.oracle_a_eff.restype = u32
        lib.oracle_a_eff.argtypes = [pp, u32]
        lib.oracle_count_less.restype = u32
        lib.oracle_count_less.argtypes = [vp, u32, u64]
        lib.oracle_classify.restype = u32
        lib.oracle_classify.argtypes = [vp, u32, u32, u64]
        lib.oracle_tree.restype = None
        lib.oracle_tree.argtypes = [vp, u32, vp]
        lib.oracle_traverse_tree.restype = u32
        lib.oracle_traverse_tree.argtypes = [vp, u32, u64]
        lib.oracle_sort.restype = vp
        lib.oracle_sort.argtypes = [vp, vp, u64, pp, ctypes.c_int]
        lib.oracle_distribute.restype = vp
        lib.oracle_distribute.argtypes = [vp, vp, u64, pp]
        lib.oracle_log_count.restype = ctypes.c_size_t
        lib.oracle_log_count.argtypes = [vp]
        lib.oracle_log_info.restype = None
        lib.oracle_log_info.argtypes = [vp, ctypes.c_size_t, vp]
        lib.oracle_log_splitters.restype = None
        lib.oracle_log_splitters.argtypes = [vp, ctypes.c_size_t, vp]
        lib.oracle_log_children.restype = None
        lib.oracle_log_children.argtypes = [vp, ctypes.c_size_t, vp]
        lib.oracle_log_free.restype = None
        lib.oracle_log_free.argtypes = [vp]
        lib.oracle_select.restype = u64
        lib.oracle_select.argtypes = [vp, u64, u64]
        for w in ("u32", "u64"):
            getattr(lib, f"libref_std_sort_{w}").restype = None
            getattr(lib, f"libref_std_sort_{w}").argtypes = [vp, u64]
            getattr(lib, f"libref_parallel_sort_{w}").restype = None
            getattr(lib, f"libref_parallel_sort_{w}").argtypes = [vp, u64, ctypes.c_int]
        _lib = lib
    return _lib


@dataclass
class Params:
    """Sample-sort parameters (P:342-352 defaults; DESIGN.md readings)."""

    k: int = 128
    a: int = 30
    M: int = 1 << 17        # P:343 ("M = 217" = 2^17)
    k_policy: int = 0       # 0 = fixed (paper), 1 = adaptive (R29)
    fill_div: int = 4
    sample_cap: int = 16384
    seed: int = 5489        # R2
    threads: int = 1        # > 1: OpenMP tasks over child buckets (same output, for timing)

    def c(self) -> _Params:
        return _Params(self.k, self.a, self.M, self.k_policy, self.fill_div, self.sample_cap, self.threads,
                       self.seed & 0xFFFFFFFFFFFFFFFF)


@dataclass
class LevelRecord:
    level: int
    kb: int
    ks: int
    eq: int
    K: int
    a_eff: int
    lo: int
    m: int
    splitters: np.ndarray = field(repr=False)
    children: np.ndarray = field(repr=False)


def _as_u64(a) -> np.ndarray:
    if isinstance(a, np.ndarray):
        return np.ascontiguousarray(a.astype(np.uint64, copy=True))
    return np.array(list(a), dtype=np.uint64)          # python ints, exact up to 2^64-1


def _ptr(a: np.ndarray | None):
    return None if a is None else a.ctypes.data_as(ctypes.c_void_p)


def _read_log(h) -> list[LevelRecord]:
    lib = _load()
    out = []
    info = np.zeros(8, dtype=np.uint64)
    for i in range(lib.oracle_log_count(h)):
        lib.oracle_log_info(h, i, _ptr(info))
        lvl, kb, ks, eq, K, a_eff, lo, m = (int(x) for x in info)
        spl = np.zeros(max(ks - 1, 0), dtype=np.uint64)
        ch = np.zeros(K, dtype=np.uint64)
        if ks > 1:
            lib.oracle_log_splitters(h, i, _ptr(spl))
        lib.oracle_log_children(h, i, _ptr(ch))
        out.append(LevelRecord(lvl, kb, ks, eq, K, a_eff, lo, m, spl, ch))
    lib.oracle_log_free(h)
    return out


def sort(keys, values=None, params: Params | None = None, log: bool = False):
    """Sample sort (Algorithm 1).  Returns (keys, values, records).

    keys/values keep their input dtype (uint32 or uint64)."""
    p = params or Params()
    kdt = np.asarray(keys).dtype
    k = _as_u64(keys)
    v = None
    vdt = None
    if values is not None:
        vdt = np.asarray(values).dtype
        v = _as_u64(values)
        assert v.shape == k.shape
    c = p.c()
    h = _load().oracle_sort(_ptr(k), _ptr(v), k.size, ctypes.byref(c), 1 if log else 0)
    recs = _read_log(h) if log else []
    return k.astype(kdt), (None if v is None else v.astype(vdt)), recs


def distribute(keys, values=None, params: Params | None = None):
    """One k-way distribution step over the whole input (Phases 1-4,
    P:251-263).  Returns (partitioned keys, values, LevelRecord)."""
    p = params or Params()
    kdt = np.asarray(keys).dtype
    k = _as_u64(keys)
    v = None if values is None else _as_u64(values)
    vdt = None if values is None else np.asarray(values).dtype
    c = p.c()
    h = _load().oracle_distribute(_ptr(k), _ptr(v), k.size, ctypes.byref(c))
    rec = _read_log(h)[0]
    return k.astype(kdt), (None if v is None else v.astype(vdt)), rec


def splitmix64(x: int) -> int:
    return int(_load().oracle_splitmix64(x & 0xFFFFFFFFFFFFFFFF))


def sample_hash(seed: int, level: int, lo: int, j: int) -> int:
    return int(_load().oracle_sample_hash(seed, level, lo, j))


def choose_kb(params: Params, m: int) -> int:
    c = params.c()
    return int(_load().oracle_choose_kb(ctypes.byref(c), m))


def a_eff(params: Params, kb: int) -> int:
    c = params.c()
    return int(_load().oracle_a_eff(ctypes.byref(c), kb))


def count_less(spl, e: int) -> int:
    s = _as_u64(spl)
    return int(_load().oracle_count_less(_ptr(s), s.size, e))


def classify(spl, eq: int, e: int) -> int:
    s = _as_u64(spl)
    return int(_load().oracle_classify(_ptr(s), s.size, eq, e))


def tree(spl) -> np.ndarray:
    """Implicit search tree bt[0..k) (bt[0] unused) from k-1 sorted splitters."""
    s = _as_u64(spl)
    k = s.size + 1
    bt = np.zeros(k, dtype=np.uint64)
    _load().oracle_tree(_ptr(s), k, _ptr(bt))
    return bt


def traverse_tree(bt, e: int) -> int:
    """Algorithm 2 literally; returns a 1-based bucket index."""
    b = _as_u64(bt)
    return int(_load().oracle_traverse_tree(_ptr(b), b.size, e))


def select(keys, r: int) -> int:
    """The rank-r element of keys (the r-th entry of the sorted output)."""
    k = _as_u64(keys)
    return int(_load().oracle_select(_ptr(k), k.size, r))


def library_sort(keys: np.ndarray, threads: int = 1) -> np.ndarray:
    """CPU library reference (not the oracle): std::sort (threads == 1) or
    __gnu_parallel::sort on `threads` threads, on a copy of keys."""
    a = np.ascontiguousarray(np.array(keys, copy=True))
    w = {np.dtype(np.uint32): "u32", np.dtype(np.uint64): "u64"}[a.dtype]
    lib = _load()
    if threads <= 1:
        getattr(lib, f"libref_std_sort_{w}")(_ptr(a), a.size)
    else:
        getattr(lib, f"libref_parallel_sort_{w}")(_ptr(a), a.size, threads)
    return a
