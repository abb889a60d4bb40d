"""Host-side checks of the C ABI (no GPU): the library loads, exports every
symbol include/gss.h declares, answers temp-size queries without touching a
device, and validates its arguments."""
import ctypes
import os
import re

import pytest

import paper_conf_ipps_leischneros10_b200 as gss
from paper_conf_ipps_leischneros10_b200 import _build

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


@pytest.fixture(scope="module")
def lib():
    _build.build()
    return gss._lib()


def declared_functions():
    src = open(os.path.join(ROOT, "include", "gss.h")).read()
    src = re.sub(r"/\*.*?\*/", "", src, flags=re.S)
    return sorted(set(re.findall(r"\b(gss_[a-z0-9_]+)\s*\(", src)))


def test_exports_every_declared_symbol(lib):
    names = declared_functions()
    assert len(names) >= 20
    for name in names:
        assert hasattr(lib, name), name


def test_status_strings(lib):
    for code, name in gss._STATUS.items():
        assert lib.gss_status_string(code).decode() == name
    assert lib.gss_version() >= 1


@pytest.mark.parametrize("kind,pairs", [("u32", False), ("u64", False), ("u32", True), ("u64", True)])
def test_temp_query_is_host_only(lib, kind, pairs):
    w = 4 if kind == "u32" else 8
    for n in (0, 1, 1000, 1 << 20, 1 << 28):
        tb = gss.temp_bytes(kind, n, pairs)
        # at least the ping-pong copy of the keys (and values) plus one id byte per key
        assert tb >= n * (w + (w if pairs else 0) + 1)
        if n >= 1 << 20:
            assert tb <= n * (w + (w if pairs else 0)) * 2 + (64 << 20) + n * 8
    assert gss.temp_bytes(kind, 1 << 20, pairs, host=True) > gss.temp_bytes(kind, 1 << 20, pairs)


def test_invalid_params_rejected(lib):
    for bad in (dict(k=3), dict(k=2048), dict(k=1), dict(M=1 << 20), dict(tile=1000), dict(k_policy=3)):
        with pytest.raises(RuntimeError, match="INVALID_VALUE"):
            gss.temp_bytes("u64", 1000, **bad)
    with pytest.raises(RuntimeError, match="NOT_SUPPORTED"):
        gss.temp_bytes("u32", 1 << 32)
    # no temp_bytes pointer
    assert lib.gss_sort_u64(None, None, 10, None, None, None, None) == 1


def test_default_params(lib):
    p = gss._Params()
    assert lib.gss_default_params(8, 8, ctypes.byref(p)) == 0
    assert (p.k, p.oversample, p.small_threshold, p.tile) == (0, 30, 8192, 0)
    assert lib.gss_default_params(4, 0, ctypes.byref(p)) == 0
    assert p.small_threshold == 16384
    assert lib.gss_default_params(3, 0, ctypes.byref(p)) == 1


def test_overlapping_buffers_rejected(lib):
    # pointer-range validation happens before any device access
    tb = ctypes.c_size_t(1 << 30)
    base = 1 << 40
    n = 1000
    rc = lib.gss_sort_u64(ctypes.c_void_p(base), ctypes.c_void_p(base + 8), n, ctypes.c_void_p(base + (1 << 20)),
                          ctypes.byref(tb), None, None)
    assert rc == 1                                     # partial overlap of in and out
    rc = lib.gss_sort_u64(ctypes.c_void_p(base), ctypes.c_void_p(base + 8 * n), n, ctypes.c_void_p(base + 100),
                          ctypes.byref(tb), None, None)
    assert rc == 1                                     # temp overlaps the input
    rc = lib.gss_sort_u64(ctypes.c_void_p(base), ctypes.c_void_p(base), n, ctypes.c_void_p(base + (1 << 20)),
                          ctypes.c_size_t(16), None, None)
    assert rc == 2                                     # temp too small


def test_product_does_not_import_oracle():
    pkg = os.path.join(ROOT, "paper_conf_ipps_leischneros10_b200")
    for dirpath, _, files in os.walk(pkg):
        for f in files:
            if f.endswith((".py", ".cu", ".cuh", ".h")):
                txt = open(os.path.join(dirpath, f)).read()
                assert "import oracle" not in txt and "from oracle" not in txt and "oracle.h" not in txt, f



def test_cxx_template_header_builds_and_exports():
    """include/gss.hpp instantiated with user comparators (tests/cxx/custom_less.cu) compiles
    for sm_100a and loads without a GPU."""
    from paper_conf_ipps_leischneros10_b200 import _build
    lib = ctypes.CDLL(_build.build_cxx_test())
    for name in ("cxx_sort_residue_u64", "cxx_sort_pairs_desc_u32_u64"):
        assert hasattr(lib, name)
