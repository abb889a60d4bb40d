"""Build libgss.so (the CUDA sample sort behind include/gss.h) for sm_100a, in tree.

Every translation unit in csrc/ (gss.cu: the C ABI; gss_inst_*.cu: one
instantiation of the sort engine each) is compiled with
`nvcc -gencode arch=compute_100a,code=sm_100a -O3 -lineinfo` in parallel, then
linked into paper_conf_ipps_leischneros10_b200/libgss.so."""
from __future__ import annotations

import glob
import os
import subprocess
import sys
from concurrent.futures import ThreadPoolExecutor

PKG = os.path.dirname(os.path.abspath(__file__))
ROOT = os.path.dirname(PKG)
CSRC = os.path.join(PKG, "csrc")
OBJ = os.path.join(PKG, "build_obj")
LIB = os.path.join(PKG, "libgss.so")
NVCC = os.environ.get("NVCC", "/usr/local/cuda/bin/nvcc")
ARCH = ["-gencode", "arch=compute_100a,code=sm_100a"]
FLAGS = ARCH + ["-O3", "-lineinfo", "-std=c++17", "--expt-relaxed-constexpr", "-Xcompiler", "-fPIC",
                "-Xptxas", "-v"] + os.environ.get("GSS_NVCC_EXTRA", "").split()   # tuning experiments (-D...)


def nccl_dirs():
    """The NCCL that torch ships (2.28.x: nccl.h + libnccl.so.2); libgss.so links it with an rpath so the
    process shares torch's copy."""
    try:
        import nvidia.nccl as nn
        base = list(nn.__path__)[0]
    except Exception:  # pragma: no cover - image without the wheel
        base = None
    if base and os.path.exists(os.path.join(base, "include", "nccl.h")):
        return os.path.join(base, "include"), os.path.join(base, "lib")
    return "/usr/include", "/usr/lib/x86_64-linux-gnu"


def sources():
    return sorted(glob.glob(os.path.join(CSRC, "*.cu")))


def deps():
    return sources() + glob.glob(os.path.join(CSRC, "*.cuh")) + [os.path.join(ROOT, "include", "gss.h")]


def stale() -> bool:
    if not os.path.exists(LIB):
        return True
    t = os.path.getmtime(LIB)
    return any(os.path.getmtime(d) > t for d in deps())


def _compile(src: str):
    obj = os.path.join(OBJ, os.path.basename(src)[:-3] + ".o")
    inc, _ = nccl_dirs()
    cmd = [NVCC, *FLAGS, "-I", inc, "-c", "-o", obj, src]
    r = subprocess.run(cmd, capture_output=True, text=True)
    return src, obj, cmd, r


def build(force: bool = False, verbose: bool = False) -> str:
    if not force and not stale():
        return LIB
    os.makedirs(OBJ, exist_ok=True)
    srcs = sources()
    with ThreadPoolExecutor(max_workers=min(len(srcs), os.cpu_count() or 4)) as ex:
        results = list(ex.map(_compile, srcs))
    log = os.path.join(PKG, "build.log")
    with open(log, "w") as f:
        for src, obj, cmd, r in results:
            f.write(" ".join(cmd) + "\n" + r.stdout + r.stderr)
    bad = [r for r in results if r[3].returncode != 0]
    if bad:
        sys.stderr.write(bad[0][3].stderr[-4000:])
        raise RuntimeError(f"nvcc failed for {[os.path.basename(b[0]) for b in bad]}; see {log}")
    _, libdir = nccl_dirs()
    cmd = [NVCC, *ARCH, "-shared", "-o", LIB + ".tmp", *[r[1] for r in results], "-L", libdir, "-l:libnccl.so.2",
           "-Xlinker", f"-rpath,{libdir}"]
    r = subprocess.run(cmd, capture_output=True, text=True)
    with open(log, "a") as f:
        f.write(" ".join(cmd) + "\n" + r.stdout + r.stderr)
    if r.returncode != 0:
        sys.stderr.write(r.stderr[-4000:])
        raise RuntimeError(f"nvcc link failed ({r.returncode}); see {log}")
    os.replace(LIB + ".tmp", LIB)
    if verbose:
        print(f"built {LIB} from {len(srcs)} translation units")
    return LIB


CXX_TEST_SRC = os.path.join(ROOT, "tests", "cxx", "custom_less.cu")
CXX_TEST_LIB = os.path.join(ROOT, "tests", "cxx", "libgss_cxx_test.so")


def build_cxx_test(force: bool = False, verbose: bool = False) -> str:
    """Compile tests/cxx/custom_less.cu (include/gss.hpp with user comparators, the comparator-only
    contract of P:52-54) into tests/cxx/libgss_cxx_test.so for sm_100a."""
    dep = [CXX_TEST_SRC, os.path.join(ROOT, "include", "gss.hpp")] + deps()
    if not force and os.path.exists(CXX_TEST_LIB) and all(os.path.getmtime(d) <= os.path.getmtime(CXX_TEST_LIB)
                                                          for d in dep):
        return CXX_TEST_LIB
    cmd = [NVCC, *FLAGS, "-I", nccl_dirs()[0], "-shared", "-o", CXX_TEST_LIB + ".tmp", CXX_TEST_SRC]
    r = subprocess.run(cmd, capture_output=True, text=True)
    if r.returncode != 0:
        sys.stderr.write(r.stderr[-4000:])
        raise RuntimeError(f"nvcc failed for {CXX_TEST_SRC}")
    os.replace(CXX_TEST_LIB + ".tmp", CXX_TEST_LIB)
    if verbose:
        print(f"built {CXX_TEST_LIB}")
    return CXX_TEST_LIB


if __name__ == "__main__":
    build(force="--force" in sys.argv, verbose=True)
