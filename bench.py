#!/usr/bin/env python3
"""Benchmark of the B200 GPU sample sort (BASELINE.json metric: Gkeys/s and % of
the HBM roofline).

    python bench.py [--gpus N] [--steps K] [--warmup W] [--impl ours|reference]
                    [--workload c4_u64_2p28|c4_u64_2p29|c4_u64_2p30|c2_u32_2p27|c3_u64_2p27|c3_kv64_2p27|c3_kv32_2p27|
                                c1_u32_2p16|c5_kv64_2p29]

One step = one full sort (every level of the k-way distribution pass plus the
in-SM bucket sorts) of the workload's synthetic input, already resident in HBM
(host<->device transfer excluded as in the paper).  Inputs are larger
than the 126 MB L2 (except C1, which is latency-bound and says so).  N > 1
runs under torchrun, one process per GPU: the distributed sample sort
(paper_conf_ipps_leischneros10_b200.dist) with weak scaling (n keys per GPU).
Rank 0 prints one JSON line.

--impl reference times the CPU oracle (oracle/, the plain sample sort written
from the paper) on the host cores on a bounded sample of the same workload.
"""
from __future__ import annotations

import argparse
import json
import os
import subprocess
import sys
import time

import numpy as np

ROOT = os.path.dirname(os.path.abspath(__file__))
sys.path.insert(0, ROOT)

import inputs  # noqa: E402

WORKLOADS = {
    # name: (n, key bits, pairs, distribution, description)
    "c4_u64_2p28": (1 << 28, 64, False, "uniform", "2^28 uniform u64 keys (BASELINE configs[3], the north-star target row)"),
    "c4_u64_2p29": (1 << 29, 64, False, "uniform", "2^29 uniform u64 keys (BASELINE configs[3] sweep)"),
    "c4_u64_2p30": (1 << 30, 64, False, "uniform", "2^30 uniform u64 keys (BASELINE configs[3] sweep)"),
    "c2_u32_2p27": (1 << 27, 32, False, "uniform", "2^27 uniform u32 keys (BASELINE configs[1])"),
    "c3_u64_2p27": (1 << 27, 64, False, "uniform", "2^27 uniform u64 keys (BASELINE configs[2])"),
    "c3_kv64_2p27": (1 << 27, 64, True, "uniform", "2^27 uniform u64 key + u64 value pairs (BASELINE configs[2])"),
    "c3_kv32_2p27": (1 << 27, 32, True, "uniform", "2^27 uniform u32 key + u32 value pairs (not a BASELINE config)"),
    "c1_u32_2p16": (1 << 16, 32, False, "uniform", "2^16 uniform u32 keys, k=128 (BASELINE configs[0]; launch-bound)"),
    "c5_kv64_2p29": (1 << 29, 64, True, "uniform", "2^29 uniform u64 key + u64 value pairs per GPU: 2^32 on 8 GPUs "
                     "(BASELINE configs[4]; distributed sample sort for N > 1)"),
}
DEFAULT_WORKLOAD = "c4_u64_2p28"
CPU_SAMPLE_N = 1 << 25          # cpu_baseline leg: one oracle sort per thread count (~5 s on one core)
REF_STEP_N = 1 << 25            # --impl reference: per-step sample on all host cores


def peaks():
    path = os.path.join(ROOT, "MEASURED_PEAKS.json")
    if os.path.exists(path):
        d = json.load(open(path))
        return float(d["hbm_gbs"]), "measured (MEASURED_PEAKS.json hbm_gbs: torch copy_, read+write)"
    return 6650.0, "fallback (B200_PROFILING.md: 6.65 TB/s)"


def auto_k(n: int, M: int) -> int:
    """The library's default k (gss.h, R29): 256, doubled while two levels would
    leave final buckets above M/2 (2^30 u64 keys: 512)."""
    k = 256
    while k < 1024 and n > k * k * (M // 2):
        k *= 2
    return k


def auto_tile(n: int) -> int:
    """The library's default tile (gss.h): 65536, halved while n < 296 tiles."""
    T = 65536
    while T > 2048 and n < T * 296:
        T //= 2
    return T


def alg_bytes(kind: str, st, wk: int, wv: int, k: int, T: int, a: int, steps: int = 1) -> float:
    """Algorithmic bytes per step of one kernel kind."""
    split = sum(st.split_elems)
    if kind == "classify":
        return split * wk                                     # Phase 2 reads every key once
    if kind == "scatter":
        return split * (2 * wk + 2 * wv)                      # Phase 4 reads and writes key + value
    if kind == "small_sort":
        return st.small_elems * 2 * (wk + wv)                 # one read, one write
    if kind == "scan":
        return split * 16.0 * k / T                           # histogram written, scanned (r+w), read
    if kind == "sample":
        return sum(st.split_buckets) * a * k * 32             # one sector per sampled key
    if kind == "copy":
        return st.eq_elems * 2 * (wk + wv)
    return 0.0


def total_alg_bytes(st, wk, wv, k, T, a):
    return sum(alg_bytes(x, st, wk, wv, k, T, a) for x in ("classify", "scatter", "small_sort", "scan", "sample", "copy"))


class ClockSampler:
    """nvidia-smi clocks and throttle reasons sampled during the timed region."""
    Q = ("clocks.sm,clocks.max.sm,clocks_event_reasons.active,clocks_event_reasons.hw_slowdown,"
         "clocks_event_reasons.hw_thermal_slowdown,clocks_event_reasons.sw_thermal_slowdown,"
         "clocks_event_reasons.sw_power_cap")

    def __init__(self, index: int):
        self.index = index
        self.p = None

    def __enter__(self):
        try:
            self.p = subprocess.Popen(["nvidia-smi", f"--query-gpu={self.Q}", "--format=csv,noheader,nounits",
                                       "-lms", "100", "-i", str(self.index)], stdout=subprocess.PIPE,
                                      stderr=subprocess.DEVNULL, text=True)
        except Exception:
            self.p = None
        time.sleep(0.3)
        return self

    def __exit__(self, *a):
        self.out = ""
        if self.p is not None:
            time.sleep(0.2)
            self.p.terminate()
            try:
                self.out, _ = self.p.communicate(timeout=5)
            except Exception:
                self.p.kill()
                self.out = ""

    def summary(self):
        rows = []
        for line in (self.out or "").strip().splitlines():
            f = [x.strip() for x in line.split(",")]
            if len(f) >= 7:
                try:
                    rows.append((float(f[0]), float(f[1]), f[2:]))
                except ValueError:
                    pass
        if not rows:
            return None
        sm = [r[0] for r in rows]
        names = ["hw_slowdown", "hw_thermal_slowdown", "sw_thermal_slowdown", "sw_power_cap"]
        reasons = sorted({names[i] for r in rows for i, v in enumerate(r[2][1:5]) if v.lower() == "active"})
        load = [s for s in sm if s > 0.5 * max(sm)]
        return {"sm_mhz": float(np.median(load or sm)), "sm_max_mhz": max(r[1] for r in rows), "reasons": reasons,
                "samples": len(rows)}


def mix_check(x: np.ndarray, y: np.ndarray) -> bool:
    """Order-independent multiset fingerprint + sortedness (result check, not timed)."""
    if not np.all(y[1:] >= y[:-1]):
        return False
    def fp(a):
        z = a.astype(np.uint64) * np.uint64(0x9E3779B97F4A7C15)
        return int(np.bitwise_xor.reduce(z ^ (z >> np.uint64(29)))), int(a.astype(np.uint64).sum(dtype=np.uint64))
    return fp(x) == fp(y)


def pairs_check(x: np.ndarray, ko: np.ndarray, vo: np.ndarray, v0: int = 0) -> bool:
    """Values are input indices (+ v0, R20): they must form a permutation and
    carry their own key: x[v - v0] == key (result check, not timed)."""
    idx = vo.astype(np.int64) - v0
    if idx.min(initial=0) < 0 or idx.max(initial=0) >= x.size:
        return False
    seen = np.zeros(x.size, dtype=bool)
    seen[idx] = True
    return bool(seen.all()) and bool(np.array_equal(x[idx], ko))


def cpu_model() -> str:
    try:
        for line in open("/proc/cpuinfo"):
            if line.startswith("model name"):
                return line.split(":", 1)[1].strip()
    except OSError:
        pass
    return "unknown"


def cpu_baseline(wl: str, x: np.ndarray, hv, params: dict) -> dict:
    """The oracle on this host's cores, on a bounded sample of the workload
    (SURVEY 8(d) d.8): all cores (OpenMP tasks per child bucket, the line's
    value), one thread, and the library sorts std::sort (1 thread) and
    __gnu_parallel::sort (all cores) as context.  Not tuned; a baseline only."""
    import oracle
    oracle.build()
    n, bits, pairs, distname, _ = WORKLOADS[wl]
    ns = min(n, CPU_SAMPLE_N)
    xs = x[:ns] if distname != "sorted" else inputs.keys(distname, ns, bits)
    vs = hv[:ns] if pairs else None
    cores = os.cpu_count() or 1
    out = {}
    for label, thr in (("all_cores", cores), ("one_thread", 1)):
        prm = oracle.Params(k=params["k"], a=30, M=params["M"], k_policy=0 if params.get("k_policy") == "fixed" else 1,
                            fill_div=4, seed=5489, threads=thr)
        t0 = time.perf_counter()
        oracle.sort(xs, vs, prm)
        out[label] = {"value": ns / (time.perf_counter() - t0) / 1e9, "threads": thr}
    lib = {}
    if not pairs:
        for label, thr in (("std_sort", 1), ("gnu_parallel_sort", cores)):
            t0 = time.perf_counter()
            oracle.library_sort(xs, thr)
            lib[label] = {"value": ns / (time.perf_counter() - t0) / 1e9, "threads": thr}
    return {"value": out["all_cores"]["value"], "unit": "Gkeys/s", "cores": cores, "kind": "oracle",
            "sample": f"first {ns} keys of this workload's input ({distname}, seed 1); one oracle sort per thread count",
            "one_thread": out["one_thread"], "library_refs": lib, "cpu_model": cpu_model()}


def workload_params(wl: str):
    """Sort parameters of a workload (the library defaults, stated explicitly so the
    JSON line and the roofline terms can name them)."""
    n, bits, pairs, _, _ = WORKLOADS[wl]
    M = 8192 if (pairs and bits == 64) else (32768 if (bits == 32 and not pairs) else 16384)   # in-SM capacity (R5)
    params = dict(k=auto_k(n, M), a=30, tile=auto_tile(n), flags=16)   # flags 16: replay the launch sequence as a CUDA graph
    if wl == "c1_u32_2p16":
        params.update(k=128, k_policy="fixed")
    params["M"] = M
    return params


def metric_name(pairs: bool) -> str:
    return f"sorting rate (Gkeys/s, {'key-value pairs' if pairs else 'keys'}); % HBM roofline"


def config_dict(wl: str, world: int, params: dict) -> dict:
    n, bits, pairs, distname, desc = WORKLOADS[wl]
    kind = f"u{bits}"
    return {"workload": wl, "description": desc, "n_per_gpu": n, "dist": distname, "key": kind,
            "values": kind if pairs else None, **{k: v for k, v in params.items()},
            "l2": "inputs larger than the 126 MB L2" if n * (bits // 8) > (256 << 20) else
            "input fits in L2 (latency-bound config)", "parallelism": f"dp{world}"}


# ---------------------------------------------------------------------------
# reference arm: the CPU oracle
# ---------------------------------------------------------------------------
def run_reference(args, wl):
    rank = int(os.environ.get("RANK", "0"))
    if rank != 0:
        return 0
    import oracle
    oracle.build()
    n, bits, pairs, dist, desc = WORKLOADS[wl]
    ns = min(n, REF_STEP_N)
    x = inputs.keys(dist, ns, bits, seed=1) if dist != "sorted" else inputs.keys(dist, ns, bits)
    v = inputs.values(ns, bits) if pairs else None
    params = workload_params(wl)
    cores = os.cpu_count() or 1
    prm = oracle.Params(k=params["k"], a=30, M=params["M"], k_policy=0 if params.get("k_policy") == "fixed" else 1,
                        fill_div=4, seed=5489, threads=cores)
    times = []
    for i in range(args.warmup + args.steps):
        t0 = time.perf_counter()
        oracle.sort(x, v, prm)
        t1 = time.perf_counter()
        if i >= args.warmup:
            times.append(t1 - t0)
    t = float(np.mean(times))
    val = ns / t / 1e9
    line = {
        "impl": "reference", "metric": metric_name(pairs), "value": val,
        "unit": "Gkeys/s", "n_gpus": args.gpus, "steps": args.steps, "warmup": args.warmup,
        "ms_per_step": t * 1e3, "higher_is_better": True, "scaling": "weak", "vs_baseline": None,
        "dtype": f"u{bits}", "data": "synthetic",
        "config": {**config_dict(wl, 1, params), "n_sample": ns},
        "cpu_baseline": {"value": val, "unit": "Gkeys/s", "cores": cores, "kind": "oracle",
                         "sample": f"first {ns} keys of the workload's generator ({dist}, seed 1), "
                                   f"{cores} threads (OpenMP tasks per child bucket)", "cpu_model": cpu_model()},
        "e2e": {"value": val, "unit": "Gkeys/s", "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0},
    }
    print(json.dumps(line), flush=True)
    return 0


# ---------------------------------------------------------------------------
# our arm
# ---------------------------------------------------------------------------
def library_ref(torch, dkeys, dvals, bits, pairs, steps, dev, stream) -> dict:
    """torch.sort (CUB's device radix sort) of the same device keys -- context for the sample sort, not part of
    it: unsigned keys sorted through the order-preserving signed view (top bit flipped outside the timing);
    pairs as sort + gather of the values by the returned permutation."""
    try:
        sd = torch.int64 if bits == 64 else torch.int32
        flip = torch.tensor(-(1 << (bits - 1)), dtype=sd, device=dev)
        ks = dkeys.view(sd) ^ flip
        def once():
            y, idx = torch.sort(ks)
            if pairs:
                dvals.view(sd).index_select(0, idx)
            return y
        for _ in range(2):
            y = once()
        torch.cuda.synchronize(dev)
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        k = max(3, min(steps, 10))
        e0.record(stream)
        for _ in range(k):
            once()
        e1.record(stream)
        torch.cuda.synchronize(dev)
        ms = e0.elapsed_time(e1) / k
        return {"what": "torch.sort (CUB device radix sort) of the same resident keys" + (" + value gather" if pairs else ""),
                "ms_per_step": round(ms, 4), "value": round(dkeys.numel() / (ms * 1e-3) / 1e9, 3), "unit": "Gkeys/s"}
    except Exception as e:  # pragma: no cover - context only
        return {"error": str(e)[:200]}


def run_single(args, wl):
    os.environ.setdefault("NCCL_DEBUG", "WARN")          # keep stdout to the one JSON line
    import torch
    import torch.distributed as dist_mod

    import paper_conf_ipps_leischneros10_b200 as gss

    world, rank, local = 1, 0, int(os.environ.get("LOCAL_RANK", "0"))
    torch.cuda.set_device(local)
    dev = torch.device("cuda", local)

    n, bits, pairs, distname, desc = WORKLOADS[wl]
    wk = bits // 8
    wv = wk if pairs else 0
    kind = f"u{bits}"
    params = workload_params(wl)
    M = params["M"]

    # input: this rank's shard of the global input (weak scaling: n keys per GPU)
    x = inputs.keys(distname, n * world, bits, seed=1, start=rank * n, count=n)
    hv = inputs.values(n, bits, start=rank * n) if pairs else None
    dkeys = torch.from_numpy(x).to(dev)
    dvals = torch.from_numpy(hv).to(dev) if pairs else None
    stream = torch.cuda.current_stream(dev)

    use_dist = False
    sorter = gss.Sorter(kind, n, pairs, device=dev, **params)
    kout = torch.empty_like(dkeys)
    vout = torch.empty_like(dvals) if pairs else None
    step = lambda: sorter(dkeys, kout, dvals, vout)  # noqa: E731

    for _ in range(args.warmup):
        step()
    torch.cuda.synchronize(dev)

    def barrier():
        if world > 1:
            dist_mod.barrier()

    with ClockSampler(local) as clk:
        barrier()
        torch.cuda.synchronize(dev)
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record(stream)
        for _ in range(args.steps):
            step()
        e1.record(stream)
        torch.cuda.synchronize(dev)
        barrier()
    ms = e0.elapsed_time(e1) / args.steps
    value = n * world / (ms * 1e-3) / 1e9

    # ---- result check (not timed) ----
    ok = mix_check(x, kout.cpu().numpy())
    if pairs:
        ok = ok and pairs_check(x, kout.cpu().numpy(), vout.cpu().numpy(), rank * n)

    # ---- per-kernel breakdown (separate profiled steps, CUDA events per launch) ----
    extra = {}
    roof = None
    gpu_launches = None
    hbm, peak_src = peaks()
    if not use_dist:
        st = sorter(dkeys, kout, dvals, vout, stats=True)
        gpu_launches = st.launches * args.steps
        prof = gss.Profiler()
        kp = max(3, min(args.steps, 10))
        for _ in range(kp):
            sorter(dkeys, kout, dvals, vout, profiler=prof)
        torch.cuda.synchronize(dev)
        per = {k: (v[0] / kp, v[1] / kp) for k, v in prof.read().items() if v[1]}
        kernels_ms = {k: round(v[0], 4) for k, v in per.items()}
        dom = max((k for k in per if k not in ("h2d", "d2h")), key=lambda k: per[k][0])
        a = params["a"]
        ab = alg_bytes(dom, st, wk, wv, params["k"], params["tile"], a)
        achieved = ab / (per[dom][0] * 1e-3) / 1e9
        traffic = None
        tpath = os.path.join(ROOT, "profiles", f"ncu_traffic_{wl}.json")
        if os.path.exists(tpath):
            tr = json.load(open(tpath))
            if dom in tr:
                traffic = tr[dom]                      # DRAM bytes per step of this kernel kind (ncu)
        roof = {"bound": "hbm", "kernel": dom, "achieved": round(achieved, 1), "peak": hbm, "unit": "GB/s",
                "frac": round(achieved / hbm, 4), "traffic": traffic, "alg_bytes_per_step": ab,
                "launches_per_step": per[dom][1], "peak_source": peak_src}
        B = total_alg_bytes(st, wk, wv, params["k"], params["tile"], a)
        extra["kernels_ms_per_step"] = kernels_ms
        extra["whole_sort_roofline"] = {"alg_bytes": B, "t_roof_ms": B / (hbm * 1e9) * 1e3,
                                        "frac": round(B / (hbm * 1e9) / (ms * 1e-3), 4),
                                        "levels": st.levels, "split_elems": st.split_elems[: max(st.levels, 1)],
                                        "small_buckets": st.small_buckets}
    # ---- GPU library context: torch.sort (CUB device radix sort) on the same resident keys ----
    if not use_dist and not args.no_library_ref:
        extra["gpu_library_ref"] = library_ref(torch, dkeys, dvals, bits, pairs, args.steps, dev, stream)
    # ---- end to end through the C ABI with host buffers ----
    e2e = None
    if not use_dist:
        hs = gss.HostPipeline(kind, n, pairs, device=dev, **params)   # overlaps H2D / sort / D2H across steps
        hk = torch.from_numpy(x).pin_memory()
        ho = torch.empty_like(hk).pin_memory()
        hvi = torch.from_numpy(hv).pin_memory() if pairs else None
        hvo = torch.empty_like(hvi).pin_memory() if pairs else None
        for _ in range(2):
            hs(hk, ho, hvi, hvo)
        ke = max(10, args.steps)                                   # pipelined steps: fill and drain amortised
        hs.flush()
        torch.cuda.synchronize(dev)
        e0.record(stream)
        for _ in range(ke):
            hs(hk, ho, hvi, hvo)
        hs.flush()
        e1.record(stream)
        torch.cuda.synchronize(dev)
        ems = e0.elapsed_time(e1) / ke
        ok = ok and bool(np.array_equal(ho.numpy(), kout.cpu().numpy()))
        if pairs:
            ok = ok and pairs_check(x, ho.numpy(), hvo.numpy(), rank * n)
        e2e = {"value": n / (ems * 1e-3) / 1e9, "unit": "Gkeys/s", "h2d_bytes_per_step": n * (wk + wv),
               "d2h_bytes_per_step": n * (wk + wv), "ms_per_step": ems,
               "path": "gss_host_pipeline_run: pinned host in/out, H2D + sort + D2H every step, steps pipelined"}

    # ---- CPU baseline: the oracle on a bounded sample (rank 0, N == 1 only) ----
    cpu = None
    if not args.no_cpu_baseline:
        cpu = cpu_baseline(wl, x, hv, params)

    if rank == 0:
        line = {
            "metric": metric_name(pairs),
            "value": round(value, 3), "unit": "Gkeys/s", "n_gpus": world, "steps": args.steps,
            "warmup": args.warmup, "ms_per_step": round(ms, 4), "higher_is_better": True, "scaling": "weak",
            "vs_baseline": None, "dtype": kind, "data": "synthetic",
            "config": config_dict(wl, world, params),
            "roofline": roof, "cpu_baseline": cpu, "e2e": e2e, "gpu_launches": gpu_launches,
            "clocks": clk.summary(), "result_check": bool(ok), **extra,
        }
        print(json.dumps(line), flush=True)
    return 0 if ok else 1

NVLINK_GBS = 770.0   # measured peer copy per direction (B200_PROFILING.md; 900 nominal)


def run_dist(args, wl):
    """N > 1 (or --force-dist): the distributed sample sort (gss_dist_*, NCCL
    over NVLink), weak scaling: n keys per GPU, n*N in total.  Device time of
    K calls on every rank (barrier + synchronize on both sides), max over ranks."""
    import torch
    import torch.distributed as dist_mod

    import paper_conf_ipps_leischneros10_b200 as gss
    from paper_conf_ipps_leischneros10_b200 import dist as gdist

    world = int(os.environ.get("WORLD_SIZE", "1"))
    rank = int(os.environ.get("RANK", "0"))
    local = int(os.environ.get("LOCAL_RANK", "0"))
    torch.cuda.set_device(local)
    dev = torch.device("cuda", local)
    if not dist_mod.is_initialized():
        os.environ.setdefault("MASTER_ADDR", "127.0.0.1")
        os.environ.setdefault("MASTER_PORT", "29533")
        dist_mod.init_process_group("nccl", rank=rank, world_size=world, device_id=dev)

    n, bits, pairs, distname, desc = WORKLOADS[wl]
    wk = bits // 8
    wv = wk if pairs else 0
    kind = f"u{bits}"
    params = workload_params(wl)
    params.pop("flags", None)                  # no graph replay: the received count varies per call
    if args.fused:
        params["flags"] = 64                   # GSS_FLAG_DIST_FUSED
    x = inputs.keys(distname, n * world, bits, seed=1, start=rank * n, count=n)
    hv = inputs.values(n, bits, start=rank * n) if pairs else None
    dkeys = torch.from_numpy(x).to(dev)
    dvals = torch.from_numpy(hv).to(dev) if pairs else None
    stream = torch.cuda.current_stream(dev)
    sorter = gdist.DistSorter(kind, n, pairs, device=dev, **params)
    step = lambda: sorter(dkeys, dvals)  # noqa: E731
    for _ in range(args.warmup):
        step()
    torch.cuda.synchronize(dev)

    def max_over_ranks(v):
        t = torch.tensor([v], device=dev, dtype=torch.float64)
        dist_mod.all_reduce(t, op=dist_mod.ReduceOp.MAX)
        return float(t.item())

    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    with ClockSampler(local) as clk:
        dist_mod.barrier()
        torch.cuda.synchronize(dev)
        e0.record(stream)
        for _ in range(args.steps):
            step()
        e1.record(stream)
        torch.cuda.synchronize(dev)
        dist_mod.barrier()
    ms = max_over_ranks(e0.elapsed_time(e1) / args.steps)
    value = n * world / (ms * 1e-3) / 1e9
    ok = sorter.verify(x, hv)
    send, recv, cuts = sorter.last_exchange()

    # per-kernel breakdown of our kernels inside the call (CUDA events per launch) and the roofline
    hbm, peak_src = peaks()
    prof = gss.Profiler()
    kp = max(3, min(args.steps, 5))
    st = None
    for i in range(kp):
        r = sorter(dkeys, dvals, profiler=prof, stats=(i == 0))
        if i == 0:
            st = r[3]
    torch.cuda.synchronize(dev)
    per = {k: (v[0] / kp, v[1] / kp) for k, v in prof.read().items() if v[1]}
    launches = int(round(sum(v[1] for v in per.values()))) + 1 + (1 if world > 1 else 0)   # + sample, splitter pick
    n_recv = sorter.n_out
    # algorithmic bytes: global level (classify w_k, scatter 2(w_k+w_v) over n) + the local sort's levels
    # and in-SM sort (from its statistics) + the all-to-all bytes that leave this GPU over NVLink
    local_sort_B = total_alg_bytes(st, wk, wv, params["k"], params["tile"], params["a"])
    B_local = n * (3 * wk + 2 * wv) + local_sort_B
    B_a2a = sum(c for q, c in enumerate(send) if q != rank) * (wk + wv)
    t_roof = B_local / (hbm * 1e9) + B_a2a / (NVLINK_GBS * 1e9)
    t_roof = max_over_ranks(t_roof)
    dom = max(per, key=lambda k: per[k][0])
    roof = {"bound": "hbm+nvlink", "kernel": dom, "achieved": None, "peak": hbm, "unit": "GB/s",
            "frac": round(t_roof / (ms * 1e-3), 4), "traffic": None, "t_roof_ms": t_roof * 1e3,
            "alg_bytes_local": B_local, "a2a_bytes_out": B_a2a, "nvlink_gbs": NVLINK_GBS, "peak_source": peak_src,
            "note": "frac = (B_local / HBM + B_a2a / NVLink) / measured step time (SURVEY 8(d) d.6), max over ranks"}
    if dom in ("classify", "scatter", "small_sort"):
        # the dominant kernel kind summed over the global partition and the local sort
        ab = {"classify": (n + sum(st.split_elems)) * wk,
              "scatter": (n + sum(st.split_elems)) * 2 * (wk + wv),
              "small_sort": st.small_elems * 2 * (wk + wv)}[dom]
        roof["achieved"] = round(ab / (per[dom][0] * 1e-3) / 1e9, 1)
        roof["kernel_frac"] = round(roof["achieved"] / hbm, 4)

    # end to end: pinned host shard -> device, distributed sort, received range -> host, every step
    hk = torch.from_numpy(x).pin_memory()
    hvi = torch.from_numpy(hv).pin_memory() if pairs else None
    hko = torch.empty(sorter.capacity, dtype=dkeys.dtype).pin_memory()
    hvo = torch.empty(sorter.capacity, dtype=dkeys.dtype).pin_memory() if pairs else None
    ke = max(3, min(args.steps, 5))
    dist_mod.barrier()
    torch.cuda.synchronize(dev)
    e0.record(stream)
    d2h = 0
    for _ in range(ke):
        dkeys.copy_(hk, non_blocking=True)
        if pairs:
            dvals.copy_(hvi, non_blocking=True)
        k, v, nr = sorter(dkeys, dvals)
        hko[:nr].copy_(k, non_blocking=True)
        if pairs:
            hvo[:nr].copy_(v, non_blocking=True)
        d2h = nr * (wk + wv)
    e1.record(stream)
    torch.cuda.synchronize(dev)
    ems = max_over_ranks(e0.elapsed_time(e1) / ke)
    e2e = {"value": n * world / (ems * 1e-3) / 1e9, "unit": "Gkeys/s", "h2d_bytes_per_step": n * (wk + wv),
           "d2h_bytes_per_step": d2h, "ms_per_step": ems,
           "path": "DistSorter (gss_dist_sort_*): pinned host shard H2D, distributed sort, received range D2H"}
    okt = torch.tensor([1 if ok else 0], device=dev)
    dist_mod.all_reduce(okt, op=dist_mod.ReduceOp.MIN)
    ok = bool(okt.item())
    if rank == 0:
        line = {
            "metric": metric_name(pairs),
            "value": round(value, 3), "unit": "Gkeys/s", "n_gpus": world, "steps": args.steps,
            "warmup": args.warmup, "ms_per_step": round(ms, 4), "higher_is_better": True, "scaling": "weak",
            "vs_baseline": None, "dtype": kind, "data": "synthetic",
            "config": {**config_dict(wl, world, params), "path": "gss_dist_sort (NCCL all-to-all-v)",
                       "n_total": n * world},
            "roofline": roof, "cpu_baseline": None, "e2e": e2e, "gpu_launches": launches * args.steps,
            "clocks": clk.summary(), "result_check": ok,
            "exchange": {"send_counts_rank0": send, "recv_counts_rank0": recv, "cuts": cuts,
                         "n_recv_rank0": n_recv},
            "kernels_ms_per_step_rank0": {k: round(v[0], 4) for k, v in per.items()},
        }
        print(json.dumps(line), flush=True)
    del sorter
    dist_mod.destroy_process_group()
    return 0 if ok else 1


def spawn_ranks(args) -> int:
    """`python bench.py --gpus N` without torchrun: launch N ranks (one process per GPU) through
    torch.distributed.run on this node and pass their output through."""
    import socket
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    port = s.getsockname()[1]
    s.close()
    cmd = [sys.executable, "-m", "torch.distributed.run", "--nnodes=1", f"--nproc-per-node={args.gpus}",
           "--master-addr", "127.0.0.1", "--master-port", str(port), os.path.abspath(__file__), *sys.argv[1:]]
    return subprocess.call(cmd)


def run_ours(args, wl):
    os.environ.setdefault("NCCL_DEBUG", "WARN")          # keep stdout to the one JSON line
    world = int(os.environ.get("WORLD_SIZE", "0"))
    if world == 0 and args.gpus > 1:
        return spawn_ranks(args)
    if max(world, 1) > 1 or args.force_dist:
        return run_dist(args, wl)
    return run_single(args, wl)


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--steps", type=int, default=10)
    ap.add_argument("--warmup", type=int, default=3)
    ap.add_argument("--impl", default="ours", choices=["ours", "reference"])
    ap.add_argument("--workload", default=DEFAULT_WORKLOAD, choices=sorted(WORKLOADS))
    ap.add_argument("--no-cpu-baseline", action="store_true")
    ap.add_argument("--no-library-ref", action="store_true", help="skip the torch.sort (CUB) context timing")
    ap.add_argument("--force-dist", action="store_true", help="use the distributed path even on one GPU")
    ap.add_argument("--fused", action="store_true", help="distributed path: fused scatter into peer windows "
                                                         "(GSS_FLAG_DIST_FUSED)")
    args = ap.parse_args()
    if args.warmup < 3 and args.impl == "ours":
        args.warmup = 3
    if args.impl == "reference":
        return run_reference(args, args.workload)
    return run_ours(args, args.workload)


if __name__ == "__main__":
    sys.exit(main())
