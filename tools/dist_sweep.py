"""Throughput on the paper's input distributions (DESIGN.md §4 readings R13-R19, R22).

One line per (key type, distribution): time per sort (CUDA events on the sort's stream, inputs resident in
HBM and larger than L2), Gkeys/s, the whole-sort algorithmic bytes of that run (bench.py's model, the run's
own level statistics) against the measured HBM peak, the level/bucket statistics, and a result check
(non-decreasing output + order-independent multiset fingerprint of the input, bench.mix_check).

usage: python tools/dist_sweep.py [--n-log 27] [--steps 5] [--types u32,u64,kv64] [--dists uniform,...] > out.jsonl
"""
import argparse
import json
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import numpy as np  # noqa: E402
import torch  # noqa: E402

import bench  # noqa: E402
import inputs  # noqa: E402
import paper_conf_ipps_leischneros10_b200 as gss  # noqa: E402

TYPES = {"u32": (32, False), "u64": (64, False), "kv32": (32, True), "kv64": (64, True)}

ap = argparse.ArgumentParser()
ap.add_argument("--n-log", type=int, default=27)
ap.add_argument("--steps", type=int, default=5)
ap.add_argument("--warmup", type=int, default=3)
ap.add_argument("--types", default="u32,u64,kv64")
ap.add_argument("--dists", default=",".join(d for d in inputs.DISTRIBUTIONS))
a = ap.parse_args()
n = 1 << a.n_log
hbm, peak_src = bench.peaks()
dev = torch.device("cuda", 0)
stream = torch.cuda.current_stream(dev)
for t in a.types.split(","):
    bits, pairs = TYPES[t]
    wk = bits // 8
    wv = wk if pairs else 0
    M = 8192 if (pairs and bits == 64) else (32768 if (bits == 32 and not pairs) else 16384)
    prm = dict(k=bench.auto_k(n, M), a=30, tile=bench.auto_tile(n), flags=16, M=M)
    s = gss.Sorter(f"u{bits}", n, pairs, device=dev, **prm)
    hv = inputs.values(n, bits) if pairs else None
    dv = torch.from_numpy(hv).to(dev) if pairs else None
    vo = torch.empty_like(dv) if pairs else None
    for d in a.dists.split(","):
        x = inputs.keys(d, n, bits, seed=1) if d != "sorted" else inputs.keys(d, n, bits)
        dk = torch.from_numpy(x).to(dev)
        ko = torch.empty_like(dk)
        for _ in range(a.warmup):
            s(dk, ko, dv, vo)
        st = s(dk, ko, dv, vo, stats=True)
        torch.cuda.synchronize(dev)
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record(stream)
        for _ in range(a.steps):
            s(dk, ko, dv, vo)
        e1.record(stream)
        torch.cuda.synchronize(dev)
        ms = e0.elapsed_time(e1) / a.steps
        ok = bench.mix_check(x, ko.cpu().numpy())
        if pairs and ok:          # values: the pairs must be the input's (key, index) pairs (R20: value = index)
            kk, vv = ko.cpu().numpy(), vo.cpu().numpy()
            idx = vv.astype(np.int64)
            ok = bool((x[idx] == kk).all()) and bool((np.bincount(idx, minlength=n) == 1).all())
        B = bench.total_alg_bytes(st, wk, wv, prm["k"], prm["tile"], 30)
        print(json.dumps({"type": t, "dist": d, "n": n, "ms": round(ms, 4), "gkeys_s": round(n / ms / 1e6, 3),
                          "whole_sort_roofline_frac": round(B / (hbm * 1e9) / (ms * 1e-3), 4),
                          "alg_bytes": B, "levels": st.levels, "small_buckets": st.small_buckets,
                          "max_small": st.max_small, "err": st.error_flags, "ok": bool(ok),
                          "params": prm, "peak_gbs": hbm, "peak_source": peak_src}), flush=True)
        del dk, ko
