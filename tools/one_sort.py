"""Run W+S sorts of a bench workload (for ncu launch lists / full captures)."""
import argparse
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import torch  # noqa: E402

import bench  # noqa: E402
import inputs  # noqa: E402
import paper_conf_ipps_leischneros10_b200 as gss  # noqa: E402

ap = argparse.ArgumentParser()
ap.add_argument("--workload", default=bench.DEFAULT_WORKLOAD)
ap.add_argument("--steps", type=int, default=1)
ap.add_argument("--warmup", type=int, default=1)
ap.add_argument("--k", type=int, default=0)                 # 0: the library default (auto)
ap.add_argument("--tile", type=int, default=0)                # 0: the library default
ap.add_argument("--M", type=int, default=0)
ap.add_argument("--fill_div", type=int, default=0)
ap.add_argument("--flags", type=int, default=0)
ap.add_argument("--cls_arrays", type=int, default=0)
ap.add_argument("--a", type=int, default=0)
args = ap.parse_args()
n, bits, pairs, dist, _ = bench.WORKLOADS[args.workload]
x = inputs.keys(dist, n, bits, seed=1)
k = torch.from_numpy(x).cuda()
v = torch.from_numpy(inputs.values(n, bits)).cuda() if pairs else None
M = args.M or (8192 if (pairs and bits == 64) else (32768 if (bits == 32 and not pairs) else 16384))
s = gss.Sorter(f"u{bits}", n, pairs, k=args.k, tile=args.tile, M=M, fill_div=args.fill_div or None, flags=args.flags,
               cls_arrays=args.cls_arrays or None, a=args.a or None)
ko = torch.empty_like(k)
vo = torch.empty_like(v) if pairs else None
for i in range(args.warmup + args.steps):
    st = s(k, ko, v, vo, stats=(i == 0))
    if i == 0:
        print("launches per sort:", st.launches, "levels:", st.levels, "split:", st.split_elems[:3],
              "small buckets:", st.small_buckets, "max small:", st.max_small)
torch.cuda.synchronize()
