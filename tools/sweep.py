"""Parameter sweep on one workload: time per sort and per-kernel breakdown.
usage: python tools/sweep.py [--workload W] cfg1 cfg2 ...   where cfg = k=256,fill_div=4,M=16384,tile=16384,flags=0"""
import argparse, json, os, sys
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import torch
import bench, inputs
import paper_conf_ipps_leischneros10_b200 as gss

ap = argparse.ArgumentParser()
ap.add_argument("--workload", default="c4_u64_2p28")
ap.add_argument("--steps", type=int, default=5)
ap.add_argument("--dist", default=None, help="override the workload's input distribution")
ap.add_argument("cfgs", nargs="*")
a = ap.parse_args()
n, bits, pairs, dist, _ = bench.WORKLOADS[a.workload]
dist = a.dist or os.environ.get("GSS_DIST") or dist
x = inputs.keys(dist, n, bits, seed=1)
k = torch.from_numpy(x).cuda()
v = torch.from_numpy(inputs.values(n, bits)).cuda() if pairs else None
ko = torch.empty_like(k); vo = torch.empty_like(v) if pairs else None
for cfg in a.cfgs or ["k=256"]:
    prm = {}
    for kv in cfg.split(","):
        kk, vv = kv.split("=")
        prm[kk] = vv if kk == "k_policy" else int(vv)
    try:
        s = gss.Sorter(f"u{bits}", n, pairs, **prm)
        for _ in range(2):
            s(k, ko, v, vo)
        st = s(k, ko, v, vo, stats=True)
        torch.cuda.synchronize()
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record()
        for _ in range(a.steps):
            s(k, ko, v, vo)
        e1.record(); torch.cuda.synchronize()
        ms = e0.elapsed_time(e1) / a.steps
        prof = gss.Profiler()
        for _ in range(3):
            s(k, ko, v, vo, profiler=prof)
        torch.cuda.synchronize()
        per = {kk: round(vv[0] / 3, 3) for kk, vv in prof.read().items() if vv[1]}
        ok = bench.mix_check(x, ko.cpu().numpy()) if a.steps else None
        print(json.dumps({"cfg": cfg, "ms": round(ms, 3), "gkeys": round(n / ms / 1e6, 2), "levels": st.levels,
                          "small_buckets": st.small_buckets, "max_small": st.max_small, "err": st.error_flags,
                          "ok": ok, "kernels": per}), flush=True)
    except Exception as e:
        print(json.dumps({"cfg": cfg, "error": str(e)}), flush=True)
