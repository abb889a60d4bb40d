"""Mismatch counts of whole sorts under parameter variants (debug aid)."""
import os, sys
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import numpy as np
import torch
import inputs
import paper_conf_ipps_leischneros10_b200 as gss

n = (1 << 20) + 4321
for bits in (32, 64):
    x = inputs.keys("uniform", n, bits, seed=1)
    ref = np.sort(x)
    kd = torch.from_numpy(x).cuda()
    for name, kw in [("default", dict(M=4096)), ("stable", dict(M=4096, flags=4)), ("k32", dict(M=4096, k=32)),
                     ("k16", dict(M=4096, k=16)), ("k64", dict(M=4096, k=64)), ("k256fixed", dict(M=4096, k_policy="fixed")),
                     ("1level", dict(M=16384, max_levels=1)), ("tile2048", dict(M=4096, tile=2048)),
                     ("bigM", dict()), ("k1024", dict(M=4096, k=1024))]:
        try:
            ko, _, st = gss.sort(kd, None, stats=True, **kw)
            torch.cuda.synchronize()
            got = ko.cpu().numpy()
            bad = int((got != ref).sum())
            print(f"u{bits} {name:10s} mismatches={bad} levels={st.levels} split={st.split_elems[:4]} err={st.error_flags}",
                  flush=True)
        except Exception as e:
            print(f"u{bits} {name} EXC {e}", flush=True)
