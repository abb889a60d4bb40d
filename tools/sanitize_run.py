"""Small sorts of every exported kind for compute-sanitizer (memcheck, racecheck,
synccheck, initcheck): several tiles, two or more levels, every in-SM size class,
the equality path, the stable / direct / recompute scatter variants and the
overflow fallback.  Each result is checked against numpy (sanitizer runs are
slow, so the sizes are small).  Usage:
    compute-sanitizer --tool racecheck python tools/sanitize_run.py
"""
import os
import sys

import numpy as np
import torch

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import inputs  # noqa: E402
import paper_conf_ipps_leischneros10_b200 as gss  # noqa: E402


def run():
    n = (1 << 17) + 333
    cases = 0
    for width in (32, 64):
        for pairs in (False, True):
            for dist, flags, extra in (("uniform", 0, {}), ("dd", 0, {}), ("and3", 4, {}), ("uniform", 8, {}),
                                       ("staggered", 1, {}), ("uniform", 0, dict(max_levels=1, k=8, k_policy="fixed")),
                                       ("and4", 512, {}), ("sorted", 0, {})):
                x = inputs.keys(dist, n, width, seed=3)
                v = inputs.values(n, width) if pairs else None
                kd = torch.from_numpy(x).cuda()
                vd = torch.from_numpy(v).cuda() if pairs else None
                ko, vo = gss.sort(kd, vd, M=2048, tile=4096, flags=flags, **extra)
                y = ko.cpu().numpy()
                assert np.array_equal(y, np.sort(x)), (width, pairs, dist, flags)
                if pairs:
                    vv = vo.cpu().numpy().astype(np.int64)
                    assert np.array_equal(np.sort(vv), np.arange(n)) and np.array_equal(x[vv], y)
                cases += 1
    print(f"sanitize_run: {cases} sorts ok", flush=True)


if __name__ == "__main__":
    run()
