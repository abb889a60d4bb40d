"""Host logic of the distributed sample sort (paper_conf_ipps_leischneros10_b200.dist)
with world_size 2 over gloo on CPU.  The per-rank kernels are replaced by CPU
stand-ins written here from the same definitions (sample positions from the
oracle's hash, stable partition by #{spl < e}), so this checks the
orchestration: splitter choice, count exchange, all-to-all-v displacements and
the global order of the concatenated result."""
import os
import socket
import sys

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


class CpuOps:
    def sample(self, keys, s, lo_global, seed):
        import oracle
        x = keys.numpy()
        n = x.size
        pos = [(oracle.sample_hash(seed, 255, lo_global, j) * n) >> 64 for j in range(s)]
        return torch.from_numpy(x[pos].copy())

    def sort(self, keys, vals=None):
        x = keys.numpy()
        order = np.argsort(x, kind="stable")
        return torch.from_numpy(x[order].copy()), (None if vals is None else torch.from_numpy(vals.numpy()[order].copy()))

    def partition_by(self, keys, vals, spl):
        x = keys.numpy()
        ids = np.searchsorted(spl.numpy(), x, side="left")
        order = np.argsort(ids, kind="stable")
        cnt = np.bincount(ids, minlength=spl.numel() + 1).astype(np.uint64)
        pv = None if vals is None else torch.from_numpy(vals.numpy()[order].copy())
        return torch.from_numpy(x[order].copy()), pv, torch.from_numpy(cnt)


def _worker(rank, world, port, n_local, dist_name, q):
    sys.path.insert(0, ROOT)
    import inputs
    from paper_conf_ipps_leischneros10_b200.dist import DistSorter
    dist.init_process_group("gloo", init_method=f"tcp://127.0.0.1:{port}", rank=rank, world_size=world)
    try:
        x = inputs.keys(dist_name, n_local * world, 64, seed=3, start=rank * n_local, count=n_local)
        v = inputs.values(n_local, 64, start=rank * n_local)
        ds = DistSorter("u64", n_local, True, device="cpu", samples_per_rank=64, ops=CpuOps())
        k, vv, nr = ds(torch.from_numpy(x), torch.from_numpy(v))
        good = ds.verify(x)
        q.put((rank, k.numpy().copy(), vv.numpy().copy(), nr, good, ds.last_counts))
    finally:
        dist.destroy_process_group()


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


@pytest.mark.parametrize("dist_name", ["uniform", "staggered"])
def test_distributed_sort_gloo_world2(dist_name):
    import inputs
    world, n_local = 2, 3000
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_worker, args=(r, world, port, n_local, dist_name, q)) for r in range(world)]
    for p in procs:
        p.start()
    res = sorted([q.get(timeout=120) for _ in range(world)], key=lambda t: t[0])
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    x = inputs.keys(dist_name, n_local * world, 64, seed=3)
    keys = np.concatenate([r[1] for r in res])
    vals = np.concatenate([r[2] for r in res]).astype(np.int64)
    np.testing.assert_array_equal(keys, np.sort(x))                 # rank r holds the r-th range
    np.testing.assert_array_equal(np.sort(vals), np.arange(x.size))  # values: a permutation ...
    np.testing.assert_array_equal(x[vals], keys)                     # ... pairing each key with its index
    assert all(r[4] for r in res)                                    # DistSorter.verify agrees
    send0, recv0 = res[0][5]
    send1, recv1 = res[1][5]
    assert recv0 == [send0[0], send1[0]] and recv1 == [send0[1], send1[1]]
    assert sum(send0) == n_local and sum(send1) == n_local
    assert abs(res[0][3] - n_local) < 0.25 * n_local                 # balanced by the sample


def test_splitter_positions():
    from paper_conf_ipps_leischneros10_b200.dist import splitter_positions
    assert splitter_positions(8 * 16384, 8) == [16384 * (i + 1) - 1 for i in range(7)]
    assert splitter_positions(10, 1) == []
