"""Host logic of the distributed sample sort (gss_dist_*) without a GPU.

1. gss_dist_plan (libgss.so, host only) against a brute-force model of the
   exchange: every element (bucket, source rank, index) placed in the global
   order, the cuts checked for balance and for never splitting a range
   bucket, and every rank's send ranges / receive counts re-derived.
2. The whole orchestration at world size 2 and 3 over gloo on CPU: each rank
   draws its shard, the hashed sample (oracle's SplitMix64), gathers and sorts
   the samples, picks the splitters S[(i+1)VS/P - 1] (R1), partitions in
   equality mode (R4), all-gathers the counts, asks gss_dist_plan for its
   send/receive ranges, exchanges with gloo point-to-point and sorts its range
   -- the same steps the CUDA path runs with NCCL.  The concatenation over
   ranks must equal the oracle's sort of the global input, and duplicate-heavy
   inputs (dd, all equal) must stay balanced (equality buckets are split).
"""
import os
import socket
import sys

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _plan(P, me, counts):
    from paper_conf_ipps_leischneros10_b200.dist import plan
    return plan(P, me, counts)


def brute_force_exchange(P, counts):
    """Model: the global order lists bucket by bucket, inside a bucket source
    rank by source rank.  Returns per element (bucket, src, local position)."""
    K = 2 * P - 1
    order = []
    loc = np.zeros(P, dtype=np.int64)
    local_start = np.concatenate([np.zeros((P, 1), dtype=np.int64), np.cumsum(counts, axis=1)], axis=1)
    for i in range(K):
        for q in range(P):
            for j in range(int(counts[q, i])):
                order.append((i, q, int(local_start[q, i]) + j))
    return order


@pytest.mark.parametrize("P", [1, 2, 3, 5, 8])
def test_plan_against_brute_force(P):
    rng = np.random.default_rng(P)
    K = 2 * P - 1
    for trial in range(30):
        counts = rng.integers(0, 40, size=(P, K)).astype(np.uint64)
        if trial % 3 == 0:
            counts[:, 1::2] = 0                       # no equality buckets (distinct splitters)
        if trial % 5 == 1 and P > 1:
            counts[:, K // 2 | 1] += 300             # one heavy equality bucket (duplicate splitters)
        order = brute_force_exchange(P, counts.astype(np.int64))
        N = len(order)
        plans = [_plan(P, me, counts) for me in range(P)]
        cuts = [int(c) for c in plans[0][0]]
        assert cuts[0] == 0 and cuts[-1] == N and all(a <= b for a, b in zip(cuts, cuts[1:]))
        for pl in plans:
            assert [int(c) for c in pl[0]] == cuts        # every rank computes the same cuts
        dest = np.zeros(N, dtype=np.int64)
        for q in range(P):
            dest[cuts[q]:cuts[q + 1]] = q
        # range buckets (even ids) are never split across ranks
        by_bucket = {}
        for g, (i, q, j) in enumerate(order):
            by_bucket.setdefault(i, set()).add(int(dest[g]))
        for i, ds in by_bucket.items():
            if i % 2 == 0:
                assert len(ds) == 1, (i, ds)
        # balance: a cut moves off its target only to the nearer end of a range bucket
        biggest_range = max([int(counts[:, i].sum()) for i in range(0, K, 2)] + [0])
        for q in range(1, P):
            assert abs(cuts[q] - (N * q) // P) <= biggest_range // 2 + 1
        # send ranges and receive counts
        for me in range(P):
            _, so, sc, rc = plans[me]
            for q in range(P):
                mine = sorted(j for g, (i, src, j) in enumerate(order) if src == me and dest[g] == q)
                assert int(sc[q]) == len(mine)
                if mine:
                    assert mine == list(range(int(so[q]), int(so[q]) + int(sc[q])))    # contiguous local range
                assert int(rc[q]) == sum(1 for g, (i, src, j) in enumerate(order) if src == q and dest[g] == me)


def test_plan_rejects_bad_arguments():
    from paper_conf_ipps_leischneros10_b200 import _lib
    from paper_conf_ipps_leischneros10_b200.dist import _bind
    lib = _bind(_lib())
    z = np.zeros(16, dtype=np.uint64)
    p = z.ctypes.data_as(__import__("ctypes").c_void_p)
    assert lib.gss_dist_plan(2, 2, 3, p, p, p, p, p) == 1       # me >= P
    assert lib.gss_dist_plan(2, 0, 2, p, p, p, p, p) == 1       # K != 2P-1
    assert lib.gss_dist_plan(0, 0, 1, p, p, p, p, p) == 1


# ---------------------------------------------------------------------------
# World size 2 / 3 over gloo: the orchestration end to end on CPU
# ---------------------------------------------------------------------------
def _worker(rank, world, port, n_local, dist_name, S, q):
    sys.path.insert(0, ROOT)
    import inputs
    import oracle
    dist.init_process_group("gloo", init_method=f"tcp://127.0.0.1:{port}", rank=rank, world_size=world)
    try:
        x = inputs.keys(dist_name, n_local * world, 64, seed=3, start=rank * n_local, count=n_local)
        v = inputs.values(n_local, 64, start=rank * n_local)
        # 1. shard starts; 2. hashed sample of the shard (R2, level tag 255)
        lo = rank * n_local
        smp = np.array([x[(oracle.sample_hash(5489, 255, lo, j) * n_local) >> 64] for j in range(S)], dtype=np.uint64)
        # 3. all-gather, identical sort, splitters S[(i+1) V S / P - 1]
        g = [torch.zeros(S, dtype=torch.int64) for _ in range(world)]
        dist.all_gather(g, torch.from_numpy(smp.view(np.int64)))
        allsmp = np.sort(np.concatenate([t.numpy().view(np.uint64) for t in g]))
        VS = world * S
        spl = np.array([allsmp[((i + 1) * VS) // world - 1] for i in range(world - 1)], dtype=np.uint64)
        # 4. equality-mode ids (R4): 2b between splitters, 2b+1 equal to splitter b; stable partition
        nspl = world - 1
        b = np.searchsorted(spl, x, side="left")
        hit = (b < nspl) & (x == spl[np.minimum(b, max(nspl - 1, 0))]) if nspl else np.zeros(x.size, bool)
        ids = 2 * b + hit
        order = np.argsort(ids, kind="stable")
        pk, pv = x[order], v[order]
        cnt = np.bincount(ids, minlength=2 * world - 1).astype(np.uint64)
        # 5. counts of every rank, the plan from libgss.so
        gc = [torch.zeros(2 * world - 1, dtype=torch.int64) for _ in range(world)]
        dist.all_gather(gc, torch.from_numpy(cnt.view(np.int64)))
        counts = np.stack([t.numpy().view(np.uint64) for t in gc])
        cuts, so, sc, rc = _plan(world, rank, counts)
        # 6. exchange (gloo point-to-point)
        reqs, bufs = [], []
        for peer in range(world):
            a, c = int(so[peer]), int(sc[peer])
            if c and peer != rank:
                reqs.append(dist.isend(torch.from_numpy(pk[a:a + c].view(np.int64).copy()), peer))
                reqs.append(dist.isend(torch.from_numpy(pv[a:a + c].view(np.int64).copy()), peer))
        for peer in range(world):
            c = int(rc[peer])
            kb, vb = torch.zeros(c, dtype=torch.int64), torch.zeros(c, dtype=torch.int64)
            if c and peer == rank:                       # the rank's own range: a local copy
                a = int(so[rank])
                assert int(sc[rank]) == c
                kb.copy_(torch.from_numpy(pk[a:a + c].view(np.int64)))
                vb.copy_(torch.from_numpy(pv[a:a + c].view(np.int64)))
            elif c:
                reqs.append(dist.irecv(kb, peer))
                reqs.append(dist.irecv(vb, peer))
            bufs.append((kb, vb))
        for r in reqs:
            r.wait()
        rk = np.concatenate([kb.numpy().view(np.uint64) for kb, _ in bufs])
        rv = np.concatenate([vb.numpy().view(np.uint64) for _, vb in bufs])
        # 7. local sort
        o = np.argsort(rk, kind="stable")
        q.put((rank, rk[o], rv[o], [int(c) for c in cuts], [int(c) for c in sc], [int(c) for c in rc]))
    finally:
        dist.destroy_process_group()


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


@pytest.mark.parametrize("world,dist_name", [(2, "uniform"), (2, "staggered"), (2, "dd"), (2, "equal"),
                                             (3, "uniform"), (3, "dd"), (3, "and5")])
def test_distributed_orchestration_gloo(world, dist_name):
    import inputs
    import oracle
    n_local = 4000
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_worker, args=(r, world, port, n_local, dist_name, 256, q)) for r in range(world)]
    for p in procs:
        p.start()
    res = sorted([q.get(timeout=180) for _ in range(world)], key=lambda t: t[0])
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    x = inputs.keys(dist_name, n_local * world, 64, seed=3)
    ok, _, _ = oracle.sort(x, None, oracle.Params(k=64, a=30, M=512, k_policy=1))
    keys = np.concatenate([r[1] for r in res])
    vals = np.concatenate([r[2] for r in res]).astype(np.int64)
    np.testing.assert_array_equal(keys, ok)                          # rank r holds the r-th range of the oracle's order
    np.testing.assert_array_equal(np.sort(vals), np.arange(x.size))  # values: a permutation ...
    np.testing.assert_array_equal(x[vals], keys)                     # ... pairing each key with its index
    sends = np.array([r[4] for r in res])
    recvs = np.array([r[5] for r in res])
    np.testing.assert_array_equal(recvs, sends.T)                    # what q sends to r is what r receives from q
    for r in res:                                                    # balanced, also with duplicates
        assert abs(len(r[1]) - n_local) <= 0.2 * n_local, [len(t[1]) for t in res]
