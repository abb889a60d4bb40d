"""GPU parity: the CUDA path (through the C ABI) against the CPU oracle.

Keys must match bit-exact; values (value = input index, R20) must form the
same multiset of (key, value) pairs; one distribution level (gss_partition)
must equal the oracle's stable partition, splitters and bucket sizes
bit-exact (R7).
"""
import os

import numpy as np
import pytest
import torch

import inputs

pytestmark = pytest.mark.gpu

DT = {32: torch.uint32, 64: torch.uint64}


@pytest.fixture(scope="module")
def gss():
    import paper_conf_ipps_leischneros10_b200 as g
    g._lib()
    return g


def to_dev(a: np.ndarray) -> torch.Tensor:
    return torch.from_numpy(np.ascontiguousarray(a)).cuda()


def to_host(t: torch.Tensor) -> np.ndarray:
    return t.cpu().numpy()


NPROC = os.cpu_count() or 1


def oracle_params(oracle_mod, k=256, M=16384, a=30, seed=5489, k_policy="adaptive", fill_div=4, threads=NPROC):
    return oracle_mod.Params(k=k, a=a, M=M, k_policy=1 if k_policy == "adaptive" else 0, fill_div=fill_div,
                             sample_cap=16384, seed=seed, threads=threads)


def _few(n, width):
    """3 distinct keys (test-side input shape, no method arithmetic)."""
    x = inputs.keys("uniform", n, width, seed=4)
    return (x % x.dtype.type(3)) * x.dtype.type(1000003)


def check_pairs(x, v_out, k_out):
    n = x.size
    vo = v_out.astype(np.int64)
    np.testing.assert_array_equal(np.sort(vo), np.arange(n))
    np.testing.assert_array_equal(x[vo], k_out)


# ---------------------------------------------------------------------------
# One level: gss_partition == oracle.distribute (a2..a6 bit-exact)
# ---------------------------------------------------------------------------
@pytest.mark.parametrize("width", [32, 64])
@pytest.mark.parametrize("dist", ["uniform", "dd", "and4", "sorted", "staggered", "equal"])
@pytest.mark.parametrize("with_vals", [False, True])
def test_partition_level_bit_exact(gss, oracle_mod, width, dist, with_vals):
    n = 5 * 2048 * 3 + 777                                  # several tiles and a ragged tail
    x = inputs.keys(dist, n, width, seed=3)
    v = inputs.values(n, width) if with_vals else None
    prm = dict(k=128, a=30, seed=77, k_policy="fixed", tile=2048)
    ko, vo, spl, off, info = gss.partition(to_dev(x), to_dev(v) if with_vals else None, **prm)
    ok, ov, rec = oracle_mod.distribute(x, v, oracle_params(oracle_mod, k=128, seed=77, k_policy="fixed", M=0))
    assert info == (rec.kb, rec.ks, rec.eq, rec.K)
    np.testing.assert_array_equal(to_host(spl).astype(np.uint64), rec.splitters)
    np.testing.assert_array_equal(to_host(off).astype(np.uint64),
                                  np.concatenate([[0], np.cumsum(rec.children)]).astype(np.uint64))
    np.testing.assert_array_equal(to_host(ko), ok)
    if with_vals:
        np.testing.assert_array_equal(to_host(vo), ov)


# ---------------------------------------------------------------------------
# Phase 2 by the radix-indexed splitter lookup (default for unsigned keys)
# against the paper's tree descent (GSS_FLAG_TREE_CLASSIFY = 512): both must
# give the oracle's ids, so the stable partition is bit-exact either way.
# Inputs aimed at the lookup's corners: keys at 0 and the type maximum, a
# dense cluster that puts many splitters into one bin (the binary-search
# path), a span of one or two key values (shift 0), the full 64-bit range
# (shift 52), below-range keys (bin 0).
# ---------------------------------------------------------------------------
def _lut_case(case, n, width, seed=11):
    rng = np.random.default_rng(seed)
    dt = np.uint32 if width == 32 else np.uint64
    mx = int(np.iinfo(dt).max)
    if case == "extremes":
        return rng.choice(np.array([0, 1, mx - 1, mx], dtype=dt), n)
    if case == "cluster":
        x = rng.integers(0, mx, n, dtype=dt, endpoint=True)
        c = rng.integers(1 << (width - 8), (1 << (width - 8)) + 3000, n, dtype=dt)
        return np.where(rng.random(n) < 0.9, c, x).astype(dt)
    if case == "narrow":
        return rng.integers(1 << (width - 2), (1 << (width - 2)) + 2, n, dtype=dt)
    if case == "full":
        x = rng.integers(0, mx, n, dtype=dt, endpoint=True)
        x[::97] = 0
        x[::89] = mx
        return x
    raise ValueError(case)


LUT_CASES = ["extremes", "cluster", "narrow", "full"]


@pytest.mark.parametrize("width", [32, 64])
@pytest.mark.parametrize("case", LUT_CASES + ["uniform", "and4", "sorted"])
@pytest.mark.parametrize("flags", [0, 512])
def test_partition_lookup_vs_tree(gss, oracle_mod, width, case, flags):
    n = 5 * 2048 * 3 + 777
    x = _lut_case(case, n, width) if case in LUT_CASES else inputs.keys(case, n, width, seed=3)
    for k in (16, 128, 1024):
        prm = dict(k=k, a=30, seed=77, k_policy="fixed", tile=2048, flags=flags)
        ko, _, spl, off, info = gss.partition(to_dev(x), None, **prm)
        ok, _, rec = oracle_mod.distribute(x, None, oracle_params(oracle_mod, k=k, seed=77, k_policy="fixed", M=0))
        assert info == (rec.kb, rec.ks, rec.eq, rec.K)
        np.testing.assert_array_equal(to_host(off).astype(np.uint64),
                                      np.concatenate([[0], np.cumsum(rec.children)]).astype(np.uint64))
        np.testing.assert_array_equal(to_host(ko), ok)


@pytest.mark.parametrize("width,pairs", [(32, False), (64, False), (64, True)])
@pytest.mark.parametrize("case", LUT_CASES)
def test_sort_lookup_corner_inputs(gss, oracle_mod, width, pairs, case):
    n = (1 << 20) + 4321
    x = _lut_case(case, n, width)
    v = inputs.values(n, width) if pairs else None
    ko, vo, st = gss.sort(to_dev(x), to_dev(v) if pairs else None, M=4096, stats=True)
    ok, _, recs = oracle_mod.sort(x, None, oracle_params(oracle_mod, M=4096), log=True)
    np.testing.assert_array_equal(to_host(ko), ok)
    if pairs:
        check_pairs(x, to_host(vo), ok)
    assert_levels_match(st, recs)


# ---------------------------------------------------------------------------
# Whole sort: keys bit-exact vs the oracle, values as a multiset
# ---------------------------------------------------------------------------
KINDS = [(32, False), (64, False), (32, True), (64, True)]


@pytest.mark.parametrize("width,pairs", KINDS)
@pytest.mark.parametrize("dist", inputs.DISTRIBUTIONS)
def test_sort_distributions(gss, oracle_mod, width, pairs, dist):
    n = (1 << 20) + 4321
    x = inputs.keys(dist, n, width, seed=1)
    v = inputs.values(n, width) if pairs else None
    M = 4096
    ko, vo, st = gss.sort(to_dev(x), to_dev(v) if pairs else None, M=M, stats=True)
    torch.cuda.synchronize()
    assert st.error_flags == 0
    ok, _, recs = oracle_mod.sort(x, None, oracle_params(oracle_mod, M=M), log=True)
    np.testing.assert_array_equal(to_host(ko), ok)
    if pairs:
        check_pairs(x, to_host(vo), ok)
    # the level structure matches the oracle's records: keys split per level
    for lvl in range(4):
        want = sum(r.m for r in recs if r.level == lvl)
        assert st.split_elems[lvl] == want, (lvl, st.split_elems[:4])
    assert st.overflow_buckets == 0


@pytest.mark.parametrize("width,pairs", KINDS)
def test_edge_sizes(gss, oracle_mod, width, pairs):
    M = 16384 if not (pairs and width == 64) else 8192
    for n in (0, 1, 2, 31, 32, 33, 2047, 2048, 2049, M - 1, M, M + 1, 3 * M + 5, 1 << 16):
        x = inputs.keys("uniform", n, width, seed=n + 1)
        v = inputs.values(n, width) if pairs else None
        ko, vo = gss.sort(to_dev(x), to_dev(v) if pairs else None)
        np.testing.assert_array_equal(to_host(ko), np.sort(x), err_msg=f"n={n}")
        if pairs:
            check_pairs(x, to_host(vo), np.sort(x))


@pytest.mark.parametrize("k,policy", [(2, "fixed"), (4, "fixed"), (128, "fixed"), (1024, "fixed"), (512, "adaptive")])
def test_k_values(gss, oracle_mod, k, policy):
    n = 300_000
    x = inputs.keys("gaussian", n, 64, seed=k)
    M = 2048
    ko, _, st = gss.sort(to_dev(x), k=k, M=M, k_policy=policy, stats=True)
    assert st.error_flags == 0
    ok, _, recs = oracle_mod.sort(x, None, oracle_params(oracle_mod, k=k, M=M, k_policy=policy), log=True)
    np.testing.assert_array_equal(to_host(ko), ok)
    if st.overflow_buckets == 0:
        for lvl in range(3):
            assert st.split_elems[lvl] == sum(r.m for r in recs if r.level == lvl)


def test_c1_config(gss, oracle_mod):
    """BASELINE configs[0]: 2^16 uniform u32, k=128, one level + small sort."""
    n = 1 << 16
    x = inputs.keys("uniform", n, 32, seed=1)
    ko, _, st = gss.sort(to_dev(x), k=128, k_policy="fixed", M=1 << 14, stats=True)
    ok, _, recs = oracle_mod.sort(x, None, oracle_params(oracle_mod, k=128, M=1 << 14, k_policy="fixed"), log=True)
    np.testing.assert_array_equal(to_host(ko), ok)
    assert st.levels == 1 and len(recs) == 1
    assert st.small_buckets == 128


def test_overflow_fallback(gss, oracle_mod):
    n = 1 << 18
    for pairs in (False, True):
        x = inputs.keys("uniform", n, 64, seed=4)
        v = inputs.values(n, 64) if pairs else None
        ko, vo, st = gss.sort(to_dev(x), to_dev(v) if pairs else None, k=16, k_policy="fixed", M=2048,
                              max_levels=1, stats=True)
        assert st.overflow_buckets > 0 and st.error_flags == 0
        np.testing.assert_array_equal(to_host(ko), np.sort(x))
        if pairs:
            check_pairs(x, to_host(vo), np.sort(x))


def test_in_place_and_descending(gss):
    n = 200_003
    x = inputs.keys("and2", n, 64, seed=5)
    t = to_dev(x)
    gss.sort(t, out=t)
    np.testing.assert_array_equal(to_host(t), np.sort(x))
    kd, _ = gss.sort(to_dev(x), descending=True)
    np.testing.assert_array_equal(to_host(kd), np.sort(x)[::-1])
    v = inputs.values(n, 64)
    tk, tv = to_dev(x), to_dev(v)
    gss.sort(tk, tv, out=tk, values_out=tv)
    check_pairs(x, to_host(tv), np.sort(x))


def test_sort_host_end_to_end(gss):
    n = 1 << 20
    for width, pairs in KINDS:
        x = inputs.keys("uniform", n, width, seed=6)
        hk = torch.from_numpy(x).pin_memory()
        hv = torch.from_numpy(inputs.values(n, width)).pin_memory() if pairs else None
        ko, vo = gss.sort_host(hk, hv)
        np.testing.assert_array_equal(ko.numpy(), np.sort(x))
        if pairs:
            check_pairs(x, vo.numpy(), np.sort(x))


def test_partition_by_and_sample(gss, oracle_mod):
    n = 123_457
    x = inputs.keys("uniform", n, 64, seed=8)
    v = inputs.values(n, 64)
    spl = np.sort(x[[5, 99, 1000, 5000, 77777, 100000, 120000]])
    ko, vo, cnt = gss.partition_by(to_dev(x), to_dev(v), to_dev(spl))
    ids = np.searchsorted(spl, x, side="left")              # #{spl < e}, ties go left
    order = np.argsort(ids, kind="stable")
    np.testing.assert_array_equal(to_host(ko), x[order])
    np.testing.assert_array_equal(to_host(vo), v[order])
    np.testing.assert_array_equal(to_host(cnt), np.bincount(ids, minlength=len(spl) + 1))
    s = gss.sample(to_dev(x), 1000, lo_global=12345, level_tag=255, seed=9)
    want = [x[(oracle_mod.sample_hash(9, 255, 12345, j) * n) >> 64] for j in range(1000)]
    np.testing.assert_array_equal(to_host(s), np.array(want, dtype=np.uint64))


def test_deterministic(gss):
    n = 1 << 20
    x = inputs.keys("dd", n, 64)
    v = inputs.values(n, 64)
    a = gss.sort(to_dev(x), to_dev(v))
    b = gss.sort(to_dev(x), to_dev(v))
    assert torch.equal(a[0], b[0]) and torch.equal(a[1], b[1])


# ---------------------------------------------------------------------------
# BASELINE sizes, in the configuration bench.py times: properties at any size
# plus sampled ranks computed one by one by the oracle.
# ---------------------------------------------------------------------------
@pytest.mark.parametrize("width,n,dist", [(64, 1 << 28, "uniform"), (32, 1 << 27, "uniform"),
                                          (32, 1 << 27, "dd"), (64, 1 << 27, "and4")])
def test_full_size(gss, oracle_mod, width, n, dist):
    x = inputs.keys(dist, n, width, seed=1)
    ko, _, st = gss.sort(to_dev(x), stats=True)
    assert st.error_flags == 0
    y = to_host(ko)
    assert np.all(y[1:] >= y[:-1])                          # non-decreasing
    # same multiset: order-independent sums of a mixing function
    def mix(a):
        z = a.astype(np.uint64) * np.uint64(0x9E3779B97F4A7C15)
        return np.bitwise_xor.reduce(z ^ (z >> np.uint64(29))), int(a.astype(np.uint64).sum(dtype=np.uint64))
    assert mix(x) == mix(y)
    for r in (0, n // 3, n - 1):
        assert int(y[r]) == oracle_mod.select(x, r)


@pytest.mark.parametrize("width,pairs", KINDS)
@pytest.mark.parametrize("dist", ["uniform", "dd", "and3", "equal", "few"])
@pytest.mark.parametrize("flags", [0, 2])
def test_bucket_sorter_variants(gss, oracle_mod, width, pairs, dist, flags):
    """Both bucket sorters give the oracle's keys: the CTA-wide merge sort
    (default) and the in-SM sample split + warp segment sorts
    (GSS_FLAG_SPLIT_SORT = 2).  'few' (3 distinct keys) drives every bucket of
    the split into its hand-back path (a sub-bucket larger than a warp)."""
    n = (1 << 19) + 77
    x = _few(n, width) if dist == "few" else inputs.keys(dist, n, width, seed=2)
    v = inputs.values(n, width) if pairs else None
    ko, vo, st = gss.sort(to_dev(x), to_dev(v) if pairs else None, flags=flags, stats=True)
    assert st.error_flags == 0
    want = oracle_mod.sort(x, None, oracle_params(oracle_mod))[0]
    np.testing.assert_array_equal(to_host(ko), want)
    if pairs:
        check_pairs(x, to_host(vo), want)


@pytest.mark.parametrize("width,pairs", KINDS)
@pytest.mark.parametrize("m", [513, 4097, 9000, 16384])
@pytest.mark.parametrize("flags", [0, 2])
def test_single_bucket(gss, oracle_mod, width, pairs, m, flags):
    """n <= M: the whole input is one in-SM bucket (no distribution level), sorted
    by the bucket sorter of its size class; sizes straddle class boundaries."""
    cap = 8192 if (pairs and width == 64) else 16384
    m = min(m, cap)
    for dist in ("uniform", "few"):
        x = _few(m, width) if dist == "few" else inputs.keys(dist, m, width, seed=3)
        v = inputs.values(m, width) if pairs else None
        ko, vo, st = gss.sort(to_dev(x), to_dev(v) if pairs else None, flags=flags, stats=True)
        assert st.error_flags == 0 and st.levels == 0
        want = oracle_mod.sort(x, None, oracle_params(oracle_mod, M=cap))[0]
        np.testing.assert_array_equal(to_host(ko), want)
        if pairs:
            check_pairs(x, to_host(vo), want)


@pytest.mark.parametrize("width,pairs", KINDS)
@pytest.mark.parametrize("dist", ["uniform", "dd", "and3", "staggered"])
def test_recompute_ids_ablation(gss, oracle_mod, width, pairs, dist):
    """GSS_FLAG_RECOMPUTE_IDS (the paper's Phase 4: re-descend the tree
    instead of reading stored ids) gives the oracle's keys through several levels."""
    n = (1 << 20) + 999
    x = inputs.keys(dist, n, width, seed=5)
    v = inputs.values(n, width) if pairs else None
    ko, vo, st = gss.sort(to_dev(x), to_dev(v) if pairs else None, M=4096, flags=1, stats=True)
    assert st.error_flags == 0 and st.levels >= 2
    want = oracle_mod.sort(x, None, oracle_params(oracle_mod, M=4096))[0]
    np.testing.assert_array_equal(to_host(ko), want)
    if pairs:
        check_pairs(x, to_host(vo), want)


def test_recompute_ids_ablation_large(gss, oracle_mod):
    """GSS_FLAG_RECOMPUTE_IDS at 2^24 keys (hundreds of tiles per CTA, a tree
    reload at every tile of level 1): sorted, same multiset, sampled ranks."""
    n = 1 << 24
    x = inputs.keys("uniform", n, 64, seed=6)
    ko, _, st = gss.sort(to_dev(x), flags=1, stats=True)
    assert st.error_flags == 0 and st.levels == 2
    y = to_host(ko)
    assert np.all(y[1:] >= y[:-1])
    np.testing.assert_array_equal(np.sort(x[::4097]), np.sort(y[np.searchsorted(y, x[::4097])]))
    for r in (0, n // 2, n - 1):
        assert int(y[r]) == oracle_mod.select(x, r)


def _dist_world1():
    import torch.distributed as dist
    os.environ.setdefault("MASTER_ADDR", "127.0.0.1")
    os.environ.setdefault("MASTER_PORT", "29561")
    if not dist.is_initialized():
        dist.init_process_group("nccl", rank=0, world_size=1, device_id=torch.device("cuda", 0))


@pytest.mark.parametrize("width,pairs", KINDS)
@pytest.mark.parametrize("dist_name", ["gaussian", "dd", "equal"])
@pytest.mark.parametrize("fused", [False, True])
def test_distributed_sorter_single_rank_nccl(gss, oracle_mod, width, pairs, dist_name, fused):
    """gss_dist_sort_* on one rank over NCCL: (n, capacity) all-gather, sample all-gather,
    sample sort, splitters, equality-mode partition, counts all-gather, plan, NCCL
    send/recv to itself (or, fused = GSS_FLAG_DIST_FUSED, the scatter writing into the
    rank's NCCL symmetric window), local sort -- keys equal the oracle's."""
    from paper_conf_ipps_leischneros10_b200.dist import DistSorter
    _dist_world1()
    n = (1 << 20) + 17
    x = inputs.keys(dist_name, n, width, seed=9)
    v = inputs.values(n, width) if pairs else None
    ds = DistSorter(f"u{width}", n, pairs, flags=64 if fused else 0)
    for _ in range(2):
        k, vv, nr = ds(to_dev(x), to_dev(v) if pairs else None)
    assert nr == n
    ok, _, _ = oracle_mod.sort(x, None, oracle_params(oracle_mod, M=4096))
    np.testing.assert_array_equal(to_host(k), ok)
    if pairs:
        check_pairs(x, to_host(vv), ok)
    assert ds.verify(x, v)
    send, recv, cuts = ds.last_exchange()
    assert send == [n] and recv == [n] and cuts == [0, n]


def test_distributed_capacity_error(gss):
    from paper_conf_ipps_leischneros10_b200.dist import DistSorter
    _dist_world1()
    n = 1 << 16
    x = inputs.keys("uniform", n, 64, seed=2)
    ds = DistSorter("u64", n, False, capacity=n - 1)
    with pytest.raises(RuntimeError, match="GSS_ERROR_CAPACITY"):
        ds(to_dev(x))


@pytest.mark.parametrize("width", [32, 64])
@pytest.mark.parametrize("nspl", [0, 1, 3, 7, 100])
def test_partition_by_eq_mode(gss, width, nspl):
    """gss_partition_by_eq: ids 2b / 2b+1 (R4 with given, possibly repeated, splitters),
    stable partition and counts bit-exact against the plain definition."""
    n = 5 * 65536 + 1234
    x = inputs.keys("and3", n, width, seed=nspl + 1)
    v = inputs.values(n, width)
    rng = np.random.default_rng(nspl)
    spl = np.sort(x[rng.integers(0, n, size=nspl)]) if nspl else x[:0]
    if nspl >= 3:
        spl[1] = spl[2]                                      # a duplicate splitter
    ko, vo, cnt = gss.partition_by(to_dev(x), to_dev(v), to_dev(spl), eq=True)
    b = np.searchsorted(spl, x, side="left")
    hit = (b < nspl) & (x == spl[np.minimum(b, max(nspl - 1, 0))]) if nspl else np.zeros(n, bool)
    ids = 2 * b + hit
    order = np.argsort(ids, kind="stable")
    np.testing.assert_array_equal(to_host(ko), x[order])
    np.testing.assert_array_equal(to_host(vo), v[order])
    np.testing.assert_array_equal(to_host(cnt), np.bincount(ids, minlength=2 * nspl + 1))


@pytest.mark.parametrize("width,pairs", KINDS)
def test_stable_flag_same_keys(gss, oracle_mod, width, pairs):
    """GSS_FLAG_STABLE (ballot-ranked stable scatter) and the default atomic-ranked scatter
    both give the oracle's keys; the level structure matches the oracle's records."""
    n = (1 << 20) + 3
    x = inputs.keys("and2", n, width, seed=4)
    v = inputs.values(n, width) if pairs else None
    M = 4096
    ok, _, recs = oracle_mod.sort(x, None, oracle_params(oracle_mod, M=M, threads=NPROC), log=True)
    for flags in (4, 0):
        ko, vo, st = gss.sort(to_dev(x), to_dev(v) if pairs else None, M=M, flags=flags, stats=True)
        np.testing.assert_array_equal(to_host(ko), ok)
        if pairs:
            check_pairs(x, to_host(vo), ok)
        assert_levels_match(st, recs)


@pytest.mark.parametrize("width,pairs", KINDS)
def test_direct_scatter_ablation(gss, oracle_mod, width, pairs):
    """GSS_FLAG_DIRECT_SCATTER (the paper's unstructured Phase 4) gives the oracle's keys."""
    n = (1 << 20) + 11
    x = inputs.keys("staggered", n, width, seed=3)
    v = inputs.values(n, width) if pairs else None
    M = 4096
    ok, _, recs = oracle_mod.sort(x, None, oracle_params(oracle_mod, M=M, threads=NPROC), log=True)
    ko, vo, st = gss.sort(to_dev(x), to_dev(v) if pairs else None, M=M, flags=8, stats=True)
    np.testing.assert_array_equal(to_host(ko), ok)
    if pairs:
        check_pairs(x, to_host(vo), ok)
    assert_levels_match(st, recs)


# ---------------------------------------------------------------------------
# The configuration bench.py times: library defaults (auto k = 256, auto tile
# T = 65536 so every tile spans 16 scatter chunks, M = the in-SM capacity),
# the persistent grids walking hundreds of tiles, and the CUDA-graph replay
# (GSS_FLAG_GRAPH) -- element by element against the oracle.
# ---------------------------------------------------------------------------
def default_M(width, pairs):
    return 8192 if (pairs and width == 64) else (32768 if (width == 32 and not pairs) else 16384)


def default_k(n, M):
    k = 256
    while k < 1024 and n > k * k * (M // 2):
        k *= 2
    return k


def assert_levels_match(st, recs):
    for lvl in range(4):
        assert st.split_elems[lvl] == sum(r.m for r in recs if r.level == lvl), (lvl, st.split_elems[:4])
    assert st.overflow_buckets == 0 and st.error_flags == 0


@pytest.mark.parametrize("width,pairs", KINDS)
@pytest.mark.parametrize("dist", ["uniform", "dd", "and4", "sorted"])
def test_bench_config_parity(gss, oracle_mod, width, pairs, dist):
    n = (1 << 25) + 777                                     # 513 tiles of 65536 keys, ragged last tile
    x = inputs.keys(dist, n, width, seed=1)
    v = inputs.values(n, width) if pairs else None
    M = default_M(width, pairs)
    ok, _, recs = oracle_mod.sort(x, None, oracle_params(oracle_mod, k=default_k(n, M), M=M, threads=NPROC),
                                  log=True)
    # library defaults, with statistics (direct launches)
    ko, vo, st = gss.sort(to_dev(x), to_dev(v) if pairs else None, stats=True)
    np.testing.assert_array_equal(to_host(ko), ok)
    if pairs:
        check_pairs(x, to_host(vo), ok)
    assert_levels_match(st, recs)
    # the bench's path: a persistent Sorter with the CUDA-graph flag; the second
    # call replays the captured graph
    kind = f"u{width}"
    s = gss.Sorter(kind, n, pairs, flags=16)
    kin, kout = to_dev(x), torch.empty(n, dtype=DT[width], device="cuda")
    vin = to_dev(v) if pairs else None
    vout = torch.empty_like(vin) if pairs else None
    for _ in range(2):
        kout.zero_()
        s(kin, kout, vin, vout)
    np.testing.assert_array_equal(to_host(kout), ok)
    if pairs:
        check_pairs(x, to_host(vout), ok)


@pytest.mark.parametrize("width,n,pairs,dist", [(64, 1 << 28, False, "uniform"), (64, 1 << 27, True, "uniform"),
                                                (64, 1 << 27, True, "and4"), (32, 1 << 27, False, "staggered")])
def test_full_size_elementwise(gss, oracle_mod, width, n, pairs, dist):
    """BASELINE configs[1-3] sizes (2^28 u64 is the north-star row) through the
    bench's Sorter + graph path, compared element by element with the oracle."""
    x = inputs.keys(dist, n, width, seed=1)
    v = inputs.values(n, width) if pairs else None
    M = default_M(width, pairs)
    s = gss.Sorter(f"u{width}", n, pairs, flags=16)
    kin = to_dev(x)
    kout = torch.empty_like(kin)
    vin = to_dev(v) if pairs else None
    vout = torch.empty_like(vin) if pairs else None
    for _ in range(2):
        s(kin, kout, vin, vout)
    got = to_host(kout)
    gv = to_host(vout) if pairs else None
    del kin, kout, vin, vout
    torch.cuda.empty_cache()
    ok, _, _ = oracle_mod.sort(x, None, oracle_params(oracle_mod, k=default_k(n, M), M=M, threads=NPROC))
    np.testing.assert_array_equal(got, ok)
    if pairs:
        check_pairs(x, gv, ok)


def test_graph_replay(gss):
    """GSS_FLAG_GRAPH: the captured launch sequence replays correctly on new data in the same buffers."""
    n = (1 << 16)
    s = gss.Sorter("u32", n, False, k=128, k_policy="fixed", flags=16)
    kin = torch.empty(n, dtype=torch.uint32, device="cuda")
    kout = torch.empty_like(kin)
    for seed in (1, 2, 3):
        x = inputs.keys("uniform", n, 32, seed=seed)
        kin.copy_(torch.from_numpy(x))
        s(kin, kout)
        np.testing.assert_array_equal(to_host(kout), np.sort(x))


@pytest.mark.parametrize("width,pairs", KINDS)
def test_host_pipeline(gss, width, pairs):
    """gss_host_pipeline_*: consecutive pipelined host-buffer sorts are each correct."""
    n = (1 << 18) + 5
    hp = gss.HostPipeline(f"u{width}", n, pairs)
    xs = [inputs.keys("uniform", n, width, seed=s) for s in (1, 2, 3, 4)]
    his = [torch.from_numpy(x).pin_memory() for x in xs]
    hos = [torch.empty_like(h).pin_memory() for h in his]
    hv = torch.from_numpy(inputs.values(n, width)).pin_memory() if pairs else None
    hvo = [torch.empty_like(hv).pin_memory() for _ in xs] if pairs else [None] * 4
    for i in range(4):
        hp(his[i], hos[i], hv, hvo[i])
    hp.flush()
    torch.cuda.synchronize()
    for i in range(4):
        np.testing.assert_array_equal(hos[i].numpy(), np.sort(xs[i]))
        if pairs:
            check_pairs(xs[i], hvo[i].numpy(), np.sort(xs[i]))


# ---------------------------------------------------------------------------
# Float keys: IEEE-754 totalOrder (gss_sort_f32 / gss_sort_f64)
# ---------------------------------------------------------------------------
def _total_order_bits(bits: np.ndarray, width: int) -> np.ndarray:
    """IEEE 754-2008 5.10 totalOrder as an unsigned integer order: negative
    numbers (sign bit set) reverse, positives follow them."""
    top = np.uint64(1) << np.uint64(width - 1)
    full = np.uint64((1 << width) - 1)
    b = bits.astype(np.uint64)
    return np.where(b & top, b ^ full, b | top)


def _from_total_order_bits(r: np.ndarray, width: int) -> np.ndarray:
    top = np.uint64(1) << np.uint64(width - 1)
    full = np.uint64((1 << width) - 1)
    return np.where(r & top, r ^ top, r ^ full)


@pytest.mark.parametrize("width", [32, 64])
def test_float_total_order(gss, oracle_mod, width):
    ft, ut = (np.float32, np.uint32) if width == 32 else (np.float64, np.uint64)
    n = (1 << 20) + 999
    rng = np.random.default_rng(width)
    x = (rng.standard_normal(n) * rng.choice([1e-30, 1.0, 1e20], n)).astype(ft)
    special = np.array([np.nan, -np.nan, np.inf, -np.inf, 0.0, -0.0, np.finfo(ft).tiny / 4,
                        -np.finfo(ft).tiny / 4, np.finfo(ft).max, -np.finfo(ft).max], dtype=ft)
    idx = rng.integers(0, n, 4096)
    x[idx] = special[rng.integers(0, special.size, idx.size)]
    x[:1000] = x[1000:2000]                                  # duplicates
    bits = x.view(ut)
    ko, _, st = gss.sort(to_dev(x), M=4096, stats=True)
    assert st.error_flags == 0
    got = to_host(ko).view(ut)
    # the oracle sorts the totalOrder images of the same bit patterns
    ranks = _total_order_bits(bits, width)
    ok, _, recs = oracle_mod.sort(ranks, None, oracle_params(oracle_mod, M=4096), log=True)
    want = _from_total_order_bits(ok.astype(np.uint64), width).astype(ut)
    np.testing.assert_array_equal(got, want)
    for lvl in range(3):
        assert st.split_elems[lvl] == sum(r.m for r in recs if r.level == lvl)
    # independent check on the ordinary numbers: numpy's float order
    y = to_host(ko)
    fin = y[np.isfinite(y) & (y != 0)]
    np.testing.assert_array_equal(fin, np.sort(x[np.isfinite(x) & (x != 0)]))
    # -NaN first, +NaN last, -0 before +0
    sgn = np.signbit(y)
    nan = np.isnan(y)
    assert np.all(nan[:int((nan & sgn).sum())]) and np.all(nan[n - int((nan & ~sgn).sum()):])
    z = np.flatnonzero(y == 0)
    assert np.all(np.diff(sgn[z].astype(np.int8)) <= 0)



# ---------------------------------------------------------------------------
# Comparator-only contract: descending order for every kind, and
# include/gss.hpp instantiated with user comparators (tests/cxx/custom_less.cu)
# ---------------------------------------------------------------------------
@pytest.mark.parametrize("width,pairs", KINDS)
@pytest.mark.parametrize("dist", ["uniform", "dd", "and4"])
def test_descending_all_kinds(gss, oracle_mod, width, pairs, dist):
    n = (1 << 20) + 99
    x = inputs.keys(dist, n, width, seed=21)
    v = inputs.values(n, width) if pairs else None
    ok, _, _ = oracle_mod.sort(x, None, oracle_params(oracle_mod, M=4096))
    ko, vo = gss.sort(to_dev(x), to_dev(v) if pairs else None, descending=True, M=4096)
    np.testing.assert_array_equal(to_host(ko), ok[::-1])
    if pairs:
        check_pairs(x, to_host(vo), ok[::-1])


@pytest.fixture(scope="module")
def cxx_lib():
    import ctypes
    from paper_conf_ipps_leischneros10_b200 import _build
    lib = ctypes.CDLL(_build.build_cxx_test())
    vp, sz = ctypes.c_void_p, ctypes.c_size_t
    lib.cxx_sort_residue_u64.restype = ctypes.c_int
    lib.cxx_sort_residue_u64.argtypes = [vp, vp, sz, vp, ctypes.POINTER(sz), vp]
    lib.cxx_sort_pairs_desc_u32_u64.restype = ctypes.c_int
    lib.cxx_sort_pairs_desc_u32_u64.argtypes = [vp, vp, vp, vp, sz, vp, ctypes.POINTER(sz), vp]
    return lib


def _cxx_call(fn, head):
    import ctypes
    tb = ctypes.c_size_t(0)
    assert fn(*head, None, ctypes.byref(tb), None) == 0
    temp = torch.empty(max(tb.value, 1), dtype=torch.uint8, device="cuda")
    s = torch.cuda.current_stream().cuda_stream
    assert fn(*head, ctypes.c_void_p(temp.data_ptr()), ctypes.byref(tb), s) == 0
    torch.cuda.synchronize()


@pytest.mark.parametrize("n", [1000, (1 << 20) + 7])
def test_gss_hpp_user_comparators(gss, cxx_lib, n):
    import ctypes
    p = lambda t: ctypes.c_void_p(t.data_ptr())  # noqa: E731
    # u64 keys by residue mod 1000003: equivalent keys form runs in any order
    x = inputs.keys("uniform", n, 64, seed=5)
    kin, kout = to_dev(x), torch.empty(n, dtype=torch.uint64, device="cuda")
    _cxx_call(cxx_lib.cxx_sort_residue_u64, (p(kin), p(kout), n))
    y = to_host(kout)
    r = y % np.uint64(1000003)
    assert np.all(r[1:] >= r[:-1])
    np.testing.assert_array_equal(np.sort(y), np.sort(x))
    # u32 keys, u64 values, descending: a key/value width pair libgss.so does not export
    k32 = inputs.keys("and2", n, 32, seed=6)
    v64 = np.arange(n, dtype=np.uint64)
    ki, vi = to_dev(k32), to_dev(v64)
    ko, vo = torch.empty_like(ki), torch.empty_like(vi)
    _cxx_call(cxx_lib.cxx_sort_pairs_desc_u32_u64, (p(ki), p(vi), p(ko), p(vo), n))
    got_k, got_v = to_host(ko), to_host(vo).astype(np.int64)
    np.testing.assert_array_equal(got_k, np.sort(k32)[::-1])
    np.testing.assert_array_equal(np.sort(got_v), np.arange(n))
    np.testing.assert_array_equal(k32[got_v], got_k)


# ---------------------------------------------------------------------------
# The paper's design alternatives as runtime ablations, each
# against the oracle: (iii) fewer Phase-2 counter arrays per CTA,
# (iv) bitonic instead of odd-even merge networks in the in-SM sort
# (P:339-341); (i) recompute ids and (ii) the direct scatter are above.
# ---------------------------------------------------------------------------
@pytest.mark.parametrize("width,pairs", KINDS)
@pytest.mark.parametrize("variant", [dict(cls_arrays=1), dict(cls_arrays=2), dict(cls_arrays=4),
                                     dict(flags=128), dict(flags=32), dict(flags=128 | 16), dict(flags=512)])
def test_ablation_variants_vs_oracle(gss, oracle_mod, width, pairs, variant):
    n = (1 << 21) + 333
    x = inputs.keys("and3", n, width, seed=31)
    v = inputs.values(n, width) if pairs else None
    M = 4096
    ok, _, recs = oracle_mod.sort(x, None, oracle_params(oracle_mod, M=M), log=True)
    graph = bool(variant.get("flags", 0) & 16)                 # the graph path ignores statistics
    if graph:
        ko, vo = gss.sort(to_dev(x), to_dev(v) if pairs else None, M=M, **variant)
        st = None
    else:
        ko, vo, st = gss.sort(to_dev(x), to_dev(v) if pairs else None, M=M, stats=True, **variant)
    np.testing.assert_array_equal(to_host(ko), ok)
    if pairs:
        check_pairs(x, to_host(vo), ok)
    if st is not None:
        assert_levels_match(st, recs)


# ---------------------------------------------------------------------------
# Cluster-wide bucket sort (GSS_FLAG_CLUSTER_SORT = 256):
# buckets between one CTA's and a cluster's capacity, against the oracle
# ---------------------------------------------------------------------------
CLUSTER_CAP = {(32, False): 8 * 512 * 32, (64, False): 8 * 512 * 16, (32, True): 8 * 512 * 16,
               (64, True): 8 * 512 * 8}
CTA_CAP = {(32, False): 32768, (64, False): 16384, (32, True): 16384, (64, True): 8192}


@pytest.mark.parametrize("width,pairs", KINDS)
@pytest.mark.parametrize("dist", ["uniform", "and4", "sorted"])
def test_cluster_sort_vs_oracle(gss, oracle_mod, width, pairs, dist):
    M = CLUSTER_CAP[(width, pairs)]
    n = 48 * (M // 2) + 555                          # level 0 at k = 64 leaves buckets of ~0.75 M > one CTA
    x = inputs.keys(dist, n, width, seed=41)
    v = inputs.values(n, width) if pairs else None
    ok, _, recs = oracle_mod.sort(x, None, oracle_params(oracle_mod, k=64, M=M, k_policy="fixed"), log=True)
    ko, vo, st = gss.sort(to_dev(x), to_dev(v) if pairs else None, k=64, k_policy="fixed", M=M, flags=256,
                          stats=True)
    np.testing.assert_array_equal(to_host(ko), ok)
    if pairs:
        check_pairs(x, to_host(vo), ok)
    assert_levels_match(st, recs)
    if dist != "and4":
        assert st.cluster_buckets > 0 and st.max_small > CTA_CAP[(width, pairs)]


@pytest.mark.parametrize("width,pairs", KINDS)
def test_cluster_sort_single_bucket(gss, width, pairs):
    """n <= M: the whole input is one bucket for one cluster (sizes around the slice boundaries)."""
    cap = CLUSTER_CAP[(width, pairs)]
    for n in (CTA_CAP[(width, pairs)] + 1, cap // 2 + 3, cap - 1, cap):
        x = inputs.keys("uniform", n, width, seed=n)
        v = inputs.values(n, width) if pairs else None
        ko, vo, st = gss.sort(to_dev(x), to_dev(v) if pairs else None, flags=256, stats=True)
        np.testing.assert_array_equal(to_host(ko), np.sort(x), err_msg=f"n={n}")
        if pairs:
            check_pairs(x, to_host(vo), np.sort(x))
        assert st.cluster_buckets == 1 and st.levels == 0



def test_error_out_flags(gss):
    """gss_params.error_out: the capacity-check flags land in a device word without a host sync,
    on the direct path and through the CUDA-graph replay; 0 for a valid result."""
    n = (1 << 20) + 5
    x = inputs.keys("and2", n, 64, seed=8)
    err = torch.full((1,), 0x7fffffff, dtype=torch.int32, device="cuda")
    ko, _ = gss.sort(to_dev(x), error_out=err)
    assert int(err.item()) == 0
    np.testing.assert_array_equal(to_host(ko), np.sort(x))
    s = gss.Sorter("u64", n, False, flags=16, error_out=err)
    kin, kout = to_dev(x), torch.empty(n, dtype=torch.uint64, device="cuda")
    for _ in range(2):
        err.fill_(0x7fffffff)
        s(kin, kout)
        assert int(err.item()) == 0
    np.testing.assert_array_equal(to_host(kout), np.sort(x))


# ---------------------------------------------------------------------------
# The fused global scatter with several destination segments (the P > 1 data path of
# GSS_FLAG_DIST_FUSED, which a world-size-1 run cannot reach: there the only segment is the
# rank's own window).  gssi_dist_level (internal export): phase 1 classifies and counts, phase 2
# scatters the equality-mode partition straight into P separate buffers through a RemoteSeg table
# whose cuts fall anywhere (inside buckets too); every bucket must arrive whole, as a multiset.
# ---------------------------------------------------------------------------
@pytest.mark.parametrize("width,pairs", KINDS)
@pytest.mark.parametrize("P", [2, 3, 8])
def test_fused_scatter_segments(gss, width, pairs, P):
    import ctypes
    lib = gss._lib()
    fn = getattr(lib, f"gssi_dist_level_u{width}")
    vp, sz, u32 = ctypes.c_void_p, ctypes.c_size_t, ctypes.c_uint32
    fn.restype = ctypes.c_int
    fn.argtypes = [vp, vp, vp, vp, sz, vp, u32, vp, vp, u32, u32, vp, ctypes.POINTER(sz), vp]
    n = 3 * 65536 + 4321
    x = inputs.keys("and3", n, width, seed=P)
    v = inputs.values(n, width)
    rng = np.random.default_rng(P)
    spl = np.sort(x[rng.integers(0, n, size=P - 1)])
    nspl = P - 1
    b = np.searchsorted(spl, x, side="left")
    ids = 2 * b + ((b < nspl) & (x == spl[np.minimum(b, nspl - 1)]))
    order = np.argsort(ids, kind="stable")
    want_k, want_v, want_ids = x[order], v[order], ids[order]
    # P segments with arbitrary cuts of the partition index space, each into its own buffer at an offset
    cuts = np.sort(np.concatenate([[0, n], rng.integers(0, n, size=P - 1)]))
    dt = DT[width]
    kin, vin = to_dev(x), to_dev(v)
    kbuf, vbuf = torch.empty_like(kin), torch.empty_like(vin)           # stand-in local output (unused)
    dspl = to_dev(spl)
    cnt = torch.zeros(2 * nspl + 1, dtype=torch.uint64, device="cuda")
    outs, offs = [], []
    seg = np.zeros((P, 4), dtype=np.uint64)                             # (lo|hi, pad, kdst, vdst) as u64 words
    w = width // 8
    for q in range(P):
        lo, hi = int(cuts[q]), int(cuts[q + 1])
        off = 7 * q + 3                                                  # arbitrary alignment of the destination
        kd = torch.zeros(hi - lo + off + 8, dtype=dt, device="cuda")
        vd = torch.zeros(hi - lo + off + 8, dtype=dt, device="cuda")
        outs.append((kd, vd)); offs.append(off)
        seg[q, 0] = np.uint64(lo | (hi << 32))
        seg[q, 2] = np.uint64((kd.data_ptr() + (off - lo) * w) % (1 << 64))
        seg[q, 3] = np.uint64((vd.data_ptr() + (off - lo) * w) % (1 << 64)) if pairs else 0
    dseg = torch.from_numpy(seg.view(np.int64)).cuda()
    head = (ctypes.c_void_p(kin.data_ptr()), ctypes.c_void_p(vin.data_ptr()) if pairs else None,
            ctypes.c_void_p(kbuf.data_ptr()), ctypes.c_void_p(vbuf.data_ptr()) if pairs else None, n,
            ctypes.c_void_p(dspl.data_ptr()), nspl, ctypes.c_void_p(cnt.data_ptr()))
    tb = sz(0)
    assert fn(*head, None, 0, 1, None, ctypes.byref(tb), None) == 0
    temp = torch.empty(max(tb.value, 1), dtype=torch.uint8, device="cuda")
    s = torch.cuda.current_stream().cuda_stream
    assert fn(*head, None, 0, 1, ctypes.c_void_p(temp.data_ptr()), ctypes.byref(tb), s) == 0
    assert fn(*head, ctypes.c_void_p(dseg.data_ptr()), P, 2, ctypes.c_void_p(temp.data_ptr()), ctypes.byref(tb), s) == 0
    torch.cuda.synchronize()
    np.testing.assert_array_equal(to_host(cnt), np.bincount(ids, minlength=2 * nspl + 1))
    got_k = np.concatenate([to_host(outs[q][0])[offs[q]:offs[q] + int(cuts[q + 1] - cuts[q])] for q in range(P)])
    got_v = np.concatenate([to_host(outs[q][1])[offs[q]:offs[q] + int(cuts[q + 1] - cuts[q])] for q in range(P)])
    # bucket by bucket, the same (key, value) multiset as the stable partition
    bounds = np.concatenate([[0], np.cumsum(np.bincount(ids, minlength=2 * nspl + 1))])
    for i in range(2 * nspl + 1):
        a, e = int(bounds[i]), int(bounds[i + 1])
        if pairs:
            np.testing.assert_array_equal(np.sort(got_v[a:e]), np.sort(want_v[a:e]))
            np.testing.assert_array_equal(x[got_v[a:e].astype(np.int64)], got_k[a:e])
        else:
            np.testing.assert_array_equal(np.sort(got_k[a:e]), np.sort(want_k[a:e]))
    for q in range(P):                                                   # nothing written outside the segments
        kd = to_host(outs[q][0])
        assert not kd[:offs[q]].any() and not kd[offs[q] + int(cuts[q + 1] - cuts[q]):].any()


@pytest.mark.parametrize("width,pairs", KINDS)
@pytest.mark.parametrize("P,dist_name", [(2, "uniform"), (4, "dd"), (8, "staggered"), (8, "equal")])
def test_distributed_steps_virtual_ranks(gss, oracle_mod, width, pairs, P, dist_name):
    """The distributed sort's device steps for P virtual ranks on one GPU, composed exactly as
    gss_dist_sort does (only the collectives are replaced by device copies): hashed samples of every
    shard (gss_sample, level tag 255, lo = shard start), the sorted gathered sample (gss_sort), the
    splitters S[(i+1)VS/P - 1], the equality-mode partition of every shard (gss_partition_by_eq), the
    exchange plan (gss_dist_plan), the exchange, the local sorts.  The concatenation over ranks equals
    the oracle's sort of the global input; duplicate-heavy inputs stay balanced."""
    from paper_conf_ipps_leischneros10_b200.dist import plan
    n_local, S = (1 << 18) + 77, 16384
    x = inputs.keys(dist_name, n_local * P, width, seed=5)
    v = inputs.values(n_local * P, width)
    shards = [(to_dev(x[r * n_local:(r + 1) * n_local]), to_dev(v[r * n_local:(r + 1) * n_local])) for r in range(P)]
    smp = torch.cat([gss.sample(k, S, lo_global=r * n_local, level_tag=255, seed=5489) for r, (k, _) in enumerate(shards)])
    ssorted, _ = gss.sort(smp)
    VS = P * S
    sdt = torch.int32 if width == 32 else torch.int64                    # (no unsigned gather on CUDA in torch)
    pos = torch.tensor([((i + 1) * VS) // P - 1 for i in range(P - 1)], dtype=torch.long, device="cuda")
    spl = ssorted.view(sdt)[pos].view(ssorted.dtype)
    parts = [gss.partition_by(k, vv if pairs else None, spl, eq=True) for k, vv in shards]
    counts = np.stack([to_host(c).astype(np.uint64) for _, _, c in parts])
    plans = [plan(P, r, counts) for r in range(P)]
    results = []
    for q in range(P):                                          # rank q receives, source-major, then sorts
        rk, rv = [], []
        for r in range(P):
            so, sc = int(plans[r][1][q]), int(plans[r][2][q])
            rk.append(parts[r][0][so:so + sc])
            if pairs:
                rv.append(parts[r][1][so:so + sc])
            assert sc == int(plans[q][3][r])                   # what r sends to q is what q expects from r
        kq = torch.cat(rk)
        vq = torch.cat(rv) if pairs else None
        ko, vo = gss.sort(kq, vq)
        results.append((to_host(ko), to_host(vo) if pairs else None))
    ok, _, _ = oracle_mod.sort(x, None, oracle_params(oracle_mod, M=4096))
    got = np.concatenate([r[0] for r in results])
    np.testing.assert_array_equal(got, ok)
    if pairs:
        check_pairs(x, np.concatenate([r[1] for r in results]), ok)
    for r in results:                                           # balanced to within a few percent
        assert abs(len(r[0]) - n_local) <= 0.1 * n_local, [len(t[0]) for t in results]
