"""Pins for the CPU oracle (oracle/oracle.c) against what the paper and the
mathematics fix -- no GPU needed.

Each test names the part of the oracle it pins and the independent fact it
uses: brute force on tiny inputs, a library sort, the paper's worked k=8
tree example, public SplitMix64 known answers, closed forms, invariants.
"""
import itertools
import random

import numpy as np
import pytest

from conftest import golden

import inputs

MASK = (1 << 64) - 1
GAMMA = 0x9E3779B97F4A7C15


def py_fmix(z):
    z &= MASK
    z = ((z ^ (z >> 30)) * 0xBF58476D1CE4E5B9) & MASK
    z = ((z ^ (z >> 27)) * 0x94D049BB133111EB) & MASK
    return z ^ (z >> 31)


# --------------------------------------------------------------------------
# RNG (R2): SplitMix64 known answers
# --------------------------------------------------------------------------
def test_splitmix64_known_answers(oracle_mod):
    kat = golden("splitmix64_kat.txt")
    seed = kat["seed"][0]
    # The sequential generator's i-th output is fmix(seed + (i+1) gamma), and
    # oracle_splitmix64(x) = fmix(x + gamma).
    for i, want in enumerate(kat["out"]):
        assert oracle_mod.splitmix64((seed + i * GAMMA) & MASK) == want
    # the input generator draws the same sequence
    w = inputs.words(np.arange(3, dtype=np.int64), 0, 1, seed)
    assert [int(x) for x in w] == kat["out"]


def test_sample_hash_composition(oracle_mod):
    # H(seed, level, lo, j) = sm(sm(sm(seed ^ (level<<56)) ^ lo) ^ j), sm pinned above
    sm = oracle_mod.splitmix64
    for seed, level, lo, j in [(5489, 0, 0, 0), (1, 3, 12345, 77), (MASK, 255, 1 << 40, 7679)]:
        want = sm(sm(sm(seed ^ (level << 56)) ^ lo) ^ j)
        assert oracle_mod.sample_hash(seed, level, lo, j) == want


# --------------------------------------------------------------------------
# Tree layout and Algorithm 2
# --------------------------------------------------------------------------
def test_tree_layout_paper_example(oracle_mod):
    g = golden("tree_k8.txt")
    k = g["k"][0]
    spl = [10 * i for i in range(1, k)]           # s_i = 10 i, distinct
    bt = oracle_mod.tree(spl)
    assert [int(x) for x in bt[1:]] == [10 * i for i in g["bt"]]
    # leaves b1..b8 left to right: bucket j holds s_{j-1} < e <= s_j
    for j in g["leaves"]:
        for e in ([10 * (j - 1) + 1, 10 * j] if j < k else [10 * (j - 1) + 1, 10 ** 6]):
            assert oracle_mod.traverse_tree(bt, e) == j


@pytest.mark.parametrize("k", [2, 4, 8, 16, 128, 256, 1024])
def test_descent_equals_count_less(oracle_mod, k):
    """Algorithm 2 (ties go left) equals #{spl < e}, also with duplicate splitters."""
    rng = random.Random(k)
    for alphabet in (3, 10, 1000, 1 << 64):
        for _ in range(20):
            spl = sorted(rng.randrange(alphabet) for _ in range(k - 1))
            bt = oracle_mod.tree(spl)
            for _ in range(20):
                e = rng.randrange(alphabet) if rng.random() < 0.7 else rng.choice(spl)
                brute = sum(1 for s in spl if s < e)             # plain definition
                assert oracle_mod.count_less(spl, e) == brute
                assert oracle_mod.traverse_tree(bt, e) - 1 == brute


def test_classify_equality_mode(oracle_mod):
    spl = [5, 5, 9]
    for e, want in [(0, 0), (5, 1), (6, 4), (9, 5), (10, 6)]:
        # b = #{spl < e}; id = 2b + [b < ns and e == spl[b]]
        assert oracle_mod.classify(spl, 1, e) == want
    assert oracle_mod.classify(spl, 0, 7) == 2


# --------------------------------------------------------------------------
# Parameters
# --------------------------------------------------------------------------
def test_choose_kb_rule(oracle_mod):
    P = oracle_mod.Params
    assert oracle_mod.choose_kb(P(k=128, k_policy=0, M=1 << 15), 1 << 16) == 128
    p = P(k=256, k_policy=1, M=1 << 14, fill_div=4)
    assert oracle_mod.choose_kb(p, 1 << 28) == 256                  # capped at k
    assert oracle_mod.choose_kb(p, 1 << 20) == 256                  # ceil(4*2^20/2^14) = 256
    assert oracle_mod.choose_kb(p, (1 << 19) + 1) == 256            # ceil(...) = 129 -> 256
    assert oracle_mod.choose_kb(p, 1 << 19) == 128
    assert oracle_mod.choose_kb(p, (1 << 14) + 1) == 8              # ceil(4.0002) = 5 -> 8
    assert oracle_mod.choose_kb(P(k=2, k_policy=1, M=4), 100) == 2  # min(k, ...)
    assert oracle_mod.a_eff(P(a=30, sample_cap=16384), 1024) == 16
    assert oracle_mod.a_eff(P(a=30, sample_cap=16384), 256) == 30


# --------------------------------------------------------------------------
# Whole sort: brute force and library sort
# --------------------------------------------------------------------------
TINY_PARAMS = [
    dict(k=2, a=1, M=1),
    dict(k=4, a=2, M=1),
    dict(k=8, a=1, M=2),
    dict(k=4, a=1, M=1, k_policy=1, fill_div=1),
    dict(k=8, a=3, M=1, k_policy=1, fill_div=2),
]


@pytest.mark.parametrize("pp", TINY_PARAMS)
def test_exhaustive_tiny(oracle_mod, pp):
    """Every sequence of length <= 6 over {0,1,2} sorts like sorted()."""
    p = oracle_mod.Params(**pp)
    for n in range(0, 7):
        for seq in itertools.product((0, 1, 2), repeat=n):
            keys = np.array(seq, dtype=np.uint64)
            out, vals, recs = oracle_mod.sort(keys, np.arange(n, dtype=np.uint64), p, log=True)
            assert out.tolist() == sorted(seq)
            # values: a permutation of [0, n) with in_key[val[i]] == out_key[i]
            assert sorted(vals.tolist()) == list(range(n))
            assert all(seq[v] == k for k, v in zip(out.tolist(), vals.tolist()))
            for r in recs:
                assert r.m > p.M


@pytest.mark.parametrize("dist", inputs.DISTRIBUTIONS)
@pytest.mark.parametrize("width", [32, 64])
def test_sort_matches_library(oracle_mod, dist, width):
    n = 50_000
    x = inputs.keys(dist, n, width, seed=7)
    p = oracle_mod.Params(k=16, a=8, M=512, seed=11)
    out, _, recs = oracle_mod.sort(x, params=p, log=True)
    assert out.dtype == x.dtype
    np.testing.assert_array_equal(out, np.sort(x))
    check_records(recs, p)


def test_random_params(oracle_mod):
    rng = np.random.default_rng(3)
    for _ in range(40):
        n = int(rng.integers(0, 20_000))
        k = int(2 ** rng.integers(1, 11))
        p = oracle_mod.Params(k=k, a=int(rng.integers(1, 40)), M=int(rng.integers(1, 3000)),
                              k_policy=int(rng.integers(0, 2)), fill_div=int(rng.integers(1, 8)),
                              seed=int(rng.integers(0, 2 ** 63)))
        alphabet = int(rng.choice([2, 17, 1000, 2 ** 32]))
        x = rng.integers(0, alphabet, size=n, dtype=np.uint64)
        out, vals, recs = oracle_mod.sort(x, np.arange(n, dtype=np.uint64), p, log=True)
        np.testing.assert_array_equal(out, np.sort(x))
        np.testing.assert_array_equal(np.sort(vals), np.arange(n, dtype=np.uint64))
        np.testing.assert_array_equal(x[vals.astype(np.int64)], out)
        check_records(recs, p)


def check_records(recs, p):
    for r in recs:
        assert r.m > p.M                                       # only buckets > M are split
        assert int(r.children.sum()) == r.m                    # a partition
        assert r.K == (2 * r.ks - 1 if r.eq else r.ks)
        assert np.all(r.splitters[:-1] <= r.splitters[1:])     # sorted sample order statistics
        if not r.eq:
            assert r.ks == r.kb
            # distinct splitters and >= 2 of them => every range child is smaller (progress)
            assert np.all(r.children < r.m)
        else:
            rng_children = r.children[0::2]
            assert np.all(rng_children < r.m)                  # splitter keys left every range child


# --------------------------------------------------------------------------
# One distribution step: stable partition, splitters from the hashed sample
# --------------------------------------------------------------------------
@pytest.mark.parametrize("dist", ["uniform", "dd", "and4", "equal", "sorted"])
def test_distribute_is_stable_partition(oracle_mod, dist):
    n = 30_000
    x = inputs.keys(dist, n, 64, seed=5)
    v = inputs.values(n, 64)
    p = oracle_mod.Params(k=64, a=10, M=100, k_policy=0, seed=99)
    out, vals, r = oracle_mod.distribute(x, v, p)
    spl = [int(s) for s in r.splitters]
    # ids by the plain definition (brute-force count), then Python's stable sort
    ids = np.searchsorted(np.array(spl, dtype=np.uint64), x, side="left").astype(np.int64)
    if r.eq:
        sp = np.array(spl + [0], dtype=np.uint64)
        hit = (ids < len(spl)) & (x == sp[np.minimum(ids, len(spl))])
        ids = 2 * ids + hit
    order = np.argsort(ids, kind="stable")
    np.testing.assert_array_equal(out, x[order])
    np.testing.assert_array_equal(vals, v[order])
    np.testing.assert_array_equal(r.children, np.bincount(ids, minlength=r.K))


def test_splitters_are_sample_order_statistics(oracle_mod):
    n = 100_000
    x = inputs.keys("uniform", n, 64, seed=2)
    p = oracle_mod.Params(k=128, a=30, M=1000, seed=5489)
    _, _, r = oracle_mod.distribute(x, None, p)
    assert (r.kb, r.ks, r.eq, r.a_eff) == (128, 128, 0, 30)
    seed = p.seed
    h0 = py_fmix((py_fmix((seed ^ (0 << 56)) + GAMMA) ^ 0) + GAMMA)   # sm(sm(seed ^ lvl) ^ lo)
    S = []
    for j in range(r.a_eff * r.kb):
        h = py_fmix((h0 ^ j) + GAMMA)
        S.append(int(x[(h * n) >> 64]))
    S.sort()
    want = [S[r.a_eff * (i + 1) - 1] for i in range(r.kb - 1)]
    assert [int(s) for s in r.splitters] == want


# --------------------------------------------------------------------------
# Special cases
# --------------------------------------------------------------------------
def test_all_equal_one_equality_bucket(oracle_mod):
    n = 10_000
    x = np.full(n, 42, dtype=np.uint64)
    p = oracle_mod.Params(k=128, a=30, M=64)
    out, _, recs = oracle_mod.sort(x, params=p, log=True)
    np.testing.assert_array_equal(out, x)
    assert len(recs) == 1
    r = recs[0]
    assert r.eq == 1 and r.ks == 64 and r.K == 127
    # every key equals every splitter: b = 0, id = 1 (the first equality bucket)
    assert int(r.children[1]) == n and int(r.children.sum()) == n


def test_sorted_and_small_cases(oracle_mod):
    p = oracle_mod.Params(k=8, a=4, M=16)
    x = np.arange(1000, dtype=np.uint64)
    out, _, _ = oracle_mod.sort(x, params=p)
    np.testing.assert_array_equal(out, x)
    for n in (0, 1, 2, 16):
        y = np.arange(n, 0, -1, dtype=np.uint64)
        out, _, recs = oracle_mod.sort(y, params=p, log=True)
        np.testing.assert_array_equal(out, np.sort(y))
        assert recs == []                                     # n <= M: no distribution level
    ext = np.array([0, MASK, 5, MASK, 0, 1], dtype=np.uint64)
    out, _, _ = oracle_mod.sort(ext, params=oracle_mod.Params(k=2, a=1, M=1))
    assert out.tolist() == sorted(ext.tolist())


def test_dd_finishes_in_equality_mode(oracle_mod):
    n = 1 << 16
    x = inputs.keys("dd", n, 32)
    p = oracle_mod.Params(k=128, a=30, M=1 << 10)
    out, _, recs = oracle_mod.sort(x, params=p, log=True)
    np.testing.assert_array_equal(out, np.sort(x))
    assert recs[0].eq == 1
    assert max(r.level for r in recs) <= 1


def test_select_is_rank(oracle_mod):
    x = inputs.keys("and3", 20_001, 64, seed=9)
    s = np.sort(x)
    for r in (0, 1, 777, 10_000, 20_000):
        assert oracle_mod.select(x, r) == int(s[r])


# --------------------------------------------------------------------------
# Equality mode (R4) splitters, recomputed from the hashed sample in Python,
# at level 0 and at level 1 (lo != 0 keys the hash); R4.
# --------------------------------------------------------------------------
def py_splitters(arr, lo, m, level, p, kb, a):
    """Sample a*kb keys of arr[lo, lo+m) at H(seed, level, lo, j) (R2), sort
    them, take S[a(i+1)-1] (R1); if two are equal or kb == 2, switch to
    equality mode with ks = max(2, kb/2) splitters S[(s/ks)(i+1)-1] (R4)."""
    h0 = py_fmix((py_fmix((p.seed ^ (level << 56)) + GAMMA) ^ lo) + GAMMA)
    s = a * kb
    S = sorted(int(arr[lo + ((py_fmix((h0 ^ j) + GAMMA) * m) >> 64)]) for j in range(s))
    spl = [S[a * (i + 1) - 1] for i in range(kb - 1)]
    eq = kb == 2 or any(spl[i] == spl[i + 1] for i in range(len(spl) - 1))
    if not eq:
        return 0, kb, spl
    ks = max(2, kb // 2)
    stride = s // ks
    return 1, ks, [S[stride * (i + 1) - 1] for i in range(ks - 1)]


@pytest.mark.parametrize("dist", ["dd", "and5", "equal", "uniform"])
def test_equality_mode_splitters_recomputed(oracle_mod, dist):
    n = 40_000
    x = inputs.keys(dist, n, 32, seed=12)
    if dist == "uniform":
        x = (x % np.uint32(7)).astype(np.uint32)                  # few distinct keys: eq mode at level 0
    p = oracle_mod.Params(k=64, a=12, M=256, k_policy=0, seed=321)
    lvl1, _, r0 = oracle_mod.distribute(x, None, p)
    eq, ks, spl = py_splitters(x, 0, n, 0, p, r0.kb, r0.a_eff)
    assert (r0.eq, r0.ks) == (eq, ks)
    assert [int(s) for s in r0.splitters] == spl
    saw_eq = r0.eq
    # level-1 buckets: the oracle's own records of the whole sort, against the
    # Python recomputation on the (separately pinned) level-0 partition
    _, _, recs = oracle_mod.sort(x, params=p, log=True)
    assert recs[0].lo == 0 and recs[0].level == 0
    for r in recs:
        if r.level != 1:
            continue
        eq, ks, spl = py_splitters(lvl1, r.lo, r.m, 1, p, r.kb, r.a_eff)
        assert (r.eq, r.ks, r.K) == (eq, ks, 2 * ks - 1 if eq else ks)
        assert [int(s) for s in r.splitters] == spl
        saw_eq |= r.eq
    assert saw_eq, "input did not exercise equality mode"


@pytest.mark.parametrize("pairs", [False, True])
def test_threads_give_identical_results(oracle_mod, pairs):
    """The OpenMP mode (tasks per child bucket, chunked Phases 2-4) gives the
    same keys, values and level records as the sequential recursion."""
    n = 600_001
    for dist in ("uniform", "dd", "and3"):
        x = inputs.keys(dist, n, 64, seed=3)
        v = inputs.values(n, 64) if pairs else None
        res = []
        for t in (1, 4):
            p = oracle_mod.Params(k=64, a=20, M=2000, k_policy=1, seed=7, threads=t)
            res.append(oracle_mod.sort(x, v, p, log=True))
        (k1, v1, r1), (k4, v4, r4) = res
        np.testing.assert_array_equal(k1, np.sort(x))
        np.testing.assert_array_equal(k1, k4)
        if pairs:
            np.testing.assert_array_equal(v1, v4)
        assert len(r1) == len(r4) and len(r1) > 1
        for a, b in zip(r1, r4):
            assert (a.level, a.lo, a.m, a.kb, a.ks, a.eq, a.K) == (b.level, b.lo, b.m, b.kb, b.ks, b.eq, b.K)
            np.testing.assert_array_equal(a.splitters, b.splitters)
            np.testing.assert_array_equal(a.children, b.children)


def test_library_references_sort(oracle_mod):
    x = inputs.keys("uniform", 100_003, 32, seed=2)
    for t in (1, 3):
        np.testing.assert_array_equal(oracle_mod.library_sort(x, t), np.sort(x))
