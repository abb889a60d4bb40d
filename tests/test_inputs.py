"""Pins for the synthetic input generators (inputs/)."""
import numpy as np
import pytest

import inputs


def test_uniform_u32_is_high_half_of_u64():
    a = inputs.keys("uniform", 1000, 64, seed=3)
    b = inputs.keys("uniform", 1000, 32, seed=3)
    np.testing.assert_array_equal(b, (a >> np.uint64(32)).astype(np.uint32))


def test_chunking_and_offsets_are_consistent():
    full = inputs.keys("bucket", 10_000, 64, seed=4)
    part = inputs.keys("bucket", 10_000, 64, seed=4, start=1234, count=5000)
    np.testing.assert_array_equal(full[1234:6234], part)


@pytest.mark.parametrize("width", [32, 64])
def test_gaussian_exact_floor_of_mean(width):
    n = 257
    g = inputs.keys("gaussian", n, width, seed=8)
    i = np.arange(n, dtype=np.int64)
    ws = [inputs.words(i, w, 4, 8) for w in range(4)]
    for t in range(n):
        xs = [int(w[t]) >> (64 - width) for w in ws]
        assert int(g[t]) == sum(xs) // 4                   # average of 4 random values


def test_dd_matches_block_rule():
    # the first p/2 blocks hold log n, the next p/4 hold log(n/2), ...
    for logn in range(4, 16):
        n = 1 << logn
        x = inputs.keys("dd", n, 32)
        for p in (2, 4, 8, 16):
            if p > n:
                continue
            blk = n // p
            for b in range(p - 1):
                # blocks [p - p/2^t, p - p/2^(t+1)) hold log2(n / 2^t)
                t = 0
                while b >= p - (p >> (t + 1)):
                    t += 1
                assert np.all(x[b * blk:(b + 1) * blk] == logn - t), (n, p, b)
        assert x[-1] == 0 and x[0] == logn


def test_staggered_slots_cover_all_once():
    p = inputs.P_GEN
    slots = sorted((2 * i - 1) if i <= p // 2 else (2 * i - p - 2) for i in range(1, p + 1))
    assert slots == list(range(p))


@pytest.mark.parametrize("width", [32, 64])
def test_staggered_and_bucket_ranges(width):
    n = 240 * 97 + 13
    H = 1 << (width - 1)
    p = inputs.P_GEN
    st = inputs.keys("staggered", n, width, seed=2).astype(object)
    bs = inputs.keys("bucket", n, width, seed=2).astype(object)
    for i in range(0, n, 37):
        r = ((i + 1) * p + n - 1) // n - 1
        assert r * n // p <= i < (r + 1) * n // p
        bi = r + 1
        slot = 2 * bi - 1 if bi <= p // 2 else 2 * bi - p - 2
        assert slot * H // p <= st[i] <= (slot + 1) * H // p - 1
        b0 = r * n // p
        blen = (r + 1) * n // p - b0
        j = ((i - b0 + 1) * p + blen - 1) // blen - 1
        assert j * blen // p <= i - b0 < (j + 1) * blen // p
        assert j * H // p <= bs[i] <= (j + 1) * H // p - 1


@pytest.mark.parametrize("r", [2, 3, 4])
def test_and_r_bit_frequency(r):
    x = inputs.keys(f"and{r}", 1 << 16, 64, seed=1)
    bits = np.unpackbits(x.view(np.uint8)).mean()
    assert abs(bits - 2.0 ** -r) < 0.01


def test_sorted_is_sorted_uniform():
    a = inputs.keys("sorted", 5000, 64)
    np.testing.assert_array_equal(a, np.sort(inputs.keys("uniform", 5000, 64)))
