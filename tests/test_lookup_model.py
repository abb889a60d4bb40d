"""Model of Phase 2's radix-indexed splitter lookup (csrc/gss_kernels.cuh lut_bin / lut_build / lut_group),
checked against the definition it replaces: Algorithm 2's descent computes b = #{splitters s < e}
(P:305-311), i.e. numpy's searchsorted(spl, e, side='left') on the sorted splitters.  The model follows
the kernel step by step (4096 bins of 2^shift key values from s_0, bin 0 below s_0, the last bin open above;
lo = #{s < bin start}, hi = #{s < bin end}; the refinement by spl[lo] and a binary search over
spl[lo+1 .. hi)), so an off-by-one in the bin arithmetic or the table shows here without a GPU."""
import numpy as np
import pytest

LUT_BITS = 12
LUT_N = 1 << LUT_BITS


def lut_bin(e: int, base: int, shift: int) -> int:
    if e < base:
        return 0
    return min((e - base) >> shift, LUT_N - 1)


def lut_build(spl: list[int]):
    base = spl[0] if spl else 0
    span = (spl[-1] - base) if spl else 0
    bl = span.bit_length()
    shift = bl - LUT_BITS if bl > LUT_BITS else 0
    cnt = [0] * LUT_N
    for s in spl:
        cnt[lut_bin(s, base, shift)] += 1
    lo, table = 0, []
    for c in cnt:
        table.append((lo, lo + c))
        lo += c
    crowd = sum(c for c in cnt if c >= 2)
    return base, shift, table, crowd * 8 <= len(spl)


def lut_lookup(e: int, spl: list[int], base: int, shift: int, table) -> int:
    lo, hi = table[lut_bin(e, base, shift)]
    b = lo
    if hi > lo:
        if spl[lo] < e:
            b = lo + 1
            l, h = b, hi                       # first index of spl[lo+1 .. hi) not below e
            while l < h:
                m = (l + h) >> 1
                if spl[m] < e:
                    l = m + 1
                else:
                    h = m
            b = l
    return b


def _check(spl, keys):
    spl = sorted(int(s) for s in spl)
    base, shift, table, _ = lut_build(spl)
    want = np.searchsorted(np.array(spl, dtype=object), np.array(keys, dtype=object), side="left")
    got = [lut_lookup(int(e), spl, base, shift, table) for e in keys]
    assert list(want) == got


@pytest.mark.parametrize("width", [32, 64])
@pytest.mark.parametrize("nspl", [1, 3, 15, 255, 1023])
def test_lookup_equals_rank_random(width, nspl):
    rng = np.random.default_rng(nspl + width)
    mx = (1 << width) - 1
    spl = [int(x) for x in rng.integers(0, mx, nspl, dtype=np.uint64 if width == 64 else np.uint32, endpoint=True)]
    keys = [int(x) for x in rng.integers(0, mx, 3000, dtype=np.uint64 if width == 64 else np.uint32, endpoint=True)]
    keys += spl + [s + 1 for s in spl if s < mx] + [s - 1 for s in spl if s > 0] + [0, mx]
    _check(spl, keys)


@pytest.mark.parametrize("width", [32, 64])
def test_lookup_corner_splitters(width):
    mx = (1 << width) - 1
    cases = [
        [0], [mx], [0, mx], [5, 5, 5, 5], [0] * 7 + [mx] * 8,          # duplicates, extremes
        [1 << (width - 1)] * 3 + [(1 << (width - 1)) + 1],              # a span of one value (shift 0)
        list(range(100, 100 + 4096 * 3, 3)),                            # span just above 12 bits
        [i * (mx // 300) for i in range(300)],                          # the full range (shift = width - 12)
        sorted((1 << k) for k in range(width)),                         # exponentially spaced: crowded low bins
    ]
    for spl in cases:
        keys = sorted(set([0, 1, mx, mx - 1] + [s for s in spl] + [min(s + 1, mx) for s in spl] +
                          [max(s - 1, 0) for s in spl] + list(range(0, 64))))
        _check(spl, keys)


def test_crowding_rule():
    """The per-bucket fallback: more than 1/8 of the splitters sharing a bin keeps the descent."""
    even = [i * 1000 for i in range(255)]
    assert lut_build(even)[3]
    expo = sorted((1 << k) for k in range(64))
    assert not lut_build(expo)[3]
