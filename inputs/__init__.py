"""Seeded synthetic inputs for GPU sample sort (shared by tests, bench, smoke).

This module holds only the input distributions; it contains none of the
sorting method's arithmetic.  The distributions are the ones the paper
evaluates on (after Helman, Bader & JaJa [7]), with the
readings R13-R19, R22 of DESIGN.md:

* element i depends only on (seed, i): ``word(i, w)`` is the (i*W + w)-th
  output of SplitMix64 seeded with ``seed`` (W = words per element), so the
  same global input is produced for any chunking or rank count;
* u32 keys take the high 32 bits of a word; u64 keys the whole word;
* P_gen = 240 generator blocks, H = 2^(w-1) (R22).

All functions return numpy arrays (uint32 or uint64).
"""
from __future__ import annotations

import numpy as np

GOLDEN = np.uint64(0x9E3779B97F4A7C15)
C1 = np.uint64(0xBF58476D1CE4E5B9)
C2 = np.uint64(0x94D049BB133111EB)
P_GEN = 240
CHUNK = 1 << 22

DISTRIBUTIONS = ("uniform", "gaussian", "bucket", "staggered", "sorted", "dd", "and2", "and3", "and4",
                 "and5", "equal")


def _fmix(z: np.ndarray) -> np.ndarray:
    with np.errstate(over="ignore"):
        z ^= z >> np.uint64(30)
        z *= C1
        z ^= z >> np.uint64(27)
        z *= C2
        z ^= z >> np.uint64(31)
    return z


def words(i: np.ndarray, w: int, W: int, seed: int) -> np.ndarray:
    """word(i, w) = fmix64(seed + (i*W + w + 1) * golden), i an int64/uint64 array."""
    j = i.astype(np.uint64) * np.uint64(W) + np.uint64(w + 1)
    with np.errstate(over="ignore"):
        z = np.uint64(seed & 0xFFFFFFFFFFFFFFFF) + j * GOLDEN
    return _fmix(z)


def _to_width(x: np.ndarray, width: int) -> np.ndarray:
    return (x >> np.uint64(32)) if width == 32 else x


def _mulhi(x: np.ndarray, rng: np.ndarray, width: int) -> np.ndarray:
    """floor(x * rng / 2^width) for w-bit x and rng <= 2^width, exactly."""
    if width == 32:
        return (x * rng) >> np.uint64(32)
    m32 = np.uint64(0xFFFFFFFF)
    s32 = np.uint64(32)
    xh, xl = x >> s32, x & m32
    rh, rl = rng >> s32, rng & m32
    with np.errstate(over="ignore"):
        mid = xh * rl + ((xl * rl) >> s32)
        mid2 = xl * rh + (mid & m32)
        return xh * rh + (mid >> s32) + (mid2 >> s32)


def _block(i: np.ndarray, n: int, p: int) -> np.ndarray:
    """Block r of element i for blocks [floor(r n/p), floor((r+1) n/p)) (R15)."""
    return ((i + 1) * p + n - 1) // n - 1


def _ranges(H: int, p: int):
    """Sub-range j = [floor(j H / p), floor((j+1) H / p) - 1] as (lo, size) tables (exact big ints)."""
    lo = [(j * H) // p for j in range(p)]
    hi = [((j + 1) * H) // p - 1 for j in range(p)]
    return (np.array(lo, dtype=np.uint64), np.array([h - l + 1 for l, h in zip(lo, hi)], dtype=np.uint64))


def _chunk(dist: str, i: np.ndarray, n: int, width: int, seed: int) -> np.ndarray:
    H = 1 << (width - 1)
    p = P_GEN
    if dist in ("uniform", "sorted"):                         # P:373 (R13), R18
        return _to_width(words(i, 0, 1, seed), width)
    if dist == "gaussian":                                    # P:374-375 (R14): floor(sum of 4 / 4), exact
        xs = [_to_width(words(i, w, 4, seed), width) for w in range(4)]
        q = sum(x >> np.uint64(2) for x in xs)
        rsum = sum(x & np.uint64(3) for x in xs)
        with np.errstate(over="ignore"):
            return q + (rsum >> np.uint64(2))
    if dist == "bucket":                                      # P:376-378 (R15)
        r = _block(i, n, p)
        b0 = (r * n) // p
        blen = ((r + 1) * n) // p - b0
        off = i - b0
        # sub-group j of the block: [floor(j len / p), floor((j+1) len / p))
        j = ((off + 1) * p + blen - 1) // blen - 1
        lo, rng = _ranges(H, p)
        x = _to_width(words(i, 0, 1, seed), width)
        return lo[j] + _mulhi(x, rng[j], width)
    if dist == "staggered":                                   # P:379-380 (R16)
        r = _block(i, n, p)
        bi = r + 1                                            # 1-based block index
        slot = np.where(bi <= p // 2, 2 * bi - 1, 2 * bi - p - 2)
        lo, rng = _ranges(H, p)
        x = _to_width(words(i, 0, 1, seed), width)
        return lo[slot] + _mulhi(x, rng[slot], width)
    if dist == "dd":                                          # P:381-383 (R17): ceil(log2(n - i))
        v = (n - i).astype(np.uint64)
        out = np.zeros(v.shape, dtype=np.uint64)
        # ceil(log2 v) = bit length of (v - 1)
        t = v - np.uint64(1)
        while True:
            nz = t > 0
            if not nz.any():
                break
            out += nz.astype(np.uint64)
            t >>= np.uint64(1)
        return out
    if dist.startswith("and"):                                # R19: AND of r words
        rr = int(dist[3:])
        x = _to_width(words(i, 0, rr, seed), width)
        for w in range(1, rr):
            x &= _to_width(words(i, w, rr, seed), width)
        return x
    if dist == "equal":
        return np.full(i.shape, np.uint64(0x5A5A5A5A5A5A5A5A) >> np.uint64(64 - width), dtype=np.uint64)
    raise ValueError(f"unknown distribution {dist!r}")


def keys(dist: str, n: int, width: int = 64, seed: int = 1, start: int = 0, count: int | None = None) -> np.ndarray:
    """Keys [start, start+count) of the n-element input of ``dist`` (uint32/uint64)."""
    assert width in (32, 64)
    count = n - start if count is None else count
    dt = np.uint32 if width == 32 else np.uint64
    out = np.empty(count, dtype=dt)
    for c0 in range(0, count, CHUNK):
        c1 = min(count, c0 + CHUNK)
        i = np.arange(start + c0, start + c1, dtype=np.int64)
        out[c0:c1] = _chunk(dist, i, n, width, seed).astype(dt)
    if dist == "sorted":
        if start != 0 or count != n:
            raise ValueError("sorted input is only defined for the whole array")
        out.sort(kind="stable")
    return out


def values(n: int, width: int = 64, start: int = 0) -> np.ndarray:
    """value_i = i, the input index (R20)."""
    return np.arange(start, start + n, dtype=np.uint32 if width == 32 else np.uint64)
