// gss_kernels.cuh -- the kernels of one k-way distribution level and the
// bucket finishers (section 4 "Algorithm Overview" P:251-275 and
// section 5 "Implementation Details" P:279-352).
//
// One level = sample (Phase 1) -> classify (Phase 2) -> scan (Phase 3) ->
// scatter (Phase 4) -> plan (the recursion of Algorithm 1, and the
// delayed bucket sorting of P:326-331).  Every kernel is persistent: a grid of
// (SMs x resident CTAs) loops over the level's work, whose size is read from
// device memory, so the host enqueues a fixed launch sequence with no
// per-level synchronisation.
#pragma once

#include <cooperative_groups.h>

#include "gss_device.cuh"

namespace gss {

constexpr int kClsThreads = 256;
#ifndef GSS_CLS_U
#define GSS_CLS_U 8                                              // keys per lane per classify group
#endif
#ifndef GSS_SCATTER_THREADS
#define GSS_SCATTER_THREADS 512
#endif
#ifndef GSS_SCATTER_MINB
#define GSS_SCATTER_MINB 2
#endif
#ifndef GSS_SCATTER_EARLY
#define GSS_SCATTER_EARLY 0
#endif
#ifndef GSS_SCATTER_SPREAD
#define GSS_SCATTER_SPREAD 0     // 1: per-id work spread over every warp -- measured slower (2^28 u64 scatter 3.16 vs 2.94 ms)
#endif
#ifndef GSS_SCATTER_PAIRFOLD
#define GSS_SCATTER_PAIRFOLD 0   // 1: two threads per id in the fold (u64 3.18 vs 3.11 ms, pairs 3.30 vs 2.99: slower)
#endif
constexpr int kScatterThreads = GSS_SCATTER_THREADS;
#ifndef GSS_SCATTER_ITER
#define GSS_SCATTER_ITER 8
#endif
#ifndef GSS_SCATTER_ITER_U32
#define GSS_SCATTER_ITER_U32 16  // 4-byte keys alone: 16 per thread (the registers and shared bytes of 8 u64 keys);
#endif                           // 2^27 u32 scatter 1.05 vs 1.14 ms (u64 at 16: 1.74 vs 1.56 ms, so 8 there)
// keys per thread per chunk; a chunk (kScatterThreads x this) is staged in shared memory: 4096 keys, 8192 for u32
#ifndef GSS_SCATTER_ITER_KV32
#define GSS_SCATTER_ITER_KV32 8
#endif
template <class Key, class Val>
constexpr int scatter_iter() {
  return sizeof(Key) == 4 ? (kHasVal<Val> ? (sizeof(Val) == 4 ? GSS_SCATTER_ITER_KV32 : GSS_SCATTER_ITER)
                                          : GSS_SCATTER_ITER_U32)
                          : GSS_SCATTER_ITER;
}
#define GSS_SCATTER_CHUNK_CONSTANTS                                  \
  constexpr int kScatterIter = scatter_iter<Key, Val>();            \
  constexpr int kChunk = kScatterThreads * kScatterIter;
constexpr int kScanCtas = 256;
constexpr int kScanThreads = 256;
constexpr int kPlanThreads = 256;
constexpr int kSampleThreads = 1024;                              // sample sort capacity 16384

// ---------------------------------------------------------------------------
// init: zero the counters, create the level-0 bucket (or the single small
// bucket when n <= M).
// ---------------------------------------------------------------------------
template <class Key, class Val, class IdT>
__global__ void k_init(Ctx<Key, Val, IdT> c) {
  uint32_t* w = reinterpret_cast<uint32_t*>(c.cnt);
  for (uint32_t i = threadIdx.x; i < sizeof(Counters) / 4; i += blockDim.x) w[i] = 0;
  __syncthreads();
  if (threadIdx.x != 0 || c.n == 0) return;
  if (c.mode == MODE_SORT && c.n <= c.M) {
    c.cnt->small_elems = c.n;
    c.cnt->max_small = c.n;
    if (c.n > c.class_cap[kNumClasses - 1]) {                  // GSS_FLAG_CLUSTER_SORT: one cluster sorts it
      c.clus[0] = Item{0, c.n, c.src0, 0};
      c.cnt->clus_count = 1;
      return;
    }
    uint32_t cls = 0;
    while (cls + 1 < kNumClasses && c.n > c.class_cap[cls]) cls++;
    c.small[cls][0] = Item{0, c.n, c.src0, 0};
    c.cnt->small_count[cls] = 1;
    c.cnt->small_elems = c.n;
    c.cnt->max_small = c.n;
    return;
  }
  uint32_t kb;
  if (c.mode == MODE_PARTITION_BY) {
    kb = 1;
    while (kb < c.given_nspl + 1) kb <<= 1;
  } else {
    kb = choose_kb(c.k, c.k_policy, c.fill_div, c.M, c.n);
  }
  uint32_t nt = (uint32_t)(((uint64_t)c.n + c.T - 1) / c.T);
  Bucket B{};
  B.lo = 0; B.m = c.n; B.tile_start = 0; B.ntiles = nt; B.kb = kb;
  B.hist_base = 0; B.spl_base = 0; B.id_base = 0;
  c.bk[0][0] = B;
  LevelCounters& L = c.cnt->lvl[0];
  const uint32_t kids = (c.mode == MODE_PARTITION_BY && c.given_eq) ? 2 * kb : kb;   // K <= kids - 1
  L.num_buckets = 1; L.num_tiles = nt; L.hist_alloc = max(kids, 3u) * nt; L.spl_alloc = 2 * kb;
  L.split_elems = c.n;
}

// ---------------------------------------------------------------------------
// Phase 1: per split bucket, a*k_b keys at hashed positions
// (with replacement, R1/R2), sorted in shared memory by one CTA; splitters
// spl[i] = S[a(i+1)-1]; equality mode if two splitters are equal or k_b == 2
// (R4), then k_s = k_b/2 splitters S[(s/k_s)(i+1)-1]; the implicit tree
// bt[j] = s_{(2q+1) k_s / 2^(d+1)}.
// ---------------------------------------------------------------------------
// NT: 1024 threads (capacity 16384 sample keys), or 512 (8192) with two CTAs per SM where a * k_max fits,
// so that the 256 sample sorts of a level with k = 256 run in one wave
template <class Key, class Val, class IdT, class Cmp, int NT = kSampleThreads>
__global__ void __launch_bounds__(NT, kSampleThreads / NT) k_sample(Ctx<Key, Val, IdT> c, uint32_t level) {
  constexpr int kSampleThreads = NT;
  extern __shared__ __align__(16) unsigned char smem_raw[];
  Key* sk = reinterpret_cast<Key*>(smem_raw);
  using Sorter = CtaSort<Key, NoVal, NT, Cmp>;
  const Cmp less;
  const uint32_t slot = level & 1;
  const uint32_t nb = c.cnt->lvl[level].num_buckets;
  const Key* src = c.keys(c.src(level));
  for (uint32_t b = blockIdx.x; b < nb; b += gridDim.x) {
    Bucket B = c.bk[slot][b];
    const uint32_t kb = B.kb;
    uint32_t a = c.a;
    if (c.sample_cap / kb < a) a = c.sample_cap / kb;
    if (a < 1) a = 1;
    const uint32_t s = a * kb;
    for (uint32_t j0 = threadIdx.x; j0 < s; j0 += 8 * kSampleThreads) {   // 8 gathers in flight
      Key g[8];
#pragma unroll
      for (int u = 0; u < 8; u++) {
        const uint32_t j = j0 + u * kSampleThreads;
        if (j < s) g[u] = src[B.lo + sample_pos(c.seed, level, B.lo, j, B.m)];
      }
#pragma unroll
      for (int u = 0; u < 8; u++) {
        const uint32_t j = j0 + u * kSampleThreads;
        if (j < s) sk[phys(j)] = g[u];
      }
    }
    Sorter::sort(sk, nullptr, (int)s, less);
    bool dup = false;
    for (uint32_t i = threadIdx.x; i + 2 < kb; i += kSampleThreads)
      dup |= !less(sk[phys(a * (i + 1) - 1)], sk[phys(a * (i + 2) - 1)]);
    const bool eq = __syncthreads_or(dup) || kb == 2;
    const uint32_t ks = eq ? max(2u, kb / 2) : kb;
    const uint32_t stride = s / ks;
    Key* tree = c.spl[slot] + B.spl_base;
    Key* spl = tree + kb;
    for (uint32_t i = threadIdx.x; i + 1 < ks; i += kSampleThreads) spl[i] = sk[phys(stride * (i + 1) - 1)];
    for (uint32_t j = threadIdx.x + 1; j < ks; j += kSampleThreads) {
      uint32_t d = ilog2(j), q = j - (1u << d);
      uint32_t idx1 = ((2 * q + 1) * ks) >> (d + 1);
      tree[j] = sk[phys(stride * idx1 - 1)];
    }
    if (threadIdx.x == 0) {
      Bucket* g = &c.bk[slot][b];
      g->ks = ks; g->eq = eq ? 1u : 0u; g->K = eq ? 2 * ks - 1 : ks; g->clamp = 0;
    }
    for (uint32_t i = threadIdx.x; i < B.ntiles; i += kSampleThreads) c.tile_bucket[slot][B.tile_start + i] = b;
    __syncthreads();
  }
}

// partition_by: the splitters are given (distributed global level).  k_s is
// the next power of two >= nspl+1; the tree is padded with copies of the
// largest splitter and ids are clamped to nspl.  With given_eq the ids follow
// the equality rule (R4): 2b for keys strictly between splitters b-1 and b,
// 2b+1 for keys equal to splitter b (K = 2 nspl + 1), so a run of equal keys
// lands in one equality bucket whatever the number of equal splitters.
template <class Key, class Val, class IdT>
__global__ void k_set_splitters(Ctx<Key, Val, IdT> c) {
  Bucket B = c.bk[0][0];
  const uint32_t nspl = c.given_nspl;
  const uint32_t ks = B.kb;
  Key* tree = c.spl[0] + B.spl_base;
  Key* spl = tree + ks;
  for (uint32_t i = threadIdx.x; i + 1 < ks; i += blockDim.x) spl[i] = c.given_spl[min(i, nspl - 1)];
  for (uint32_t j = threadIdx.x + 1; j < ks; j += blockDim.x) {
    uint32_t d = ilog2(j), q = j - (1u << d);
    uint32_t idx1 = ((2 * q + 1) * ks) >> (d + 1);
    tree[j] = c.given_spl[min(idx1 - 1, nspl - 1)];
  }
  if (threadIdx.x == 0) {
    Bucket* g = &c.bk[0][0];
    g->ks = ks; g->eq = c.given_eq; g->K = c.given_eq ? 2 * nspl + 1 : nspl + 1; g->clamp = 1;
  }
  for (uint32_t i = threadIdx.x; i < B.ntiles; i += blockDim.x) c.tile_bucket[0][B.tile_start + i] = 0;
}

// ---------------------------------------------------------------------------
// Phase 2: bucket id of every key by the tree descent,
// stored (u8/u16) for Phase 4, and the per-tile histogram written bucket-major
// hist[id * p + t] (R6).  Counters: one k-array per warp (the paper's 8
// per-group arrays) in shared memory, then their vector sum
// (P:320-321).
// ---------------------------------------------------------------------------
// Shared-memory access by 32-bit shared-window address.
template <class Key>
__device__ __forceinline__ Key ld_shared(uint32_t a) {
  if constexpr (sizeof(Key) == 8) {
    unsigned long long x;
    asm volatile("ld.shared.u64 %0, [%1];" : "=l"(x) : "r"(a));
    return bit_cast_dev<Key>(x);
  } else {
    uint32_t x;
    asm volatile("ld.shared.u32 %0, [%1];" : "=r"(x) : "r"(a));
    return bit_cast_dev<Key>(x);
  }
}
// Two adjacent keys (a 2W-byte aligned pair) by one shared load.
template <class Key>
__device__ __forceinline__ void ld_shared_pair(uint32_t a, Key& x0, Key& x1) {
  if constexpr (sizeof(Key) == 8) {
    unsigned long long u0, u1;
    asm volatile("ld.shared.v2.u64 {%0, %1}, [%2];" : "=l"(u0), "=l"(u1) : "r"(a));
    x0 = bit_cast_dev<Key>(u0); x1 = bit_cast_dev<Key>(u1);
  } else {
    uint32_t u0, u1;
    asm volatile("ld.shared.v2.u32 {%0, %1}, [%2];" : "=r"(u0), "=r"(u1) : "r"(a));
    x0 = bit_cast_dev<Key>(u0); x1 = bit_cast_dev<Key>(u1);
  }
}
#ifndef GSS_CLS_PAIRLOAD
#define GSS_CLS_PAIRLOAD 0
#endif

__device__ __forceinline__ void red_shared_add(uint32_t a, uint32_t v) {
  asm volatile("red.shared.add.u32 [%0], %1;" ::"r"(a), "r"(v));
}

// Tree layout in shared memory.  Levels 0..4 (nodes 1..31) stay in plain
// Eytzinger order: a warp touches at most 16 distinct nodes of one level, all
// inside 128 B, so those loads are conflict-free broadcasts.  Levels 5..7
// (nodes 32..255) are where 32 lanes hit up to 32 different nodes; there every
// node is replicated once per bank group (128 B per node: 32 copies of a u32
// key, 16 of a u64 key) and lane l reads copy l mod (128/w), so a warp's load
// is conflict-free whatever the keys are.  Levels >= 8 (k > 256) fall back to
// the plain order.
constexpr uint32_t kTopLevels = 5;
constexpr uint32_t kRepEnd = 8;
constexpr uint32_t kRepNodes = (1u << kRepEnd) - (1u << kTopLevels);    // 224
template <class Key>
constexpr uint32_t rep_copies() { return 128u / sizeof(Key); }
template <class Key>
constexpr size_t cls_smem_bytes(uint32_t kmax) {
  return (size_t)kmax * sizeof(Key) * 2 + (size_t)kRepNodes * 128 + (size_t)(kClsThreads / 32) * kmax * 4 +
         (size_t)(kClsThreads / 32) * (32 * GSS_CLS_U) * 2 + (size_t)(1u << 12) * 4 + 64 * 4;   // + lookup table, scan scratch
}

// One level of Algorithm 2 (j := 2j + (e > bt[j])) on a node address
// a = base + step*j: a' = 2a - base + step*[bt[j] < e]  (the doubling on the
// FMA pipe, the comparison and select on the ALU pipe).
template <class Key, class Cmp>
__device__ __forceinline__ uint32_t descend_step(uint32_t a, Key e, uint32_t s0, uint32_t s1, Cmp less) {
  const Key x = ld_shared<Key>(a);
  const uint32_t t = less(x, e) ? s1 : s0;
  uint32_t r;
  asm("mad.lo.u32 %0, %1, 2, %2;" : "=r"(r) : "r"(a), "r"(t));
  return r;
}

// Bucket ids of U keys per lane: the whole descent (plain top levels,
// bank-replicated middle levels, plain deep levels), then the id rule of the
// tile's mode (0: range buckets, 1: equality mode R4, 2: clamped ids of
// partition_by, 3: partition_by in equality mode).
template <int MODE, int U, class Key, class Cmp>
__device__ __forceinline__ void descend_group(const Key (&e)[U], uint32_t (&id)[U], uint32_t tree_s, uint32_t rep_b,
                                              const Key* spl, uint32_t logk, uint32_t ks, uint32_t K, Cmp less) {
  constexpr uint32_t W = sizeof(Key);
  const uint32_t r0 = 0u - rep_b, r1 = 128u - rep_b;         // replicated region steps (per lane)
  const uint32_t d1 = min(logk, kTopLevels), d2 = min(logk, kRepEnd);
  // plain region: r = W*j relative to the tree, r' = 2r + W*[bt[j] < e]
  uint32_t r[U];
#pragma unroll
  for (int u = 0; u < U; u++) r[u] = W;
  uint32_t d = 0;
#if GSS_CLS_PAIRLOAD
  // two levels per round trip: node j and both children (2j, 2j+1 are adjacent: one 2W-byte load)
  // are loaded together, so the dependent chain has one shared-memory latency per two levels
  for (; d + 2 <= d1; d += 2) {
#pragma unroll
    for (int u = 0; u < U; u++) {
      const Key x = ld_shared<Key>(tree_s + r[u]);
      Key c0, c1;
      ld_shared_pair<Key>(tree_s + 2 * r[u], c0, c1);
      const bool p1 = less(x, e[u]);
      const bool p2 = less(p1 ? c1 : c0, e[u]);
      r[u] = 4 * r[u] + (p1 ? 2 * W : 0u) + (p2 ? W : 0u);
    }
  }
#endif
  for (; d < d1; d++) {
#pragma unroll
    for (int u = 0; u < U; u++) {
      const Key x = ld_shared<Key>(tree_s + r[u]);
      const uint32_t t = less(x, e[u]) ? W : 0u;
      asm("mad.lo.u32 %0, %1, 2, %2;" : "=r"(r[u]) : "r"(r[u]), "r"(t));
    }
  }
  if (logk > kTopLevels) {
    // replicated region: absolute a = rep_b + 128 j
    uint32_t a[U];
#pragma unroll
    for (int u = 0; u < U; u++) a[u] = rep_b + (128u / W) * r[u];
    for (uint32_t d = kTopLevels; d < d2; d++) {
#pragma unroll
      for (int u = 0; u < U; u++) a[u] = descend_step(a[u], e[u], r0, r1, less);
    }
#pragma unroll
    for (int u = 0; u < U; u++) r[u] = (a[u] - rep_b) / (128u / W);
    for (uint32_t d = kRepEnd; d < logk; d++) {
#pragma unroll
      for (int u = 0; u < U; u++) {
        const Key x = ld_shared<Key>(tree_s + r[u]);
        const uint32_t t = less(x, e[u]) ? W : 0u;
        asm("mad.lo.u32 %0, %1, 2, %2;" : "=r"(r[u]) : "r"(r[u]), "r"(t));
      }
    }
  }
#pragma unroll
  for (int u = 0; u < U; u++) {
    const uint32_t b = r[u] / W - (1u << logk);
    if constexpr (MODE == 1) {
      // equality bucket of splitter b (b < ks-1 and e == spl[b]: ties go left, so e <= spl[b])
      const uint32_t bb = min(b, ks - 2);
      id[u] = 2 * b + ((b + 1 < ks && !less(e[u], spl[bb])) ? 1u : 0u);
    } else if constexpr (MODE == 2) {
      id[u] = min(b, K - 1);
    } else if constexpr (MODE == 3) {
      // given splitters in equality mode (distributed global level): nspl = (K-1)/2
      // real splitters, the padded tree slots copy the largest; range id 2b, equality id 2b+1
      const uint32_t nspl = K >> 1, bc = min(b, nspl);
      id[u] = 2 * bc + ((bc < nspl && !less(e[u], spl[min(bc, nspl - 1)])) ? 1u : 0u);
    } else {
      id[u] = b;
    }
  }
}

// ---------------------------------------------------------------------------
// Radix-indexed splitter lookup: an exact replacement of the descent for
// unsigned keys under operator< (the same id b = #{splitters s < e} that
// Algorithm 2 computes).  The bucket's splitter range
// [s_0, s_{ks-2}] is cut into kLutN bins of 2^shift key values each (keys
// below s_0 fall into bin 0, keys above the range into the last, open bin);
// lut[i] = lo | hi << 16 with lo = #{s < start of bin i} and hi = #{s < end
// of bin i}.  A key of bin i has lo <= b <= hi: when lo == hi -- every bin
// without a splitter, i.e. all but at most ks-1 of the kLutN -- the single
// shared load is the whole classification; otherwise spl[lo] decides between
// lo and lo+1, and a bin holding two or more splitters (rare unless the keys
// cluster in value) finishes with a binary search over spl[lo+1 .. hi).  On
// B200 the 8-level descent is issue-bound (~65 instructions per u64 key); the
// lookup needs about a third of that.  GSS_FLAG_TREE_CLASSIFY keeps the
// paper's descent for every key (ablation).
// ---------------------------------------------------------------------------
constexpr uint32_t kLutBits = 12, kLutN = 1u << kLutBits;
template <class Key, class Cmp>
constexpr bool lut_ok() { return std::is_same<Cmp, Less>::value && std::is_unsigned<Key>::value; }

template <class Key>
__device__ __forceinline__ uint32_t lut_bin(Key e, Key base, uint32_t shift) {
  const Key q = (Key)(e - base) >> shift;
  const uint32_t i = q > (Key)(kLutN - 1) ? kLutN - 1 : (uint32_t)q;
  return e < base ? 0u : i;
}

// Builds lut[0..kLutN) from the nspl sorted splitters in shared memory; every
// thread of the kClsThreads-thread CTA calls it (begins and ends with a barrier).
// Returns whether the table pays for this bucket: false when more than 1/8 of
// the splitters share a bin with another one (keys clustered in value, e.g.
// AND-ed random words, whose splitters crowd the low bins) -- those buckets
// keep the descent.
template <class Key>
__device__ __forceinline__ bool lut_build(uint32_t* lut, const Key* spl, uint32_t nspl, Key& base, uint32_t& shift,
                                          uint32_t* s_warp) {
  constexpr uint32_t PER = kLutN / kClsThreads;
  static_assert(PER * kClsThreads == kLutN, "bins per thread");
  __syncthreads();                                             // spl[] is loaded
  base = nspl ? spl[0] : Key(0);
  const Key span = nspl ? (Key)(spl[nspl - 1] - base) : Key(0);
  uint32_t bl = 0;
  if constexpr (sizeof(Key) == 8) bl = span ? 64u - (uint32_t)__clzll((long long)span) : 0u;
  else bl = span ? 32u - (uint32_t)__clz((int)span) : 0u;
  shift = bl > kLutBits ? bl - kLutBits : 0u;
#pragma unroll
  for (uint32_t j = 0; j < PER; j++) lut[threadIdx.x + j * kClsThreads] = 0;
  if (threadIdx.x == 0) s_warp[63] = 0;
  __syncthreads();
  for (uint32_t j = threadIdx.x; j < nspl; j += kClsThreads) atomicAdd(lut + lut_bin(spl[j], base, shift), 1u);
  __syncthreads();
  uint32_t cnt[PER], tot = 0, crowd = 0;
#pragma unroll
  for (uint32_t j = 0; j < PER; j++) {
    cnt[j] = lut[threadIdx.x * PER + j];
    tot += cnt[j];
    crowd += cnt[j] >= 2 ? cnt[j] : 0u;
  }
  if (crowd) atomicAdd(s_warp + 63, crowd);
  uint32_t lo = block_exclusive_scan<kClsThreads>(tot, s_warp, nullptr);   // ends with a barrier
#pragma unroll
  for (uint32_t j = 0; j < PER; j++) {
    lut[threadIdx.x * PER + j] = lo | ((lo + cnt[j]) << 16);
    lo += cnt[j];
  }
  const bool good = s_warp[63] * 8 <= nspl;
  __syncthreads();
  return good;
}

// Bucket ids of U keys per lane by the lookup, then the id rule of the tile's
// mode (0: range buckets, 1: equality mode R4), as in descend_group.
template <int MODE, int U, class Key>
__device__ __forceinline__ void lut_group(const Key (&e)[U], uint32_t (&id)[U], uint32_t lut_s, const Key* spl,
                                          Key base, uint32_t shift, uint32_t ks) {
  uint32_t b[U], slow = 0;
#pragma unroll
  for (int u = 0; u < U; u++) {
    uint32_t ent;
    asm volatile("ld.shared.u32 %0, [%1];" : "=r"(ent) : "r"(lut_s + 4u * lut_bin(e[u], base, shift)));
    const uint32_t lo = ent & 0xffffu, hi = ent >> 16;
    b[u] = lo;
    if (hi > lo) {
      const bool gt = spl[lo] < e[u];
      b[u] = lo + (gt ? 1u : 0u);
      if (gt && hi > lo + 1) slow |= 1u << u;
    }
  }
  if (__any_sync(kFull, slow)) {
#pragma unroll
    for (int u = 0; u < U; u++) {
      if (slow & (1u << u)) {
        // first index of spl[b .. hi) not below e (the bin's remaining splitters)
        uint32_t l = b[u], h;
        {
          uint32_t ent;
          asm volatile("ld.shared.u32 %0, [%1];" : "=r"(ent) : "r"(lut_s + 4u * lut_bin(e[u], base, shift)));
          h = ent >> 16;
        }
        while (l < h) {
          const uint32_t m = (l + h) >> 1;
          if (spl[m] < e[u]) l = m + 1; else h = m;
        }
        b[u] = l;
      }
    }
  }
#pragma unroll
  for (int u = 0; u < U; u++) {
    if constexpr (MODE == 1) {
      const uint32_t bb = min(b[u], ks - 2);
      id[u] = 2 * b[u] + ((b[u] + 1 < ks && !(e[u] < spl[bb])) ? 1u : 0u);
    } else {
      id[u] = b[u];
    }
  }
}

// Where a tile's ids come from: the descent (tree_s, rep_b, logk) or the lookup (lut_s, base, shift).
template <class Key>
struct ClsSrc {
  uint32_t tree_s, rep_b, logk, lut_s, shift;
  Key base;
  bool use_lut;                      // this bucket classifies by the lookup (else the descent)
};

// Warp-contiguous groups: warp w of the CTA handles keys [g + 256 w, g + 256 w
// + 256) of each 2048-key group g, lane l the keys 32u + l (coalesced loads);
// the warp stages its 256 ids in shared memory and writes them as one 8-byte
// store per lane.  Full groups run without bounds tests; the next group's
// keys are loaded before this group descends.
#ifndef GSS_CLS_L2PF
#define GSS_CLS_L2PF 3   // groups ahead of the L2 prefetch in Phase 2 (0: none)
#endif
template <int MODE, bool STORE, bool LUT, class Key, class IdT, class Cmp>
__device__ __forceinline__ void classify_tile(const Key* __restrict__ src, IdT* __restrict__ tids, uint32_t beg,
                                              uint32_t len, const ClsSrc<Key>& cs, const Key* spl,
                                              uint32_t ks, uint32_t K, uint32_t wc_s, IdT* wid, Cmp less) {
  auto ids_of = [&](const Key (&e)[GSS_CLS_U], uint32_t (&id)[GSS_CLS_U]) {
    if constexpr (LUT) {
#ifndef GSS_CLS_LUT_ONLY
#define GSS_CLS_LUT_ONLY 0   // experiment: no per-bucket fallback to the descent in the lookup instantiation
#endif
      if (GSS_CLS_LUT_ONLY || cs.use_lut) lut_group<MODE>(e, id, cs.lut_s, spl, cs.base, cs.shift, ks);
      else descend_group<MODE>(e, id, cs.tree_s, cs.rep_b, spl, cs.logk, ks, K, less);
    } else {
      descend_group<MODE>(e, id, cs.tree_s, cs.rep_b, spl, cs.logk, ks, K, less);
    }
  };
  constexpr int U = GSS_CLS_U;                                 // keys per lane per group
  constexpr uint32_t G = U * kClsThreads;                      // keys per group
  const int lane = threadIdx.x & 31, w = threadIdx.x >> 5;
  const uint32_t off = (uint32_t)w * (32 * U) + lane;
  const Key* sp = src + beg + off;
  const uint32_t nfull = len / G;
  Key nx[U];
  if (nfull) {
#pragma unroll
    for (int u = 0; u < U; u++) nx[u] = sp[u * 32];
  }
  for (uint32_t g = 0; g < nfull; g++) {
    Key e[U];
#pragma unroll
    for (int u = 0; u < U; u++) e[u] = nx[u];
    if (g + 1 < nfull) {
#pragma unroll
      for (int u = 0; u < U; u++) nx[u] = sp[(g + 1) * G + u * 32];
    }
#if GSS_CLS_L2PF
    // the warp's keys of group g + GSS_CLS_L2PF pulled into L2 (one 128-byte line per lane): the register
    // prefetch above then waits for L2 rather than DRAM, without holding more registers
    if (g + GSS_CLS_L2PF < nfull && lane * 128u < U * 32u * (uint32_t)sizeof(Key))
      asm volatile("prefetch.global.L2 [%0];" ::"l"(reinterpret_cast<const char*>(sp - lane) +
                                                  ((size_t)(g + GSS_CLS_L2PF) * G) * sizeof(Key) + lane * 128u));
#endif
    uint32_t id[U];
    ids_of(e, id);
#pragma unroll
    for (int u = 0; u < U; u++) {
      red_shared_add(wc_s + 4 * id[u], 1u);
      if constexpr (STORE) wid[u * 32 + lane] = (IdT)id[u];
    }
    if constexpr (!STORE) continue;                            // GSS_FLAG_RECOMPUTE_IDS: Phase 4 re-descends
    __syncwarp();
    // lane l writes ids [l*U, l*U + U) of the warp's 256 (U * sizeof(IdT) bytes)
    IdT* gp = tids + g * G + (uint32_t)w * (32 * U) + lane * U;
    if constexpr (U * sizeof(IdT) == 4) {
      *reinterpret_cast<uint32_t*>(gp) = *reinterpret_cast<const uint32_t*>(wid + lane * U);
    } else if constexpr (U * sizeof(IdT) == 8) {
      *reinterpret_cast<uint2*>(gp) = *reinterpret_cast<const uint2*>(wid + lane * U);
    } else if constexpr (U * sizeof(IdT) == 32) {
      *reinterpret_cast<uint4*>(gp) = *reinterpret_cast<const uint4*>(wid + lane * U);
      *reinterpret_cast<uint4*>(gp + 16 / sizeof(IdT)) = *reinterpret_cast<const uint4*>(wid + lane * U + 16 / sizeof(IdT));
    } else {
      static_assert(U * sizeof(IdT) == 16, "ids per lane: 4, 8, 16 or 32 bytes");
      *reinterpret_cast<uint4*>(gp) = *reinterpret_cast<const uint4*>(wid + lane * U);
    }
    __syncwarp();
  }
  // tail group: bounds-tested
  const uint32_t tb = nfull * G;
  if (tb < len) {
    Key e[U];
#pragma unroll
    for (int u = 0; u < U; u++) {
      const uint32_t i = tb + off + u * 32;
      if (i < len) e[u] = src[beg + i];
      else e[u] = src[beg];
    }
    uint32_t id[U];
    ids_of(e, id);
#pragma unroll
    for (int u = 0; u < U; u++) {
      const uint32_t i = tb + off + u * 32;
      if (i < len) {
        red_shared_add(wc_s + 4 * id[u], 1u);
        if constexpr (STORE) tids[i] = (IdT)id[u];
      }
    }
  }
}

// Persistent: CTA b classifies the contiguous tile range [b*per, (b+1)*per),
// so consecutive tiles mostly share a bucket and its tree stays in shared
// memory.
// PART: the partition_by modes (2, 3) only; else the sort modes (0, 1): each
// instantiation holds only the descents it runs (their registers add up).
template <class Key, class Val, class IdT, class Cmp, bool PART = false, bool LUT = false>
#ifndef GSS_CLS_MINB
#define GSS_CLS_MINB 2
#endif
__global__ void __launch_bounds__(kClsThreads, GSS_CLS_MINB) k_classify(Ctx<Key, Val, IdT> c, uint32_t level, uint32_t kmax) {
  extern __shared__ __align__(16) unsigned char smem_raw[];
  constexpr uint32_t REP = rep_copies<Key>();
  Key* tree = reinterpret_cast<Key*>(smem_raw);
  Key* spl = tree + kmax;
  Key* rep = spl + kmax;                                       // kRepNodes x REP keys
  uint32_t* wcnt = reinterpret_cast<uint32_t*>(rep + kRepNodes * REP);
  constexpr int NW = kClsThreads / 32;
  IdT* wid0 = reinterpret_cast<IdT*>(wcnt + NW * kmax);
  IdT* wid = wid0 + (threadIdx.x >> 5) * (32 * GSS_CLS_U);                                      // per-warp id staging
  uint32_t* lut = reinterpret_cast<uint32_t*>(wid0 + NW * (32 * GSS_CLS_U));                    // kLutN entries
  uint32_t* s_scan = lut + kLutN;
  const Cmp less;
  const uint32_t slot = level & 1;
  const uint32_t nt = c.cnt->lvl[level].num_tiles;
  const Key* src = c.keys(c.src(level));
  const int w = threadIdx.x >> 5;
  const uint32_t per = (nt + gridDim.x - 1) / gridDim.x;
  const uint32_t t0 = blockIdx.x * per, t1 = min(nt, t0 + per);
  // Counter arrays (the paper splits contention over 8 arrays).  Default: one per warp (8 per CTA,
  // 32 threads each, as in the paper); gss_params.cls_arrays = 1/2/4 shares arrays between warps (SURVEY
  // NEXT-4 iii, an ablation)
  const uint32_t narr = c.cls_arrays;                          // 1, 2, 4 or 8 (= NW)
  const uint32_t wc_s = (uint32_t)__cvta_generic_to_shared(wcnt + (w / (NW / narr)) * kmax);
  const uint32_t tree_s = (uint32_t)__cvta_generic_to_shared(tree);
  // node j of levels 5..7 is read by this lane at rep_b + 128 j
  const uint32_t rep_b = (uint32_t)__cvta_generic_to_shared(rep) - (1u << kTopLevels) * 128u +
                         (threadIdx.x % REP) * (uint32_t)sizeof(Key);
  // the radix-indexed lookup replaces the descent for unsigned keys under operator< (not for partition_by)
  constexpr bool kLut = LUT && lut_ok<Key, Cmp>() && !PART;
  ClsSrc<Key> cs;
  cs.tree_s = tree_s; cs.rep_b = rep_b; cs.lut_s = (uint32_t)__cvta_generic_to_shared(lut);
  cs.shift = 0; cs.base = Key(0); cs.logk = 0; cs.use_lut = false;
  uint32_t cur = 0xffffffffu;
  for (uint32_t t = t0; t < t1; t++) {
    const uint32_t b = c.tile_bucket[slot][t];
    const Bucket B = c.bk[slot][b];
    __syncthreads();                                           // previous tile's counters are read
    if (b != cur) {
      const Key* g = c.spl[slot] + B.spl_base;
      for (uint32_t j = threadIdx.x + 1; j < B.ks; j += kClsThreads) tree[j] = g[j];
      for (uint32_t j = threadIdx.x; j + 1 < B.ks; j += kClsThreads) spl[j] = g[B.kb + j];
      if constexpr (kLut) cs.use_lut = lut_build(lut, spl, B.ks - 1, cs.base, cs.shift, s_scan);
      if (B.ks > (1u << kTopLevels)) {
        const uint32_t nrep = (min(B.ks, 1u << kRepEnd) - (1u << kTopLevels)) * REP;
        for (uint32_t q = threadIdx.x; q < nrep; q += kClsThreads) rep[q] = g[(1u << kTopLevels) + q / REP];
      }
      cur = b;
    }
    for (uint32_t j = threadIdx.x; j < narr * kmax; j += kClsThreads) wcnt[j] = 0;
    __syncthreads();
    const uint32_t tl = t - B.tile_start;
    const uint32_t beg = B.lo + tl * c.T;
    const uint32_t len = min(c.T, B.m - tl * c.T);
    cs.logk = ilog2(B.ks);
    IdT* tids = c.ids + B.id_base + tl * c.T;                  // 16-byte aligned per tile
    if constexpr (PART) {
      if (B.eq) classify_tile<3, true, false>(src, tids, beg, len, cs, spl, B.ks, B.K, wc_s, wid, less);
      else classify_tile<2, true, false>(src, tids, beg, len, cs, spl, B.ks, B.K, wc_s, wid, less);
    } else if (c.recompute) {
      if (B.eq) classify_tile<1, false, kLut>(src, tids, beg, len, cs, spl, B.ks, B.K, wc_s, wid, less);
      else classify_tile<0, false, kLut>(src, tids, beg, len, cs, spl, B.ks, B.K, wc_s, wid, less);
    } else if constexpr (kLut) {
      if (B.eq) classify_tile<1, true, true>(src, tids, beg, len, cs, spl, B.ks, B.K, wc_s, wid, less);
      else classify_tile<0, true, true>(src, tids, beg, len, cs, spl, B.ks, B.K, wc_s, wid, less);
    } else if (B.eq) {
      classify_tile<1, true, false>(src, tids, beg, len, cs, spl, B.ks, B.K, wc_s, wid, less);
    } else {
      classify_tile<0, true, false>(src, tids, beg, len, cs, spl, B.ks, B.K, wc_s, wid, less);
    }
    __syncthreads();
    uint32_t* hist = c.hist[slot] + B.hist_base;
    for (uint32_t id = threadIdx.x; id < B.K; id += kClsThreads) {
      uint32_t s = 0;
#pragma unroll
      for (int q = 0; q < NW; q++) s += (uint32_t)q < narr ? wcnt[q * kmax + id] : 0u;
      hist[id * B.ntiles + tl] = s;
    }
  }
}

// ---------------------------------------------------------------------------
// Phase 3: exclusive prefix sum over the level's whole histogram
// table (every bucket's K x p rows, bucket-major).  Each bucket later
// subtracts the scan value at its own first entry, so one unsegmented scan
// serves all buckets of the level.
// ---------------------------------------------------------------------------
template <class Key, class Val, class IdT>
__global__ void __launch_bounds__(kScanThreads) k_scan_reduce(Ctx<Key, Val, IdT> c, uint32_t level) {
  __shared__ unsigned long long s_red[kScanThreads / 32];
  const uint32_t L = c.cnt->lvl[level].hist_alloc;
  const uint32_t chunk = (L + gridDim.x - 1) / gridDim.x;
  const uint32_t lo = min(L, blockIdx.x * chunk), hi = min(L, lo + chunk);
  const uint32_t* h = c.hist[level & 1];
  uint64_t s = 0;
  for (uint32_t i = lo + threadIdx.x; i < hi; i += kScanThreads) s += h[i];
  s = block_sum_u64<kScanThreads>(s, s_red);
  if (threadIdx.x == 0) c.scan_part[blockIdx.x] = (uint32_t)s;
}

template <class Key, class Val, class IdT>
__global__ void __launch_bounds__(kScanThreads) k_scan_final(Ctx<Key, Val, IdT> c, uint32_t level) {
  __shared__ unsigned long long s_red[kScanThreads / 32];
  __shared__ uint32_t s_warp[kScanThreads / 32];
  __shared__ uint32_t s_total;
  constexpr int PER = 8;
  const uint32_t L = c.cnt->lvl[level].hist_alloc;
  const uint32_t chunk = (L + gridDim.x - 1) / gridDim.x;
  const uint32_t lo = min(L, blockIdx.x * chunk), hi = min(L, lo + chunk);
  uint64_t pre = 0;
  for (uint32_t i = threadIdx.x; i < blockIdx.x; i += kScanThreads) pre += c.scan_part[i];
  uint32_t carry = (uint32_t)block_sum_u64<kScanThreads>(pre, s_red);
  uint32_t* h = c.hist[level & 1];
  for (uint32_t base = lo; base < hi; base += kScanThreads * PER) {
    uint32_t x[PER], sum = 0;
    const uint32_t i0 = base + threadIdx.x * PER;
#pragma unroll
    for (int j = 0; j < PER; j++) {
      x[j] = (i0 + j < hi) ? h[i0 + j] : 0u;
      sum += x[j];
    }
    uint32_t ex = block_exclusive_scan<kScanThreads>(sum, s_warp, &s_total);
    uint32_t run = carry + ex;
#pragma unroll
    for (int j = 0; j < PER; j++) {
      if (i0 + j < hi) h[i0 + j] = run;
      run += x[j];
    }
    carry += s_total;
    __syncthreads();
  }
}

// ---------------------------------------------------------------------------
// Phase 4: every key goes to its bucket's global offset plus its
// rank among the tile's keys of that bucket.  Ranks are stable (R7): a warp
// ranks 32 consecutive keys with __match_any_sync and per-warp counters.
// The tile is then reordered by bucket in shared memory (the presorting the
// paper tried, re-adopted for B200) so each bucket's run is
// written with coalesced stores.
// ---------------------------------------------------------------------------
template <class Key, class Val, class IdT>
struct ScatterSmem {
  // splitter tree, sorted splitters and bank-replicated middle levels, as in
  // k_classify (only with GSS_FLAG_RECOMPUTE_IDS)
  __host__ __device__ static size_t tree_bytes(uint32_t kmax) {
    return (size_t)kmax * sizeof(Key) * 2 + (size_t)kRepNodes * 128;
  }
  static size_t bytes(uint32_t kmax, bool recompute = false) {
    GSS_SCATTER_CHUNK_CONSTANTS
    size_t b = recompute ? tree_bytes(kmax) : 0;
    b += (size_t)kmax * 4 * 3;                                  // gbase, ctot, delta
    b += (size_t)(kScatterThreads / 32) * kmax * 4;             // per-warp counters
    b += 64;                                                    // scan scratch
    b = (b + 15) & ~size_t(15);
    b += (size_t)kChunk * sizeof(Key);
    if (kHasVal<Val>) b += (size_t)kChunk * sizeof(Val);
    b += (size_t)kChunk * sizeof(IdT);                          // staged ids
    return b;
  }
};

// Predicated shared-memory atomic add (no branch, 32-bit shared address).
__device__ __forceinline__ uint32_t atom_add_shared_if(uint32_t pred, uint32_t saddr, uint32_t v) {
  uint32_t old = 0;
  asm volatile(
      "{\n\t.reg .pred p;\n\tsetp.ne.u32 p, %1, 0;\n\t@p atom.shared.add.u32 %0, [%2], %3;\n\t}"
      : "+r"(old)
      : "r"(pred), "r"(saddr), "r"(v)
      : "memory");
  return old;
}

// Ranks of a thread's ITER keys within (warp, id) from the warp's counters: iid[it] becomes
// (rank << 16) | id (or stays the empty marker).  One shared atomic per key -- except when all the
// warp's keys of the chunk hold one id (sorted input, long runs of equal keys), where 32 atomics per
// step on one address would serialise: then lane 0 adds 32*ITER and item (it, lane) takes rank
// it*32 + lane (deterministic either way).  2^27 u32 sorted: 3.80 -> 3.11 ms per sort; dd 1.89 -> 1.54.
#ifndef GSS_WARP_UNIFORM_RANK
#define GSS_WARP_UNIFORM_RANK 1
#endif
template <int ITER>
__device__ __forceinline__ void rank_in_warp(uint32_t (&iid)[ITER], uint32_t wc_s, int lane) {
  if constexpr (GSS_WARP_UNIFORM_RANK) {
    const uint32_t first = __shfl_sync(kFull, iid[0], 0);
    bool same = first != 0xffffffffu;
#pragma unroll
    for (int it = 0; it < ITER; it++) same = same && iid[it] == first;
    if (__all_sync(kFull, same)) {
      uint32_t base = 0;
      if (lane == 0) base = atom_add_shared_if(1u, wc_s + 4 * first, 32u * ITER);
      base = __shfl_sync(kFull, base, 0);
#pragma unroll
      for (int it = 0; it < ITER; it++) iid[it] = ((base + 32u * it + (uint32_t)lane) << 16) | first;
      return;
    }
  }
#pragma unroll
  for (int it = 0; it < ITER; it++) {
    const uint32_t r = atom_add_shared_if(iid[it] != 0xffffffffu ? 1u : 0u, wc_s + 4 * (iid[it] & 0xffffu), 1u);
    iid[it] = iid[it] == 0xffffffffu ? iid[it] : (r << 16) | iid[it];
  }
}

// Phase 4 kernel.  Persistent: the CTA walks its tiles (blockIdx.x, +gridDim.x,
// ...) chunk by chunk; the keys, values and ids of the next chunk are loaded
// into registers before the current chunk's runs are written out, so the
// global-load latency overlaps the write phase and the barriers.
// RECOMP (GSS_FLAG_RECOMPUTE_IDS, the paper's choice): no stored
// ids; every key re-descends its bucket's splitter tree (same layout and
// descent as k_classify) when its chunk is ranked.
template <class Key, class Val, class IdT, class Cmp, bool STABLE, bool RECOMP = false>
__global__ void __launch_bounds__(kScatterThreads, GSS_SCATTER_MINB) k_scatter(Ctx<Key, Val, IdT> c, uint32_t level, uint32_t kmax) {
  extern __shared__ __align__(16) unsigned char smem_raw[];
  // the stable ranking (partitions, GSS_FLAG_STABLE) keeps 8 keys per thread: at 16 it spills (224 B stack);
  // the shared allocation (ScatterSmem) is sized for the larger chunk
  constexpr int kScatterIter = STABLE ? GSS_SCATTER_ITER : scatter_iter<Key, Val>();
  constexpr int kChunk = kScatterThreads * kScatterIter;
  constexpr int NW = kScatterThreads / 32;
  constexpr uint32_t REP = rep_copies<Key>();
  Key* tree = reinterpret_cast<Key*>(smem_raw);
  Key* spl = tree + kmax;
  Key* rep = spl + kmax;
  const size_t tb = RECOMP ? ScatterSmem<Key, Val, IdT>::tree_bytes(kmax) : 0;
  const uint32_t tree_s = (uint32_t)__cvta_generic_to_shared(tree);
  const uint32_t rep_b = (uint32_t)__cvta_generic_to_shared(rep) - (1u << kTopLevels) * 128u +
                         (threadIdx.x % REP) * (uint32_t)sizeof(Key);
  uint32_t* gbase = reinterpret_cast<uint32_t*>(smem_raw + tb);
  uint32_t* ctot = gbase + kmax;
  uint32_t* delta = ctot + kmax;
  uint32_t* wcnt = delta + kmax;
  uint32_t* s_warp = wcnt + NW * kmax;
  size_t off = tb + (((size_t)(kmax * 3 + NW * kmax) * 4 + 64 + 15) & ~size_t(15));
  Key* skeys = reinterpret_cast<Key*>(smem_raw + off);
  off += (size_t)kChunk * sizeof(Key);
  Val* svals = reinterpret_cast<Val*>(smem_raw + off);
  if constexpr (kHasVal<Val>) off += (size_t)kChunk * sizeof(Val);
  IdT* sids = reinterpret_cast<IdT*>(smem_raw + off);
  const Cmp less;

  const uint32_t slot = level & 1;
  const uint32_t nt = c.cnt->lvl[level].num_tiles;
  const uint32_t sb = c.src(level), db = c.dst(level);
  const Key* ksrc = c.keys(sb);
  Key* kdst = c.wkeys(db);
  const Val* vsrc = nullptr;
  Val* vdst = nullptr;
  if constexpr (kHasVal<Val>) { vsrc = c.vals(sb); vdst = c.wvals(db); }
  const IdT* idsrc = c.ids;
  const int lane = threadIdx.x & 31, w = threadIdx.x >> 5;
  const uint32_t ltmask = lanemask_lt();
  uint32_t* wc = wcnt + w * kmax;
  const uint32_t wc_s = (uint32_t)__cvta_generic_to_shared(wc);
  const uint32_t q0 = w * (32 * kScatterIter) + lane;

  uint32_t t = blockIdx.x;
  if (t >= nt) return;
  // per-tile state kept in registers: start, length, id base, K (the
  // histogram row is re-read from the bucket record when a tile starts)
  uint32_t beg, len, K, idb;
  uint32_t tmode = 0, tks = 0, cur_b = 0xffffffffu, next_b = 0;   // RECOMP: id rule and tree of the tile's bucket
  auto tile_info = [&](uint32_t tt) {
    const uint32_t bi = c.tile_bucket[slot][tt];
    const Bucket B = c.bk[slot][bi];
    const uint32_t tl = tt - B.tile_start;
    beg = B.lo + tl * c.T;
    len = min(c.T, B.m - tl * c.T);
    K = B.K;
    idb = B.id_base + tl * c.T;
    next_b = bi;
  };
  // RECOMP: the tile's tree into shared memory (a barrier must precede and follow)
  auto load_tree = [&](uint32_t bi) {
    const Bucket B = c.bk[slot][bi];
    const Key* g = c.spl[slot] + B.spl_base;
    for (uint32_t j = threadIdx.x + 1; j < B.ks; j += kScatterThreads) tree[j] = g[j];
    for (uint32_t j = threadIdx.x; j + 1 < B.ks; j += kScatterThreads) spl[j] = g[B.kb + j];
    if (B.ks > (1u << kTopLevels)) {
      const uint32_t nrep = (min(B.ks, 1u << kRepEnd) - (1u << kTopLevels)) * REP;
      for (uint32_t q = threadIdx.x; q < nrep; q += kScatterThreads) rep[q] = g[(1u << kTopLevels) + q / REP];
    }
    tmode = B.eq ? 1u : (B.clamp ? 2u : 0u);
    tks = B.ks;
    cur_b = bi;
  };
  auto load_gbase = [&](uint32_t tt) {
    const Bucket B = c.bk[slot][c.tile_bucket[slot][tt]];
    const uint32_t tl = tt - B.tile_start;
    const uint32_t* hist = c.hist[slot] + B.hist_base;
    const uint32_t hb = hist[0];
    for (uint32_t id = threadIdx.x; id < B.K; id += kScatterThreads)
      gbase[id] = hist[id * B.ntiles + tl] - hb + B.lo;
  };
  tile_info(t);
  load_gbase(t);
  if constexpr (RECOMP) {
    load_tree(next_b);
    __syncthreads();
  }
  // prefetch registers: the chunk to process next
  Key pk[kScatterIter];
  Val pv[kScatterIter];
  uint32_t pid[kScatterIter];
  auto load_chunk = [&](uint32_t cbeg, uint32_t cid, uint32_t clen) {
#pragma unroll
    for (int it = 0; it < kScatterIter; it++) {
      const uint32_t q = q0 + it * 32;
      pid[it] = 0xffffffffu;
      if (q < clen) {
        pk[it] = ksrc[cbeg + q];
        if constexpr (RECOMP) pid[it] = 0u;                     // id computed when the chunk is ranked
        else pid[it] = idsrc[cid + q];
        if constexpr (kHasVal<Val>) pv[it] = vsrc[cbeg + q];
      }
    }
  };
  uint32_t c0 = 0;
  load_chunk(beg, idb, min((uint32_t)kChunk, len));
#ifdef GSS_SCATTER_PHASES
  unsigned long long ph[6] = {0, 0, 0, 0, 0, 0}, tp = clock64();
  uint32_t nchunks = 0;
#define GSS_PH(i) do { const unsigned long long tn = clock64(); ph[i] += tn - tp; tp = tn; } while (0)
#else
#define GSS_PH(i) do {} while (0)
#endif
  for (;;) {
    const uint32_t clen = min((uint32_t)kChunk, len - c0);
    Key kk[kScatterIter];
    Val vv[kScatterIter];
    uint32_t iid[kScatterIter];                                    // id; after ranking (rank << 16) | id
#pragma unroll
    for (int it = 0; it < kScatterIter; it++) {
      kk[it] = pk[it];
      iid[it] = pid[it];
      if constexpr (kHasVal<Val>) vv[it] = pv[it];
    }
    if constexpr (RECOMP) {
      // re-descend (Algorithm 2) with the tile mode's id rule
      uint32_t id[kScatterIter];
      const uint32_t logk = ilog2(tks);
      if (tmode == 1) descend_group<1>(kk, id, tree_s, rep_b, spl, logk, tks, K, less);
      else if (tmode == 2) descend_group<2>(kk, id, tree_s, rep_b, spl, logk, tks, K, less);
      else descend_group<0>(kk, id, tree_s, rep_b, spl, logk, tks, K, less);
#pragma unroll
      for (int it = 0; it < kScatterIter; it++) iid[it] = iid[it] == 0xffffffffu ? iid[it] : id[it];
    }
    const uint32_t cur_K = K, cur_clen = clen;
    bool new_tile = false;
    bool done = false;
#if GSS_SCATTER_EARLY
    // advance and prefetch the next chunk at once: its loads overlap this whole chunk
    c0 += kChunk;
    if (c0 >= len) {
      t += gridDim.x;
      c0 = 0;
      if (t >= nt) done = true;
      else {
        tile_info(t);
        new_tile = true;
      }
    }
    if (!done) load_chunk(beg + c0, idb + c0, min((uint32_t)kChunk, len - c0));
#endif
    for (uint32_t id = lane; id < cur_K; id += 32) wc[id] = 0;
    __syncwarp();
    if constexpr (STABLE) {
      // Stable ranks (R7): peer masks of lanes holding the same bucket id, one
      // ballot per id bit; the lowest lane of each group adds the group size to
      // the warp's counter, so ranks follow lane order.
      constexpr int NBITS = sizeof(IdT) == 1 ? 8 : 10;
      uint32_t peers[kScatterIter], old[kScatterIter];
#pragma unroll
      for (int it = 0; it < kScatterIter; it++) {
        const uint32_t id = iid[it];
        uint32_t pm = __ballot_sync(kFull, id != 0xffffffffu);
#pragma unroll
        for (int bit = 0; bit < NBITS; bit++) {
          const bool on = (id >> bit) & 1u;
          const uint32_t bal = __ballot_sync(kFull, on);
          pm &= on ? bal : ~bal;
        }
        peers[it] = pm;
      }
#pragma unroll
      for (int it = 0; it < kScatterIter; it++) {
        const uint32_t lead = (iid[it] != 0xffffffffu && (peers[it] & ltmask) == 0) ? 1u : 0u;
        old[it] = atom_add_shared_if(lead, wc_s + 4 * (iid[it] & 0xffffu), (uint32_t)__popc(peers[it]));
        __syncwarp();
      }
#pragma unroll
      for (int it = 0; it < kScatterIter; it++) {
        const uint32_t r = __popc(peers[it] & ltmask) + __shfl_sync(kFull, old[it], __ffs(peers[it]) - 1);
        iid[it] = iid[it] == 0xffffffffu ? iid[it] : (r << 16) | iid[it];
      }
    } else {
      // One shared-memory atomic per key on the warp's own counters: ranks are
      // unique within (warp, id) in any order, so the level is a partition
      // whose within-bucket order is the hardware's atomic order.
      rank_in_warp<kScatterIter>(iid, wc_s, lane);
    }
    __syncthreads();
    GSS_PH(0);
    // chunk totals per id, exclusive scan over ids, then every warp's start
    // within each id folded into its counter (one lookup per key below)
#if GSS_SCATTER_PAIRFOLD
    if (2 * cur_K <= (uint32_t)kScatterThreads) {
      // two threads per id, each folding half of the warps' counters (its
      // 8 loads in flight at once); the pair's halves meet by a shuffle
      constexpr int HW = NW / 2;
      const uint32_t id = threadIdx.x >> 1, h = threadIdx.x & 1;
      uint32_t x[HW], sh = 0;
      if (id < cur_K) {
#pragma unroll
        for (int q = 0; q < HW; q++) { x[q] = wcnt[(h * HW + q) * kmax + id]; sh += x[q]; }
      }
      const uint32_t so = __shfl_xor_sync(kFull, sh, 1);
      const uint32_t tot = sh + so;
      const uint32_t ex0 = block_exclusive_scan<kScatterThreads>(h == 0 && id < cur_K ? tot : 0u, s_warp, nullptr);
      const uint32_t ex = h == 0 ? ex0 : ex0 - tot;             // the id's run start (same for both halves)
      if (id < cur_K) {
        uint32_t run = ex + (h ? so : 0u);
#pragma unroll
        for (int q = 0; q < HW; q++) { wcnt[(h * HW + q) * kmax + id] = run; run += x[q]; }
        if (h == 0) {
          delta[id] = gbase[id] - ex;                           // global index = delta + staged position
          gbase[id] += tot;
        }
      }
    } else
#endif
    {
      // id owners spread over every warp (thread i * threads/kmax owns id i), in thread order for the scan
      const bool spread = GSS_SCATTER_SPREAD && kmax <= (uint32_t)kScatterThreads;
      const uint32_t sstride = spread ? (uint32_t)kScatterThreads / kmax : 1u;
      const uint32_t per = spread ? ((threadIdx.x % sstride) == 0 ? 1u : 0u)
                                  : (cur_K + kScatterThreads - 1) / kScatterThreads;
      const uint32_t i0 = spread ? threadIdx.x / sstride : threadIdx.x * per;
      uint32_t tsum = 0;
      for (uint32_t j = 0; j < per; j++) {
        const uint32_t id = i0 + j;
        if (id < cur_K) {
          uint32_t tt = 0;
#pragma unroll
          for (int q = 0; q < NW; q++) tt += wcnt[q * kmax + id];
          ctot[id] = tt;
          tsum += tt;
        }
      }
      uint32_t ex = block_exclusive_scan<kScatterThreads>(tsum, s_warp, nullptr);
      for (uint32_t j = 0; j < per; j++) {
        const uint32_t id = i0 + j;
        if (id < cur_K) {
          uint32_t run = ex;
#pragma unroll
          for (int q = 0; q < NW; q++) {
            const uint32_t x = wcnt[q * kmax + id];
            wcnt[q * kmax + id] = run;
            run += x;
          }
          delta[id] = gbase[id] - ex;                         // global index = delta + staged position
          gbase[id] += ctot[id];
          ex = run;
        }
      }
    }
    __syncthreads();
    GSS_PH(1);
#pragma unroll
    for (int it = 0; it < kScatterIter; it++) {
      if (iid[it] != 0xffffffffu) {
        const uint32_t id = iid[it] & 0xffffu;
        const uint32_t pos = wc[id] + (iid[it] >> 16);
        skeys[pos] = kk[it];
        if constexpr (kHasVal<Val>) svals[pos] = vv[it];
        sids[pos] = (IdT)id;
      }
    }
    __syncthreads();
    GSS_PH(2);
#if !GSS_SCATTER_EARLY
    // advance and prefetch the next chunk (possibly of the next tile)
    c0 += kChunk;
    if (c0 >= len) {
      t += gridDim.x;
      c0 = 0;
      if (t >= nt) done = true;
      else {
        tile_info(t);
        new_tile = true;
      }
    }
    if (!done) load_chunk(beg + c0, idb + c0, min((uint32_t)kChunk, len - c0));
#endif
    // write this chunk's bucket runs
#pragma unroll 4
    for (uint32_t q = threadIdx.x; q < cur_clen; q += kScatterThreads) {
      const uint32_t d = delta[sids[q]] + q;
      kdst[d] = skeys[q];
      if constexpr (kHasVal<Val>) vdst[d] = svals[q];
    }
    __syncthreads();
    GSS_PH(3);
#ifdef GSS_SCATTER_PHASES
    nchunks++;
    if (done && threadIdx.x == 0 && (blockIdx.x == 0 || blockIdx.x == 100))
      printf("scatter phases block %d chunks %u: rank %llu scan %llu reorder %llu write %llu (cycles per chunk)\n",
             blockIdx.x, nchunks, ph[0] / nchunks, ph[1] / nchunks, ph[2] / nchunks, ph[3] / nchunks);
#endif
    if (done) break;
    if (new_tile) {
      load_gbase(t);
      if constexpr (RECOMP) {
        if (next_b != cur_b) {
          __syncthreads();                                     // every key of the old tile is ranked
          load_tree(next_b);
          __syncthreads();                                     // the new tree is complete before the next descent
        }
      }
    }
  }
}

// ---------------------------------------------------------------------------
// Phase 4 with bulk-copy stores (the default sort scatter on B200).  The
// chunk is ranked and reordered by bucket id in shared memory as in
// k_scatter, but the bucket runs leave shared memory through the TMA bulk-copy
// engine (cp.async.bulk.global.shared::cta, SASS UBLKCP) instead of per-key
// LDS + STG: one thread per bucket id issues its run's 16-byte-aligned middle
// as one asynchronous copy and stores at most A-1 head and A-1 tail elements
// itself (A = 16 / key bytes).  Each run's staging slot is placed so that it
// has the same alignment modulo 16 bytes as its global destination, which
// costs at most A-1 slots per id.  The copies of chunk c drain while chunk
// c+1 is ranked (NBUF = 2 staging buffers; 1 where shared memory is short).
// Per chunk: 5 barriers (the paper's presorting, with the write
// phase handed to the copy engine).
// ---------------------------------------------------------------------------
__device__ __forceinline__ void bulk_s2g(void* gdst, uint32_t ssrc, uint32_t bytes) {
  asm volatile("cp.async.bulk.global.shared::cta.bulk_group [%0], [%1], %2;" ::"l"(gdst), "r"(ssrc), "r"(bytes)
               : "memory");
}
__device__ __forceinline__ void bulk_commit() { asm volatile("cp.async.bulk.commit_group;" ::: "memory"); }
template <int N>
__device__ __forceinline__ void bulk_wait_read() { asm volatile("cp.async.bulk.wait_group.read %0;" ::"n"(N) : "memory"); }
__device__ __forceinline__ void bulk_wait_all() { asm volatile("cp.async.bulk.wait_group 0;" ::: "memory"); }
__device__ __forceinline__ void fence_proxy_async_smem() { asm volatile("fence.proxy.async.shared::cta;" ::: "memory"); }

// Exclusive scan of one value per thread with two barriers (no trailing
// barrier: the caller's next barrier protects s_part).
template <int NT>
__device__ __forceinline__ uint32_t block_exclusive_scan2(uint32_t x, uint32_t* s_warp) {
  const int lane = threadIdx.x & 31, w = threadIdx.x >> 5;
  uint32_t inc = x;
#pragma unroll
  for (int o = 1; o < 32; o <<= 1) {
    const uint32_t y = __shfl_up_sync(kFull, inc, o);
    if (lane >= o) inc += y;
  }
  if (lane == 31) s_warp[w] = inc;
  __syncthreads();
  if (w == 0) {
    const uint32_t v = lane < NT / 32 ? s_warp[lane] : 0;
    uint32_t vi = v;
#pragma unroll
    for (int o = 1; o < 32; o <<= 1) {
      const uint32_t y = __shfl_up_sync(kFull, vi, o);
      if (lane >= o) vi += y;
    }
    if (lane < NT / 32) s_warp[32 + lane] = vi - v;
  }
  __syncthreads();
  return s_warp[32 + w] + inc - x;
}

// The segment holding partition index i (segments are sorted and cover the partition).
__device__ __forceinline__ const RemoteSeg* find_seg(const RemoteSeg* seg, uint32_t nseg, uint32_t i) {
  uint32_t q = 0;
  while (q + 1 < nseg && i >= seg[q].hi) q++;
  return seg + q;
}

template <class Key, class Val, class IdT>
struct ScatterBulkSmem {
  static constexpr uint32_t A = 16 / sizeof(Key);            // keys per 16 bytes
  __host__ __device__ static uint32_t stage_len(uint32_t kmax) {
    constexpr uint32_t C = (uint32_t)kScatterThreads * (uint32_t)scatter_iter<Key, Val>();
    return C + kmax * (A - 1) + A;
  }
  __host__ __device__ static size_t head_bytes(uint32_t kmax) {
    return (((size_t)kmax * 3 + (size_t)(kScatterThreads / 32) * kmax) * 4 + 64 * 4 + 15) & ~size_t(15);
  }
  __host__ __device__ static size_t key_bytes(uint32_t kmax) { return ((size_t)stage_len(kmax) * sizeof(Key) + 15) & ~size_t(15); }
  __host__ __device__ static size_t val_bytes(uint32_t kmax) {
    return kHasVal<Val> ? (((size_t)stage_len(kmax) * sizeof(Val) + 15) & ~size_t(15)) : 0;
  }
  static size_t bytes(uint32_t kmax, int nbuf) { return head_bytes(kmax) + (size_t)nbuf * (key_bytes(kmax) + val_bytes(kmax)); }
};

template <class Key, class Val, class IdT, int NBUF, bool CTA_CNT = false>
__global__ void __launch_bounds__(kScatterThreads, GSS_SCATTER_MINB)
    k_scatter_bulk(Ctx<Key, Val, IdT> c, uint32_t level, uint32_t kmax) {
  extern __shared__ __align__(16) unsigned char smem_raw[];
  constexpr int kScatterIter = scatter_iter<Key, Val>();
  constexpr int kChunk = kScatterThreads * kScatterIter;
  constexpr int NW = kScatterThreads / 32;
  using SM = ScatterBulkSmem<Key, Val, IdT>;
  constexpr uint32_t A = SM::A;
  // CTA_CNT (ablation, keys only): one counter set per CTA -- no per-warp fold (2^28 u64: 2.75 vs 2.92 ms for
  // the two levels), but ranks follow the hardware's atomic order across warps, so the order of keys inside a
  // bucket, hence the next level's sample and splitters, vary from run to run (final keys do not).  Default:
  // per-warp counters folded in a fixed order, deterministic intermediates that match the oracle's level
  // records.
  uint32_t* gbase = reinterpret_cast<uint32_t*>(smem_raw);       // next global index of each id (this tile)
  uint32_t* rstart = gbase + kmax;                                // staging slot of each id's run (this chunk)
  uint32_t* rlen = rstart + kmax;                                 // run length of each id (this chunk)
  uint32_t* wcnt = rlen + kmax;                                   // per-warp counters, then per-warp offsets
  uint32_t* s_warp = wcnt + NW * kmax;                            // 64 words of scan scratch
  Key* stage_k = reinterpret_cast<Key*>(smem_raw + SM::head_bytes(kmax));
  Val* stage_v = reinterpret_cast<Val*>(smem_raw + SM::head_bytes(kmax) + (size_t)NBUF * SM::key_bytes(kmax));
  const uint32_t SL = SM::stage_len(kmax);

  const uint32_t slot = level & 1;
  const uint32_t nt = c.cnt->lvl[level].num_tiles;
  const uint32_t sb = c.src(level), db = c.dst(level);
  const Key* ksrc = c.keys(sb);
  Key* kdst = c.wkeys(db);
  const Val* vsrc = nullptr;
  Val* vdst = nullptr;
  if constexpr (kHasVal<Val>) { vsrc = c.vals(sb); vdst = c.wvals(db); }
  const IdT* idsrc = c.ids;
  const int lane = threadIdx.x & 31, w = threadIdx.x >> 5;
  uint32_t* wc = CTA_CNT ? wcnt : wcnt + w * kmax;
  const uint32_t wc_s = (uint32_t)__cvta_generic_to_shared(wc);
  const uint32_t q0 = w * (32 * kScatterIter) + lane;

  uint32_t t = blockIdx.x;
  if (t >= nt) return;
  uint32_t beg, len, K, idb;
  auto tile_info = [&](uint32_t tt) {
    const Bucket B = c.bk[slot][c.tile_bucket[slot][tt]];
    const uint32_t tl = tt - B.tile_start;
    beg = B.lo + tl * c.T;
    len = min(c.T, B.m - tl * c.T);
    K = B.K;
    idb = B.id_base + tl * c.T;
  };
  // ids owned by this thread in the scan and the write phase, fixed for the
  // kernel (gbase, rstart, rlen of an id are only touched by its owner).
  // With kmax <= threads, id i belongs to thread i * (threads / kmax): the
  // owners (and their serialised bulk copies) are spread over every warp,
  // in thread order, as the scan requires.
  const bool spread = GSS_SCATTER_SPREAD && kmax <= (uint32_t)kScatterThreads;
  const uint32_t sstride = spread ? (uint32_t)kScatterThreads / kmax : 1u;
  const uint32_t per = spread ? ((threadIdx.x % sstride) == 0 ? 1u : 0u)
                              : (kmax + kScatterThreads - 1) / kScatterThreads;
  const uint32_t i0 = spread ? threadIdx.x / sstride : threadIdx.x * per;
  auto load_gbase = [&](uint32_t tt) {                            // owner threads only: no barrier needed
    const Bucket B = c.bk[slot][c.tile_bucket[slot][tt]];
    const uint32_t tl = tt - B.tile_start;
    const uint32_t* hist = c.hist[slot] + B.hist_base;
    const uint32_t hb = hist[0];
    for (uint32_t j = 0; j < per; j++) {
      const uint32_t id = i0 + j;
      if (id < B.K) gbase[id] = hist[id * B.ntiles + tl] - hb + B.lo;
    }
  };
  tile_info(t);
  load_gbase(t);
  Key pk[kScatterIter];
  Val pv[kScatterIter];
  uint32_t pid[kScatterIter];
  auto load_chunk = [&](uint32_t cbeg, uint32_t cid, uint32_t clen) {
#pragma unroll
    for (int it = 0; it < kScatterIter; it++) {
      const uint32_t q = q0 + it * 32;
      pid[it] = 0xffffffffu;
      if (q < clen) {
        pk[it] = ksrc[cbeg + q];
        pid[it] = idsrc[cid + q];
        if constexpr (kHasVal<Val>) pv[it] = vsrc[cbeg + q];
      }
    }
  };
  uint32_t c0 = 0, buf = 0;
  load_chunk(beg, idb, min((uint32_t)kChunk, len));
  if constexpr (CTA_CNT) {
    for (uint32_t id = threadIdx.x; id < kmax; id += kScatterThreads) wcnt[id] = 0;
    __syncthreads();
  }
  for (;;) {
    Key kk[kScatterIter];
    Val vv[kScatterIter];
    uint32_t iid[kScatterIter];
#pragma unroll
    for (int it = 0; it < kScatterIter; it++) {
      kk[it] = pk[it];
      iid[it] = pid[it];
      if constexpr (kHasVal<Val>) vv[it] = pv[it];
    }
    const uint32_t cur_K = K;
    if constexpr (!CTA_CNT) {
      for (uint32_t id = lane; id < cur_K; id += 32) wc[id] = 0;
      __syncwarp();
    }
    // ranks within (warp, id): one shared atomic per key on the warp's own counters
    rank_in_warp<kScatterIter>(iid, wc_s, lane);
    // the staging buffer written below was last read by the copies issued NBUF chunks ago
    bulk_wait_read<NBUF - 1>();
    __syncthreads();                                                // B1: counters complete
    // chunk totals per id, aligned run slots, every warp's start inside each run
    uint32_t tsum = 0;
    for (uint32_t j = 0; j < per; j++) {
      const uint32_t id = i0 + j;
      if (id < cur_K) {
        uint32_t tt = 0;
        if constexpr (CTA_CNT) {
          tt = wcnt[id];
          wcnt[id] = 0;                                           // reset for the next chunk (its atomics follow B3)
        } else {
#pragma unroll
          for (int q = 0; q < NW; q++) tt += wcnt[q * kmax + id];
        }
        rlen[id] = tt;
        tsum += tt + (A - 1);
      }
    }
    uint32_t ex = block_exclusive_scan2<kScatterThreads>(tsum, s_warp);
    for (uint32_t j = 0; j < per; j++) {
      const uint32_t id = i0 + j;
      if (id < cur_K) {
        const uint32_t L = rlen[id];
        uint32_t dal = gbase[id];                                   // destination element index (mod A)
        if (c.nremote) {
          const RemoteSeg* sg = find_seg(c.remote, c.nremote, dal);
          dal = (uint32_t)(reinterpret_cast<uintptr_t>(reinterpret_cast<Key*>(sg->kdst) + dal) / sizeof(Key));
        }
        const uint32_t st = ex + ((dal - ex) & (A - 1));            // staging slot == destination (mod A)
        rstart[id] = st;
        if constexpr (!CTA_CNT) {
          uint32_t run = st;
#pragma unroll
          for (int q = 0; q < NW; q++) {
            const uint32_t x = wcnt[q * kmax + id];
            wcnt[q * kmax + id] = run;
            run += x;
          }
        }
        ex += L + (A - 1);
      }
    }
    __syncthreads();                                                // B2: run slots known
    Key* sk = stage_k + (size_t)buf * (SM::key_bytes(kmax) / sizeof(Key));
    Val* sv = nullptr;
    if constexpr (kHasVal<Val>) sv = stage_v + (size_t)buf * (SM::val_bytes(kmax) / sizeof(Val));
#pragma unroll
    for (int it = 0; it < kScatterIter; it++) {
      if (iid[it] != 0xffffffffu) {
        const uint32_t pos = (CTA_CNT ? rstart[iid[it] & 0xffffu] : wc[iid[it] & 0xffffu]) + (iid[it] >> 16);
        sk[pos] = kk[it];
        if constexpr (kHasVal<Val>) sv[pos] = vv[it];
      }
    }
    fence_proxy_async_smem();                                       // generic-proxy stores -> bulk copies
    __syncthreads();                                                // B3: the chunk is staged
    // advance and prefetch the next chunk (possibly of the next tile)
    bool done = false, new_tile = false;
    c0 += kChunk;
    if (c0 >= len) {
      t += gridDim.x;
      c0 = 0;
      if (t >= nt) done = true;
      else { tile_info(t); new_tile = true; }
    }
    if (!done) load_chunk(beg + c0, idb + c0, min((uint32_t)kChunk, len - c0));
    // write this chunk's runs: head / tail elements by the owner, the aligned middle by the copy engine
    const uint32_t sk_s = (uint32_t)__cvta_generic_to_shared(sk);
    uint32_t sv_s = 0;
    if constexpr (kHasVal<Val>) sv_s = (uint32_t)__cvta_generic_to_shared(sv);
    // one piece of one array: dst[0..cnt) <- staging[so..so+cnt): head / tail
    // elements by this thread, the 16-byte-aligned middle by one bulk copy
    auto put1 = [&](auto* d, const auto* stg, uint32_t stg_s, uint32_t so, uint32_t cnt) {
      constexpr uint32_t W = (uint32_t)sizeof(*d), AW = 16u / W;
      const uint32_t mis = (uint32_t)(reinterpret_cast<uintptr_t>(d) & 15u) / W;
      uint32_t head = min(cnt, (AW - mis) & (AW - 1));
      // the staging slot matches the destination modulo 16 bytes (else: element by element)
      if (((stg_s + (so + head) * W) & 15u) != 0) head = cnt;
      const uint32_t mid_end = head + ((cnt - head) & ~(AW - 1));
      for (uint32_t h = 0; h < head; h++) d[h] = stg[so + h];
      if (mid_end > head) bulk_s2g(d + head, stg_s + (so + head) * W, (mid_end - head) * W);
      for (uint32_t h = mid_end; h < cnt; h++) d[h] = stg[so + h];
    };
    auto put = [&](Key* dk, Val* dv, uint32_t so, uint32_t cnt) {
      put1(dk, sk, sk_s, so, cnt);
      if constexpr (kHasVal<Val>) put1(dv, sv, sv_s, so, cnt);
    };
    for (uint32_t j = 0; j < per; j++) {
      const uint32_t id = i0 + j;
      if (id >= cur_K) break;
      const uint32_t L = rlen[id];
      if (!L) continue;
      const uint32_t g = gbase[id], st = rstart[id];
#ifndef GSS_SCATTER_NOWRITE
#define GSS_SCATTER_NOWRITE 0   // diagnostic (wrong output): the write phase skipped, to time everything else
#endif
      if (GSS_SCATTER_NOWRITE) {
      } else if (!c.nremote) {
        put(kdst + g, kHasVal<Val> ? vdst + g : nullptr, st, L);
      } else {
        // fused exchange: the run goes to the GPUs owning its partition indices
        for (uint32_t done = 0; done < L;) {
          const RemoteSeg* sg = find_seg(c.remote, c.nremote, g + done);
          const uint32_t cnt = min(L - done, sg->hi - (g + done));
          put(reinterpret_cast<Key*>(sg->kdst) + g + done,
              kHasVal<Val> ? reinterpret_cast<Val*>(sg->vdst) + g + done : nullptr, st + done, cnt);
          done += cnt;
        }
      }
      gbase[id] = g + L;
    }
    bulk_commit();
    if constexpr (NBUF == 2) buf ^= 1u;
    if (done) break;
    if (new_tile) load_gbase(t);
  }
  bulk_wait_all();
  if (c.nremote) __threadfence_system();                          // peer stores visible before the exchange barrier
}

// ---------------------------------------------------------------------------
// Phase 4, warp-specialised (keys without values; the default for 8-byte
// keys).  The single-role scatter (k_scatter_bulk) runs every phase of a chunk
// in all 16 warps between CTA barriers; its write phase -- one warp-serialised
// bulk copy per bucket run -- was a quarter of its instructions (ncu source
// page, profiles/r02_*), and the global loads of the next chunk were exposed
// at the top of every chunk.  Here warp 15 (the I/O warp) moves the data and
// warps 0..14 (the rank warps) count and reorder:
//  * the I/O warp loads each chunk (C = 15 x 256 keys and their ids) into
//    shared memory by cp.async.bulk global -> shared, completing on an
//    mbarrier (full[b], b = chunk parity); two chunk buffers, so chunk c+1 is
//    in flight while chunk c is ranked;
//  * the rank warps read their 8 keys per lane from the buffer, rank them on
//    per-warp counters (one shared atomic per key; two ids share a 32-bit
//    word, 16 bits each), fold and scan the counters among themselves (named
//    barrier 1, 480 threads), and stage the chunk grouped by bucket id in the
//    SAME buffer (every rank warp has read it before the first barrier), each
//    key with its global destination index in a parallel array; then they
//    arrive on named barrier 2+b without waiting;
//  * the I/O warp syncs on 2+b and streams the staged chunk out in slot order,
//    32 consecutive slots per store instruction (runs are contiguous, so the
//    stores coalesce per bucket run), then loads chunk c+2 into the buffer.
// Ranks within (warp, id) follow item order and the warps are folded in
// order, so each level is a stable partition exactly as in k_scatter_bulk
// (the oracle's level records hold).  GSS kFlagScatterNoWs: the single-role
// kernel (ablation).
// ---------------------------------------------------------------------------
namespace wsync {
__device__ __forceinline__ void bar_sync(uint32_t id, uint32_t n) {
  asm volatile("bar.sync %0, %1;" ::"r"(id), "r"(n) : "memory");
}
__device__ __forceinline__ void bar_arrive(uint32_t id, uint32_t n) {
  asm volatile("bar.arrive %0, %1;" ::"r"(id), "r"(n) : "memory");
}
__device__ __forceinline__ void mbar_init(uint32_t a, uint32_t cnt) {
  asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(a), "r"(cnt) : "memory");
}
__device__ __forceinline__ void mbar_arrive_tx(uint32_t a, uint32_t tx) {
  asm volatile("{\n\t.reg .b64 st;\n\tmbarrier.arrive.expect_tx.shared::cta.b64 st, [%0], %1;\n\t}" ::"r"(a), "r"(tx)
               : "memory");
}
__device__ __forceinline__ void mbar_wait(uint32_t a, uint32_t parity) {
  asm volatile(
      "{\n\t.reg .pred p;\n\tLAB_WAIT:\n\t"
      "mbarrier.try_wait.parity.shared::cta.b64 p, [%0], %1;\n\t"
      "@!p bra LAB_WAIT;\n\t}" ::"r"(a), "r"(parity)
      : "memory");
}
__device__ __forceinline__ void bulk_g2s(uint32_t sdst, const void* gsrc, uint32_t bytes, uint32_t mbar) {
  asm volatile("cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];" ::"r"(sdst),
               "l"(gsrc), "r"(bytes), "r"(mbar)
               : "memory");
}
}  // namespace wsync

#ifndef GSS_SCATTER_IO_WARPS
#define GSS_SCATTER_IO_WARPS 2   // one I/O warp could not keep up with the stores (rank warps waited on it)
#endif
#ifndef GSS_WS_FOLD2
#define GSS_WS_FOLD2 0   // 1: two threads per id pair in the fold (measured slower: u32 0.88 vs 0.83 ms, sorted u64 1.84 vs 1.63)
#endif
#ifndef GSS_SCATTER_ITER_WS_KV
#define GSS_SCATTER_ITER_WS_KV 4   // 16-byte pairs: keys per lane (the values double the chunk buffers)
#endif
template <class Key, class Val, class IdT, int NIO_ = GSS_SCATTER_IO_WARPS, bool ONE_ = false>
struct ScatterWsSmem {
  static constexpr uint32_t NIO = NIO_;                                    // I/O warps
  static constexpr uint32_t NR = kScatterThreads / 32 - NIO;               // rank warps
  static constexpr bool KV = kHasVal<Val>;
  // ONE_: one CTA per SM with the whole shared memory (16-byte pairs at 8 keys per lane)
  static constexpr uint32_t ITER =                                         // keys per lane
      KV ? (sizeof(Key) + sizeof(Val) <= 8 || ONE_ ? GSS_SCATTER_ITER : GSS_SCATTER_ITER_WS_KV)
         : (sizeof(Key) == 4 ? GSS_SCATTER_ITER_U32 : GSS_SCATTER_ITER) * (ONE_ ? 2 : 1);
  static constexpr uint32_t C = NR * 32 * ITER;                            // keys per chunk
  static constexpr uint32_t A = 16 / sizeof(Key);
  static constexpr uint32_t VS = KV ? (uint32_t)sizeof(Val) : 0u;          // value bytes
  static constexpr uint32_t AV = KV ? 16u / VS : 1u;
  static constexpr size_t al(size_t x) { return (x + 15) & ~size_t(15); }
  static constexpr size_t ink_bytes() { return al((size_t)(C + A) * sizeof(Key)); }
  static constexpr size_t inv_bytes() { return KV ? al((size_t)(C + AV) * VS) : 0; }
  static constexpr size_t in_bytes() { return ink_bytes() + inv_bytes() + al((size_t)C * sizeof(IdT)); }
  static constexpr size_t stage_bytes() {
    return al((size_t)C * sizeof(Key)) + (KV ? al((size_t)C * VS) : 0) + al((size_t)C * sizeof(IdT));
  }
  // counters NR x kmax/2 words; gbase kmax; delta 2 x kmax; scan 64 words; 2 mbarriers
  __host__ __device__ static size_t head_bytes(uint32_t kmax) {
    return al(((size_t)NR * ((kmax + 1) / 2) + 3 * (size_t)kmax + 64) * 4 + 32);
  }
  __host__ __device__ static size_t bytes(uint32_t kmax) { return 2 * in_bytes() + stage_bytes() + head_bytes(kmax); }
};

template <class Key, class Val, class IdT, int NIO = GSS_SCATTER_IO_WARPS, bool ONE = false>
__global__ void __launch_bounds__(kScatterThreads, ONE ? 1 : 2)
    k_scatter_ws(Ctx<Key, Val, IdT> c, uint32_t level, uint32_t kmax) {
  extern __shared__ __align__(16) unsigned char smem_raw[];
  using SM = ScatterWsSmem<Key, Val, IdT, NIO, ONE>;
  constexpr bool KV = SM::KV;
  constexpr uint32_t NR = SM::NR, ITER = SM::ITER, C = SM::C, A = SM::A, AV = SM::AV, NRT = NR * 32,
                     NIOT = SM::NIO * 32;
  // named barriers: 1 the rank warps; 2 staged (rank warps arrive, I/O syncs); 3 staging free (I/O arrives,
  // rank warps sync); 4+b input buffer b read (rank warps arrive, I/O syncs)
  constexpr uint32_t BAR_RANK = 1, BAR_STAGED = 2, BAR_FREE = 3, BAR_IN = 4;
  // input buffer b (selected arithmetically: no local-memory arrays)
  auto ink = [&](uint32_t b) { return reinterpret_cast<Key*>(smem_raw + b * SM::in_bytes()); };
  auto inv = [&](uint32_t b) { return reinterpret_cast<Val*>(smem_raw + b * SM::in_bytes() + SM::ink_bytes()); };
  auto ini = [&](uint32_t b) {
    return reinterpret_cast<IdT*>(smem_raw + b * SM::in_bytes() + SM::ink_bytes() + SM::inv_bytes());
  };
  Key* stk = reinterpret_cast<Key*>(smem_raw + 2 * SM::in_bytes());
  Val* stv = reinterpret_cast<Val*>(smem_raw + 2 * SM::in_bytes() + SM::al((size_t)C * sizeof(Key)));
  IdT* sti = reinterpret_cast<IdT*>(smem_raw + 2 * SM::in_bytes() + SM::al((size_t)C * sizeof(Key)) +
                                    (KV ? SM::al((size_t)C * SM::VS) : 0));
  const uint32_t KH = (kmax + 1) / 2;
  uint32_t* cnt = reinterpret_cast<uint32_t*>(smem_raw + 2 * SM::in_bytes() + SM::stage_bytes());
  uint32_t* gbase = cnt + NR * KH;                       // next global index of each id (owner threads)
  uint32_t* delta = gbase + kmax;                        // per chunk parity: destination - staging slot of each id
  uint32_t* s_warp = delta + 2 * kmax;                   // 64 words
  const uint32_t mbar_0 = ((uint32_t)__cvta_generic_to_shared(s_warp + 64) + 7) & ~7u;
  auto mbar = [&](uint32_t b) { return mbar_0 + 8 * b; };

  const uint32_t slot = level & 1;
  const uint32_t nt = c.cnt->lvl[level].num_tiles;
  const Key* ksrc = c.keys(c.src(level));
  Key* kdst = c.wkeys(c.dst(level));
  const Val* vsrc = nullptr;
  Val* vdst = nullptr;
  if constexpr (KV) { vsrc = c.vals(c.src(level)); vdst = c.wvals(c.dst(level)); }
  const IdT* idsrc = c.ids;
  const int lane = threadIdx.x & 31, w = threadIdx.x >> 5;
  if (blockIdx.x >= nt) return;
  if (threadIdx.x == 0) {
    wsync::mbar_init(mbar(0), 1);
    wsync::mbar_init(mbar(1), 1);
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
  }
  __syncthreads();

  // The chunk sequence of this CTA: tiles blockIdx.x, +gridDim.x, ...; chunks of C keys inside each tile.
  struct Cursor {
    uint32_t t, c0, beg, len, K, idb;
    bool valid;
  };
  auto tile_at = [&](Cursor& u) {
    const Bucket B = c.bk[slot][c.tile_bucket[slot][u.t]];
    const uint32_t tl = u.t - B.tile_start;
    u.beg = B.lo + tl * c.T;
    u.len = min(c.T, B.m - tl * c.T);
    u.K = B.K;
    u.idb = B.id_base + tl * c.T;
  };
  auto advance = [&](Cursor& u) {                        // new tile: u.c0 == 0
    u.c0 += C;
    if (u.c0 >= u.len) {
      u.t += gridDim.x;
      u.c0 = 0;
      u.valid = u.t < nt;
      if (u.valid) tile_at(u);
    }
  };
  Cursor cur;
  cur.t = blockIdx.x; cur.c0 = 0; cur.valid = true;
  tile_at(cur);

  if (w >= (int)NR) {
    // ------------------------------ I/O warps ------------------------------
    // warp NR loads; every I/O thread stores (slot io, io + NIOT, ...)
    const uint32_t io = threadIdx.x - NRT;
    const bool loader = w == (int)NR;
    auto load = [&](const Cursor& u, uint32_t b) {
      const uint32_t clen = min(C, u.len - u.c0);
      const uint32_t g0 = u.beg + u.c0;
      const uint32_t sh = g0 & (A - 1);                  // element q lives in slot q + sh (16-byte phase of g0)
      const uint32_t h = min(clen, (A - sh) & (A - 1));  // head elements before the aligned middle
      const uint32_t mid = (clen - h) & ~(A - 1);
      const uint32_t ib = (clen * (uint32_t)sizeof(IdT)) & ~15u;   // id bytes by bulk copy (16-byte aligned start)
      Key* bk = ink(b);
      IdT* bi = ini(b);
      for (uint32_t q = lane; q < h; q += 32) bk[q + sh] = ksrc[g0 + q];
      for (uint32_t q = h + mid + lane; q < clen; q += 32) bk[q + sh] = ksrc[g0 + q];
      for (uint32_t q = ib / (uint32_t)sizeof(IdT) + lane; q < clen; q += 32) bi[q] = idsrc[u.idb + u.c0 + q];
      uint32_t shv = 0, hv = 0, midv = 0;
      if constexpr (KV) {                                // values: their own 16-byte phase
        shv = g0 & (AV - 1);
        hv = min(clen, (AV - shv) & (AV - 1));
        midv = (clen - hv) & ~(AV - 1);
        Val* bv = inv(b);
        for (uint32_t q = lane; q < hv; q += 32) bv[q + shv] = vsrc[g0 + q];
        for (uint32_t q = hv + midv + lane; q < clen; q += 32) bv[q + shv] = vsrc[g0 + q];
      }
      __syncwarp();
      if (lane == 0) {
        fence_proxy_async_smem();                        // the buffer's generic accesses before the async writes
        wsync::mbar_arrive_tx(mbar(b), mid * (uint32_t)sizeof(Key) + ib + midv * SM::VS);
        if constexpr (KV) {
          if (midv)
            wsync::bulk_g2s((uint32_t)__cvta_generic_to_shared(inv(b) + hv + shv), vsrc + g0 + hv, midv * SM::VS,
                            mbar(b));
        }
        if (mid)
          wsync::bulk_g2s((uint32_t)__cvta_generic_to_shared(bk + h + sh), ksrc + g0 + h, mid * (uint32_t)sizeof(Key),
                          mbar(b));
        if (ib) wsync::bulk_g2s((uint32_t)__cvta_generic_to_shared(bi), idsrc + u.idb + u.c0, ib, mbar(b));
      }
    };
    Cursor ld = cur;                                     // load cursor: two chunks ahead
    if (loader) load(ld, 0);
    advance(ld);
    if (ld.valid && loader) load(ld, 1);
    for (uint32_t k = 0;; k++) {
      const uint32_t b = k & 1;
      const uint32_t clen = min(C, cur.len - cur.c0);
      wsync::bar_sync(BAR_IN + b, kScatterThreads);      // the rank warps have read input buffer b (chunk k)
      if (ld.valid) advance(ld);
      if (ld.valid && loader) load(ld, b);               // chunk k+2
      wsync::bar_sync(BAR_STAGED, kScatterThreads);      // chunk k staged
      // the staged chunk in slot order: 32 consecutive slots per store (runs are contiguous), four in flight
      const uint32_t* dl = delta + b * kmax;
      uint32_t s = io;
      for (; s + 3 * NIOT < clen; s += 4 * NIOT) {
        Key x[4];
        uint32_t y[4];
#pragma unroll
        for (int u = 0; u < 4; u++) { x[u] = stk[s + NIOT * u]; y[u] = s + NIOT * u + dl[sti[s + NIOT * u]]; }
#pragma unroll
        for (int u = 0; u < 4; u++) kdst[y[u]] = x[u];
        if constexpr (KV) {
#pragma unroll
          for (int u = 0; u < 4; u++) vdst[y[u]] = stv[s + NIOT * u];
        }
      }
      for (; s < clen; s += NIOT) {
        const uint32_t y = s + dl[sti[s]];
        kdst[y] = stk[s];
        if constexpr (KV) vdst[y] = stv[s];
      }
      __syncwarp();
      wsync::bar_arrive(BAR_FREE, kScatterThreads);      // the staging buffer may be rewritten
      advance(cur);
      if (!cur.valid) break;
    }
    return;
  }

  // ------------------------------ rank warps ------------------------------
  const uint32_t* wc = cnt + w * KH;
  const uint32_t wc_s = (uint32_t)__cvta_generic_to_shared(wc);
  const uint32_t own = threadIdx.x;                      // owner of ids 2*own, 2*own+1
  for (uint32_t k = 0;; k++) {
    const uint32_t b = k & 1;
    const uint32_t K = cur.K, KP = (K + 1) / 2;
    // owner of id pair (2pp, 2pp+1): thread pp, or threads 2pp (hh = 0) and 2pp+1 (hh = 1) where 2 KP
    // threads exist (the fold below); gbase of a pair is read and written by its hh = 0 thread only
    const bool two = GSS_WS_FOLD2 && 2 * KP <= NRT;      // block-uniform
    const uint32_t pp = two ? own >> 1 : own, hh = two ? (own & 1) : 0u;
    const bool act = pp < KP;
    if (cur.c0 == 0 && act && hh == 0) {                 // a new tile: the global start of each id in it
      const Bucket B = c.bk[slot][c.tile_bucket[slot][cur.t]];
      const uint32_t tl = cur.t - B.tile_start;
      const uint32_t* hist = c.hist[slot] + B.hist_base;
      const uint32_t hb = hist[0];
#pragma unroll
      for (uint32_t j = 0; j < 2; j++) {
        const uint32_t id = 2 * pp + j;
        if (id < K) gbase[id] = hist[id * B.ntiles + tl] - hb + B.lo;
      }
    }
    const uint32_t clen = min(C, cur.len - cur.c0);
    const uint32_t sh = (cur.beg + cur.c0) & (A - 1), shv = (cur.beg + cur.c0) & (AV - 1);
    for (uint32_t j = lane; j < KP; j += 32) cnt[w * KH + j] = 0;
    wsync::mbar_wait(mbar(b), (k >> 1) & 1);
    Key kk[ITER];
    Val vv[ITER];
    uint32_t iid[ITER];
    {
      const Key* bk = ink(b);
      const IdT* bi = ini(b);
#pragma unroll
      for (uint32_t it = 0; it < ITER; it++) {
        const uint32_t q = w * (32 * ITER) + it * 32 + lane;
        iid[it] = 0xffffffffu;
        if (q < clen) {
          kk[it] = bk[q + sh];
          if constexpr (KV) vv[it] = inv(b)[q + shv];
          iid[it] = bi[q];
        }
      }
    }
    __syncwarp();
    wsync::bar_arrive(BAR_IN + b, kScatterThreads);      // input buffer b may be refilled
    // ranks within (warp, id): packed counters, two ids per word
    {
      const uint32_t first = __shfl_sync(kFull, iid[0], 0);
      bool same = first != 0xffffffffu;
#pragma unroll
      for (uint32_t it = 0; it < ITER; it++) same = same && iid[it] == first;
      if (__all_sync(kFull, same)) {
        uint32_t base = 0;
        if (lane == 0) base = atom_add_shared_if(1u, wc_s + 4 * (first >> 1), (32u * ITER) << (16 * (first & 1)));
        base = (__shfl_sync(kFull, base, 0) >> (16 * (first & 1))) & 0xffffu;
#pragma unroll
        for (uint32_t it = 0; it < ITER; it++) iid[it] = ((base + 32u * it + (uint32_t)lane) << 16) | first;
      } else {
#pragma unroll
        for (uint32_t it = 0; it < ITER; it++) {
          const uint32_t id = iid[it] & 0xffffu, hs = 16 * (id & 1);
          const uint32_t r = atom_add_shared_if(iid[it] != 0xffffffffu ? 1u : 0u, wc_s + 4 * (id >> 1), 1u << hs);
          iid[it] = iid[it] == 0xffffffffu ? iid[it] : (((r >> hs) & 0xffffu) << 16) | id;
        }
      }
    }
    wsync::bar_sync(BAR_RANK, NRT);                      // counters complete
    // owners: chunk totals of ids 2p, 2p+1 (runs packed in id order), every warp's start in them.  Two
    // adjacent threads per pair (each folding half of the rank warps' counters) where 2 * KP threads exist,
    // which halves the serial fold between the barriers; else one thread per pair.
    const uint32_t qa = two ? hh * (NR / 2) : 0u, qb = two ? (hh ? NR : NR / 2) : NR;
    uint32_t a0 = 0, a1 = 0;                              // this thread's warps
    if (act) {
#pragma unroll 7
      for (uint32_t q = qa; q < qb; q++) {
        const uint32_t x = cnt[q * KH + pp];
        a0 += x & 0xffffu;
        a1 += x >> 16;
      }
    }
    uint32_t b0 = 0, b1 = 0;                              // the partner's warps
    if (two) {
      b0 = __shfl_xor_sync(kFull, a0, 1);
      b1 = __shfl_xor_sync(kFull, a1, 1);
    }
    const uint32_t L0 = a0 + b0, L1 = a1 + b1;
    const uint32_t tsum = (act && hh == 0) ? L0 + L1 : 0u;   // an odd K's missing id counts 0
    uint32_t ex;
    {
      uint32_t inc = tsum;
#pragma unroll
      for (int o = 1; o < 32; o <<= 1) {
        const uint32_t y = __shfl_up_sync(kFull, inc, o);
        if (lane >= o) inc += y;
      }
      if (lane == 31) s_warp[w] = inc;
      wsync::bar_sync(BAR_RANK, NRT);
      if (w == 0) {
        const uint32_t v = lane < (int)NR ? s_warp[lane] : 0u;
        uint32_t vi = v;
#pragma unroll
        for (int o = 1; o < 32; o <<= 1) {
          const uint32_t y = __shfl_up_sync(kFull, vi, o);
          if (lane >= o) vi += y;
        }
        if (lane < (int)NR) s_warp[32 + lane] = vi - v;
      }
      wsync::bar_sync(BAR_RANK, NRT);
      ex = s_warp[32 + w] + inc - tsum;
    }
    if (two) ex = __shfl_sync(kFull, ex, lane & ~1);     // the pair's base (its even thread's prefix)
    if (act) {
      const uint32_t st0 = ex, st1 = ex + L0;
      const uint32_t id0 = 2 * pp;
      if (hh == 0) {
        uint32_t* dl = delta + b * kmax;
        dl[id0] = gbase[id0] - st0;
        gbase[id0] += L0;
        if (id0 + 1 < K) {
          dl[id0 + 1] = gbase[id0 + 1] - st1;
          gbase[id0 + 1] += L1;
        }
      }
      uint32_t r0 = st0 + (hh ? b0 : 0u), r1 = st1 + (hh ? b1 : 0u);
#pragma unroll 7
      for (uint32_t q = qa; q < qb; q++) {
        const uint32_t x = cnt[q * KH + pp];
        cnt[q * KH + pp] = r0 | (r1 << 16);
        r0 += x & 0xffffu;
        r1 += x >> 16;
      }
    }
    if (k > 0) wsync::bar_sync(BAR_FREE, kScatterThreads);   // the I/O warp has written chunk k-1 out
    wsync::bar_sync(BAR_RANK, NRT);                      // run slots known
#pragma unroll
    for (uint32_t it = 0; it < ITER; it++) {
      if (iid[it] != 0xffffffffu) {
        const uint32_t id = iid[it] & 0xffffu;
        const uint32_t pos = ((wc[id >> 1] >> (16 * (id & 1))) & 0xffffu) + (iid[it] >> 16);
        stk[pos] = kk[it];
        if constexpr (KV) stv[pos] = vv[it];
        sti[pos] = (IdT)id;
      }
    }
    wsync::bar_arrive(BAR_STAGED, kScatterThreads);
    advance(cur);
    if (!cur.valid) break;
  }
  wsync::bar_sync(BAR_FREE, kScatterThreads);            // matches the I/O warp's last arrival
}

// ---------------------------------------------------------------------------
// Phase 4, default variant (R7: a partition, not stable).  Every key takes
// its rank within (chunk, id) from one shared-memory atomic on the CTA's
// counter for its id; warp 0 scans the K chunk totals into staged run
// offsets and staged -> global displacements; the chunk is reordered by id in
// shared memory and each bucket run is written with coalesced stores.  One
// counter set per CTA (not per warp) keeps the per-chunk bookkeeping at K
// counters.  CTA b handles the contiguous tile range [b*per, (b+1)*per); the
// next chunk's keys, values and ids are loaded into registers before the
// current chunk's runs are written out.
template <class Key, class Val, class IdT>
struct ScatterFastSmem {
  // staging of the current chunk's keys in natural order frees their
  // registers for the next chunk's loads (not for 16-byte pairs: smem)
#ifndef GSS_SCATTER_STAGE
#define GSS_SCATTER_STAGE 0      // staging measured slower on B200 (3.40 vs 3.13 ms per 2^28 u64 sort)
#endif
  static constexpr bool kStage = GSS_SCATTER_STAGE && (!kHasVal<Val> || sizeof(Key) + sizeof(Val) <= 8);
  static size_t bytes(uint32_t kmax) {
    GSS_SCATTER_CHUNK_CONSTANTS
    size_t b = (size_t)kmax * 4 * 3;                            // cnt/off, delta, gbase
    b = (b + 15) & ~size_t(15);
    b += (size_t)kChunk * sizeof(Key) * (kStage ? 2 : 1);
    if (kHasVal<Val>) b += (size_t)kChunk * sizeof(Val) * (kStage ? 2 : 1);
    b += (size_t)kChunk * sizeof(IdT);
    return b;
  }
};

template <class Key, class Val, class IdT, class Cmp>
__global__ void __launch_bounds__(kScatterThreads, GSS_SCATTER_MINB)
    k_scatter_fast(Ctx<Key, Val, IdT> c, uint32_t level, uint32_t kmax) {
  extern __shared__ __align__(16) unsigned char smem_raw[];
  GSS_SCATTER_CHUNK_CONSTANTS
  constexpr bool STAGE = ScatterFastSmem<Key, Val, IdT>::kStage;
  uint32_t* cnt = reinterpret_cast<uint32_t*>(smem_raw);          // chunk counts, then run offsets
  uint32_t* delta = cnt + kmax;
  uint32_t* gbase = delta + kmax;
  size_t o = ((size_t)kmax * 12 + 15) & ~size_t(15);
  Key* skeys = reinterpret_cast<Key*>(smem_raw + o);
  o += (size_t)kChunk * sizeof(Key);
  Val* svals = reinterpret_cast<Val*>(smem_raw + o);
  if constexpr (kHasVal<Val>) o += (size_t)kChunk * sizeof(Val);
  Key* tkeys = reinterpret_cast<Key*>(smem_raw + o);              // staging (natural order)
  if constexpr (STAGE) o += (size_t)kChunk * sizeof(Key);
  Val* tvals = reinterpret_cast<Val*>(smem_raw + o);
  if constexpr (STAGE && kHasVal<Val>) o += (size_t)kChunk * sizeof(Val);
  IdT* sids = reinterpret_cast<IdT*>(smem_raw + o);

  const uint32_t slot = level & 1;
  const uint32_t nt = c.cnt->lvl[level].num_tiles;
  const uint32_t sb = c.src(level), db = c.dst(level);
  const Key* ksrc = c.keys(sb);
  Key* kdst = c.wkeys(db);
  const Val* vsrc = nullptr;
  Val* vdst = nullptr;
  if constexpr (kHasVal<Val>) { vsrc = c.vals(sb); vdst = c.wvals(db); }
  const IdT* idsrc = c.ids;
  const int lane = threadIdx.x & 31, w = threadIdx.x >> 5;
  const uint32_t cnt_s = (uint32_t)__cvta_generic_to_shared(cnt);
  const uint32_t q0 = w * (32 * kScatterIter) + lane;
  const uint32_t per = (nt + gridDim.x - 1) / gridDim.x;
  uint32_t t = blockIdx.x * per;
  const uint32_t t_end = min(nt, t + per);
  if (t >= t_end) return;

  // per-tile state kept in registers: start, length, id base, K (the
  // histogram row is re-read from the bucket record when a tile starts)
  uint32_t beg, len, K, idb;
  auto tile_info = [&](uint32_t tt) {
    const Bucket B = c.bk[slot][c.tile_bucket[slot][tt]];
    const uint32_t tl = tt - B.tile_start;
    beg = B.lo + tl * c.T;
    len = min(c.T, B.m - tl * c.T);
    K = B.K;
    idb = B.id_base + tl * c.T;
  };
  auto load_gbase = [&](uint32_t tt) {
    const Bucket B = c.bk[slot][c.tile_bucket[slot][tt]];
    const uint32_t tl = tt - B.tile_start;
    const uint32_t* hist = c.hist[slot] + B.hist_base;
    const uint32_t hb = hist[0];
    for (uint32_t id = threadIdx.x; id < B.K; id += kScatterThreads)
      gbase[id] = hist[id * B.ntiles + tl] - hb + B.lo;
  };
  tile_info(t);
  load_gbase(t);
  for (uint32_t id = threadIdx.x; id < kmax; id += kScatterThreads) cnt[id] = 0;
  Key pk[kScatterIter];
  Val pv[kScatterIter];
  uint32_t pid[kScatterIter];                                      // id, or 0xffffffff past the chunk end
  auto load_chunk = [&](uint32_t cbeg, uint32_t cid, uint32_t clen) {
#pragma unroll
    for (int it = 0; it < kScatterIter; it++) {
      const uint32_t q = q0 + it * 32;
      pid[it] = 0xffffffffu;
      if (q < clen) {
        pk[it] = ksrc[cbeg + q];
        pid[it] = idsrc[cid + q];
        if constexpr (kHasVal<Val>) pv[it] = vsrc[cbeg + q];
      }
    }
  };
  uint32_t c0 = 0;
  load_chunk(beg, idb, min((uint32_t)kChunk, len));
  __syncthreads();                                                 // gbase and counters initialised
#ifdef GSS_SCATTER_PHASES
  unsigned long long ph[6] = {0, 0, 0, 0, 0, 0}, tp = clock64();
  uint32_t nchunks = 0;
#endif
  for (;;) {
    const uint32_t clen = min((uint32_t)kChunk, len - c0);
    uint32_t ir[kScatterIter];                                     // (rank << 16) | id; 0xffffffff = none
    Key kk[kScatterIter];
    Val vv[kScatterIter];
#pragma unroll
    for (int it = 0; it < kScatterIter; it++) {
      ir[it] = pid[it];
      if constexpr (STAGE) {
        // the keys (and values) wait in shared memory in natural order
        if (ir[it] != 0xffffffffu) {
          tkeys[q0 + it * 32] = pk[it];
          if constexpr (kHasVal<Val>) tvals[q0 + it * 32] = pv[it];
        }
      } else {
        kk[it] = pk[it];
        if constexpr (kHasVal<Val>) vv[it] = pv[it];
      }
    }
    // 1. rank within (chunk, id): one shared atomic per key on the CTA's counter
#pragma unroll
    for (int it = 0; it < kScatterIter; it++) {
      const uint32_t id = ir[it] & 0xffffu;
      const uint32_t r = atom_add_shared_if(ir[it] != 0xffffffffu ? 1u : 0u, cnt_s + 4 * id, 1u);
      ir[it] = ir[it] == 0xffffffffu ? ir[it] : (r << 16) | id;
    }
    // advance and, with staging, prefetch the next chunk now: its loads
    // overlap the scan, the reorder and the write-out of this one
    const uint32_t cur_clen = clen, cur_K = K;
#ifdef GSS_EXP_SEQWRITE
    const uint32_t cur_beg = beg + c0;
#endif
    bool new_tile = false, done = false;
    c0 += kChunk;
    if (c0 >= len) {
      t++;
      c0 = 0;
      if (t >= t_end) done = true;
      else { tile_info(t); new_tile = true; }
    }
    if constexpr (STAGE) {
      if (!done) load_chunk(beg + c0, idb + c0, min((uint32_t)kChunk, len - c0));
    }
    __syncthreads();
    GSS_PH(0);
    // 2. warp 0: exclusive scan of the K chunk totals -> staged run offsets
    //    (cnt), staged -> global displacement (delta); gbase advances
    if (w == 0) {
      uint32_t run = 0;
      for (uint32_t id0 = 0; id0 < cur_K; id0 += 32 * 8) {
        const uint32_t ib = id0 + lane * 8;
        uint32_t x[8], sum = 0;
#pragma unroll
        for (int j = 0; j < 8; j++) {
          x[j] = ib + j < cur_K ? cnt[ib + j] : 0u;
          sum += x[j];
        }
        uint32_t inc = sum;
#pragma unroll
        for (int sh = 1; sh < 32; sh <<= 1) {
          const uint32_t y = __shfl_up_sync(kFull, inc, sh);
          if (lane >= sh) inc += y;
        }
        uint32_t ex = run + inc - sum;
#pragma unroll
        for (int j = 0; j < 8; j++) {
          if (ib + j < cur_K) {
            cnt[ib + j] = ex;
            delta[ib + j] = gbase[ib + j] - ex;
            gbase[ib + j] += x[j];
          }
          ex += x[j];
        }
        run += __shfl_sync(kFull, inc, 31);
      }
    }
    __syncthreads();
    GSS_PH(1);
    // 3. reorder the chunk by id in shared memory
#pragma unroll
    for (int it = 0; it < kScatterIter; it++) {
      if (ir[it] != 0xffffffffu) {
        const uint32_t id = ir[it] & 0xffffu;
        const uint32_t pos = cnt[id] + (ir[it] >> 16);
        if constexpr (STAGE) {
          skeys[pos] = tkeys[q0 + it * 32];
          if constexpr (kHasVal<Val>) svals[pos] = tvals[q0 + it * 32];
        } else {
          skeys[pos] = kk[it];
          if constexpr (kHasVal<Val>) svals[pos] = vv[it];
        }
        sids[pos] = (IdT)id;
      }
    }
    if constexpr (!STAGE) {
      if (!done) load_chunk(beg + c0, idb + c0, min((uint32_t)kChunk, len - c0));
    }
    __syncthreads();
    GSS_PH(2);
    // 4. write this chunk's bucket runs; clear the counters for the next chunk
#pragma unroll 4
    for (uint32_t q = threadIdx.x; q < cur_clen; q += kScatterThreads) {
#ifdef GSS_EXP_SEQWRITE
      const uint32_t d = cur_beg + q;                              // diagnostic: plain copy (wrong result)
#else
      const uint32_t d = delta[sids[q]] + q;
#endif
      kdst[d] = skeys[q];
      if constexpr (kHasVal<Val>) vdst[d] = svals[q];
    }
    for (uint32_t id = threadIdx.x; id < cur_K; id += kScatterThreads) cnt[id] = 0;
#ifdef GSS_SCATTER_PHASES
    { const unsigned long long tn = clock64(); ph[3] += tn - tp; tp = tn; }
    nchunks++;
    if (done && threadIdx.x == 0 && (blockIdx.x == 0 || blockIdx.x == 100))
      printf("fast scatter phases block %d chunks %u: rank %llu scan %llu reorder %llu write %llu (cycles per chunk)\n",
             blockIdx.x, nchunks, ph[0] / nchunks, ph[1] / nchunks, ph[2] / nchunks, ph[3] / nchunks);
#endif
    if (done) break;
    if (new_tile) {
      // gbase is rewritten only after every thread has left steps 2-4
      __syncthreads();
      load_gbase(t);
    }
    __syncthreads();
  }
}

// Phase 4 as the paper describes it: every key goes
// straight from registers to its global position; the position is the tile's
// offset for its bucket plus a shared-memory atomic cursor (the per-block
// counters of P:312-317).  No staging and no barriers inside a tile; the
// within-bucket order is the atomics' order (a valid partition, not stable).
// A warp whose 32 keys share one bucket (sorted input) takes one atomic.
constexpr int kDirectThreads = 256;
template <class Key, class Val, class IdT, class Cmp>
__global__ void __launch_bounds__(kDirectThreads, 4) k_scatter_direct(Ctx<Key, Val, IdT> c, uint32_t level) {
  extern __shared__ __align__(16) unsigned char smem_raw[];
  uint32_t* cursor = reinterpret_cast<uint32_t*>(smem_raw);
  const uint32_t cur_s = (uint32_t)__cvta_generic_to_shared(cursor);
  const uint32_t slot = level & 1;
  const uint32_t nt = c.cnt->lvl[level].num_tiles;
  const uint32_t sb = c.src(level), db = c.dst(level);
  const Key* ksrc = c.keys(sb);
  Key* kdst = c.wkeys(db);
  const Val* vsrc = nullptr;
  Val* vdst = nullptr;
  if constexpr (kHasVal<Val>) { vsrc = c.vals(sb); vdst = c.wvals(db); }
  const int lane = threadIdx.x & 31;
  const uint32_t ltmask = lanemask_lt();
  constexpr int U = 8;
  for (uint32_t t = blockIdx.x; t < nt; t += gridDim.x) {
    const uint32_t b = c.tile_bucket[slot][t];
    const Bucket B = c.bk[slot][b];
    const uint32_t tl = t - B.tile_start;
    const uint32_t beg = B.lo + tl * c.T;
    const uint32_t len = min(c.T, B.m - tl * c.T);
    const uint32_t* hist = c.hist[slot] + B.hist_base;
    const uint32_t hb = hist[0];
    __syncthreads();
    for (uint32_t id = threadIdx.x; id < B.K; id += kDirectThreads) cursor[id] = hist[id * B.ntiles + tl] - hb + B.lo;
    __syncthreads();
    const Key* ks = ksrc + beg;
    const IdT* is = c.ids + B.id_base + tl * c.T;
    const Val* vs = nullptr;
    if constexpr (kHasVal<Val>) vs = vsrc + beg;
    for (uint32_t w0 = threadIdx.x & ~31u; w0 < len; w0 += U * kDirectThreads) {   // warp-uniform trip count
      const uint32_t i0 = w0 + lane;
      Key kk[U];
      Val vv[U];
      uint32_t id[U];
#pragma unroll
      for (int u = 0; u < U; u++) {
        const uint32_t i = i0 + u * kDirectThreads;
        id[u] = 0xffffffffu;
        if (i < len) {
          kk[u] = ks[i];
          id[u] = is[i];
          if constexpr (kHasVal<Val>) vv[u] = vs[i];
        }
      }
#pragma unroll
      for (int u = 0; u < U; u++) {
        const uint32_t myid = id[u];
        const uint32_t first = __shfl_sync(kFull, myid, 0);
        uint32_t d;
        if (__all_sync(kFull, myid == first) && first != 0xffffffffu) {
          // the whole warp in one bucket: one atomic, lane order
          uint32_t base = 0;
          if (lane == 0) base = atomicAdd(&cursor[first], 32u);
          d = __shfl_sync(kFull, base, 0) + (uint32_t)__popc(ltmask);
        } else {
          d = atom_add_shared_if(myid != 0xffffffffu ? 1u : 0u, cur_s + 4 * (myid & 0xffffu), 1u);
        }
        if (myid != 0xffffffffu) {
          kdst[d] = kk[u];
          if constexpr (kHasVal<Val>) vdst[d] = vv[u];
        }
      }
    }
  }
}

// ---------------------------------------------------------------------------
// Recursion (Algorithm 1) with delayed small sorts: every
// child of every bucket split at this level becomes a next-level bucket
// (m > M), an in-SM sort item (m <= M), a final equality bucket (R4), or --
// past the last launched level -- an overflow item.
// ---------------------------------------------------------------------------
// Warp-aggregated append of `cnt` items per lane to a list with counter
// *ctr: returns each lane's first slot (lanes with cnt == 0 get garbage).
// All 32 lanes must call it.
__device__ __forceinline__ uint32_t warp_append(uint32_t* ctr, uint32_t cnt) {
  const int lane = threadIdx.x & 31;
  uint32_t incl = cnt;
#pragma unroll
  for (int o = 1; o < 32; o <<= 1) {
    uint32_t y = __shfl_up_sync(kFull, incl, o);
    if (lane >= o) incl += y;
  }
  const uint32_t total = __shfl_sync(kFull, incl, 31);
  uint32_t base = 0;
  if (lane == 0 && total) base = atomicAdd(ctr, total);
  base = __shfl_sync(kFull, base, 0);
  return base + incl - cnt;
}

__device__ __forceinline__ uint64_t warp_sum64(uint64_t x) {
#pragma unroll
  for (int o = 16; o > 0; o >>= 1) x += __shfl_xor_sync(kFull, x, o);
  return x;
}
__device__ __forceinline__ uint32_t warp_max32(uint32_t x) {
#pragma unroll
  for (int o = 16; o > 0; o >>= 1) x = max(x, __shfl_xor_sync(kFull, x, o));
  return x;
}

template <class Key, class Val, class IdT>
__global__ void __launch_bounds__(kPlanThreads) k_plan(Ctx<Key, Val, IdT> c, uint32_t level) {
  const uint32_t slot = level & 1;
  const uint32_t nb = c.cnt->lvl[level].num_buckets;
  const uint32_t db = c.dst(level);
  const uint32_t next = level + 1;
  const int lane = threadIdx.x & 31;
  const uint32_t cap_last = c.class_cap[kNumClasses - 1];
  for (uint32_t b = blockIdx.x; b < nb; b += gridDim.x) {
    const Bucket B = c.bk[slot][b];
    const uint32_t* hist = c.hist[slot] + B.hist_base;
    const uint32_t hb = hist[0];
    for (uint32_t id0 = 0; id0 < B.K; id0 += kPlanThreads) {         // uniform trip count
      const uint32_t id = id0 + threadIdx.x;
      uint32_t start = 0, m = 0;
      if (id < B.K) {
        start = hist[id * B.ntiles] - hb + B.lo;
        const uint32_t end = (id + 1 < B.K) ? hist[(id + 1) * B.ntiles] - hb + B.lo : B.lo + B.m;
        m = end - start;
      }
      const bool is_eq = m && B.eq && (id & 1);
      // categories: small-sort class, copy (big equality bucket), next level, overflow
      const bool to_small = m && ((is_eq && db != BUF_OUT && m <= cap_last) || (!is_eq && m <= c.M));
      const bool to_copy = is_eq && db != BUF_OUT && m > cap_last;
      const bool to_next = m && !is_eq && m > c.M && next < c.L;
      const bool to_ovf = m && !is_eq && m > c.M && next >= c.L;
      // equality-bucket statistics
      {
        const uint64_t e_cnt = warp_sum64(is_eq ? 1 : 0), e_el = warp_sum64(is_eq ? m : 0);
        if (lane == 0 && e_cnt) {
          atomicAdd(&c.cnt->eq_buckets, (unsigned long long)e_cnt);
          atomicAdd(&c.cnt->eq_elems, (unsigned long long)e_el);
        }
      }
      // buckets above one CTA's capacity (only with GSS_FLAG_CLUSTER_SORT, where M may exceed it): the
      // cluster-wide sort
      const bool to_clus = to_small && m > cap_last;
      if (__any_sync(kFull, to_clus)) {
        const uint32_t i = warp_append(&c.cnt->clus_count, to_clus ? 1u : 0u);
        if (to_clus) {
          if (i < c.cap_clus) c.clus[i] = Item{start, m, db, 0};
          else atomicOr(&c.cnt->err, 16u);
        }
      }
      // in-SM sort lists, one per size class
      uint32_t cls = 0;
      while (cls + 1 < kNumClasses && m > c.class_cap[cls]) cls++;
      for (int q = 0; q < kNumClasses; q++) {
        const bool mine = to_small && !to_clus && cls == (uint32_t)q;
        if (!__any_sync(kFull, mine)) continue;
        const uint32_t i = warp_append(&c.cnt->small_count[q], mine ? 1u : 0u);
        if (mine) {
          if (i < c.cap_small[q]) c.small[q][i] = Item{start, m, db, 0};
          else atomicOr(&c.cnt->err, 1u);
        }
      }
      {
        const uint64_t s_el = warp_sum64(to_small ? m : 0);
        const uint32_t s_max = warp_max32(to_small ? m : 0);
        if (lane == 0 && s_el) {
          atomicAdd(&c.cnt->small_elems, (unsigned long long)s_el);
          atomicMax(&c.cnt->max_small, (unsigned long long)s_max);
        }
      }
      if (__any_sync(kFull, to_copy)) {
        const uint32_t nt = to_copy ? (uint32_t)(((uint64_t)m + c.T - 1) / c.T) : 0;
        const uint32_t i = warp_append(&c.cnt->copy_count, nt);
        if (to_copy) {
          if (i + nt <= c.cap_copy) {
            for (uint32_t q = 0; q < nt; q++) c.copy[i + q] = Item{start + q * c.T, min(c.T, m - q * c.T), db, 0};
          } else {
            atomicOr(&c.cnt->err, 2u);
          }
        }
      }
      if (__any_sync(kFull, to_next)) {
        LevelCounters& NL = c.cnt->lvl[next];
        const uint32_t kb = to_next ? choose_kb(c.k, c.k_policy, c.fill_div, c.M, m) : 0;
        const uint32_t nt = to_next ? (uint32_t)(((uint64_t)m + c.T - 1) / c.T) : 0;
        const uint32_t bi = warp_append(&NL.num_buckets, to_next ? 1u : 0u);
        const uint32_t ts = warp_append(&NL.num_tiles, nt);
        const uint32_t hbn = warp_append(&NL.hist_alloc, to_next ? max(kb, 3u) * nt : 0u);
        const uint32_t sbn = warp_append(&NL.spl_alloc, 2 * kb);
        const uint32_t ib = warp_append(&NL.id_alloc, to_next ? (m + 15u) & ~15u : 0u);
        const uint64_t el = warp_sum64(to_next ? m : 0);
        if (lane == 0 && el) atomicAdd(&NL.split_elems, (unsigned long long)el);
        if (to_next) {
          if (bi < c.cap_buckets && ts + nt <= c.cap_tiles && hbn + max(kb, 3u) * nt <= c.cap_hist &&
              sbn + 2 * kb <= c.cap_spl) {
            Bucket nbk{};
            nbk.lo = start; nbk.m = m; nbk.tile_start = ts; nbk.ntiles = nt; nbk.kb = kb;
            nbk.hist_base = hbn; nbk.spl_base = sbn;
            nbk.id_base = ib;                                     // 16-element aligned, disjoint per bucket
            c.bk[next & 1][bi] = nbk;
          } else {
            atomicOr(&c.cnt->err, 4u);
          }
        }
      }
      if (__any_sync(kFull, to_ovf)) {
        const uint32_t i = warp_append(&c.cnt->ovf_count, to_ovf ? 1u : 0u);
        const uint64_t el = warp_sum64(to_ovf ? m : 0);
        if (lane == 0 && el) atomicAdd(&c.cnt->ovf_elems, (unsigned long long)el);
        if (to_ovf) {
          if (i < c.cap_ovf) c.ovf[i] = Item{start, m, db, 0};
          else atomicOr(&c.cnt->err, 8u);
        }
      }
    }
  }
}

// ---------------------------------------------------------------------------
// Sorting buckets: one CTA per bucket of at most M keys; the
// bucket is loaded to shared memory, sorted by CtaSort, written to keys_out.
// ---------------------------------------------------------------------------
// keys per thread of the bucket sorter (32 items per thread measured slower
// on B200: register pressure outweighs the saved merge round), i.e. the
// CtaSort default
#ifndef GSS_U32_ITEMS
#define GSS_U32_ITEMS 32
#endif
// 4-byte keys without values may hold 32 per thread (same 32 registers as
// 16 eight-byte keys): one merge round fewer and half the searches per key
template <class Key, class Val>
constexpr int small_items() { return (sizeof(Key) == 4 && !kHasVal<Val>) ? GSS_U32_ITEMS : sort_items<Key, Val>(); }
constexpr int kSmallMaxThreads = 1024;

// ---------------------------------------------------------------------------
// In-SM bucket sort, one CTA per bucket.  Both kernels below
// serve every size class with one instantiation: the block has
// class_warps(cls) warps (blockDim.x, chosen by the host).
// ---------------------------------------------------------------------------

// Block-wide merge sort: the bucket is loaded to shared memory, each thread
// sorts ITEMS keys with the odd-even merge network, then merge-path rounds
// across the whole CTA (CtaSort).  Used for the one-warp class (where it is
// a warp sort), for the buckets the in-SM split hands back (cls ==
// kNumClasses, 1024 threads), and for every class unless GSS_FLAG_SPLIT_SORT.
template <class Key, class Val>
__host__ __device__ constexpr size_t block_sort_smem_bytes(int nt) {
  return (size_t)padded_len(nt * small_items<Key, Val>()) * (sizeof(Key) + (kHasVal<Val> ? sizeof(Val) : 0));
}

#ifndef GSS_SMALL_L2PF
#define GSS_SMALL_L2PF 1     // the next bucket of the CTA prefetched into L2 (8-byte keys alone)
#endif
#ifndef GSS_SMALL_DIRECT
#define GSS_SMALL_DIRECT 1   // bucket keys read by the sorting threads straight into registers: 2^27 u32 in-SM
#endif                       // sort 1.61 -> 1.52 ms, u64 pairs 4.47 -> 4.33, u32 pairs 2.63 -> 2.56; 8-byte keys
                             // alone keep the cp.async staging (4.76 vs 4.83 ms)
#ifndef GSS_SMALL_CPASYNC
#define GSS_SMALL_CPASYNC 1   // 8-byte keys: 4.83 vs 4.96 ms (2^28 u64), pairs 4.45 vs 4.57; 4-byte copies lose (2.15 vs 1.58)
#endif
// MAXT: the widest CTA the instantiation serves.  The ablation kFlagSmallNarrow gives classes of up to 20
// warps MAXT = 640 with two resident CTAs guaranteed, which caps the registers at 48 (from 60): four 10-warp
// CTAs per SM instead of three -- measured no faster (2^28 u64 4.98 vs 4.90 ms).
constexpr int kSmallNarrowThreads = 640;
template <class Key, class Val, class IdT, class Cmp, bool BITONIC = false, int MAXT = kSmallMaxThreads>
__global__ void __launch_bounds__(MAXT, MAXT <= kSmallNarrowThreads ? 2 : 1)
    k_small_block(Ctx<Key, Val, IdT> c, uint32_t cls) {
  extern __shared__ __align__(16) unsigned char smem_raw[];
  constexpr int ITEMS = small_items<Key, Val>();
  using Sorter = CtaSort<Key, Val, kSmallMaxThreads, Cmp, ITEMS, BITONIC>;
  const int nt = (int)blockDim.x;
  Key* sk = reinterpret_cast<Key*>(smem_raw);
  Val* sv = reinterpret_cast<Val*>(smem_raw + (size_t)padded_len(nt * ITEMS) * sizeof(Key));
  const Cmp less;
  const bool fb = cls == (uint32_t)kNumClasses;
  const uint32_t ni = fb ? min(c.cnt->fb_count, c.cap_fb) : min(c.cnt->small_count[cls], c.cap_small[cls]);
  const Item* list = fb ? c.fb : c.small[cls];
  for (uint32_t i = blockIdx.x; i < ni; i += gridDim.x) {
    const Item I = list[i];
    const uint32_t m = I.m;
    const Key* src = c.keys(I.buf) + I.lo;
    const Val* vs = nullptr;
    if constexpr (kHasVal<Val>) vs = c.vals(I.buf) + I.lo;
#if GSS_SMALL_L2PF
    // the CTA's next bucket pulled into L2 while this one is sorted (its cp.async load then waits for L2, not
    // DRAM): 8-byte keys alone (2^28 u64 in-SM sort 4.76 -> 4.74 ms; 2^27 u32 1.52 -> 1.56, so not there)
    if (sizeof(Key) == 8 && !kHasVal<Val> && i + gridDim.x < ni) {
      const Item J = list[i + gridDim.x];
      const char* nk = reinterpret_cast<const char*>(c.keys(J.buf) + J.lo);
      const uint32_t lines = (uint32_t)(((size_t)J.m * sizeof(Key) + 127) / 128);
      for (uint32_t q = threadIdx.x; q < lines; q += nt) asm volatile("prefetch.global.L2 [%0];" ::"l"(nk + 128 * (size_t)q));
      if constexpr (kHasVal<Val>) {
        const char* nv = reinterpret_cast<const char*>(c.vals(J.buf) + J.lo);
        const uint32_t vl = (uint32_t)(((size_t)J.m * sizeof(Val) + 127) / 128);
        for (uint32_t q = threadIdx.x; q < vl; q += nt) asm volatile("prefetch.global.L2 [%0];" ::"l"(nv + 128 * (size_t)q));
      }
    }
#endif
    if constexpr (GSS_SMALL_DIRECT && !Sorter::WB && !(sizeof(Key) == 8 && !kHasVal<Val>)) {
      // the threads read their first items straight from global memory (no shared-memory staging)
      Sorter::sort(sk, sv, (int)m, less, nt, src, vs);
    } else {
    if constexpr (GSS_SMALL_CPASYNC && sizeof(Key) == 8) {
    // the bucket goes global -> shared by asynchronous copies (no registers,
    // every copy of the thread in flight at once)
    for (uint32_t q = threadIdx.x; q < m; q += nt) {
      asm volatile("cp.async.ca.shared.global [%0], [%1], %2;" ::"r"((uint32_t)__cvta_generic_to_shared(sk + phys(q))),
                   "l"(src + q), "n"(sizeof(Key)));
      if constexpr (kHasVal<Val>)
        asm volatile("cp.async.ca.shared.global [%0], [%1], %2;" ::"r"((uint32_t)__cvta_generic_to_shared(sv + phys(q))),
                     "l"(vs + q), "n"(sizeof(Val)));
    }
    asm volatile("cp.async.wait_all;" ::: "memory");
    } else {
    // load the bucket with LU independent loads in flight per thread
    constexpr int LU = 4;
    for (uint32_t q0 = threadIdx.x; q0 < m; q0 += LU * nt) {
      Key tk[LU];
      Val tv[LU];
#pragma unroll
      for (int u = 0; u < LU; u++) {
        const uint32_t q = q0 + u * nt;
        if (q < m) {
          tk[u] = src[q];
          if constexpr (kHasVal<Val>) tv[u] = vs[q];
        }
      }
#pragma unroll
      for (int u = 0; u < LU; u++) {
        const uint32_t q = q0 + u * nt;
        if (q < m) {
          sk[phys(q)] = tk[u];
          if constexpr (kHasVal<Val>) sv[phys(q)] = tv[u];
        }
      }
    }
    }
    Sorter::sort(sk, sv, (int)m, less, nt);
    }
    for (uint32_t q = threadIdx.x; q < m; q += nt) c.kout[I.lo + q] = sk[phys(q)];
    if constexpr (kHasVal<Val>)
      for (uint32_t q = threadIdx.x; q < m; q += nt) c.vout[I.lo + q] = sv[phys(q)];
    if (nt == 32) __syncwarp(); else __syncthreads();
  }
}

// ---------------------------------------------------------------------------
// Cluster-wide bucket sort (GSS_FLAG_CLUSTER_SORT): buckets
// larger than one CTA's shared memory -- the range where the paper falls
// back to a global-memory quicksort before its M = 2^17 --
// are sorted by a cluster of kClusterCtas CTAs (one per SM) through
// distributed shared memory.  CTA r loads slice [s_r, s_r+1) of the bucket
// (s_r = floor(r m / CL)), sorts it with CtaSort, then log2(CL) merge rounds
// pair ever larger groups of slices: each CTA produces the output positions of
// its own slice by a merge-path search and a sequential merge whose operands
// are read from the other CTAs' shared memory (ld through
// cluster.map_shared_rank), into its second buffer; a cluster barrier
// separates the rounds.  Ties take A first; the sort stays unstable.
// ---------------------------------------------------------------------------
constexpr int kClusterCtas = 8;
constexpr int kClusterThreads = 512;
template <class Key, class Val>
constexpr uint32_t cluster_slice() { return (uint32_t)kClusterThreads * (uint32_t)small_items<Key, Val>(); }
template <class Key, class Val>
constexpr uint32_t cluster_capacity() { return (uint32_t)kClusterCtas * cluster_slice<Key, Val>(); }
template <class Key, class Val>
constexpr size_t cluster_smem_bytes() {
  return 2 * (size_t)padded_len((int)cluster_slice<Key, Val>()) * (sizeof(Key) + (kHasVal<Val> ? sizeof(Val) : 0)) + 256;
}

template <class Key, class Val, class IdT, class Cmp>
__global__ void __cluster_dims__(kClusterCtas, 1, 1) __launch_bounds__(kClusterThreads, 1)
    k_small_cluster(Ctx<Key, Val, IdT> c) {
  extern __shared__ __align__(16) unsigned char smem_raw[];
  namespace cg = cooperative_groups;
  cg::cluster_group cl = cg::this_cluster();
  constexpr int CL = kClusterCtas;
  constexpr int ITEMS = small_items<Key, Val>();
  constexpr uint32_t C = cluster_slice<Key, Val>();
  constexpr int PL = padded_len((int)C);
  using Sorter = CtaSort<Key, Val, kClusterThreads, Cmp, ITEMS>;
  const Cmp less;
  const uint32_t r = cl.block_rank();
  Key* kb[2];
  Val* vb[2];
  kb[0] = reinterpret_cast<Key*>(smem_raw);
  kb[1] = kb[0] + PL;
  vb[0] = reinterpret_cast<Val*>(smem_raw + 2 * (size_t)PL * sizeof(Key));
  vb[1] = vb[0] + (kHasVal<Val> ? PL : 0);
  uint32_t* s_sl = reinterpret_cast<uint32_t*>(smem_raw + cluster_smem_bytes<Key, Val>() - 256);   // CL+1 slice starts
  const uint32_t ni = min(c.cnt->clus_count, c.cap_clus);
  const uint32_t ncl = gridDim.x / CL;
  for (uint32_t i = blockIdx.x / CL; i < ni; i += ncl) {
    const Item I = c.clus[i];
    const uint32_t m = I.m;
    if (threadIdx.x <= (uint32_t)CL) s_sl[threadIdx.x] = (uint32_t)(((uint64_t)threadIdx.x * m) / CL);
    __syncthreads();
    const uint32_t s0 = s_sl[r], len = s_sl[r + 1] - s0;
    const Key* src = c.keys(I.buf) + I.lo;
    const Val* vsrc = nullptr;
    if constexpr (kHasVal<Val>) vsrc = c.vals(I.buf) + I.lo;
    for (uint32_t q = threadIdx.x; q < len; q += kClusterThreads) {
      kb[0][phys(q)] = src[s0 + q];
      if constexpr (kHasVal<Val>) vb[0][phys(q)] = vsrc[s0 + q];
    }
    Sorter::sort(kb[0], vb[0], (int)len, less);                    // the CTA's slice, ascending
    cl.sync();                                                      // every slice sorted
    uint32_t cur = 0;
    // the bucket position pos lives in CTA owner(pos) at local slot pos - s_owner
    auto owner = [&](uint32_t pos) -> uint32_t {
      uint32_t o = (uint32_t)(((uint64_t)CL * (pos + 1) + m - 1) / m) - 1;
      return min(o, (uint32_t)CL - 1);
    };
    auto ldk = [&](uint32_t pos) -> Key {
      const uint32_t o = owner(pos);
      const Key* rk = cl.map_shared_rank(kb[cur], o);
      return rk[phys(pos - s_sl[o])];
    };
    auto ldv = [&](uint32_t pos) -> Val {
      const uint32_t o = owner(pos);
      const Val* rv = cl.map_shared_rank(vb[cur], o);
      return rv[phys(pos - s_sl[o])];
    };
    for (int w = 1; w < CL; w *= 2) {
      const uint32_t g = r / (2 * w);
      const uint32_t a0 = s_sl[g * 2 * w], b0 = s_sl[min(g * 2 * w + w, (uint32_t)CL)];
      const uint32_t b1 = s_sl[min(g * 2 * w + 2 * w, (uint32_t)CL)];
      const uint32_t aLen = b0 - a0, bLen = b1 - b0;
      Key* ok = kb[cur ^ 1];
      Val* ov = vb[cur ^ 1];
      for (uint32_t o0 = threadIdx.x * ITEMS; o0 < len; o0 += kClusterThreads * ITEMS) {
        const uint32_t cnt = min((uint32_t)ITEMS, len - o0);
        const uint32_t d = s0 - a0 + o0;                            // output diagonal inside the pair
        // j = number of A keys among the first d outputs (A first on ties):
        // the smallest j in [lo, hi) with B[d-1-j] < A[j], else hi
        uint32_t lo = d > bLen ? d - bLen : 0, hi = min(d, aLen);
        while (lo < hi) {
          const uint32_t mid = (lo + hi) >> 1;
          if (less(ldk(b0 + d - 1 - mid), ldk(a0 + mid))) hi = mid;
          else lo = mid + 1;
        }
        uint32_t xa = lo, xb = d - lo;
        Key ka{}, kbk{};
        Val va{}, vbv{};
        if (xa < aLen) { ka = ldk(a0 + xa); if constexpr (kHasVal<Val>) va = ldv(a0 + xa); }
        if (xb < bLen) { kbk = ldk(b0 + xb); if constexpr (kHasVal<Val>) vbv = ldv(b0 + xb); }
        for (uint32_t j = 0; j < cnt; j++) {
          const bool ta = xb >= bLen || (xa < aLen && !less(kbk, ka));
          ok[phys(o0 + j)] = ta ? ka : kbk;
          if constexpr (kHasVal<Val>) ov[phys(o0 + j)] = ta ? va : vbv;
          if (ta) {
            if (++xa < aLen) { ka = ldk(a0 + xa); if constexpr (kHasVal<Val>) va = ldv(a0 + xa); }
          } else {
            if (++xb < bLen) { kbk = ldk(b0 + xb); if constexpr (kHasVal<Val>) vbv = ldv(b0 + xb); }
          }
        }
      }
      cl.sync();                                                    // every read of this round's input is done
      cur ^= 1;
    }
    for (uint32_t q = threadIdx.x; q < len; q += kClusterThreads) {
      c.kout[I.lo + s0 + q] = kb[cur][phys(q)];
      if constexpr (kHasVal<Val>) c.vout[I.lo + s0 + q] = vb[cur][phys(q)];
    }
    cl.sync();                                                      // buffers free for the next bucket
  }
}

// ---------------------------------------------------------------------------
// GSS_FLAG_SPLIT_SORT (ablation) for classes of two or more warps: one more sample-sort split inside
// the SM -- the paper's "sample sort based" chunk sorter,
// re-derived for B200 -- so that no merge round ever spans more than one
// warp (those rounds need a block barrier each and the longest merge-path
// searches):
//   B. warp 0 draws S = 128 (or 256) sample keys at hashed positions (R2,
//      level tag 254), sorts them in registers (bitonic network, shuffles) and
//      lays the k2 - 1 splitters out as the implicit tree
//   C. every key (streamed from global memory) descends the tree
//      (Algorithm 2; ties go left, R3); its sub-bucket id is kept
//      in shared memory and the sub-bucket sizes are counted with shared atomics
//   D. warp 0: sub-bucket offsets; consecutive sub-buckets are packed greedily
//      into segments of at most WCAP keys (one warp's sort capacity), each
//      starting at a 16-aligned shared slot
//   E. every key (read again: L2 hits) takes the next slot of its sub-bucket
//      (one shared atomic; the order inside a sub-bucket is irrelevant)
//   F. each warp merge-sorts whole segments with warp barriers only and writes
//      them out: sub-buckets are ordered ranges, so the concatenation of the
//      sorted segments is the sorted bucket.
// A sub-bucket larger than WCAP (heavy duplicates) or more than kMaxSegs
// segments hands the bucket to k_small_block (the fb list).
// ---------------------------------------------------------------------------
constexpr int kSubMaxK = 256;            // sub-buckets per bucket (power of two; ids are u8)
constexpr int kMaxSegs = 128;            // warp segments per bucket
constexpr int kSegSlack = 16 * kMaxSegs; // alignment slack (slots)

// keys per lane of the segment sorter: 16 for 4-byte keys, else 8 (64 registers)
#ifndef GSS_SEG_ITEMS_WIDE
#define GSS_SEG_ITEMS_WIDE 16
#endif
template <class Key, class Val>
constexpr int seg_items() { return (sizeof(Key) + (kHasVal<Val> ? sizeof(Val) : 0)) > 8 ? 8 : GSS_SEG_ITEMS_WIDE; }

// Dynamic shared memory of the split sorter for a class of capacity cap:
// key (+ value) slots plus alignment slack, and one u8 sub-bucket id per key.
template <class Key, class Val>
__host__ __device__ constexpr size_t small_smem_bytes(uint32_t cap) {
  return (size_t)padded_len((int)cap + kSegSlack) * (sizeof(Key) + (kHasVal<Val> ? sizeof(Val) : 0)) + cap;
}

// Bitonic sort of 32 * P keys held P per lane in registers (lane l holds
// sorted positions l*P .. l*P + P - 1 afterwards): in-lane compare-exchanges
// for strides < P, shuffles across lanes for the others.  Used for the
// split's sample (the sample sort "fits in shared memory", P:347-349 --
// here it fits in one warp's registers).
template <int P, class Key, class Cmp>
__device__ __forceinline__ void warp_bitonic_sort(Key (&x)[P], Cmp less) {
  const int lane = threadIdx.x & 31;
#pragma unroll
  for (int k = 2; k <= 32 * P; k <<= 1) {
#pragma unroll
    for (int j = k >> 1; j > 0; j >>= 1) {
      if (j >= P) {
        const int lj = j / P;
        const bool lower = (lane & lj) == 0;
#pragma unroll
        for (int i = 0; i < P; i++) {
          const bool up = ((lane * P + i) & k) == 0;
          const Key y = __shfl_xor_sync(kFull, x[i], lj);
          const bool take = (lower == up) ? less(y, x[i]) : less(x[i], y);
          x[i] = take ? y : x[i];
        }
      } else {
#pragma unroll
        for (int i = 0; i < P; i++) {
          if ((i & j) == 0) {
            const bool up = ((lane * P + i) & k) == 0;
            const bool sw = up ? less(x[i + j], x[i]) : less(x[i], x[i + j]);
            const Key a = sw ? x[i + j] : x[i], b = sw ? x[i] : x[i + j];
            x[i] = a;
            x[i + j] = b;
          }
        }
      }
    }
  }
}

// Warp 0 of the split: S = 32 * P sample keys at hashed positions (R2, level
// tag 254), sorted in registers; splitter i = S[(i + 1) * S / k2] goes to
// node j of the implicit tree (D1) via a shared staging array.
template <int P, class Key, class Cmp>
__device__ __forceinline__ void split_splitters(const Key* src, uint64_t seed, uint64_t lo, uint32_t m, uint32_t k2,
                                                Key* stage, Key* tree) {
  const int lane = threadIdx.x & 31;
  Key x[P];
#pragma unroll
  for (int i = 0; i < P; i++) x[i] = src[sample_pos(seed, 254, lo, (uint64_t)(lane * P + i), m)];
  warp_bitonic_sort<P>(x, Cmp());
#pragma unroll
  for (int i = 0; i < P; i++) stage[lane * P + i] = x[i];
  __syncwarp();
  const uint32_t r = (32u * P) / k2;                      // oversampling
  for (uint32_t j = lane + 1; j < k2; j += 32) {
    const uint32_t d = ilog2(j), q = j - (1u << d);
    const uint32_t si = ((2 * q + 1) * k2) >> (d + 1);    // splitter index + 1
    tree[j] = stage[si * r];
  }
}

template <class Key>
struct SmallSplitShared {
  Key tree[kSubMaxK];                    // tree[1 .. k2-1]
  uint32_t cnt[kSubMaxK];                // sub-bucket sizes, then slot cursors
  uint32_t pre[kSubMaxK + 1];            // exclusive prefix of the sizes
  uint32_t nxt[kSubMaxK];                // greedy packing: first sub-bucket after a segment started here
  int32_t mark[kSubMaxK];                // segment index at a segment's first sub-bucket, else -1
  uint32_t seg_smem[kMaxSegs], seg_out[kMaxSegs], seg_len[kMaxSegs];
  uint32_t nseg, fallback;
};

// At most kSplitMaxThreads threads: the 16-key-per-lane segment sort of
// 8-byte keys needs about 72 registers; larger classes get more segments
// per warp (the keys are streamed, so the block size is free).
constexpr int kSplitMaxThreads = 448;

template <class Key, class Val, class IdT, class Cmp>
__global__ void __launch_bounds__(kSplitMaxThreads, 2)
    k_small(Ctx<Key, Val, IdT> c, uint32_t cls) {
  extern __shared__ __align__(16) unsigned char smem_raw[];
  __shared__ SmallSplitShared<Key> sh;
  constexpr int ITEMS = small_items<Key, Val>();
  constexpr int WITEMS = seg_items<Key, Val>();
  constexpr uint32_t WCAP = 32 * WITEMS;                   // one warp's sort capacity
  constexpr uint32_t kSubMean = WCAP / 4;                  // target keys per sub-bucket
  using WSort = CtaSort<Key, Val, 32, Cmp, WITEMS>;
  const int nt = (int)blockDim.x;
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5, nw = nt >> 5;
  const uint32_t cap = c.class_cap[cls];
  const size_t slots = (size_t)padded_len((int)cap + kSegSlack);
  Key* sk = reinterpret_cast<Key*>(smem_raw);
  Val* sv = reinterpret_cast<Val*>(smem_raw + slots * sizeof(Key));
  uint8_t* sid = smem_raw + slots * (sizeof(Key) + (kHasVal<Val> ? sizeof(Val) : 0));
  const Cmp less;
  const uint32_t ni = min(c.cnt->small_count[cls], c.cap_small[cls]);
  const Item* list = c.small[cls];
  for (uint32_t i = blockIdx.x; i < ni; i += gridDim.x) {
    const Item I = list[i];
    const uint32_t m = I.m;
    const Key* src = c.keys(I.buf) + I.lo;
    const Val* vs = nullptr;
    if constexpr (kHasVal<Val>) vs = c.vals(I.buf) + I.lo;
    // ---- A. clear the sub-bucket tables
    uint32_t k2 = 2;
    while (k2 < (uint32_t)kSubMaxK && k2 * kSubMean < m) k2 <<= 1;
    for (uint32_t j = threadIdx.x; j < k2; j += nt) {
      sh.cnt[j] = 0;
      sh.mark[j] = -1;
    }
    // ---- B. warp 0: sample, sort it in registers, splitter tree
    if (warp == 0) {
      if (k2 <= 128) split_splitters<4, Key, Cmp>(src, c.seed, I.lo, m, k2, sk, sh.tree);
      else split_splitters<8, Key, Cmp>(src, c.seed, I.lo, m, k2, sk, sh.tree);
    }
    __syncthreads();
    // ---- C. descend (Algorithm 2), count, keep the id (keys streamed from
    // global memory, GR per thread in flight; no keys held across barriers)
    {
      const uint32_t logk = ilog2(k2);
      constexpr int GR = 4;
      for (uint32_t q0 = threadIdx.x; q0 < m; q0 += GR * nt) {
        Key e[GR];
        uint32_t jj[GR];
#pragma unroll
        for (int u = 0; u < GR; u++) {
          const uint32_t q = q0 + u * nt;
          if (q < m) e[u] = src[q];
          jj[u] = 1;
        }
        for (uint32_t d = 0; d < logk; d++) {
#pragma unroll
          for (int u = 0; u < GR; u++) jj[u] = 2 * jj[u] + (less(sh.tree[jj[u]], e[u]) ? 1u : 0u);
        }
#pragma unroll
        for (int u = 0; u < GR; u++) {
          const uint32_t q = q0 + u * nt;
          if (q < m) {
            const uint32_t id = jj[u] - k2;
            sid[q] = (uint8_t)id;
            red_shared_add((uint32_t)__cvta_generic_to_shared(&sh.cnt[id]), 1u);
          }
        }
      }
    }
    __syncthreads();
    // ---- D. offsets, greedy segments, slot cursors (warp 0; lane l owns
    // sub-buckets [l*PER, l*PER + PER))
    if (warp == 0) {
      constexpr int PER = kSubMaxK / 32;
      const uint32_t j0 = lane * PER, j1 = min(j0 + PER, k2);
      uint32_t sum = 0, mx = 0;
#pragma unroll 1
      for (uint32_t j = j0; j < j1; j++) { const uint32_t x = sh.cnt[j]; sum += x; mx = max(mx, x); }
      uint32_t incl = sum;
#pragma unroll
      for (int o = 1; o < 32; o <<= 1) {
        const uint32_t y = __shfl_up_sync(kFull, incl, o);
        if (lane >= o) incl += y;
      }
      uint32_t run = incl - sum;
#pragma unroll 1
      for (uint32_t j = j0; j < j1; j++) { sh.pre[j] = run; run += sh.cnt[j]; }
      if (lane == 0) sh.pre[k2] = m;
      mx = warp_max32(mx);
      __syncwarp();
      bool fb = mx > WCAP;
      if (!fb) {
#pragma unroll 1
        for (uint32_t j = j0; j < j1; j++) {
          const uint32_t target = sh.pre[j] + WCAP;
          uint32_t lo = j + 1, hi = k2;                    // largest e with pre[e] <= target
          while (lo < hi) {
            const uint32_t mid = (lo + hi + 1) >> 1;
            if (sh.pre[mid] <= target) lo = mid; else hi = mid - 1;
          }
          sh.nxt[j] = lo;
        }
        __syncwarp();
        if (lane == 0) {
          uint32_t sb = 0, n = 0, slot = 0;
          while (sb < k2 && n < (uint32_t)kMaxSegs) {
            const uint32_t e = sh.nxt[sb];
            const uint32_t len = sh.pre[e] - sh.pre[sb];
            sh.seg_smem[n] = slot; sh.seg_out[n] = sh.pre[sb]; sh.seg_len[n] = len;
            sh.mark[sb] = (int32_t)n;
            slot += (len + 15u) & ~15u;
            n++;
            sb = e;
          }
          sh.nseg = n;
          sh.fallback = sb < k2 ? 1u : 0u;
        }
        __syncwarp();
        fb = sh.fallback != 0;
      }
      if (fb) {
        if (lane == 0) {
          sh.fallback = 1;
          const uint32_t slot = atomicAdd(&c.cnt->fb_count, 1u);
          if (slot < c.cap_fb) c.fb[slot] = I;
          else atomicOr(&c.cnt->err, 16u);
        }
      } else {
        // segment of sub-bucket j = the last mark at or before j (prefix max)
        int32_t gm = -1;
#pragma unroll 1
        for (uint32_t j = j0; j < j1; j++) gm = max(gm, sh.mark[j]);
#pragma unroll
        for (int o = 1; o < 32; o <<= 1) {
          const int32_t y = __shfl_up_sync(kFull, gm, o);
          if (lane >= o) gm = max(gm, y);
        }
        int32_t g = __shfl_up_sync(kFull, gm, 1);
        if (lane == 0) g = -1;
#pragma unroll 1
        for (uint32_t j = j0; j < j1; j++) {
          g = max(g, sh.mark[j]);
          sh.cnt[j] = sh.seg_smem[g] + sh.pre[j] - sh.seg_out[g];
        }
      }
    }
    __syncthreads();
    if (sh.fallback) {                                     // k_small_block sorts it later
      __syncthreads();
      continue;
    }
    // ---- E. every key (and value) takes the next slot of its sub-bucket
    {
      constexpr int GR = 4;
      for (uint32_t q0 = threadIdx.x; q0 < m; q0 += GR * nt) {
        Key e[GR];
        Val v[GR];
#pragma unroll
        for (int u = 0; u < GR; u++) {
          const uint32_t q = q0 + u * nt;
          if (q < m) {
            e[u] = src[q];
            if constexpr (kHasVal<Val>) v[u] = vs[q];
          }
        }
#pragma unroll
        for (int u = 0; u < GR; u++) {
          const uint32_t q = q0 + u * nt;
          if (q < m) {
            const uint32_t pos = atomicAdd(&sh.cnt[sid[q]], 1u);
            sk[phys(pos)] = e[u];
            if constexpr (kHasVal<Val>) sv[phys(pos)] = v[u];
          }
        }
      }
    }
    __syncthreads();
    // ---- F. warps sort whole segments and write them out
    {
      Key* kout = c.kout + I.lo;
      Val* vout = nullptr;
      if constexpr (kHasVal<Val>) vout = c.vout + I.lo;
      const uint32_t nseg = sh.nseg;
      for (uint32_t g = warp; g < nseg; g += nw) {
        const uint32_t base = sh.seg_smem[g], len = sh.seg_len[g], out = sh.seg_out[g];
        Key* gk = sk + phys(base);                         // base is 16-aligned: phys(base + r) = phys(base) + phys(r)
        Val* gv = nullptr;
        if constexpr (kHasVal<Val>) gv = sv + phys(base);
        if (len > 1) WSort::sort(gk, gv, (int)len, less);
        for (uint32_t r = lane; r < len; r += 32) {
          kout[out + r] = gk[phys(r)];
          if constexpr (kHasVal<Val>) vout[out + r] = gv[phys(r)];
        }
      }
    }
    __syncthreads();
  }
}

// Final equality buckets larger than the in-SM capacity that did not end in
// keys_out: moved tile by tile.
// dst[0..m) = src[0..m) by one CTA: 16-byte vectors (source and destination share their alignment:
// the same index of two 256-byte aligned buffers) with four in flight per thread, scalar ends.
template <class T>
__device__ __forceinline__ void cta_copy(T* __restrict__ dst, const T* __restrict__ src, uint32_t m) {
  constexpr uint32_t A = 16 / sizeof(T);
  const uint32_t mis = (uint32_t)((reinterpret_cast<uintptr_t>(src) & 15u) / sizeof(T));
  const uint32_t head = min(m, (A - mis) & (A - 1));
  const uint32_t nv = (m - head) / A;
  for (uint32_t q = threadIdx.x; q < head; q += blockDim.x) dst[q] = src[q];
  const uint4* vs = reinterpret_cast<const uint4*>(src + head);
  uint4* vd = reinterpret_cast<uint4*>(dst + head);
  constexpr int U = 4;
  for (uint32_t q0 = threadIdx.x; q0 < nv; q0 += U * blockDim.x) {
    uint4 t[U];
#pragma unroll
    for (int u = 0; u < U; u++) {
      const uint32_t q = q0 + u * blockDim.x;
      if (q < nv) t[u] = vs[q];
    }
#pragma unroll
    for (int u = 0; u < U; u++) {
      const uint32_t q = q0 + u * blockDim.x;
      if (q < nv) vd[q] = t[u];
    }
  }
  for (uint32_t q = head + nv * A + threadIdx.x; q < m; q += blockDim.x) dst[q] = src[q];
}

template <class Key, class Val, class IdT>
__global__ void k_copy(Ctx<Key, Val, IdT> c) {
  const uint32_t ni = min(c.cnt->copy_count, c.cap_copy);
  for (uint32_t i = blockIdx.x; i < ni; i += gridDim.x) {
    const Item I = c.copy[i];
    cta_copy(c.kout + I.lo, c.keys(I.buf) + I.lo, I.m);
    if constexpr (kHasVal<Val>) cta_copy(c.vout + I.lo, c.vals(I.buf) + I.lo, I.m);
  }
}

// ---------------------------------------------------------------------------
// Fallback for buckets still larger than M after the last launched level
// (only reachable with adversarial inputs or a small max_levels): one CTA
// sorts the bucket with in-SM sorted runs and global merge-path passes that
// ping-pong between the bucket's ranges in the two buffers.
// ---------------------------------------------------------------------------
template <class Key, class Val, class Cmp>
__device__ void merge_pass_global(const Key* __restrict__ ks, const Val* __restrict__ vs, Key* __restrict__ kd,
                                  Val* __restrict__ vd, uint32_t m, uint32_t w, int nt, Cmp less) {
  for (uint32_t o = threadIdx.x; o < m; o += nt) {
    const uint32_t ps = (o / (2 * w)) * (2 * w);
    const uint32_t aLen = min(w, m - ps);
    const uint32_t bLen = (m - ps > w) ? min(w, m - ps - w) : 0;
    const uint32_t diag = o - ps;
    uint32_t lo = diag > bLen ? diag - bLen : 0, hi = min(diag, aLen);
    while (lo < hi) {
      uint32_t mid = (lo + hi) >> 1;
      if (less(ks[ps + w + diag - 1 - mid], ks[ps + mid])) hi = mid; else lo = mid + 1;
    }
    const uint32_t ai = lo, bi = diag - lo;
    bool takeA = (bi >= bLen) || (ai < aLen && !less(ks[ps + w + bi], ks[ps + ai]));
    const uint32_t from = takeA ? ps + ai : ps + w + bi;
    kd[o] = ks[from];
    if constexpr (kHasVal<Val>) vd[o] = vs[from];
  }
}

template <class Key, class Val, class IdT, class Cmp, int NT>
__global__ void __launch_bounds__(NT, 1) k_overflow(Ctx<Key, Val, IdT> c) {
  extern __shared__ __align__(16) unsigned char smem_raw[];
  using Sorter = CtaSort<Key, Val, NT, Cmp>;
  Key* sk = reinterpret_cast<Key*>(smem_raw);
  Val* sv = reinterpret_cast<Val*>(smem_raw + (size_t)Sorter::PL * sizeof(Key));
  const Cmp less;
  const uint32_t ni = min(c.cnt->ovf_count, c.cap_ovf);
  constexpr uint32_t CH = Sorter::C;
  for (uint32_t i = blockIdx.x; i < ni; i += gridDim.x) {
    const Item I = c.ovf[i];
    uint32_t cur = I.buf, oth = (I.buf == BUF_TMP) ? BUF_OUT : BUF_TMP;
    Key* kx = c.wkeys(cur);
    Val* vx = nullptr;
    if constexpr (kHasVal<Val>) vx = c.wvals(cur);
    for (uint32_t c0 = 0; c0 < I.m; c0 += CH) {
      const uint32_t len = min(CH, I.m - c0);
      for (uint32_t q = threadIdx.x; q < len; q += NT) sk[phys(q)] = kx[I.lo + c0 + q];
      if constexpr (kHasVal<Val>)
        for (uint32_t q = threadIdx.x; q < len; q += NT) sv[phys(q)] = vx[I.lo + c0 + q];
      Sorter::sort(sk, sv, (int)len, less);
      for (uint32_t q = threadIdx.x; q < len; q += NT) kx[I.lo + c0 + q] = sk[phys(q)];
      if constexpr (kHasVal<Val>)
        for (uint32_t q = threadIdx.x; q < len; q += NT) vx[I.lo + c0 + q] = sv[phys(q)];
      __syncthreads();
    }
    for (uint32_t w = CH; w < I.m; w *= 2) {
      const Val* vs = nullptr;
      Val* vd = nullptr;
      if constexpr (kHasVal<Val>) { vs = c.wvals(cur) + I.lo; vd = c.wvals(oth) + I.lo; }
      merge_pass_global<Key, Val, Cmp>(c.wkeys(cur) + I.lo, vs, c.wkeys(oth) + I.lo, vd, I.m, w, NT,
                                       less);
      __syncthreads();
      uint32_t tmp = cur; cur = oth; oth = tmp;
    }
    if (cur != BUF_OUT) {
      for (uint32_t q = threadIdx.x; q < I.m; q += NT) c.kout[I.lo + q] = c.wkeys(cur)[I.lo + q];
      if constexpr (kHasVal<Val>)
        for (uint32_t q = threadIdx.x; q < I.m; q += NT) c.vout[I.lo + q] = c.wvals(cur)[I.lo + q];
    }
    __syncthreads();
  }
}

// gss_partition outputs: splitters, K+1 bucket boundaries, {kb, ks, eq, K}.
template <class Key, class Val, class IdT>
__global__ void k_partition_out(Ctx<Key, Val, IdT> c, Key* spl_out, uint64_t* off_out, uint32_t* info_out,
                                uint64_t* counts_out) {
  const Bucket B = c.bk[0][0];
  const uint32_t* hist = c.hist[0] + B.hist_base;
  const uint32_t hb = hist[0];
  if (threadIdx.x == 0 && info_out) {
    info_out[0] = B.kb; info_out[1] = B.ks; info_out[2] = B.eq; info_out[3] = B.K;
  }
  if (spl_out)
    for (uint32_t i = threadIdx.x; i + 1 < B.ks; i += blockDim.x) spl_out[i] = c.spl[0][B.spl_base + B.kb + i];
  for (uint32_t id = threadIdx.x; id <= B.K; id += blockDim.x) {
    uint64_t s = id < B.K ? (uint64_t)(hist[id * B.ntiles] - hb) : (uint64_t)B.m;
    if (off_out) off_out[id] = s;
    if (counts_out && id < B.K) {
      uint64_t e = id + 1 < B.K ? (uint64_t)(hist[(id + 1) * B.ntiles] - hb) : (uint64_t)B.m;
      counts_out[id] = e - s;
    }
  }
}

// gss_sample: s keys at hashed positions (the distributed global sample).
template <class Key>
__global__ void k_gather_sample(const Key* keys, uint64_t n, uint64_t lo_global, uint32_t level, uint64_t seed,
                                Key* out, uint64_t s) {
  for (uint64_t j = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; j < s; j += (uint64_t)gridDim.x * blockDim.x)
    out[j] = keys[sample_pos(seed, level, lo_global, j, n)];
}

}  // namespace gss
