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

#include "gss_device.cuh"

namespace gss {

constexpr int kClsThreads = 256;
constexpr int kScatterThreads = 256;
constexpr int kScatterIter = 8;                                   // keys per thread per chunk
constexpr int kChunk = kScatterThreads * kScatterIter;            // 2048 keys staged per chunk
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
  uint32_t nt = (c.n + c.T - 1) / c.T;
  Bucket B{};
  B.lo = 0; B.m = c.n; B.tile_start = 0; B.ntiles = nt; B.kb = kb;
  B.hist_base = 0; B.spl_base = 0;
  c.bk[0][0] = B;
  LevelCounters& L = c.cnt->lvl[0];
  L.num_buckets = 1; L.num_tiles = nt; L.hist_alloc = max(kb, 3u) * nt; L.spl_alloc = 2 * kb;
  L.split_elems = c.n;
}

// ---------------------------------------------------------------------------
// Phase 1: per split bucket, a*k_b keys at hashed positions
// (with replacement, R1/R2), sorted in shared memory by one CTA; splitters
// spl[i] = S[a(i+1)-1]; equality mode if two splitters are equal or k_b == 2
// (R4), then k_s = k_b/2 splitters S[(s/k_s)(i+1)-1]; the implicit tree
// bt[j] = s_{(2q+1) k_s / 2^(d+1)}.
// ---------------------------------------------------------------------------
template <class Key, class Val, class IdT, class Cmp>
__global__ void __launch_bounds__(kSampleThreads, 1) k_sample(Ctx<Key, Val, IdT> c, uint32_t level) {
  extern __shared__ __align__(16) unsigned char smem_raw[];
  Key* sk = reinterpret_cast<Key*>(smem_raw);
  using Sorter = CtaSort<Key, NoVal, kSampleThreads, Cmp>;
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
    for (uint32_t j = threadIdx.x; j < s; j += kSampleThreads)
      sk[phys(j)] = src[B.lo + sample_pos(c.seed, level, B.lo, j, B.m)];
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
// largest splitter and ids are clamped to nspl.
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
    g->ks = ks; g->eq = 0; g->K = nspl + 1; g->clamp = 1;
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
template <int LOGK, class Key, class IdT, class Cmp>
__device__ __forceinline__ void classify_tile(const Key* __restrict__ src, IdT* __restrict__ ids, uint32_t beg,
                                              uint32_t len, const Key* tree, const Key* spl, uint32_t ks,
                                              uint32_t K, bool eq, bool clamp, uint32_t* wc, Cmp less) {
  constexpr int U = 4;
  for (uint32_t i0 = threadIdx.x; i0 < len; i0 += U * kClsThreads) {
    Key e[U];
#pragma unroll
    for (int u = 0; u < U; u++) {
      uint32_t i = i0 + u * kClsThreads;
      if (i < len) e[u] = src[beg + i];
    }
#pragma unroll
    for (int u = 0; u < U; u++) {
      uint32_t i = i0 + u * kClsThreads;
      if (i < len) {
        uint32_t b = descend<LOGK>(tree, e[u], less);
        uint32_t id;
        if (eq) id = 2 * b + ((b + 1 < ks && !less(e[u], spl[b])) ? 1u : 0u);
        else id = clamp ? min(b, K - 1) : b;
        ids[beg + i] = (IdT)id;
        atomicAdd(&wc[id], 1u);
      }
    }
  }
}

template <class Key, class Val, class IdT, class Cmp>
__global__ void __launch_bounds__(kClsThreads) k_classify(Ctx<Key, Val, IdT> c, uint32_t level, uint32_t kmax) {
  extern __shared__ __align__(16) unsigned char smem_raw[];
  Key* tree = reinterpret_cast<Key*>(smem_raw);
  Key* spl = tree + kmax;
  uint32_t* wcnt = reinterpret_cast<uint32_t*>(spl + kmax);
  constexpr int NW = kClsThreads / 32;
  const Cmp less;
  const uint32_t slot = level & 1;
  const uint32_t nt = c.cnt->lvl[level].num_tiles;
  const Key* src = c.keys(c.src(level));
  const int w = threadIdx.x >> 5;
  uint32_t cur = 0xffffffffu;
  for (uint32_t t = blockIdx.x; t < nt; t += gridDim.x) {
    const uint32_t b = c.tile_bucket[slot][t];
    const Bucket B = c.bk[slot][b];
    if (b != cur) {
      for (uint32_t j = threadIdx.x + 1; j < B.ks; j += kClsThreads) tree[j] = c.spl[slot][B.spl_base + j];
      for (uint32_t j = threadIdx.x; j + 1 < B.ks; j += kClsThreads) spl[j] = c.spl[slot][B.spl_base + B.kb + j];
      cur = b;
    }
    for (uint32_t j = threadIdx.x; j < NW * kmax; j += kClsThreads) wcnt[j] = 0;
    __syncthreads();
    const uint32_t tl = t - B.tile_start;
    const uint32_t beg = B.lo + tl * c.T;
    const uint32_t len = min(c.T, B.m - tl * c.T);
    uint32_t* wc = wcnt + w * kmax;
    const bool eq = B.eq != 0, clamp = B.clamp != 0;
    switch (ilog2(B.ks)) {
#define GSS_CLS_CASE(L) \
  case L: classify_tile<L>(src, c.ids, beg, len, tree, spl, B.ks, B.K, eq, clamp, wc, less); break;
      GSS_CLS_CASE(0) GSS_CLS_CASE(1) GSS_CLS_CASE(2) GSS_CLS_CASE(3) GSS_CLS_CASE(4) GSS_CLS_CASE(5)
      GSS_CLS_CASE(6) GSS_CLS_CASE(7) GSS_CLS_CASE(8) GSS_CLS_CASE(9) GSS_CLS_CASE(10)
#undef GSS_CLS_CASE
      default: break;
    }
    __syncthreads();
    uint32_t* hist = c.hist[slot] + B.hist_base;
    for (uint32_t id = threadIdx.x; id < B.K; id += kClsThreads) {
      uint32_t s = 0;
#pragma unroll
      for (int q = 0; q < NW; q++) s += wcnt[q * kmax + id];
      hist[id * B.ntiles + tl] = s;
    }
    __syncthreads();
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
template <class Key, class Val>
struct ScatterSmem {
  static size_t bytes(uint32_t kmax) {
    size_t b = 0;
    b += (size_t)kmax * 4 * 3;                                  // gbase, ctot, cstart
    b += (size_t)(kScatterThreads / 32) * kmax * 4;             // per-warp counters
    b += 64;                                                    // scan scratch
    b = (b + 15) & ~size_t(15);
    b += (size_t)kChunk * sizeof(Key);
    if (kHasVal<Val>) b += (size_t)kChunk * sizeof(Val);
    b += (size_t)kChunk * 2;                                    // staged ids (u16)
    return b;
  }
};

template <class Key, class Val, class IdT, class Cmp>
__global__ void __launch_bounds__(kScatterThreads) k_scatter(Ctx<Key, Val, IdT> c, uint32_t level, uint32_t kmax) {
  extern __shared__ __align__(16) unsigned char smem_raw[];
  constexpr int NW = kScatterThreads / 32;
  uint32_t* gbase = reinterpret_cast<uint32_t*>(smem_raw);
  uint32_t* ctot = gbase + kmax;
  uint32_t* cstart = ctot + kmax;
  uint32_t* wcnt = cstart + kmax;
  uint32_t* s_warp = wcnt + NW * kmax;
  size_t off = ((size_t)(kmax * 3 + NW * kmax) * 4 + 64 + 15) & ~size_t(15);
  Key* skeys = reinterpret_cast<Key*>(smem_raw + off);
  off += (size_t)kChunk * sizeof(Key);
  Val* svals = reinterpret_cast<Val*>(smem_raw + off);
  if constexpr (kHasVal<Val>) off += (size_t)kChunk * sizeof(Val);
  uint16_t* sids = reinterpret_cast<uint16_t*>(smem_raw + off);

  const uint32_t slot = level & 1;
  const uint32_t nt = c.cnt->lvl[level].num_tiles;
  const uint32_t sb = c.src(level), db = c.dst(level);
  const Key* ksrc = c.keys(sb);
  Key* kdst = c.wkeys(db);
  const Val* vsrc = nullptr;
  Val* vdst = nullptr;
  if constexpr (kHasVal<Val>) { vsrc = c.vals(sb); vdst = c.wvals(db); }
  const int lane = threadIdx.x & 31, w = threadIdx.x >> 5;
  const uint32_t ltmask = lanemask_lt();

  for (uint32_t t = blockIdx.x; t < nt; t += gridDim.x) {
    const uint32_t b = c.tile_bucket[slot][t];
    const Bucket B = c.bk[slot][b];
    const uint32_t tl = t - B.tile_start;
    const uint32_t beg = B.lo + tl * c.T;
    const uint32_t len = min(c.T, B.m - tl * c.T);
    const uint32_t* hist = c.hist[slot] + B.hist_base;
    const uint32_t hb = hist[0];
    for (uint32_t id = threadIdx.x; id < B.K; id += kScatterThreads) gbase[id] = hist[id * B.ntiles + tl] - hb + B.lo;
    const uint32_t K = B.K;
    for (uint32_t c0 = 0; c0 < len; c0 += kChunk) {
      const uint32_t clen = min((uint32_t)kChunk, len - c0);
      uint32_t* wc = wcnt + w * kmax;
      for (uint32_t id = lane; id < K; id += 32) wc[id] = 0;
      __syncwarp();
      Key kk[kScatterIter];
      Val vv[kScatterIter];
      uint32_t iid[kScatterIter], rk[kScatterIter];
#pragma unroll
      for (int it = 0; it < kScatterIter; it++) {
        const uint32_t q = w * (32 * kScatterIter) + it * 32 + lane;
        iid[it] = 0xffffffffu;
        if (q < clen) {
          kk[it] = ksrc[beg + c0 + q];
          iid[it] = c.ids[beg + c0 + q];
          if constexpr (kHasVal<Val>) vv[it] = vsrc[beg + c0 + q];
        }
      }
#pragma unroll
      for (int it = 0; it < kScatterIter; it++) {
        const uint32_t id = iid[it];
        const uint32_t peers = __match_any_sync(kFull, id);
        const uint32_t lt = __popc(peers & ltmask);
        uint32_t cv = 0;
        if (id != 0xffffffffu) cv = wc[id];
        rk[it] = cv + lt;
        __syncwarp();
        if (id != 0xffffffffu && lt == 0) wc[id] = cv + __popc(peers);
        __syncwarp();
      }
      __syncthreads();
      for (uint32_t id = threadIdx.x; id < K; id += kScatterThreads) {
        uint32_t run = 0;
#pragma unroll
        for (int q = 0; q < NW; q++) {
          uint32_t x = wcnt[q * kmax + id];
          wcnt[q * kmax + id] = run;
          run += x;
        }
        ctot[id] = run;
      }
      __syncthreads();
      {
        // exclusive scan of ctot over ids -> cstart (each thread owns a run of ids)
        const uint32_t per = (K + kScatterThreads - 1) / kScatterThreads;
        const uint32_t i0 = threadIdx.x * per;
        uint32_t s = 0;
        for (uint32_t j = 0; j < per; j++)
          if (i0 + j < K) s += ctot[i0 + j];
        uint32_t ex = block_exclusive_scan<kScatterThreads>(s, s_warp, nullptr);
        for (uint32_t j = 0; j < per; j++)
          if (i0 + j < K) { cstart[i0 + j] = ex; ex += ctot[i0 + j]; }
      }
      __syncthreads();
#pragma unroll
      for (int it = 0; it < kScatterIter; it++) {
        const uint32_t id = iid[it];
        if (id != 0xffffffffu) {
          const uint32_t pos = cstart[id] + wc[id] + rk[it];
          skeys[pos] = kk[it];
          if constexpr (kHasVal<Val>) svals[pos] = vv[it];
          sids[pos] = (uint16_t)id;
        }
      }
      __syncthreads();
      for (uint32_t q = threadIdx.x; q < clen; q += kScatterThreads) {
        const uint32_t id = sids[q];
        const uint32_t d = gbase[id] + (q - cstart[id]);
        kdst[d] = skeys[q];
        if constexpr (kHasVal<Val>) vdst[d] = svals[q];
      }
      __syncthreads();
      for (uint32_t id = threadIdx.x; id < K; id += kScatterThreads) gbase[id] += ctot[id];
      __syncthreads();
    }
  }
}

// ---------------------------------------------------------------------------
// Recursion (Algorithm 1) with delayed small sorts: every
// child of every bucket split at this level becomes a next-level bucket
// (m > M), an in-SM sort item (m <= M), a final equality bucket (R4), or --
// past the last launched level -- an overflow item.
// ---------------------------------------------------------------------------
template <class Key, class Val, class IdT>
__device__ __forceinline__ void push_small(const Ctx<Key, Val, IdT>& c, uint32_t lo, uint32_t m, uint32_t buf) {
  uint32_t cls = 0;
  while (cls + 1 < kNumClasses && m > c.class_cap[cls]) cls++;
  uint32_t i = atomicAdd(&c.cnt->small_count[cls], 1u);
  if (i < c.cap_small[cls]) c.small[cls][i] = Item{lo, m, buf, 0};
  else atomicOr(&c.cnt->err, 1u);
  atomicAdd(&c.cnt->small_elems, (unsigned long long)m);
  atomicMax(&c.cnt->max_small, (unsigned long long)m);
}

template <class Key, class Val, class IdT>
__global__ void __launch_bounds__(kPlanThreads) k_plan(Ctx<Key, Val, IdT> c, uint32_t level) {
  const uint32_t slot = level & 1;
  const uint32_t nb = c.cnt->lvl[level].num_buckets;
  const uint32_t db = c.dst(level);
  const uint32_t next = level + 1;
  for (uint32_t b = blockIdx.x; b < nb; b += gridDim.x) {
    const Bucket B = c.bk[slot][b];
    const uint32_t* hist = c.hist[slot] + B.hist_base;
    const uint32_t hb = hist[0];
    for (uint32_t id = threadIdx.x; id < B.K; id += kPlanThreads) {
      const uint32_t start = hist[id * B.ntiles] - hb + B.lo;
      const uint32_t end = (id + 1 < B.K) ? hist[(id + 1) * B.ntiles] - hb + B.lo : B.lo + B.m;
      const uint32_t m = end - start;
      if (m == 0) continue;
      const bool is_eq = B.eq && (id & 1);
      if (is_eq) {
        atomicAdd(&c.cnt->eq_buckets, 1ull);
        atomicAdd(&c.cnt->eq_elems, (unsigned long long)m);
        if (db == BUF_OUT) continue;                       // all keys equal and already in place
        if (m <= c.class_cap[kNumClasses - 1]) {
          push_small(c, start, m, db);
        } else {
          uint32_t nt = (m + c.T - 1) / c.T;
          uint32_t i = atomicAdd(&c.cnt->copy_count, nt);
          if (i + nt <= c.cap_copy) {
            for (uint32_t q = 0; q < nt; q++) c.copy[i + q] = Item{start + q * c.T, min(c.T, m - q * c.T), db, 0};
          } else {
            atomicOr(&c.cnt->err, 2u);
          }
        }
      } else if (m <= c.M) {
        push_small(c, start, m, db);
      } else if (next < c.L) {
        const uint32_t kb = choose_kb(c.k, c.k_policy, c.fill_div, c.M, m);
        const uint32_t nt = (m + c.T - 1) / c.T;
        LevelCounters& NL = c.cnt->lvl[next];
        const uint32_t bi = atomicAdd(&NL.num_buckets, 1u);
        const uint32_t ts = atomicAdd(&NL.num_tiles, nt);
        const uint32_t hbn = atomicAdd(&NL.hist_alloc, max(kb, 3u) * nt);
        const uint32_t sbn = atomicAdd(&NL.spl_alloc, 2 * kb);
        atomicAdd(&NL.split_elems, (unsigned long long)m);
        if (bi < c.cap_buckets && ts + nt <= c.cap_tiles && hbn + max(kb, 3u) * nt <= c.cap_hist &&
            sbn + 2 * kb <= c.cap_spl) {
          Bucket nbk{};
          nbk.lo = start; nbk.m = m; nbk.tile_start = ts; nbk.ntiles = nt; nbk.kb = kb;
          nbk.hist_base = hbn; nbk.spl_base = sbn;
          c.bk[next & 1][bi] = nbk;
        } else {
          atomicOr(&c.cnt->err, 4u);
        }
      } else {
        uint32_t i = atomicAdd(&c.cnt->ovf_count, 1u);
        if (i < c.cap_ovf) c.ovf[i] = Item{start, m, db, 0};
        else atomicOr(&c.cnt->err, 8u);
        atomicAdd(&c.cnt->ovf_elems, (unsigned long long)m);
      }
    }
  }
}

// ---------------------------------------------------------------------------
// Sorting buckets: one CTA per bucket of at most M keys; the
// bucket is loaded to shared memory, sorted by CtaSort, written to keys_out.
// ---------------------------------------------------------------------------
template <class Key, class Val, class IdT, class Cmp, int NT>
__global__ void __launch_bounds__(NT, 1) k_small(Ctx<Key, Val, IdT> c, uint32_t cls) {
  extern __shared__ __align__(16) unsigned char smem_raw[];
  using Sorter = CtaSort<Key, Val, NT, Cmp>;
  Key* sk = reinterpret_cast<Key*>(smem_raw);
  Val* sv = reinterpret_cast<Val*>(smem_raw + (size_t)Sorter::PL * sizeof(Key));
  const Cmp less;
  const uint32_t ni = min(c.cnt->small_count[cls], c.cap_small[cls]);
  for (uint32_t i = blockIdx.x; i < ni; i += gridDim.x) {
    const Item I = c.small[cls][i];
    const Key* src = c.keys(I.buf);
    for (uint32_t q = threadIdx.x; q < I.m; q += NT) sk[phys(q)] = src[I.lo + q];
    if constexpr (kHasVal<Val>) {
      const Val* vs = c.vals(I.buf);
      for (uint32_t q = threadIdx.x; q < I.m; q += NT) sv[phys(q)] = vs[I.lo + q];
    }
    Sorter::sort(sk, sv, (int)I.m, less);
    for (uint32_t q = threadIdx.x; q < I.m; q += NT) c.kout[I.lo + q] = sk[phys(q)];
    if constexpr (kHasVal<Val>)
      for (uint32_t q = threadIdx.x; q < I.m; q += NT) c.vout[I.lo + q] = sv[phys(q)];
    __syncthreads();
  }
}

// Final equality buckets larger than the in-SM capacity that did not end in
// keys_out: moved tile by tile.
template <class Key, class Val, class IdT>
__global__ void k_copy(Ctx<Key, Val, IdT> c) {
  const uint32_t ni = min(c.cnt->copy_count, c.cap_copy);
  for (uint32_t i = blockIdx.x; i < ni; i += gridDim.x) {
    const Item I = c.copy[i];
    const Key* ks = c.keys(I.buf);
    for (uint32_t q = threadIdx.x; q < I.m; q += blockDim.x) c.kout[I.lo + q] = ks[I.lo + q];
    if constexpr (kHasVal<Val>) {
      const Val* vs = c.vals(I.buf);
      for (uint32_t q = threadIdx.x; q < I.m; q += blockDim.x) c.vout[I.lo + q] = vs[I.lo + q];
    }
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
