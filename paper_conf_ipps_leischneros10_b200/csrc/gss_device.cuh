// gss_device.cuh -- device-side data structures and primitives of the B200
// GPU sample sort (Leischner, Osipov & Sanders, IPDPS 2010; PAPER.md P:<line>).
//
// Written for sm_100a.  Everything here is integer work: unsigned compares,
// moves, counting and scans; no tensor cores (nothing is a contraction).
#pragma once

#include <cstdint>
#include <type_traits>
#include <cuda_runtime.h>

namespace gss {

// In-SM sort size classes (R8): class i holds the buckets sorted by a CTA of
// class_warps(i) warps, i.e. up to class_warps(i) * 32 * sort_items keys:
// 1..8 warps one by one, then 10, 12, 16, 24, 32.  Fine classes keep most
// threads of a bucket's CTA busy (with power-of-two classes a bucket just
// above a class boundary left half of its CTA idle at every merge barrier);
// few enough that the empty ones cost little in launch-bound sorts.
constexpr int kNumClasses = 13;
__host__ __device__ constexpr int class_warps(int i) {
  return i < 8 ? i + 1 : (i == 8 ? 10 : (i == 9 ? 12 : (i == 10 ? 16 : (i == 11 ? 24 : 32))));
}
constexpr int kMaxLevels = 16;        // distribution levels launched at most
constexpr uint32_t kFull = 0xffffffffu;

enum Buf : uint32_t { BUF_IN = 0, BUF_TMP = 1, BUF_OUT = 2 };
enum Mode : uint32_t { MODE_SORT = 0, MODE_PARTITION = 1, MODE_PARTITION_BY = 2 };

struct NoVal {};
template <class V> constexpr bool kHasVal = !std::is_same<V, NoVal>::value;

// Bit-exact reinterpretation (keys may be floating point).
template <class T, class U>
__device__ __forceinline__ T bit_cast_dev(const U& u) {
  static_assert(sizeof(T) == sizeof(U), "size mismatch");
  T t;
  memcpy(&t, &u, sizeof(T));
  return t;
}

// Keys are ordered only through a comparator.
struct Less {
  template <class T> __device__ __forceinline__ bool operator()(const T& a, const T& b) const { return a < b; }
};
struct Greater {
  template <class T> __device__ __forceinline__ bool operator()(const T& a, const T& b) const { return b < a; }
};
// Orders under which equivalent keys are bit-identical, so that a copy of a
// key is indistinguishable from the key (the in-SM sort's bounds-free merge
// and padding rely on it; any other comparator takes the safe paths).
template <class Cmp> struct BitwiseOrder : std::false_type {};
template <> struct BitwiseOrder<Less> : std::true_type {};
template <> struct BitwiseOrder<Greater> : std::true_type {};

// IEEE-754 total order for floating-point keys: -NaN < -inf < ... < -0 < +0 <
// ... < +inf < +NaN, i.e. a strict weak (in fact total) order on bit patterns.
struct TotalLess {
  __device__ __forceinline__ static uint32_t rank(float x) {
    const uint32_t b = bit_cast_dev<uint32_t>(x);
    return b ^ ((b >> 31) ? 0xffffffffu : 0x80000000u);
  }
  __device__ __forceinline__ static unsigned long long rank(double x) {
    const unsigned long long b = bit_cast_dev<unsigned long long>(x);
    return b ^ ((b >> 63) ? 0xffffffffffffffffull : 0x8000000000000000ull);
  }
  template <class T> __device__ __forceinline__ bool operator()(const T& a, const T& b) const {
    return rank(a) < rank(b);
  }
};
template <> struct BitwiseOrder<TotalLess> : std::true_type {};     // rank() is a bijection on bit patterns

// A bucket being split at some level (one row of the paper's k x p table
// per tile).
struct Bucket {
  uint32_t lo, m;          // range [lo, lo+m) of the level's source buffer
  uint32_t tile_start;     // first level-global tile index
  uint32_t ntiles;         // p = ceil(m / T)
  uint32_t kb;             // k_b: buckets asked for (R29)
  uint32_t ks;             // range buckets: k_b, or k_b/2 in equality mode (R4)
  uint32_t K;              // bucket ids: ks, or 2 ks - 1 in equality mode
  uint32_t eq;             // equality mode
  uint32_t hist_base;      // start of this bucket's K x ntiles histogram (bucket-major)
  uint32_t spl_base;       // start of its splitter storage: tree[kb] then sorted spl[kb]
  uint32_t clamp;          // partition_by: ids are min(b, K-1)
  uint32_t id_base;        // start of its stored bucket ids (16-byte aligned; tile t at id_base + t*T)
};

// A destination segment of a partition whose output goes to other GPUs
// (the fused global level of the distributed sort): partition indices
// [lo, hi) are stored at kdst[i] / vdst[i] (pointers pre-offset by -lo, into a
// peer's NCCL symmetric window).
struct RemoteSeg {
  uint32_t lo, hi, pad0, pad1;
  void* kdst;
  void* vdst;
};

struct Item {              // a final bucket (small sort / copy / overflow work)
  uint32_t lo, m, buf, pad;
};

struct LevelCounters {
  uint32_t num_buckets, num_tiles, hist_alloc, spl_alloc;
  unsigned long long split_elems;
  uint32_t id_alloc, pad;  // stored bucket ids: each bucket's range rounded up to 16 elements
};

struct Counters {
  LevelCounters lvl[kMaxLevels + 1];
  uint32_t small_count[kNumClasses];
  uint32_t copy_count, ovf_count, err, fb_count;   // fb: buckets the in-SM split hands to the block sort
  unsigned long long small_elems, max_small, eq_buckets, eq_elems, ovf_elems;
  uint32_t clus_count, pad_c;                       // buckets for the cluster-wide sort (GSS_FLAG_CLUSTER_SORT)
};

// Everything a kernel needs, passed by value.
template <class Key, class Val, class IdT>
struct Ctx {
  const Key* kin; Key* ktmp; Key* kout;
  const Val* vin; Val* vtmp; Val* vout;
  IdT* ids;
  Counters* cnt;
  Bucket* bk[2];
  uint32_t* tile_bucket[2];
  uint32_t* hist[2];
  Key* spl[2];
  Item* small[kNumClasses];
  Item* copy;
  Item* ovf;
  Item* fb;
  Item* clus;                        // buckets above one CTA's capacity, sorted by a thread-block cluster
  uint32_t* scan_part;
  const Key* given_spl;              // MODE_PARTITION_BY
  uint32_t given_nspl;
  uint32_t given_eq;                 // MODE_PARTITION_BY in equality mode (ids 2b / 2b+1)
  uint32_t cls_arrays;               // Phase-2 counter arrays per CTA (8 = one per warp)
  const RemoteSeg* remote;           // MODE_PARTITION_BY, phase 2: destinations on other GPUs
  uint32_t nremote;
  uint32_t n, M, T, k, a, k_policy, fill_div, sample_cap, L, mode, dst0, src0, stable;
  uint32_t recompute;                // GSS_FLAG_RECOMPUTE_IDS: no stored ids, Phase 4 re-descends
  uint32_t lut;                      // radix-indexed splitter lookup in Phase 2 (off: GSS_FLAG_TREE_CLASSIFY)
  uint32_t cap_buckets, cap_tiles, cap_hist, cap_spl, cap_copy, cap_ovf, cap_fb, cap_clus;
  uint32_t cap_small[kNumClasses];
  uint32_t class_cap[kNumClasses];
  uint64_t seed;

  __device__ __forceinline__ uint32_t dst(uint32_t l) const {
    uint32_t other = dst0 == BUF_TMP ? BUF_OUT : BUF_TMP;
    return (l & 1) ? other : dst0;
  }
  __device__ __forceinline__ uint32_t src(uint32_t l) const { return l == 0 ? src0 : dst(l - 1); }
  __device__ __forceinline__ const Key* keys(uint32_t b) const {
    return b == BUF_IN ? kin : (b == BUF_TMP ? ktmp : kout);
  }
  __device__ __forceinline__ Key* wkeys(uint32_t b) const { return b == BUF_TMP ? ktmp : kout; }
  __device__ __forceinline__ const Val* vals(uint32_t b) const {
    return b == BUF_IN ? vin : (b == BUF_TMP ? vtmp : vout);
  }
  __device__ __forceinline__ Val* wvals(uint32_t b) const { return b == BUF_TMP ? vtmp : vout; }
};

// --------------------------------------------------------------------------
// Sample positions: SplitMix64 counter hash (R2, replacing the paper's LCG
// seeded by a CPU Mersenne Twister).
// --------------------------------------------------------------------------
__device__ __forceinline__ uint64_t splitmix64(uint64_t x) {
  uint64_t z = x + 0x9E3779B97F4A7C15ull;
  z = (z ^ (z >> 30)) * 0xBF58476D1CE4E5B9ull;
  z = (z ^ (z >> 27)) * 0x94D049BB133111EBull;
  return z ^ (z >> 31);
}
__device__ __forceinline__ uint64_t sample_pos(uint64_t seed, uint32_t level, uint64_t lo, uint64_t j,
                                               uint64_t m) {
  uint64_t h = splitmix64(splitmix64(splitmix64(seed ^ ((uint64_t)level << 56)) ^ lo) ^ j);
  return __umul64hi(h, m);
}

// k_b rule: the paper's fixed k or the adaptive R29 rule.
__device__ __host__ __forceinline__ uint32_t choose_kb(uint32_t k, uint32_t policy, uint32_t f, uint64_t M,
                                                       uint64_t m) {
  if (policy == 2) return k;
  uint64_t want = (f * m + M - 1) / M;
  uint32_t kb = 1;
  while (kb < want && kb < k) kb <<= 1;
  if (kb < 4) kb = 4;
  if (kb > k) kb = k;
  return kb;
}

__device__ __forceinline__ uint32_t ilog2(uint32_t x) { return 31 - __clz(x); }
__device__ __forceinline__ uint32_t lanemask_lt() {
  uint32_t r;
  asm("mov.u32 %0, %%lanemask_lt;" : "=r"(r));
  return r;
}

// --------------------------------------------------------------------------
// Block-wide exclusive scan of one value per thread (NT threads).
// --------------------------------------------------------------------------
template <int NT>
__device__ __forceinline__ uint32_t block_exclusive_scan(uint32_t x, uint32_t* s_warp, uint32_t* total) {
  const int lane = threadIdx.x & 31, w = threadIdx.x >> 5;
  uint32_t inc = x;
#pragma unroll
  for (int o = 1; o < 32; o <<= 1) {
    uint32_t y = __shfl_up_sync(kFull, inc, o);
    if (lane >= o) inc += y;
  }
  if (lane == 31) s_warp[w] = inc;
  __syncthreads();
  if (w == 0) {
    uint32_t v = lane < NT / 32 ? s_warp[lane] : 0;
    uint32_t vi = v;
#pragma unroll
    for (int o = 1; o < 32; o <<= 1) {
      uint32_t y = __shfl_up_sync(kFull, vi, o);
      if (lane >= o) vi += y;
    }
    if (lane < NT / 32) s_warp[lane] = vi - v;
    if (lane == NT / 32 - 1 && total) *total = vi;
  }
  __syncthreads();
  uint32_t r = s_warp[w] + inc - x;
  __syncthreads();
  return r;
}

template <int NT>
__device__ __forceinline__ uint64_t block_sum_u64(uint64_t x, unsigned long long* s_red) {
  const int lane = threadIdx.x & 31, w = threadIdx.x >> 5;
#pragma unroll
  for (int o = 16; o > 0; o >>= 1) x += __shfl_xor_sync(kFull, x, o);
  if (lane == 0) s_red[w] = x;
  __syncthreads();
  uint64_t r = 0;
#pragma unroll
  for (int i = 0; i < NT / 32; i++) r += s_red[i];
  __syncthreads();
  return r;
}

// --------------------------------------------------------------------------
// In-SM sort of up to NT*kItems keys (+ values) held in shared memory
// (P:326-341): each thread sorts kItems keys with Batcher's odd-even merge
// network [2], then log2(m / kItems) rounds of merge-path merges
// through shared memory.  Shared layout: element i at i + i/16 (conflict-free
// blocked access).
// --------------------------------------------------------------------------
// rounded up to 4 slots so that a value array placed after the key array stays 16-byte aligned
__host__ __device__ constexpr int padded_len(int c) { return (c + c / 16 + 1 + 3) & ~3; }
__device__ __forceinline__ int phys(int i) { return i + (i >> 4); }

#ifndef GSS_SEARCH_UNROLL
#define GSS_SEARCH_UNROLL 2   // merge-path search steps per loop iteration
#endif
constexpr int kSearchUnroll = GSS_SEARCH_UNROLL;
#ifndef GSS_FAST_KV
#define GSS_FAST_KV 0      // 1: PTX merge step for key-value pairs (measured slower: 4.69 vs 4.57 ms, 2^27 u64 pairs)
#endif
#ifndef GSS_SEARCH_CLZ
#define GSS_SEARCH_CLZ 0   // 1: search steps bounded by each lane's own range (unbalanced last pairs)
#endif

// sk[phys(i)] as a volatile shared load: issued unconditionally (the
// compiler may not turn a select on its result into a branch around it)
template <class T>
__device__ __forceinline__ T lds_key(const T* sk, int i) {
  const uint32_t s = (uint32_t)__cvta_generic_to_shared(sk + phys(i));
  if constexpr (sizeof(T) == 8) {
    unsigned long long x;
    asm volatile("ld.volatile.shared.u64 %0, [%1];" : "=l"(x) : "r"(s));
    return bit_cast_dev<T>(x);
  } else {
    uint32_t x;
    asm volatile("ld.volatile.shared.u32 %0, [%1];" : "=r"(x) : "r"(s));
    return bit_cast_dev<T>(x);
  }
}

// a = *p if pred, else b = *p: one predicated shared-memory load per target
template <class T>
__device__ __forceinline__ void load_pred(T& a, T& b, const T* p, bool pred) {
  const uint32_t s = (uint32_t)__cvta_generic_to_shared(p);
  if constexpr (sizeof(T) == 8) {
    unsigned long long x = bit_cast_dev<unsigned long long>(a), y = bit_cast_dev<unsigned long long>(b);
    asm volatile("{\n\t.reg .pred q;\n\tsetp.ne.u32 q, %2, 0;\n\t@q ld.shared.u64 %0, [%3];\n\t"
                 "@!q ld.shared.u64 %1, [%3];\n\t}"
                 : "+l"(x), "+l"(y)
                 : "r"((uint32_t)pred), "r"(s));
    a = bit_cast_dev<T>(x); b = bit_cast_dev<T>(y);
  } else if constexpr (sizeof(T) == 4) {
    uint32_t x = bit_cast_dev<uint32_t>(a), y = bit_cast_dev<uint32_t>(b);
    asm volatile("{\n\t.reg .pred q;\n\tsetp.ne.u32 q, %2, 0;\n\t@q ld.shared.u32 %0, [%3];\n\t"
                 "@!q ld.shared.u32 %1, [%3];\n\t}"
                 : "+r"(x), "+r"(y)
                 : "r"((uint32_t)pred), "r"(s));
    a = bit_cast_dev<T>(x); b = bit_cast_dev<T>(y);
  }
}

template <class Key, class Val, class Cmp>
__device__ __forceinline__ void cmp_swap(Key& a, Key& b, Val& va, Val& vb, Cmp less) {
  bool s = less(b, a);
  Key lo = s ? b : a, hi = s ? a : b;
  a = lo; b = hi;
  if constexpr (kHasVal<Val>) {
    Val l = s ? vb : va, h = s ? va : vb;
    va = l; vb = h;
  }
}

// Batcher odd-even merge sort network on k[LO .. LO+N), compile-time indices.
template <int LO, int N, int R, class Key, class Val, class Cmp>
__device__ __forceinline__ void oem_merge(Key* k, Val* v, Cmp less) {
  constexpr int step = R * 2;
  if constexpr (step < N) {
    oem_merge<LO, N, step>(k, v, less);
    oem_merge<LO + R, N, step>(k, v, less);
#pragma unroll
    for (int i = LO + R; i + R < LO + N; i += step) cmp_swap(k[i], k[i + R], v[i], v[i + R], less);
  } else {
    cmp_swap(k[LO], k[LO + R], v[LO], v[LO + R], less);
  }
}
template <int LO, int N, class Key, class Val, class Cmp>
__device__ __forceinline__ void oem_sort(Key* k, Val* v, Cmp less) {
  if constexpr (N > 1) {
    oem_sort<LO, N / 2>(k, v, less);
    oem_sort<LO + N / 2, N / 2>(k, v, less);
    oem_merge<LO, N, 1>(k, v, less);
  }
}

// Bitonic sort network on k[0 .. N) (N a power of two), compile-time indices:
// the alternative the paper measured against odd-even merge;
// selected with GSS_FLAG_BITONIC_NET (ablation).
template <int N, class Key, class Val, class Cmp>
__device__ __forceinline__ void bitonic_sort_regs(Key* k, Val* v, Cmp less) {
#pragma unroll
  for (int size = 2; size <= N; size <<= 1) {
#pragma unroll
    for (int stride = size >> 1; stride > 0; stride >>= 1) {
#pragma unroll
      for (int i = 0; i < N; i++) {
        const int j = i ^ stride;
        if (j > i) {
          if ((i & size) == 0) cmp_swap(k[i], k[j], v[i], v[j], less);
          else cmp_swap(k[j], k[i], v[j], v[i], less);
        }
      }
    }
  }
}

// BITONIC: the ablation GSS_FLAG_BITONIC_NET (runtime flag, u64 keys only)
template <int N, bool BITONIC, class Key, class Val, class Cmp>
__device__ __forceinline__ void thread_sort_net(Key* k, Val* v, Cmp less) {
  if constexpr (BITONIC) bitonic_sort_regs<N>(k, v, less);
  else oem_sort<0, N>(k, v, less);
}

// Bitonic merges across the 32 lanes of a warp, in registers (no shared
// memory, no warp barrier): every lane holds ITEMS keys sorted ascending
// (blocked: lane l has slots [l*ITEMS, (l+1)*ITEMS)); step s merges pairs of
// sorted runs of ITEMS*2^s keys (groups of 2^s lanes) into ascending runs of
// twice that length: a flip stage (slot g against slot L-1-g of the merged
// group, the lower slot keeps the minimum) followed by half-cleaners with
// strides L/4 .. 1, across lanes (shuffles) while the stride is >= ITEMS and
// inside the lane's registers below.  After the five steps the warp's
// 32*ITEMS keys are sorted ascending.  The paper's bitonic alternative
// (P:339-341), applied across lanes where the odd-even merge sort's merge-path
// rounds would cost shared-memory round trips and warp barriers.
template <int ITEMS, class Key, class Cmp>
__device__ __forceinline__ void warp_bitonic_merges(Key (&k)[ITEMS], int lane, Cmp less) {
#pragma unroll
  for (int s = 0; s < 5; s++) {
    const int gmask = (2 << s) - 1;
    const bool lower = (lane & (1 << s)) == 0;
#pragma unroll
    for (int i = 0; i < ITEMS / 2; i++) {
      const int j = ITEMS - 1 - i;
      const Key yi = __shfl_xor_sync(kFull, k[j], gmask);      // partner slot ITEMS-1-i for my slot i
      const Key yj = __shfl_xor_sync(kFull, k[i], gmask);      // partner slot i for my slot j
      const bool ti = lower ? less(yi, k[i]) : less(k[i], yi);
      const bool tj = lower ? less(yj, k[j]) : less(k[j], yj);
      k[i] = ti ? yi : k[i];
      k[j] = tj ? yj : k[j];
    }
#pragma unroll
    for (int dl = (1 << s) >> 1; dl >= 1; dl >>= 1) {
      const bool lo = (lane & dl) == 0;
#pragma unroll
      for (int i = 0; i < ITEMS; i++) {
        const Key y = __shfl_xor_sync(kFull, k[i], dl);
        const bool t = lo ? less(y, k[i]) : less(k[i], y);
        k[i] = t ? y : k[i];
      }
    }
#pragma unroll
    for (int d = ITEMS / 2; d >= 1; d >>= 1) {
#pragma unroll
      for (int i = 0; i < ITEMS; i++) {
        if ((i & d) == 0) {
          const bool sw = less(k[i + d], k[i]);
          const Key a = sw ? k[i + d] : k[i], b = sw ? k[i] : k[i + d];
          k[i] = a;
          k[i + d] = b;
        }
      }
    }
  }
}

// Stable odd-even transposition sort (only for the one partial thread).
template <int N, class Key, class Val, class Cmp>
__device__ __forceinline__ void transposition_sort(Key* k, Val* v, Cmp less) {
#pragma unroll
  for (int r = 0; r < N; r++) {
#pragma unroll
    for (int i = r & 1; i + 1 < N; i += 2) {
      bool s = less(k[i + 1], k[i]);
      Key a = s ? k[i + 1] : k[i], b = s ? k[i] : k[i + 1];
      k[i] = a; k[i + 1] = b;
      if constexpr (kHasVal<Val>) {
        Val x = s ? v[i + 1] : v[i], y = s ? v[i] : v[i + 1];
        v[i] = x; v[i + 1] = y;
      }
    }
  }
}

// keys per thread of the in-SM sort: 16, or 8 for 16-byte pairs (register budget)
template <class Key, class Val>
constexpr int sort_items() {
  return (kHasVal<Val> && sizeof(Key) + sizeof(Val) > 8) ? 8 : 16;
}

// Runs of every round are stored so that each merge pair reads as one
// bitonic sequence: run r is kept ascending when r is even and descending when
// r is odd.  A merge then walks A upwards from its left end and B downwards
// from the right end of the pair, and reading past the end of either run
// lands on a key that can never be taken wrongly:
//  * past A's end lies B's largest key (B is stored descending right after A);
//  * past B's smallest key lies A's largest key.
// Keys only: A is taken iff a < b (B wins ties), so an exhausted A (its
// "next" is max B >= every b) is never taken, and an exhausted B's stand-in
// (an A key >= the current a) is taken only when it equals the
// current a -- the same key value.  With values the stand-ins must never be
// taken: A wins ties (B's stand-in is >= a, so A is taken) and A carries one
// index test.  Either way the merge loop has no per-step bounds tests.
template <class Key, class Val, int NT, class Cmp, int ITEMS_ = sort_items<Key, Val>(), bool BITONIC = false>
struct CtaSort {
  static constexpr int ITEMS = ITEMS_;
  static constexpr int C = NT * ITEMS;
  static constexpr int PL = padded_len(C);
  static constexpr bool KV = kHasVal<Val>;
  // SAFE: the merge never takes a stand-in key and partial threads keep their
  // items apart from the pads -- needed with values, and with comparators whose
  // equivalent keys need not be bit-identical (user comparators, gss.hpp)
  static constexpr bool SAFE = KV || !BitwiseOrder<Cmp>::value;
  // keys-only unsigned keys under operator<: the merge step in PTX
  static constexpr bool kFastMerge = !KV && std::is_same<Cmp, Less>::value && std::is_unsigned<Key>::value &&
                                     (sizeof(Key) == 4 || sizeof(Key) == 8);
  __device__ static __forceinline__ void fast_step(Key& out, Key& ka, Key& kb, int& xa, int& xb, uint32_t sb) {
#ifndef GSS_MERGE_ONELOAD
#define GSS_MERGE_ONELOAD 1   // 0: two complementary predicated loads (2^28 u64 in-SM sort 4.89 vs 4.79 ms)
#endif
#ifndef GSS_MERGE_ONELOAD32
#define GSS_MERGE_ONELOAD32 0 // 4-byte keys: 1 measured slower (2^27 u32 in-SM sort 1.63 vs 1.61 ms)
#endif
    if constexpr (GSS_MERGE_ONELOAD && sizeof(Key) == 8) {
      // one shared load with every lane active (the consumed head's successor), then selects: one
      // instruction of up to 32 random 8-byte addresses instead of two complementary predicated ones
      unsigned long long o, a = ka, b = kb;
      asm volatile(
          "{\n\t.reg .pred p;\n\t.reg .u32 x, t;\n\t.reg .u64 y;\n\t"
          "setp.ge.u64 p, %1, %2;\n\t"
          "selp.b64 %0, %2, %1, p;\n\t"
          "@!p add.s32 %3, %3, 1;\n\t"
          "@p add.s32 %4, %4, -1;\n\t"
          "selp.b32 x, %4, %3, p;\n\t"
          "shr.s32 t, x, 4;\n\t"
          "add.s32 t, t, x;\n\t"
          "mad.lo.u32 t, t, 8, %5;\n\t"
          "ld.volatile.shared.u64 y, [t];\n\t"
          "selp.b64 %1, %1, y, p;\n\t"
          "selp.b64 %2, y, %2, p;\n\t}"
          : "=l"(o), "+l"(a), "+l"(b), "+r"(xa), "+r"(xb)
          : "r"(sb));
      out = (Key)o; ka = (Key)a; kb = (Key)b;
    } else if constexpr (GSS_MERGE_ONELOAD32 && sizeof(Key) == 4) {
      uint32_t o, a = ka, b = kb;
      asm volatile(
          "{\n\t.reg .pred p;\n\t.reg .u32 x, t, y;\n\t"
          "setp.ge.u32 p, %1, %2;\n\t"
          "selp.b32 %0, %2, %1, p;\n\t"
          "@!p add.s32 %3, %3, 1;\n\t"
          "@p add.s32 %4, %4, -1;\n\t"
          "selp.b32 x, %4, %3, p;\n\t"
          "shr.s32 t, x, 4;\n\t"
          "add.s32 t, t, x;\n\t"
          "mad.lo.u32 t, t, 4, %5;\n\t"
          "ld.volatile.shared.u32 y, [t];\n\t"
          "selp.b32 %1, %1, y, p;\n\t"
          "selp.b32 %2, y, %2, p;\n\t}"
          : "=r"(o), "+r"(a), "+r"(b), "+r"(xa), "+r"(xb)
          : "r"(sb));
      out = (Key)o; ka = (Key)a; kb = (Key)b;
    } else if constexpr (sizeof(Key) == 8) {
      unsigned long long o, a = ka, b = kb;
      asm volatile(
          "{\n\t.reg .pred p;\n\t.reg .u32 x, t;\n\t"
          "setp.ge.u64 p, %1, %2;\n\t"
          "selp.b64 %0, %2, %1, p;\n\t"
          "@!p add.s32 %3, %3, 1;\n\t"
          "@p add.s32 %4, %4, -1;\n\t"
          "selp.b32 x, %4, %3, p;\n\t"
          "shr.s32 t, x, 4;\n\t"
          "add.s32 t, t, x;\n\t"
          "mad.lo.u32 t, t, 8, %5;\n\t"
          "@!p ld.volatile.shared.u64 %1, [t];\n\t"
          "@p ld.volatile.shared.u64 %2, [t];\n\t}"
          : "=l"(o), "+l"(a), "+l"(b), "+r"(xa), "+r"(xb)
          : "r"(sb));
      out = (Key)o; ka = (Key)a; kb = (Key)b;
    } else {
      uint32_t o, a = ka, b = kb;
      asm volatile(
          "{\n\t.reg .pred p;\n\t.reg .u32 x, t;\n\t"
          "setp.ge.u32 p, %1, %2;\n\t"
          "selp.b32 %0, %2, %1, p;\n\t"
          "@!p add.s32 %3, %3, 1;\n\t"
          "@p add.s32 %4, %4, -1;\n\t"
          "selp.b32 x, %4, %3, p;\n\t"
          "shr.s32 t, x, 4;\n\t"
          "add.s32 t, t, x;\n\t"
          "mad.lo.u32 t, t, 4, %5;\n\t"
          "@!p ld.volatile.shared.u32 %1, [t];\n\t"
          "@p ld.volatile.shared.u32 %2, [t];\n\t}"
          : "=r"(o), "+r"(a), "+r"(b), "+r"(xa), "+r"(xb)
          : "r"(sb));
      out = (Key)o; ka = (Key)a; kb = (Key)b;
    }
  }
  // key-value pairs of unsigned keys under operator< with a value of the
  // key's width: the merge step in PTX (A wins ties; A carries the index test)
  static constexpr bool kFastMergeKV = KV && std::is_same<Cmp, Less>::value && std::is_unsigned<Key>::value &&
                                       (sizeof(Key) == 4 || sizeof(Key) == 8) && sizeof(Val) == sizeof(Key);
  __device__ static __forceinline__ void fast_step_kv(Key& ok, Val& ov, Key& ka, Key& kb, Val& va, Val& vb, int& xa,
                                                      int& xb, int ae, uint32_t sbk, uint32_t sbv) {
    if constexpr (sizeof(Key) == 8) {
      unsigned long long o, w, a = ka, b = kb, c = bit_cast_dev<unsigned long long>(va),
                               d = bit_cast_dev<unsigned long long>(vb);
      asm volatile(
          "{\n\t.reg .pred p, r;\n\t.reg .u32 x, t, u;\n\t"
          "setp.le.u64 p, %2, %3;\n\t"
          "setp.lt.s32 r, %6, %8;\n\t"
          "and.pred p, p, r;\n\t"
          "selp.b64 %0, %2, %3, p;\n\t"
          "selp.b64 %1, %4, %5, p;\n\t"
          "@p add.s32 %6, %6, 1;\n\t"
          "@!p add.s32 %7, %7, -1;\n\t"
          "selp.b32 x, %6, %7, p;\n\t"
          "shr.s32 t, x, 4;\n\t"
          "add.s32 t, t, x;\n\t"
          "mad.lo.u32 u, t, 8, %10;\n\t"
          "mad.lo.u32 t, t, 8, %9;\n\t"
          "@p ld.volatile.shared.u64 %2, [t];\n\t"
          "@!p ld.volatile.shared.u64 %3, [t];\n\t"
          "@p ld.volatile.shared.u64 %4, [u];\n\t"
          "@!p ld.volatile.shared.u64 %5, [u];\n\t}"
          : "=l"(o), "=l"(w), "+l"(a), "+l"(b), "+l"(c), "+l"(d), "+r"(xa), "+r"(xb)
          : "r"(ae), "r"(sbk), "r"(sbv));
      ok = (Key)o; ov = bit_cast_dev<Val>(w); ka = (Key)a; kb = (Key)b;
      va = bit_cast_dev<Val>(c); vb = bit_cast_dev<Val>(d);
    } else {
      uint32_t o, w, a = ka, b = kb, c = bit_cast_dev<uint32_t>(va), d = bit_cast_dev<uint32_t>(vb);
      asm volatile(
          "{\n\t.reg .pred p, r;\n\t.reg .u32 x, t, u;\n\t"
          "setp.le.u32 p, %2, %3;\n\t"
          "setp.lt.s32 r, %6, %8;\n\t"
          "and.pred p, p, r;\n\t"
          "selp.b32 %0, %2, %3, p;\n\t"
          "selp.b32 %1, %4, %5, p;\n\t"
          "@p add.s32 %6, %6, 1;\n\t"
          "@!p add.s32 %7, %7, -1;\n\t"
          "selp.b32 x, %6, %7, p;\n\t"
          "shr.s32 t, x, 4;\n\t"
          "add.s32 t, t, x;\n\t"
          "mad.lo.u32 u, t, 4, %10;\n\t"
          "mad.lo.u32 t, t, 4, %9;\n\t"
          "@p ld.volatile.shared.u32 %2, [t];\n\t"
          "@!p ld.volatile.shared.u32 %3, [t];\n\t"
          "@p ld.volatile.shared.u32 %4, [u];\n\t"
          "@!p ld.volatile.shared.u32 %5, [u];\n\t}"
          : "=r"(o), "=r"(w), "+r"(a), "+r"(b), "+r"(c), "+r"(d), "+r"(xa), "+r"(xb)
          : "r"(ae), "r"(sbk), "r"(sbv));
      ok = (Key)o; ov = bit_cast_dev<Val>(w); ka = (Key)a; kb = (Key)b;
      va = bit_cast_dev<Val>(c); vb = bit_cast_dev<Val>(d);
    }
  }

  static constexpr size_t smem_bytes() {
    return (size_t)PL * sizeof(Key) + (kHasVal<Val> ? (size_t)PL * sizeof(Val) : 0);
  }

  // ITEMS outputs of the merge of pair (A = run at ps of aLen keys, B = run at
  // ps + aLen of bLen keys, stored descending), starting at output diag.
  __device__ static __forceinline__ void merge_items(const Key* sk, const Val* sv, int ps, int aLen, int bLen,
                                                     int diag, Key* k, Val* v, Cmp less) {
    const int bEnd = ps + aLen + bLen - 1;                   // B's smallest key
    int ia;
    // Merge-path search as binary lifting with a fixed number of steps (the
    // pair width w = max(aLen, ...) is a power of two, the same for every lane
    // of the round): no data-dependent trip count, no divergence.
    const int w = aLen;                                       // aLen == w for every pair with a B run
    if constexpr (SAFE) {
      // number of A keys among the first diag outputs, A first on ties:
      // smallest j in [lo, hi) with B[diag-1-j] < A[j], else hi
      const int lo = max(0, diag - bLen), hi = min(diag, aLen);
      int j = lo;
#if GSS_SEARCH_CLZ
      for (int st = hi > lo ? 1 << (31 - __clz(hi - lo)) : 0; st > 0; st >>= 1) {
#else
#pragma unroll kSearchUnroll
      for (int st = w; st > 0; st >>= 1) {
#endif
        const int pr = j + st - 1;
        const int pc = min(pr, hi - 1);
        // clamped probe addresses: the loads stay inside the pair even when its range is empty
        // (hi == 0), where the result is discarded -- no read of a slot another warp may be storing
        const Key b = lds_key(sk, max(bEnd - (diag - 1 - pc), ps + aLen)), a = lds_key(sk, max(ps + pc, ps));
        j = (pr < hi) & !less(b, a) ? pr + 1 : j;
      }
      ia = j;
    } else {
      // number of B keys among the first diag outputs, B first on ties:
      // smallest j in [lo, hi) with A[diag-1-j] < B[j], else hi
      const int lo = max(0, diag - aLen), hi = min(diag, bLen);
      int j = lo;
#if GSS_SEARCH_CLZ
      for (int st = hi > lo ? 1 << (31 - __clz(hi - lo)) : 0; st > 0; st >>= 1) {
#else
#pragma unroll kSearchUnroll
      for (int st = w; st > 0; st >>= 1) {
#endif
        const int pr = j + st - 1;
        const int pc = min(pr, hi - 1);
        // clamped probe addresses: inside the pair even when its range is empty (hi == 0, result discarded)
        const Key a = lds_key(sk, min(ps + diag - 1 - pc, ps + aLen - 1)), b = lds_key(sk, min(bEnd - pc, bEnd));
        j = (pr < hi) & !less(a, b) ? pr + 1 : j;
      }
      ia = diag - j;
    }
    int xa = ps + ia, xb = bEnd - (diag - ia);
    const int ae = ps + aLen;
    Key ka = sk[phys(xa)], kb = sk[phys(xb)];
    if constexpr (kFastMerge) {
      // one compare, the output select, the index step and a predicated load
      // straight into the consumed head per output
      const uint32_t sb = (uint32_t)__cvta_generic_to_shared(sk);
#pragma unroll
      for (int i = 0; i < ITEMS; i++) {
        if (i + 1 < ITEMS) fast_step(k[i], ka, kb, xa, xb, sb);
        else k[i] = ka < kb ? ka : kb;
      }
      return;
    }
    Val va, vb;
    if constexpr (KV) { va = sv[phys(xa)]; vb = sv[phys(xb)]; }
#if GSS_FAST_KV
    if constexpr (kFastMergeKV) {
      const uint32_t sbk = (uint32_t)__cvta_generic_to_shared(sk), sbv = (uint32_t)__cvta_generic_to_shared(sv);
#pragma unroll
      for (int i = 0; i < ITEMS; i++) {
        if (i + 1 < ITEMS) {
          fast_step_kv(k[i], v[i], ka, kb, va, vb, xa, xb, ae, sbk, sbv);
        } else {
          const bool p = (xa < ae) && !(kb < ka);
          k[i] = p ? ka : kb;
          v[i] = p ? va : vb;
        }
      }
      return;
    }
#endif
#pragma unroll
    for (int i = 0; i < ITEMS; i++) {
      bool p;
      if constexpr (SAFE) p = (xa < ae) && !less(kb, ka);
      else p = less(ka, kb);
      k[i] = p ? ka : kb;
      if constexpr (KV) v[i] = p ? va : vb;
      if (i + 1 < ITEMS) {
        const int nx = p ? xa + 1 : xb - 1;
        xa = p ? nx : xa;
        xb = p ? xb : nx;
        const Key y = sk[phys(nx)];
        ka = p ? y : ka;
        kb = p ? kb : y;
        if constexpr (KV) {
          const Val z = sv[phys(nx)];
          va = p ? z : va;
          vb = p ? vb : z;
        }
      }
    }
  }

  // A single warp (NT == 32, or a 32-thread block) sorts on its own: only warp barriers.
  __device__ static __forceinline__ void bar(int nt) {
    if (NT == 32 || nt == 32) __syncwarp(); else __syncthreads();
  }

  // cnt items of a run [rs, rs + rlen) starting at run offset o, ascending or descending
  __device__ static __forceinline__ void store_run(Key* sk, Val* sv, const Key* k, const Val* v, int cnt, int rs,
                                                   int rlen, int o, bool desc) {
    // ascending: slots rs+o .. rs+o+ITEMS-1; descending: rs+rlen-o-ITEMS .. rs+rlen-o-1
    constexpr int RUN = ITEMS < 16 ? ITEMS : 16;                 // slots per padded row segment
    if (cnt == ITEMS && (((desc ? rs + rlen - o : rs + o)) & (RUN - 1)) == 0) {
      // the ITEMS slots fill whole padded rows (or lie in one): consecutive
      // addresses per row, immediate offsets
      if (desc) {
#pragma unroll
        for (int r = 0; r < ITEMS / RUN; r++) {
          const int q = phys(rs + rlen - 1 - o - r * RUN);
#pragma unroll
          for (int i = 0; i < RUN; i++) {
            sk[q - i] = k[r * RUN + i];
            if constexpr (KV) sv[q - i] = v[r * RUN + i];
          }
        }
      } else {
#pragma unroll
        for (int r = 0; r < ITEMS / RUN; r++) {
          const int q = phys(rs + o + r * RUN);
#pragma unroll
          for (int i = 0; i < RUN; i++) {
            sk[q + i] = k[r * RUN + i];
            if constexpr (KV) sv[q + i] = v[r * RUN + i];
          }
        }
      }
      return;
    }
#pragma unroll
    for (int i = 0; i < ITEMS; i++) {
      if (i < cnt) {
        const int q = desc ? rs + rlen - 1 - (o + i) : rs + o + i;
        sk[phys(q)] = k[i];
        if constexpr (KV) sv[phys(q)] = v[i];
      }
    }
  }

  // Sorts sk[phys(0..m)) (and sv) in place; 0 <= m <= nt * ITEMS.  Every
  // thread of the nt-thread block (nt <= NT; nt = NT unless the caller sizes
  // the block at run time), or every lane of the warp when NT == 32, must
  // call it.  Begins and ends with a barrier.
  // keys only, bit-identical equivalents: the first five merge rounds run
  // across the warp's registers (warp_bitonic_merges) instead of through
  // shared memory
#ifndef GSS_WARP_BITONIC
#define GSS_WARP_BITONIC 0   // 1: measured 2x slower (2^28 u64 in-SM sort 8.35 vs 4.91 ms; 2^27 u32 3.24 vs 1.61)
#endif
  static constexpr bool WB = GSS_WARP_BITONIC && !KV && BitwiseOrder<Cmp>::value && !BITONIC;

  // gk / gv (optional): the m keys (values) are read from global memory straight into the threads'
  // registers instead of from sk / sv: thread t < m / ITEMS takes items t, t + m/ITEMS, t + 2 m/ITEMS, ...
  // (every load instruction coalesced across the warp), the remainder goes to thread m / ITEMS.  Which keys
  // a thread starts with is immaterial (it sorts them); the runs keep the layout of the shared-memory path.
  __device__ static void sort(Key* sk, Val* sv, int m, Cmp less, int nt = NT, const Key* gk = nullptr,
                              const Val* gv = nullptr) {
    bar(nt);
    const int t = NT == 32 ? (threadIdx.x & 31) : threadIdx.x;
    const int base = t * ITEMS;
    const int cnt = min(max(m - base, 0), ITEMS);
    Key k[ITEMS];
    Val v[ITEMS];
    int w0 = ITEMS;                                      // width of the runs the merge-path rounds start from
    if constexpr (WB) {
      const int lane = threadIdx.x & 31;
      const int wbase = base - lane * ITEMS;             // the warp's first slot
      const int wcount = min(max(m - wbase, 0), 32 * ITEMS);
      if (wcount > 0) {                                  // warp-uniform
        bool has = cnt > 0;
        Key mx{};
#pragma unroll
        for (int i = 0; i < ITEMS; i++) {
          if (i < cnt) {
            k[i] = sk[phys(base + i)];
            if (i == 0 || less(mx, k[i])) mx = k[i];
          }
        }
        // pads: copies of the warp's largest key (indistinguishable from it), so the warp's real keys
        // come out as its first wcount sorted slots
#pragma unroll
        for (int o = 16; o > 0; o >>= 1) {
          const Key y = __shfl_xor_sync(kFull, mx, o);
          const bool hy = __shfl_xor_sync(kFull, has, o);
          if (hy && (!has || less(mx, y))) mx = y;
          has = has || hy;
        }
#pragma unroll
        for (int i = 0; i < ITEMS; i++)
          if (i >= cnt) k[i] = mx;
        thread_sort_net<ITEMS, BITONIC>(k, v, less);
        warp_bitonic_merges<ITEMS>(k, lane, less);
        const int my = min(max(wcount - lane * ITEMS, 0), ITEMS);
        __syncwarp();
        if (my > 0) store_run(sk, sv, k, v, my, wbase, wcount, lane * ITEMS, ((wbase / (32 * ITEMS)) & 1) != 0);
      }
      w0 = 32 * ITEMS;
    } else if (cnt > 0) {
      if (gk) {
        const int nf = m / ITEMS;                          // full threads
        const int g0 = t < nf ? t : nf * ITEMS, gs = t < nf ? nf : 1;
#pragma unroll
        for (int i = 0; i < ITEMS; i++) {
          if (i < cnt) {
            k[i] = gk[g0 + i * gs];
            if constexpr (KV) v[i] = gv[g0 + i * gs];
          }
        }
      } else {
#pragma unroll
        for (int i = 0; i < ITEMS; i++) {
          if (i < cnt) {
            k[i] = sk[phys(base + i)];
            if constexpr (KV) v[i] = sv[phys(base + i)];
          }
        }
      }
      // A partial thread pads with copies of its largest item: after sorting,
      // its first cnt outputs are exactly its real items because every pad is
      // indistinguishable from that item (same key, and the same value for
      // pairs).  Only pairs with a repeated largest key need the stable
      // transposition network instead (pads last, real items first).
      bool stable_path = false;
      if (cnt < ITEMS) {
        Key mx = k[0];
        Val vmx = v[0];
#pragma unroll
        for (int i = 1; i < ITEMS; i++)
          if (i < cnt && less(mx, k[i])) { mx = k[i]; vmx = v[i]; }
        if constexpr (SAFE) {
          int reps = 0;
#pragma unroll
          for (int i = 0; i < ITEMS; i++)
            if (i < cnt && !less(k[i], mx)) reps++;
          stable_path = reps > 1;
        }
#pragma unroll
        for (int i = 0; i < ITEMS; i++) {
          if (i >= cnt) {
            k[i] = mx;
            v[i] = vmx;
          }
        }
      }
      if constexpr (SAFE) {
        if (stable_path) transposition_sort<ITEMS>(k, v, less);
        else thread_sort_net<ITEMS, BITONIC>(k, v, less);
      } else {
        thread_sort_net<ITEMS, BITONIC>(k, v, less);
      }
    }
    if constexpr (!WB) {
      __syncwarp();
      if (cnt > 0) store_run(sk, sv, k, v, cnt, base, cnt, 0, (t & 1) != 0);   // run t: descending if t is odd
    }
    // Rounds whose merged pairs (2w keys) lie inside one warp's 32*ITEMS keys
    // only synchronise the warp; wider rounds synchronise the block.
    for (int w = w0; w < m; w *= 2) {
      const bool blk = NT > 32 && nt > 32 && 2 * w > 32 * ITEMS;
      auto round_bar = [&]() {
        if (blk) __syncthreads(); else __syncwarp();
      };
      round_bar();
      const int ps = base & ~(2 * w - 1);                // w is a power of two
      const int aLen = min(w, m - ps);
      const int bLen = max(0, min(w, m - ps - w));
      if (cnt > 0) {
        if (bLen > 0) {
          merge_items(sk, sv, ps, aLen, bLen, base - ps, k, v, less);
        } else {
#pragma unroll
          for (int i = 0; i < ITEMS; i++) {               // a lone last run: already in place and ascending
            if (i < cnt) {
              k[i] = sk[phys(base + i)];
              if constexpr (KV) v[i] = sv[phys(base + i)];
            }
          }
        }
      }
      round_bar();
      if (cnt > 0) store_run(sk, sv, k, v, cnt, ps, aLen + bLen, base - ps, (base & (2 * w)) != 0);
    }
    bar(nt);
  }
};

// --------------------------------------------------------------------------
// Branch-free descent of the implicit splitter tree (Algorithm 2):
// j := 1; repeat log k times j := 2j + (e > bt[j]); bucket = j - k.  The
// comparison is less(bt[j], e) and becomes a predicated add.
// --------------------------------------------------------------------------
template <int LOGK, class Key, class Cmp>
__device__ __forceinline__ uint32_t descend(const Key* __restrict__ tree, Key e, Cmp less) {
  uint32_t j = 1;
#pragma unroll
  for (int d = 0; d < LOGK; d++) j = 2 * j + (less(tree[j], e) ? 1u : 0u);
  return j - (1u << LOGK);
}

}  // namespace gss
