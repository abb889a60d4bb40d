#pragma once
// Shared by the translation units of libgss.so: gss.cu (the C ABI) and gss_inst_*.cu (one
// instantiation of the sort engine each, compiled in parallel).
// gss_impl.cuh -- host orchestration of the B200 GPU
// sample sort.  One call enqueues a fixed, data-independent launch sequence
// (init, then per level: sample, classify, scan x2, scatter, plan; then the
// in-SM sorts, largest size class first, copy, overflow) on the
// caller's stream; all data-dependent work lists live in device memory.
#include <algorithm>
#include <atomic>
#include <cstdio>
#include <cstring>
#include <mutex>
#include <vector>

#include "../../include/gss.h"
#include "gss_kernels.cuh"

using namespace gss;

struct gss_profiler {
  struct Rec { int kind; cudaEvent_t a, b; };
  std::vector<Rec> recs;
  std::vector<cudaEvent_t> pool;
  double ms[GSS_KERNEL_KINDS];
  uint64_t launches[GSS_KERNEL_KINDS];
  cudaEvent_t get() {
    if (!pool.empty()) { cudaEvent_t e = pool.back(); pool.pop_back(); return e; }
    cudaEvent_t e = nullptr;
    cudaEventCreate(&e);
    return e;
  }
};

namespace gssh {

inline constexpr uint32_t kVersion = 1;
inline constexpr uint32_t kFlagScatterCtaCounters = 1u << 30;   // ablation: ranks from one counter set per CTA (k_scatter_fast)
inline constexpr uint32_t kFlagScatterBulk = 1u << 29;          // ablation: bulk-copy scatter for 4-byte keys too
inline constexpr uint32_t kFlagSampleFull = 1u << 25;          // ablation: 1024-thread sample sorts always
inline constexpr uint32_t kFlagScatterWsOne = 1u << 26;         // ablation: keys alone through the one-CTA/SM form too
inline constexpr uint32_t kFlagScatterNoWs = 1u << 27;          // ablation: the single-role bulk scatter (k_scatter_bulk)
inline constexpr uint32_t kFlagSmallNarrow = 1u << 28;          // ablation: 48-register block sort for classes <= 20 warps
                                                                // (2^28 u64: 4.98 vs 4.90 ms -- occupancy is not the limit)

inline size_t align_up(size_t x, size_t a = 256) { return (x + a - 1) / a * a; }

struct DeviceInfo {
  int dev = -1, sms = 0, major = 0, minor = 0;
};

inline gss_status device_info(DeviceInfo* out) {
  static std::mutex mu;
  static DeviceInfo cache[64];
  int dev = 0;
  if (cudaGetDevice(&dev) != cudaSuccess) { cudaGetLastError(); return GSS_ERROR_CUDA; }
  std::lock_guard<std::mutex> g(mu);
  if (dev < 0 || dev >= 64) return GSS_ERROR_CUDA;
  if (cache[dev].dev != dev) {
    DeviceInfo d;
    d.dev = dev;
    if (cudaDeviceGetAttribute(&d.sms, cudaDevAttrMultiProcessorCount, dev) != cudaSuccess ||
        cudaDeviceGetAttribute(&d.major, cudaDevAttrComputeCapabilityMajor, dev) != cudaSuccess ||
        cudaDeviceGetAttribute(&d.minor, cudaDevAttrComputeCapabilityMinor, dev) != cudaSuccess) {
      cudaGetLastError();
      return GSS_ERROR_CUDA;
    }
    cache[dev] = d;
  }
  *out = cache[dev];
  if (out->major != 10 || out->minor != 0) return GSS_ERROR_NOT_SUPPORTED;   // sm_100a code only
  return GSS_SUCCESS;
}

// Resolved parameters.
struct Cfg {
  uint32_t k, a, T, L, k_policy, fill_div, flags, kmax, nclass, cls_arrays;
  uint64_t M, seed;
  uint32_t* error_out;
  uint32_t class_cap[kNumClasses];
};

template <class Key, class Val>
constexpr uint32_t max_small_capacity() {
  return 32u * 32u * (uint32_t)small_items<Key, Val>();        // a 32-warp CTA
}

template <class Key, class Val>
gss_status resolve(const gss_params* up, uint64_t n, Cfg* c, uint32_t kmin_given) {
  gss_params p{};
  if (up) p = *up;
  c->a = p.oversample ? p.oversample : 30;
  // GSS_FLAG_CLUSTER_SORT: buckets up to a thread-block cluster's capacity are final (NEXT-2)
  const uint32_t cap = (p.flags & GSS_FLAG_CLUSTER_SORT) ? cluster_capacity<Key, Val>() : max_small_capacity<Key, Val>();
  c->M = p.small_threshold ? p.small_threshold : cap;
  if (c->M > cap) return GSS_ERROR_INVALID_VALUE;
  // default k (R29): 256, raised to 512 / 1024 when two levels of 256 would
  // leave final buckets above M/2 (measured: 2^30 u64 keys 42.7 ms at k = 512
  // against 46.1 ms at k = 256, whose last level needs a third split)
  if (p.k) {
    c->k = p.k;
  } else {
    c->k = 256;
    while (c->k < 1024 && (double)n > (double)c->k * c->k * (double)(c->M / 2)) c->k *= 2;
  }
  if (c->k < 2 || c->k > 1024 || (c->k & (c->k - 1))) return GSS_ERROR_INVALID_VALUE;
  // default tile: 65536 keys, halved (down to 2048) while the input has fewer
  // than 296 tiles (two CTAs per SM of a B200) so small sorts stay parallel
  if (p.tile) {
    c->T = p.tile;
  } else {
    c->T = 65536;
    while (c->T > 2048 && n < (uint64_t)c->T * 296) c->T /= 2;
  }
  if (c->T < 2048 || c->T % 2048 || c->T > (1u << 24)) return GSS_ERROR_INVALID_VALUE;
  c->k_policy = p.k_policy ? p.k_policy : 1;
  if (c->k_policy > 2) return GSS_ERROR_INVALID_VALUE;
  c->fill_div = p.fill_div ? p.fill_div : 4;
  c->seed = p.seed ? p.seed : 5489;
  c->flags = p.flags;
  c->error_out = p.error_out;
  c->cls_arrays = p.cls_arrays ? p.cls_arrays : 8;
  if (c->cls_arrays != 1 && c->cls_arrays != 2 && c->cls_arrays != 4 && c->cls_arrays != 8) return GSS_ERROR_INVALID_VALUE;
  // size classes (R8): class i = buckets a CTA of class_warps(i) warps sorts
  c->nclass = kNumClasses;
  for (int i = 0; i < kNumClasses; i++) c->class_cap[i] = (uint32_t)(class_warps(i) * 32 * small_items<Key, Val>());
  if (c->class_cap[kNumClasses - 1] != max_small_capacity<Key, Val>()) return GSS_ERROR_NOT_SUPPORTED;
  c->kmax = std::max<uint32_t>(std::max(c->k, kmin_given), 4u);
  // levels: expected depth with children up to 2x the mean, plus one spare level
  if (p.max_levels) {
    c->L = std::min<uint32_t>(p.max_levels, kMaxLevels);
  } else {
    uint64_t m = n;
    uint32_t L = 0;
    while (m > c->M && L < kMaxLevels) {
      uint32_t kb = choose_kb(c->k, c->k_policy, c->fill_div, c->M, m);
      m = kb >= 4 ? (2 * m + kb - 1) / kb : (3 * m + 3) / 4;
      L++;
    }
    c->L = L ? std::min<uint32_t>(L + 1, kMaxLevels) : 0;
  }
  return GSS_SUCCESS;
}

// Workspace layout inside the caller's temp buffer.
template <class Key, class Val, class IdT>
struct Layout {
  size_t off_cnt, off_ktmp, off_vtmp, off_ids, off_bk[2], off_tb[2], off_hist[2], off_spl[2], off_small[kNumClasses],
      off_copy, off_ovf, off_fb, off_clus, off_scan, off_hin_k, off_hin_v, off_hout_k, off_hout_v, total;
  uint32_t cap_buckets, cap_tiles, cap_hist, cap_spl, cap_copy, cap_ovf, cap_fb, cap_clus, cap_small[kNumClasses];

  void compute(uint64_t n, const Cfg& c, int mode, bool host_io) {
    const uint64_t M = mode == MODE_SORT ? c.M : 0;
    cap_buckets = mode == MODE_SORT ? (uint32_t)(n / (M + 1) + 1) : 1;
    cap_tiles = (uint32_t)((n + c.T - 1) / c.T + cap_buckets);
    cap_hist = std::max(c.kmax, 3u) * cap_tiles;
    cap_spl = 2 * c.kmax * cap_buckets;
    const uint64_t children = (uint64_t)std::max<uint32_t>(c.L, 1) * cap_buckets * std::max(c.kmax, 3u) + 1;
    for (int i = 0; i < kNumClasses; i++) {
      uint64_t lower = i == 0 ? 0 : c.class_cap[i - 1];
      uint64_t cap = std::min<uint64_t>(children, n / (lower + 1) + 1);
      cap_small[i] = (i < (int)c.nclass) ? (uint32_t)cap : 0;
    }
    cap_copy = (uint32_t)(n / c.T + n / (c.class_cap[kNumClasses - 1] + 1) + 2);
    cap_ovf = cap_buckets;
    cap_fb = mode == MODE_SORT ? (uint32_t)(n / (c.class_cap[0] + 1) + 1) : 1;   // buckets of the split classes
    cap_clus = (mode == MODE_SORT && M > c.class_cap[kNumClasses - 1])
                   ? (uint32_t)(n / (c.class_cap[kNumClasses - 1] + 1) + 1) : 1;
    size_t o = 0;
    auto take = [&](size_t bytes) { size_t r = o; o = align_up(o + bytes); return r; };
    off_hin_k = off_hout_k = off_hin_v = off_hout_v = 0;
    if (host_io) {
      off_hin_k = take(n * sizeof(Key));
      off_hout_k = take(n * sizeof(Key));
      if (kHasVal<Val>) {
        off_hin_v = take(n * sizeof(Val));
        off_hout_v = take(n * sizeof(Val));
      }
    }
    off_cnt = take(sizeof(Counters));
    off_ktmp = take(n * sizeof(Key));
    off_vtmp = kHasVal<Val> ? take(n * sizeof(Val)) : 0;
    off_ids = take((n + 16 * ((size_t)cap_buckets + 2)) * sizeof(IdT));   // per-bucket 16-aligned id ranges
    for (int s = 0; s < 2; s++) {
      off_bk[s] = take((size_t)cap_buckets * sizeof(Bucket));
      off_tb[s] = take((size_t)cap_tiles * 4);
      off_hist[s] = take((size_t)cap_hist * 4);
      off_spl[s] = take((size_t)cap_spl * sizeof(Key));
    }
    for (int i = 0; i < kNumClasses; i++) off_small[i] = take((size_t)cap_small[i] * sizeof(Item));
    off_copy = take((size_t)cap_copy * sizeof(Item));
    off_ovf = take((size_t)cap_ovf * sizeof(Item));
    off_fb = take((size_t)cap_fb * sizeof(Item));
    off_clus = take((size_t)cap_clus * sizeof(Item));
    off_scan = take(kScanCtas * 4);
    total = o;
  }
};

inline bool ranges_overlap(const void* a, size_t na, const void* b, size_t nb) {
  if (!a || !b || !na || !nb) return false;
  uintptr_t x = (uintptr_t)a, y = (uintptr_t)b;
  return x < y + nb && y < x + na;
}
// identical or disjoint
inline bool same_or_disjoint(const void* a, size_t na, const void* b, size_t nb) {
  return a == b || !ranges_overlap(a, na, b, nb);
}

template <class F>
gss_status launch(gss_profiler* prof, int kind, cudaStream_t s, uint32_t* count, F&& f) {
  cudaEvent_t a = nullptr, b = nullptr;
  if (prof) {
    a = prof->get();
    b = prof->get();
    cudaEventRecord(a, s);
  }
  f();
  cudaError_t e = cudaGetLastError();
  if (prof) {
    cudaEventRecord(b, s);
    prof->recs.push_back({kind, a, b});
  }
  if (count) (*count)++;
  return e == cudaSuccess ? GSS_SUCCESS : GSS_ERROR_CUDA;
}

// Opt in to the dynamic shared memory a kernel needs and ask for the largest
// shared-memory carveout, so that several CTAs share an SM.
template <class K>
gss_status set_smem(K kernel, size_t bytes) {
  if (bytes > 48 * 1024) {
    if (cudaFuncSetAttribute(kernel, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)bytes) != cudaSuccess) {
      cudaGetLastError();
      return GSS_ERROR_CUDA;
    }
  }
  if (cudaFuncSetAttribute(kernel, cudaFuncAttributePreferredSharedMemoryCarveout, cudaSharedmemCarveoutMaxShared) !=
      cudaSuccess) {
    cudaGetLastError();
    return GSS_ERROR_CUDA;
  }
  return GSS_SUCCESS;
}

// Per-device cache of a grid size (the occupancy query costs host time on
// launch-bound sorts).  Racing threads store the same value.
struct GridCache {
  std::atomic<int> g[64];
  int get(int dev) const { return dev >= 0 && dev < 64 ? g[dev].load(std::memory_order_relaxed) : 0; }
  void put(int dev, int v) { if (dev >= 0 && dev < 64) g[dev].store(v, std::memory_order_relaxed); }
};

template <class K>
int grid_for(K kernel, int threads, size_t smem, int sms, int cap = 1 << 30) {
  int per = 0;
  if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per, kernel, threads, smem) != cudaSuccess) {
    cudaGetLastError();
    per = 1;
  }
  return std::max(1, std::min(cap, std::max(per, 1) * sms));
}

#define GSS_TRY(...)                            \
  do {                                          \
    gss_status _s = (__VA_ARGS__);              \
    if (_s != GSS_SUCCESS) return _s;           \
  } while (0)

template <class Key, class Val, class IdT, class Cmp>
struct Engine {
  using C = Ctx<Key, Val, IdT>;

  static C make_ctx(unsigned char* base, const Layout<Key, Val, IdT>& lay, const Cfg& cfg, uint64_t n, int mode) {
    C c{};
    c.ktmp = reinterpret_cast<Key*>(base + lay.off_ktmp);
    if constexpr (kHasVal<Val>) c.vtmp = reinterpret_cast<Val*>(base + lay.off_vtmp);
    c.ids = reinterpret_cast<IdT*>(base + lay.off_ids);
    c.cnt = reinterpret_cast<Counters*>(base + lay.off_cnt);
    for (int s = 0; s < 2; s++) {
      c.bk[s] = reinterpret_cast<Bucket*>(base + lay.off_bk[s]);
      c.tile_bucket[s] = reinterpret_cast<uint32_t*>(base + lay.off_tb[s]);
      c.hist[s] = reinterpret_cast<uint32_t*>(base + lay.off_hist[s]);
      c.spl[s] = reinterpret_cast<Key*>(base + lay.off_spl[s]);
    }
    for (int i = 0; i < kNumClasses; i++) {
      c.small[i] = reinterpret_cast<Item*>(base + lay.off_small[i]);
      c.cap_small[i] = lay.cap_small[i];
      c.class_cap[i] = cfg.class_cap[i];
    }
    c.copy = reinterpret_cast<Item*>(base + lay.off_copy);
    c.ovf = reinterpret_cast<Item*>(base + lay.off_ovf);
    c.fb = reinterpret_cast<Item*>(base + lay.off_fb);
    c.clus = reinterpret_cast<Item*>(base + lay.off_clus);
    c.scan_part = reinterpret_cast<uint32_t*>(base + lay.off_scan);
    c.n = (uint32_t)n;
    c.M = (uint32_t)cfg.M;
    c.T = cfg.T; c.k = cfg.k; c.a = cfg.a; c.k_policy = cfg.k_policy; c.fill_div = cfg.fill_div;
    c.sample_cap = 16384;
    c.L = mode == MODE_SORT ? cfg.L : 1;
    c.mode = mode;
    c.stable = ((cfg.flags & GSS_FLAG_STABLE) || mode != MODE_SORT) ? 1u : 0u;   // partitions stay stable (R7 probe)
    c.recompute = (!c.stable && (cfg.flags & GSS_FLAG_RECOMPUTE_IDS) && !(cfg.flags & GSS_FLAG_DIRECT_SCATTER) &&
                   !(cfg.flags & kFlagScatterCtaCounters)) ? 1u : 0u;
    c.lut = (cfg.flags & GSS_FLAG_TREE_CLASSIFY) ? 0u : 1u;
    c.cap_buckets = lay.cap_buckets; c.cap_tiles = lay.cap_tiles; c.cap_hist = lay.cap_hist;
    c.cap_spl = lay.cap_spl; c.cap_copy = lay.cap_copy; c.cap_ovf = lay.cap_ovf;
    c.cap_fb = lay.cap_fb;
    c.cap_clus = lay.cap_clus;
    c.seed = cfg.seed;
    c.cls_arrays = cfg.cls_arrays;
    return c;
  }

  // In-SM sorts of one size class: the block merge sort (k_small_block) by
  // default; with GSS_FLAG_SPLIT_SORT the sample split + warp segment sorts
  // (k_small) for classes of two or more warps.  cls == kNumClasses: the
  // block merge sort of the buckets the split handed back (1024 threads).
  static gss_status launch_small(C& c, const Cfg& cfg, int cls, const DeviceInfo& di, cudaStream_t s,
                                 gss_profiler* prof, uint32_t* count) {
    const bool fb = cls == kNumClasses;
    const int nt = fb ? kSmallMaxThreads : class_warps(cls) * 32;
    if (!fb && nt > 32 && (cfg.flags & GSS_FLAG_SPLIT_SORT)) {
      auto kern = k_small<Key, Val, IdT, Cmp>;
      const int ns = std::min(nt, kSplitMaxThreads);
      const size_t smem = small_smem_bytes<Key, Val>(cfg.class_cap[cls]);
      GSS_TRY(set_smem(kern, small_smem_bytes<Key, Val>(cfg.class_cap[kNumClasses - 1])));
      static GridCache grid[kNumClasses];
      int g = grid[cls].get(di.dev);
      if (!g) { g = grid_for(kern, ns, smem, di.sms); grid[cls].put(di.dev, g); }
      return launch(prof, GSS_K_SMALL_SORT, s, count, [&] { kern<<<g, ns, smem, s>>>(c, (uint32_t)cls); });
    }
    auto kern = k_small_block<Key, Val, IdT, Cmp>;
    // ablation: register-capped instantiation for the narrower classes (not for 4-byte keys with values: it spills)
    constexpr bool kNarrowOk = !(kHasVal<Val> && sizeof(Key) == 4);
    const bool narrow = kNarrowOk && nt <= kSmallNarrowThreads && (cfg.flags & kFlagSmallNarrow);
    if constexpr (kNarrowOk) {
      if (narrow) kern = k_small_block<Key, Val, IdT, Cmp, false, kSmallNarrowThreads>;
    }
    if constexpr (sizeof(Key) == 8 && !kHasVal<Val> && std::is_same<Cmp, Less>::value) {
      if (cfg.flags & GSS_FLAG_BITONIC_NET) kern = k_small_block<Key, Val, IdT, Cmp, true>;   // ablation
    }
    const size_t smem = block_sort_smem_bytes<Key, Val>(nt);
    GSS_TRY(set_smem(kern, block_sort_smem_bytes<Key, Val>(narrow ? kSmallNarrowThreads : kSmallMaxThreads)));
    static GridCache grid[4][kNumClasses + 1];
    const int gv = ((cfg.flags & GSS_FLAG_BITONIC_NET) ? 1 : 0) + (narrow ? 2 : 0);
    int g = grid[gv][cls].get(di.dev);
    if (!g) { g = grid_for(kern, nt, smem, di.sms); grid[gv][cls].put(di.dev, g); }
    return launch(prof, GSS_K_SMALL_SORT, s, count, [&] { kern<<<g, nt, smem, s>>>(c, (uint32_t)cls); });
  }

  // The whole launch sequence.  mode: sort / partition / partition_by.
  static gss_status run(C& c, const Cfg& cfg, int mode, const DeviceInfo& di, cudaStream_t s, gss_profiler* prof,
                        uint32_t* count, uint32_t phase = 0) {
    if (phase != 2)
      GSS_TRY(launch(prof, GSS_K_INIT, s, count, [&] { k_init<Key, Val, IdT><<<1, 256, 0, s>>>(c); }));
    const uint32_t kmax = cfg.kmax;
    // kernels and their shared-memory sizes
    // the sample sort CTA: 512 threads (two per SM) when every bucket's a * k_b sample fits 8192 keys
    const bool half_sample = (uint64_t)cfg.a * kmax <= 8192 && !(cfg.flags & kFlagSampleFull);
    auto ks = half_sample ? k_sample<Key, Val, IdT, Cmp, kSampleThreads / 2> : k_sample<Key, Val, IdT, Cmp>;
    const int nt_sample = half_sample ? kSampleThreads / 2 : kSampleThreads;
    const size_t sm_sample = half_sample ? CtaSort<Key, NoVal, kSampleThreads / 2, Cmp>::smem_bytes()
                                         : CtaSort<Key, NoVal, kSampleThreads, Cmp>::smem_bytes();
    auto kc = mode == MODE_PARTITION_BY ? k_classify<Key, Val, IdT, Cmp, true> : k_classify<Key, Val, IdT, Cmp, false>;
    if constexpr (lut_ok<Key, Cmp>()) {
      if (mode != MODE_PARTITION_BY && c.lut) kc = k_classify<Key, Val, IdT, Cmp, false, true>;   // radix-indexed lookup
    }
    const size_t sm_cls = cls_smem_bytes<Key>(kmax);
    auto ksc = c.stable ? k_scatter<Key, Val, IdT, Cmp, true>
                        : (c.recompute ? k_scatter<Key, Val, IdT, Cmp, false, true> : k_scatter<Key, Val, IdT, Cmp, false>);
    const size_t sm_sc = ScatterSmem<Key, Val, IdT>::bytes(kmax, c.recompute != 0);
    GSS_TRY(set_smem(ks, sm_sample));
    GSS_TRY(set_smem(kc, sm_cls));
    GSS_TRY(set_smem(ksc, sm_sc));
    static GridCache gc_sample[2], gc_plan;
    int g_sample = gc_sample[half_sample].get(di.dev), g_plan = gc_plan.get(di.dev);
    if (!g_sample) { g_sample = grid_for(ks, nt_sample, sm_sample, di.sms); gc_sample[half_sample].put(di.dev, g_sample); }
    if (!g_plan) { g_plan = grid_for(k_plan<Key, Val, IdT>, kPlanThreads, 0, di.sms); gc_plan.put(di.dev, g_plan); }
    const int g_cls = grid_for(kc, kClsThreads, sm_cls, di.sms);
    const int g_sc = grid_for(ksc, kScatterThreads, sm_sc, di.sms);
    auto ksf = k_scatter_fast<Key, Val, IdT, Cmp>;
    const size_t sm_sf = ScatterFastSmem<Key, Val, IdT>::bytes(kmax);
    GSS_TRY(set_smem(ksf, sm_sf));
    const int g_sf = grid_for(ksf, kScatterThreads, sm_sf, di.sms);
    // default sort scatter: bulk-copy stores, two staging buffers when two CTAs still fit an SM
    using SBS = ScatterBulkSmem<Key, Val, IdT>;
    const bool bulk2 = SBS::bytes(kmax, 2) <= 113 * 1024;
    auto ksb = bulk2 ? k_scatter_bulk<Key, Val, IdT, 2> : k_scatter_bulk<Key, Val, IdT, 1>;
    if constexpr (!kHasVal<Val>) {
      if (cfg.flags & kFlagScatterCtaCounters)   // ablation: one counter set per CTA (nondeterministic intermediates)
        ksb = bulk2 ? k_scatter_bulk<Key, Val, IdT, 2, true> : k_scatter_bulk<Key, Val, IdT, 1, true>;
    }
    const size_t sm_sb = SBS::bytes(kmax, bulk2 ? 2 : 1);
    GSS_TRY(set_smem(ksb, sm_sb));
    const int g_sb = grid_for(ksb, kScatterThreads, sm_sb, di.sms);
    // bulk copies pay for 8-byte keys alone (2^28 u64: 2.92 vs 3.11 ms for the two levels); with values
    // they do not (2^27 u64 pairs 3.02 vs 2.99 ms; 2^29 pairs, k = 512, one staging buffer: 18.0 vs 16.8 ms),
    // nor for 4-byte keys, where the per-run copies (one warp-serialised UBLKCP each) cost more than the
    // coalesced per-key stores they replace (2^27 u32: 1.26 vs 1.05 ms); those keep GSS_FLAG_SCATTER_REGS
    const bool bulk_default = sizeof(Key) == 8 && !kHasVal<Val>;
    const bool use_bulk = c.nremote || (!c.stable && !c.recompute && (bulk_default || (cfg.flags & kFlagScatterBulk)) &&
                          !(cfg.flags & (GSS_FLAG_DIRECT_SCATTER | GSS_FLAG_SCATTER_REGS)) &&
                          !((cfg.flags & kFlagScatterCtaCounters) && kHasVal<Val>));
    // warp-specialised scatter: keys without values on the bulk path, local destinations, shared memory for
    // two chunk buffers at this kmax (k <= 512)
    bool use_ws = false;
    auto kws = k_scatter_bulk<Key, Val, IdT, 1>;
    size_t sm_ws = 0;
    int g_ws = 0;
    {
      // keys alone and 8-byte pairs: 14 rank + 2 I/O warps, two CTAs per SM; where their chunk buffers do not
      // fit (k = 512 with 16-bit ids; 4-byte keys, 16 per lane), 12 + 4 (shorter chunks).  16-byte pairs: two
      // CTAs per SM would leave 4 keys per lane, which measured slower than the single-role kernel (2^27 u64
      // pairs 3.64 vs 3.01 ms; u32 keys 0.83 vs 1.06, u32 pairs 1.94 vs 2.01,
      // profiles/r02_ab_scatter_ws_kinds.log), so they run one CTA per SM (profiles/r02_ab_scatter_ws_pairs.log)
      constexpr size_t kWsMax = 113 * 1024;
      constexpr bool kWsKind = !kHasVal<Val> || sizeof(Key) + sizeof(Val) <= 8;
      const bool ok0 = !c.nremote && !c.stable && !c.recompute && kmax <= 512 &&
                       !(cfg.flags & (GSS_FLAG_DIRECT_SCATTER | GSS_FLAG_SCATTER_REGS | kFlagScatterCtaCounters |
                                      kFlagScatterNoWs));
      const bool ok = kWsKind && ok0;
      if ((!kWsKind || (cfg.flags & kFlagScatterWsOne)) && ok0 &&
          ScatterWsSmem<Key, Val, IdT, GSS_SCATTER_IO_WARPS, true>::bytes(kmax) <= 227 * 1024) {
        // 16-byte pairs: one CTA per SM with the whole shared memory and 8 keys per lane (2^27 u64 pairs:
        // scatter 3.02 -> 2.57 ms, 2^29 at k = 512 16.7 -> 15.1; with two CTAs and 4 keys per lane it lost)
        use_ws = true;
        sm_ws = ScatterWsSmem<Key, Val, IdT, GSS_SCATTER_IO_WARPS, true>::bytes(kmax);
        kws = k_scatter_ws<Key, Val, IdT, GSS_SCATTER_IO_WARPS, true>;
      } else if (ok && ScatterWsSmem<Key, Val, IdT>::bytes(kmax) <= kWsMax) {
        use_ws = true;
        sm_ws = ScatterWsSmem<Key, Val, IdT>::bytes(kmax);
        kws = k_scatter_ws<Key, Val, IdT>;
      } else if (ok && ScatterWsSmem<Key, Val, IdT, 4>::bytes(kmax) <= kWsMax) {
        use_ws = true;
        sm_ws = ScatterWsSmem<Key, Val, IdT, 4>::bytes(kmax);
        kws = k_scatter_ws<Key, Val, IdT, 4>;
      }
      if (use_ws) {
        GSS_TRY(set_smem(kws, sm_ws));
        g_ws = grid_for(kws, kScatterThreads, sm_ws, di.sms);
      }
    }
    auto ksd = k_scatter_direct<Key, Val, IdT, Cmp>;
    const size_t sm_sd = (size_t)kmax * 4;
    GSS_TRY(set_smem(ksd, sm_sd));
    const int g_sd = grid_for(ksd, kDirectThreads, sm_sd, di.sms);
    for (uint32_t l = 0; l < c.L; l++) {
      if (phase != 2) {
      if (mode == MODE_PARTITION_BY) {
        GSS_TRY(launch(prof, GSS_K_SAMPLE, s, count, [&] { k_set_splitters<Key, Val, IdT><<<1, 256, 0, s>>>(c); }));
      } else {
        GSS_TRY(launch(prof, GSS_K_SAMPLE, s, count, [&] { ks<<<g_sample, nt_sample, sm_sample, s>>>(c, l); }));
      }
      GSS_TRY(launch(prof, GSS_K_CLASSIFY, s, count, [&] { kc<<<g_cls, kClsThreads, sm_cls, s>>>(c, l, kmax); }));
      GSS_TRY(launch(prof, GSS_K_SCAN, s, count,
                     [&] { k_scan_reduce<Key, Val, IdT><<<kScanCtas, kScanThreads, 0, s>>>(c, l); }));
      GSS_TRY(launch(prof, GSS_K_SCAN, s, count,
                     [&] { k_scan_final<Key, Val, IdT><<<kScanCtas, kScanThreads, 0, s>>>(c, l); }));
      }
      if (phase == 1) continue;                                   // the scatter follows in phase 2
      // default and stable ranks (R7, GSS_FLAG_STABLE): k_scatter with per-warp counters (deterministic);
      // ablations: k_scatter_fast (one counter set per CTA: atomic order across warps is not
      // deterministic) and the paper's direct scatter (k_scatter_direct)
      if (use_ws) {
        GSS_TRY(launch(prof, GSS_K_SCATTER, s, count, [&] { kws<<<g_ws, kScatterThreads, sm_ws, s>>>(c, l, kmax); }));
      } else if (use_bulk) {
        GSS_TRY(launch(prof, GSS_K_SCATTER, s, count, [&] { ksb<<<g_sb, kScatterThreads, sm_sb, s>>>(c, l, kmax); }));
      } else if (c.stable || !(cfg.flags & (GSS_FLAG_DIRECT_SCATTER | kFlagScatterCtaCounters))) {
        GSS_TRY(launch(prof, GSS_K_SCATTER, s, count, [&] { ksc<<<g_sc, kScatterThreads, sm_sc, s>>>(c, l, kmax); }));
      } else if (cfg.flags & kFlagScatterCtaCounters) {
        GSS_TRY(launch(prof, GSS_K_SCATTER, s, count, [&] { ksf<<<g_sf, kScatterThreads, sm_sf, s>>>(c, l, kmax); }));
      } else {
        GSS_TRY(launch(prof, GSS_K_SCATTER, s, count,
                       [&] { ksd<<<g_sd, kDirectThreads, sm_sd, s>>>(c, l); }));
      }
      if (mode == MODE_SORT)
        GSS_TRY(launch(prof, GSS_K_PLAN, s, count, [&] { k_plan<Key, Val, IdT><<<g_plan, kPlanThreads, 0, s>>>(c, l); }));
    }
    if (mode != MODE_SORT) return GSS_SUCCESS;
    if (cfg.M > cfg.class_cap[kNumClasses - 1]) {
      // the largest buckets first: thread-block clusters of kClusterCtas CTAs (GSS_FLAG_CLUSTER_SORT)
      auto kcl = k_small_cluster<Key, Val, IdT, Cmp>;
      constexpr size_t sm_cl = cluster_smem_bytes<Key, Val>();
      GSS_TRY(set_smem(kcl, sm_cl));
      const int g_cl = std::max(1, di.sms / kClusterCtas) * kClusterCtas;
      GSS_TRY(launch(prof, GSS_K_SMALL_SORT, s, count, [&] { kcl<<<g_cl, kClusterThreads, sm_cl, s>>>(c); }));
    }
    // in-SM sorts, largest class first (buckets "ordered by size"; R8)
    for (int cls = (int)cfg.nclass - 1; cls >= 0; cls--) GSS_TRY(launch_small(c, cfg, cls, di, s, prof, count));
    if (cfg.flags & GSS_FLAG_SPLIT_SORT) GSS_TRY(launch_small(c, cfg, kNumClasses, di, s, prof, count));
    GSS_TRY(launch(prof, GSS_K_COPY, s, count, [&] { k_copy<Key, Val, IdT><<<di.sms * 4, 256, 0, s>>>(c); }));
    constexpr int NTO = 1024;
    auto ko = k_overflow<Key, Val, IdT, Cmp, NTO>;
    const size_t sm_ovf = CtaSort<Key, Val, NTO, Cmp>::smem_bytes();
    GSS_TRY(set_smem(ko, sm_ovf));
    GSS_TRY(launch(prof, GSS_K_OVERFLOW, s, count, [&] { ko<<<di.sms, NTO, sm_ovf, s>>>(c); }));
    if (cfg.error_out) {
      // the capacity-check flags of this sort (0 = the result is valid), stream ordered, no host sync
      if (cudaMemcpyAsync(cfg.error_out, &c.cnt->err, sizeof(uint32_t), cudaMemcpyDeviceToDevice, s) != cudaSuccess) {
        cudaGetLastError();
        return GSS_ERROR_CUDA;
      }
    }
    return GSS_SUCCESS;
  }
};

inline void fill_stats(const Counters& h, uint32_t L, uint32_t launches, gss_stats* st) {
  memset(st, 0, sizeof(*st));
  st->launches = launches;
  st->levels_launched = L;
  st->error_flags = h.err;
  for (uint32_t l = 0; l < kMaxLevels && l < 16; l++) {
    st->split_elems[l] = h.lvl[l].split_elems;
    st->split_buckets[l] = h.lvl[l].num_buckets;
    if (h.lvl[l].num_buckets) st->levels = l + 1;
  }
  for (int i = 0; i < kNumClasses; i++) st->small_buckets += h.small_count[i];
  st->small_elems = h.small_elems;
  st->max_small = h.max_small;
  st->eq_buckets = h.eq_buckets;
  st->eq_elems = h.eq_elems;
  st->overflow_buckets = h.ovf_count;
  st->overflow_elems = h.ovf_elems;
  st->cluster_buckets = h.clus_count;
}

// Cache of instantiated launch graphs (GSS_FLAG_GRAPH), keyed by everything
// the captured kernels bake in: entry point, device, n, buffers, parameters.
struct GraphKey {
  const void* fn;
  int dev;
  uint64_t n;
  const void* p[6];
  uint32_t cfg[8];
  uint64_t seed;
  bool operator==(const GraphKey& o) const { return memcmp(this, &o, sizeof(GraphKey)) == 0; }
};
struct GraphEntry {
  GraphKey key;
  cudaGraphExec_t exec;
};
inline std::mutex g_graph_mu;
inline std::vector<GraphEntry> g_graphs;
inline constexpr size_t kGraphCacheSize = 16;

inline cudaStream_t capture_stream(int dev) {
  static cudaStream_t streams[64] = {};
  std::lock_guard<std::mutex> g(g_graph_mu);
  if (dev < 0 || dev >= 64) return nullptr;
  if (!streams[dev] && cudaStreamCreateWithFlags(&streams[dev], cudaStreamNonBlocking) != cudaSuccess) {
    cudaGetLastError();
    streams[dev] = nullptr;
  }
  return streams[dev];
}

inline cudaGraphExec_t graph_lookup(const GraphKey& k) {
  std::lock_guard<std::mutex> g(g_graph_mu);
  for (auto& e : g_graphs)
    if (e.key == k) return e.exec;
  return nullptr;
}
inline void graph_insert(const GraphKey& k, cudaGraphExec_t exec) {
  std::lock_guard<std::mutex> g(g_graph_mu);
  if (g_graphs.size() >= kGraphCacheSize) {
    cudaGraphExecDestroy(g_graphs.front().exec);
    g_graphs.erase(g_graphs.begin());
  }
  g_graphs.push_back({k, exec});
}

// Shared driver of every entry point.
struct IO {
  const void* kin; const void* vin; void* kout; void* vout;
  const void* h_kin; const void* h_vin; void* h_kout; void* h_vout;   // host variants
  // partition outputs
  void* spl_out; uint64_t* off_out; uint32_t* info_out; uint64_t* counts_out;
  const void* given_spl; uint32_t given_nspl; uint32_t given_eq;
  // distributed global level (internal): phase 1 = classify + counts, phase 2 = the scatter
  // of the same temp state to remote segments; unstable = non-stable (bulk) scatter
  uint32_t phase, unstable, nremote;
  const void* remote;
};

template <class Key, class Val, class Cmp>
gss_status drive(IO io, size_t n, void* temp, size_t* temp_bytes, void* stream, const gss_params* up, int mode,
                 bool host_io) {
  if (!temp_bytes) return GSS_ERROR_INVALID_VALUE;
  if (n >= (1ull << 32) - 16384) return GSS_ERROR_NOT_SUPPORTED;
  uint32_t kgiven = 0;
  if (mode == MODE_PARTITION_BY) {
    if (io.given_nspl > 1023) return GSS_ERROR_INVALID_VALUE;
    kgiven = 1;
    while (kgiven < io.given_nspl + 1) kgiven <<= 1;
    if (io.given_eq) kgiven *= 2;                               // K = 2 nspl + 1 counters
  }
  Cfg cfg;
  GSS_TRY(resolve<Key, Val>(up, n, &cfg, kgiven));
  auto run_id = [&](auto id_tag) -> gss_status {
    using IdT = decltype(id_tag);
    Layout<Key, Val, IdT> lay;
    lay.compute(n, cfg, mode, host_io);
    // every element offset, tile start and 16-aligned id offset is a u32
    if ((uint64_t)n + cfg.T >= (1ull << 32) || (uint64_t)n + 16ull * ((uint64_t)lay.cap_buckets + 2) >= (1ull << 32))
      return GSS_ERROR_NOT_SUPPORTED;
    if (!temp) { *temp_bytes = lay.total; return GSS_SUCCESS; }
    if (*temp_bytes < lay.total) return GSS_ERROR_TEMP_TOO_SMALL;
    if (n == 0) {
      if (up && up->stats) { memset(up->stats, 0, sizeof(gss_stats)); up->stats->levels_launched = 0; }
      return GSS_SUCCESS;
    }
    const size_t kb = n * sizeof(Key), vb = kHasVal<Val> ? n * sizeof(Val) : 0;
    if (host_io) {
      if (!io.h_kin || !io.h_kout || (kHasVal<Val> && (!io.h_vin || !io.h_vout))) return GSS_ERROR_INVALID_VALUE;
    } else {
      if (!io.kin || !io.kout || (kHasVal<Val> && (!io.vin || !io.vout))) return GSS_ERROR_INVALID_VALUE;
      if (!same_or_disjoint(io.kin, kb, io.kout, kb)) return GSS_ERROR_INVALID_VALUE;
      if (kHasVal<Val>) {
        if (!same_or_disjoint(io.vin, vb, io.vout, vb)) return GSS_ERROR_INVALID_VALUE;
        if (ranges_overlap(io.kin, kb, io.vin, vb) || ranges_overlap(io.kout, kb, io.vout, vb) ||
            ranges_overlap(io.kin, kb, io.vout, vb) || ranges_overlap(io.kout, kb, io.vin, vb))
          return GSS_ERROR_INVALID_VALUE;
      }
      const void* bufs[4] = {io.kin, io.kout, io.vin, io.vout};
      const size_t lens[4] = {kb, kb, vb, vb};
      for (int i = 0; i < 4; i++)
        if (ranges_overlap(temp, lay.total, bufs[i], lens[i])) return GSS_ERROR_INVALID_VALUE;
    }
    if ((uintptr_t)temp % 256) return GSS_ERROR_INVALID_VALUE;
    DeviceInfo di;
    GSS_TRY(device_info(&di));
    cudaStream_t s = reinterpret_cast<cudaStream_t>(stream);
    gss_profiler* prof = up ? up->profiler : nullptr;
    unsigned char* base = reinterpret_cast<unsigned char*>(temp);
    using Eng = Engine<Key, Val, IdT, Cmp>;
    auto c = Eng::make_ctx(base, lay, cfg, n, mode);
    uint32_t count = 0;
    const Key* kin = reinterpret_cast<const Key*>(io.kin);
    Key* kout = reinterpret_cast<Key*>(io.kout);
    const Val* vin = reinterpret_cast<const Val*>(io.vin);
    Val* vout = reinterpret_cast<Val*>(io.vout);
    if (host_io) {
      kin = reinterpret_cast<const Key*>(base + lay.off_hin_k);
      kout = reinterpret_cast<Key*>(base + lay.off_hout_k);
      if constexpr (kHasVal<Val>) {
        vin = reinterpret_cast<const Val*>(base + lay.off_hin_v);
        vout = reinterpret_cast<Val*>(base + lay.off_hout_v);
      }
      GSS_TRY(launch(prof, GSS_K_H2D, s, nullptr, [&] {
        cudaMemcpyAsync(const_cast<Key*>(kin), io.h_kin, kb, cudaMemcpyHostToDevice, s);
        if (kHasVal<Val>) cudaMemcpyAsync(const_cast<Val*>(vin), io.h_vin, vb, cudaMemcpyHostToDevice, s);
      }));
    }
    c.kin = kin; c.kout = kout;
    if constexpr (kHasVal<Val>) { c.vin = vin; c.vout = vout; }
    c.src0 = BUF_IN;
    c.dst0 = BUF_TMP;
    if (mode != MODE_SORT) {
      c.dst0 = BUF_OUT;
      if ((const void*)kin == (const void*)kout) {
        // the scatter cannot run in place: stage the input in the temp buffer first
        GSS_TRY(launch(prof, GSS_K_COPY, s, nullptr, [&] {
          cudaMemcpyAsync(c.ktmp, kin, kb, cudaMemcpyDeviceToDevice, s);
          if constexpr (kHasVal<Val>) cudaMemcpyAsync(c.vtmp, vin, vb, cudaMemcpyDeviceToDevice, s);
        }));
        c.src0 = BUF_TMP;
        c.dst0 = BUF_OUT;
      }
      c.given_spl = reinterpret_cast<const Key*>(io.given_spl);
      c.given_nspl = io.given_nspl;
      c.given_eq = io.given_eq ? 1u : 0u;
      if (io.unstable) c.stable = 0;
      c.remote = reinterpret_cast<const RemoteSeg*>(io.remote);
      c.nremote = io.nremote;
    }
    if ((cfg.flags & GSS_FLAG_GRAPH) && mode == MODE_SORT && !host_io && !prof && !(up && up->stats)) {
      // replay (or capture once) the whole launch sequence as a CUDA graph
      GraphKey key;
      memset(&key, 0, sizeof(key));
      key.fn = reinterpret_cast<const void*>(&Eng::run);
      key.dev = di.dev;
      key.n = n;
      key.p[0] = io.kin; key.p[1] = io.kout; key.p[2] = io.vin; key.p[3] = io.vout; key.p[4] = temp;
      key.p[5] = cfg.error_out;
      key.cfg[0] = cfg.k; key.cfg[1] = cfg.a; key.cfg[2] = cfg.T; key.cfg[3] = cfg.L; key.cfg[4] = cfg.k_policy;
      key.cfg[5] = cfg.fill_div | (cfg.cls_arrays << 24); key.cfg[6] = cfg.flags; key.cfg[7] = (uint32_t)cfg.M;
      key.seed = cfg.seed;
      cudaGraphExec_t exec = graph_lookup(key);
      if (!exec) {
        // capture on a private non-blocking stream (the caller's may be the legacy
        // default stream, which cannot be captured); the graph replays on `s`
        cudaGraph_t g = nullptr;
        cudaStream_t cs = capture_stream(di.dev);
        if (!cs || cudaStreamBeginCapture(cs, cudaStreamCaptureModeThreadLocal) != cudaSuccess) {
          cudaGetLastError();
          return GSS_ERROR_CUDA;
        }
        const gss_status st = Eng::run(c, cfg, mode, di, cs, nullptr, &count);
        const cudaError_t ce = cudaStreamEndCapture(cs, &g);
        if (st != GSS_SUCCESS || ce != cudaSuccess) {
          cudaGetLastError();
          if (g) cudaGraphDestroy(g);
          return st != GSS_SUCCESS ? st : GSS_ERROR_CUDA;
        }
        if (cudaGraphInstantiate(&exec, g, 0) != cudaSuccess) {
          cudaGetLastError();
          cudaGraphDestroy(g);
          return GSS_ERROR_CUDA;
        }
        cudaGraphDestroy(g);
        graph_insert(key, exec);
      }
      if (cudaGraphLaunch(exec, s) != cudaSuccess) { cudaGetLastError(); return GSS_ERROR_CUDA; }
      return GSS_SUCCESS;
    }
    GSS_TRY(Eng::run(c, cfg, mode, di, s, prof, &count, io.phase));
    if (mode != MODE_SORT && io.phase != 2) {
      GSS_TRY(launch(prof, GSS_K_OTHER, s, &count, [&] {
        k_partition_out<Key, Val, IdT><<<1, 256, 0, s>>>(c, reinterpret_cast<Key*>(io.spl_out), io.off_out,
                                                          io.info_out, io.counts_out);
      }));
    }
    if (host_io) {
      GSS_TRY(launch(prof, GSS_K_D2H, s, nullptr, [&] {
        cudaMemcpyAsync(io.h_kout, kout, kb, cudaMemcpyDeviceToHost, s);
        if (kHasVal<Val>) cudaMemcpyAsync(io.h_vout, vout, vb, cudaMemcpyDeviceToHost, s);
      }));
    }
    if (up && up->stats) {
      Counters h;
      if (cudaStreamSynchronize(s) != cudaSuccess) { cudaGetLastError(); return GSS_ERROR_CUDA; }
      if (cudaMemcpy(&h, c.cnt, sizeof(Counters), cudaMemcpyDeviceToHost) != cudaSuccess) {
        cudaGetLastError();
        return GSS_ERROR_CUDA;
      }
      fill_stats(h, c.L, count, up->stats);
    }
    return GSS_SUCCESS;
  };
  if (cfg.kmax <= 256) return run_id(uint8_t{});
  return run_id(uint16_t{});
}

inline IO io_dev(const void* kin, const void* vin, void* kout, void* vout) {
  IO io{};
  io.kin = kin; io.vin = vin; io.kout = kout; io.vout = vout;
  return io;
}
inline IO io_host(const void* kin, const void* vin, void* kout, void* vout) {
  IO io{};
  io.h_kin = kin; io.h_vin = vin; io.h_kout = kout; io.h_vout = vout;
  return io;
}

#define GSS_DRIVE_SIG(K, V, C) \
  gss_status drive<K, V, C>(IO, size_t, void*, size_t*, void*, const gss_params*, int, bool)
#define GSS_FOR_EACH_INSTANCE(X) \
  X(uint32_t, NoVal, Less)       \
  X(uint64_t, NoVal, Less)       \
  X(uint32_t, uint32_t, Less)    \
  X(uint64_t, uint64_t, Less)    \
  X(uint64_t, NoVal, Greater)    \
  X(uint32_t, NoVal, Greater)    \
  X(uint32_t, uint32_t, Greater) \
  X(uint64_t, uint64_t, Greater) \
  X(float, NoVal, TotalLess)     \
  X(double, NoVal, TotalLess)
#ifndef GSS_INSTANTIATING
#define GSS_EXTERN_INSTANCE(K, V, C) extern template GSS_DRIVE_SIG(K, V, C);
GSS_FOR_EACH_INSTANCE(GSS_EXTERN_INSTANCE)
#endif

}  // namespace gssh
