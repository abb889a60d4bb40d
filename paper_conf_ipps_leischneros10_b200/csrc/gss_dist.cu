// gss_dist.cu -- distributed sample sort across GPUs, one process per GPU,
// NCCL over NVLink/NVSwitch.
//
// The paper is single-GPU; it names distributed memory as sample sort's home
// and argues that large random samples give
// splitters that balance the parts.  One call on rank r of P:
//
//  1. all-gather (n_local, out_capacity) of every rank (one host sync): the
//     global shard starts, the total N, and every rank's capacity, so every
//     rank takes the same decisions below (no rank can stop alone);
//  2. sample S keys of the local shard at hashed positions (R2, level tag 255,
//     lo = the shard's global start) -- gss_sample;
//  3. all-gather the samples; every rank sorts the identical gathered sample
//     (gss_sort) and picks the identical P-1 global splitters
//     spl[i] = S[(i+1) V S / P - 1] (R1; V = ranks with keys);
//  4. partition the shard by the splitters in equality mode (R4 applied to the
//     global level: id 2b = keys strictly between splitters b-1 and b, id
//     2b+1 = keys equal to splitter b) -- gss_partition_by_eq (stable);
//  5. all-gather the 2P-1 bucket counts of every rank (one host sync) and
//     compute the exchange plan on the host (gss_dist_plan): rank q owns the
//     global positions [cut_q, cut_{q+1}); a cut falls on a range-bucket
//     boundary, or anywhere inside an equality bucket (all its keys are
//     equal, so splitting it keeps the order) -- duplicate-heavy inputs stay
//     balanced;
//  6. grouped ncclSend / ncclRecv of keys (and values): the all-to-all-v,
//     received source-major into keys_out;
//  7. sort the received range in place (gss_sort).
// Rank r ends with the r-th contiguous range of the global sorted order.
//
// GSS_FLAG_DIST_FUSED fuses steps 4 and 6: the partition is
// only classified and counted before the plan (gssi_dist_level phase 1); after
// the plan, its scatter kernel (phase 2, the bulk-copy scatter) stores every
// bucket run straight into the receiving GPU's NCCL symmetric window
// (ncclMemAlloc + ncclCommWindowRegister; peer addresses from
// ncclGetPeerPointer over NVLink), so the exchange overlaps the scatter's HBM
// traffic and the partitioned shard is never written locally.  A one-element
// ncclAllReduce then orders every peer's stores before the local sort, which
// reads the window and writes keys_out.
#include <cuda_runtime.h>
#include <nccl.h>
#include <nccl_device.h>

#include <algorithm>
#include <cstring>
#include <new>
#include <vector>

#include "../../include/gss.h"

extern "C" {
gss_status gssi_dist_level_u32(const uint32_t* ki, const uint32_t* vi, uint32_t* kb, uint32_t* vb, size_t n,
                               const uint32_t* spl, uint32_t nspl, uint64_t* counts, const void* remote,
                               uint32_t nremote, uint32_t phase, void* t, size_t* tb, void* s);
gss_status gssi_dist_level_u64(const uint64_t* ki, const uint64_t* vi, uint64_t* kb, uint64_t* vb, size_t n,
                               const uint64_t* spl, uint32_t nspl, uint64_t* counts, const void* remote,
                               uint32_t nremote, uint32_t phase, void* t, size_t* tb, void* s);
}


namespace {

constexpr uint32_t kDistSamples = 16384;   // per rank (balance: max/mean load ~1.01 at P = 8)
constexpr uint32_t kDistTag = 255;         // level tag of the global sample (R2)

inline size_t align_up(size_t x, size_t a = 256) { return (x + a - 1) / a * a; }

template <class Key>
__global__ void k_pick_splitters(const Key* sorted, uint64_t vs, uint32_t P, Key* spl) {
  for (uint32_t i = threadIdx.x; i + 1 < P; i += blockDim.x) spl[i] = sorted[((uint64_t)(i + 1) * vs) / P - 1];
}

// every rank's window base as this GPU addresses it (LSA team over NVLink)
__global__ void k_peer_ptrs(ncclWindow_t wk, ncclWindow_t wv, int P, void** out) {
  for (int q = threadIdx.x; q < P; q += blockDim.x) {
    out[q] = ncclGetPeerPointer(wk, 0, q);
    out[P + q] = wv ? ncclGetPeerPointer(wv, 0, q) : nullptr;
  }
}

template <class Key> struct KeyOps;
template <> struct KeyOps<uint32_t> {
  static constexpr ncclDataType_t nccl = ncclUint32;
  static gss_status level(const uint32_t* ki, const uint32_t* vi, uint32_t* kb, uint32_t* vb, size_t n,
                          const uint32_t* spl, uint32_t nspl, uint64_t* cnt, const void* rem, uint32_t nrem,
                          uint32_t phase, void* t, size_t* tb, void* s) {
    return gssi_dist_level_u32(ki, vi, kb, vb, n, spl, nspl, cnt, rem, nrem, phase, t, tb, s);
  }
  static gss_status sort(const uint32_t* ki, uint32_t* ko, size_t n, void* t, size_t* tb, void* s, const gss_params* p) {
    return gss_sort_u32(ki, ko, n, t, tb, s, p);
  }
  static gss_status sort_pairs(const uint32_t* ki, const uint32_t* vi, uint32_t* ko, uint32_t* vo, size_t n, void* t,
                               size_t* tb, void* s, const gss_params* p) {
    return gss_sort_pairs_u32(ki, vi, ko, vo, n, t, tb, s, p);
  }
  static gss_status sample(const uint32_t* k, size_t n, uint64_t lo, uint64_t seed, uint32_t* out, size_t s, void* st) {
    return gss_sample_u32(k, n, lo, kDistTag, seed, out, s, st);
  }
  static gss_status part(const uint32_t* ki, const uint32_t* vi, uint32_t* ko, uint32_t* vo, size_t n,
                         const uint32_t* spl, uint32_t nspl, uint64_t* cnt, void* t, size_t* tb, void* s) {
    return gss_partition_by_eq_u32(ki, vi, ko, vo, n, spl, nspl, cnt, t, tb, s);
  }
};
template <> struct KeyOps<uint64_t> {
  static constexpr ncclDataType_t nccl = ncclUint64;
  static gss_status level(const uint64_t* ki, const uint64_t* vi, uint64_t* kb, uint64_t* vb, size_t n,
                          const uint64_t* spl, uint32_t nspl, uint64_t* cnt, const void* rem, uint32_t nrem,
                          uint32_t phase, void* t, size_t* tb, void* s) {
    return gssi_dist_level_u64(ki, vi, kb, vb, n, spl, nspl, cnt, rem, nrem, phase, t, tb, s);
  }
  static gss_status sort(const uint64_t* ki, uint64_t* ko, size_t n, void* t, size_t* tb, void* s, const gss_params* p) {
    return gss_sort_u64(ki, ko, n, t, tb, s, p);
  }
  static gss_status sort_pairs(const uint64_t* ki, const uint64_t* vi, uint64_t* ko, uint64_t* vo, size_t n, void* t,
                               size_t* tb, void* s, const gss_params* p) {
    return gss_sort_pairs_u64(ki, vi, ko, vo, n, t, tb, s, p);
  }
  static gss_status sample(const uint64_t* k, size_t n, uint64_t lo, uint64_t seed, uint64_t* out, size_t s, void* st) {
    return gss_sample_u64(k, n, lo, kDistTag, seed, out, s, st);
  }
  static gss_status part(const uint64_t* ki, const uint64_t* vi, uint64_t* ko, uint64_t* vo, size_t n,
                         const uint64_t* spl, uint32_t nspl, uint64_t* cnt, void* t, size_t* tb, void* s) {
    return gss_partition_by_eq_u64(ki, vi, ko, vo, n, spl, nspl, cnt, t, tb, s);
  }
};

#define DTRY(...)                         \
  do {                                    \
    gss_status _s = (__VA_ARGS__);        \
    if (_s != GSS_SUCCESS) return _s;     \
  } while (0)
#define NTRY(...)                                     \
  do {                                                \
    if ((__VA_ARGS__) != ncclSuccess) return GSS_ERROR_NCCL; \
  } while (0)
#define CTRY(...)                                                      \
  do {                                                                 \
    if ((__VA_ARGS__) != cudaSuccess) { cudaGetLastError(); return GSS_ERROR_CUDA; } \
  } while (0)

}  // namespace

struct gss_dist {
  ncclComm_t comm = nullptr;
  int rank = 0, P = 1, dev = 0;
  uint64_t* h_buf = nullptr;       // pinned staging of the small exchanges and the segment table
  size_t h_cap = 0;
  std::vector<uint64_t> send_cnt, recv_cnt, cuts;   // the last call's exchange plan
  // fused exchange: symmetric receive windows (keys, values) of wcap elements
  void* wk = nullptr;
  void* wv = nullptr;
  ncclWindow_t win_k = nullptr, win_v = nullptr;
  size_t wcap = 0, welem = 0;
  std::vector<void*> peer_k, peer_v;                  // every rank's window, as seen from this GPU
};

namespace {

// Symmetric receive windows of at least cap elements of w bytes (keys, and values when kv), registered
// collectively (every rank calls with the same cap), and every rank's window address as seen here.
gss_status ensure_windows(gss_dist* d, size_t cap, size_t w, bool kv, void** d_ptrs, cudaStream_t s) {
  if (d->wk && d->wcap >= cap && d->welem == w && (!kv || d->wv)) return GSS_SUCCESS;
  CTRY(cudaStreamSynchronize(s));
  if (d->win_k) ncclCommWindowDeregister(d->comm, d->win_k);
  if (d->win_v) ncclCommWindowDeregister(d->comm, d->win_v);
  if (d->wk) ncclMemFree(d->wk);
  if (d->wv) ncclMemFree(d->wv);
  d->wk = d->wv = nullptr;
  d->win_k = d->win_v = nullptr;
  d->wcap = 0;
  const size_t bytes = align_up(std::max<size_t>(cap, 1) * w, (size_t)1 << 21);
  NTRY(ncclMemAlloc(&d->wk, bytes));
  NTRY(ncclCommWindowRegister(d->comm, d->wk, bytes, &d->win_k, NCCL_WIN_COLL_SYMMETRIC));
  if (kv) {
    NTRY(ncclMemAlloc(&d->wv, bytes));
    NTRY(ncclCommWindowRegister(d->comm, d->wv, bytes, &d->win_v, NCCL_WIN_COLL_SYMMETRIC));
  }
  k_peer_ptrs<<<1, 64, 0, s>>>(d->win_k, d->win_v, d->P, d_ptrs);
  CTRY(cudaGetLastError());
  std::vector<void*> h(2 * (size_t)d->P);
  CTRY(cudaMemcpyAsync(h.data(), d_ptrs, h.size() * sizeof(void*), cudaMemcpyDeviceToHost, s));
  CTRY(cudaStreamSynchronize(s));
  d->peer_k.assign(h.begin(), h.begin() + d->P);
  d->peer_v.assign(h.begin() + d->P, h.end());
  d->wcap = bytes / w;
  d->welem = w;
  return GSS_SUCCESS;
}

gss_status host_buf(gss_dist* d, size_t words) {
  if (d->h_cap >= words) return GSS_SUCCESS;
  if (d->h_buf) cudaFreeHost(d->h_buf);
  d->h_buf = nullptr;
  d->h_cap = 0;
  CTRY(cudaMallocHost(&d->h_buf, words * sizeof(uint64_t)));
  d->h_cap = words;
  return GSS_SUCCESS;
}

template <class Key, class Val>
struct DistLayout {
  size_t off_meta, off_meta_all, off_smp, off_smp_all, off_smp_sorted, off_smp_temp, off_spl, off_cnt, off_cnt_all,
      off_part_k, off_part_v, off_part_temp, off_sort_temp, off_peer, off_seg, off_one, total;
  size_t smp_temp, part_temp, sort_temp;
};

inline bool fused_mode(const gss_params* p) { return p && (p->flags & GSS_FLAG_DIST_FUSED); }

// Host view of the internal sub-calls' parameters: the caller's method
// parameters, without statistics (only the local sort reports them).
inline gss_params sub_params(const gss_params* p, bool keep_stats) {
  gss_params q{};
  if (p) q = *p;
  if (!keep_stats) { q.stats = nullptr; q.error_out = nullptr; }
  q.flags &= ~GSS_FLAG_GRAPH;   // the buffers of the sub-calls change with the received count
  return q;
}

template <class Key, class Val>
gss_status dist_layout(int P, size_t n_local, size_t cap, const gss_params* p, DistLayout<Key, Val>* L) {
  constexpr bool KV = !std::is_same<Val, void>::value;
  using Ops = KeyOps<Key>;
  const size_t S = kDistSamples, PS = (size_t)P * S;
  gss_params sp = sub_params(p, false);
  size_t tb = 0;
  DTRY(Ops::sort(nullptr, nullptr, PS, nullptr, &tb, nullptr, &sp));
  L->smp_temp = tb;
  tb = 0;
  // the query must name the instantiation: a non-null value pointer selects the key-value one
  const Key* vsel = KV ? reinterpret_cast<const Key*>(alignof(Key)) : nullptr;
  const bool fused = fused_mode(p);
  if (fused)
    DTRY(Ops::level(nullptr, vsel, nullptr, nullptr, n_local, nullptr, (uint32_t)(P - 1), nullptr, nullptr, 0, 1,
                    nullptr, &tb, nullptr));
  else
    DTRY(Ops::part(nullptr, vsel, nullptr, nullptr, n_local, nullptr, (uint32_t)(P - 1), nullptr, nullptr, &tb, nullptr));
  L->part_temp = tb;
  tb = 0;
  if constexpr (KV) DTRY(Ops::sort_pairs(nullptr, nullptr, nullptr, nullptr, cap, nullptr, &tb, nullptr, &sp));
  else DTRY(Ops::sort(nullptr, nullptr, cap, nullptr, &tb, nullptr, &sp));
  L->sort_temp = tb;
  size_t o = 0;
  auto take = [&](size_t b) { size_t r = o; o = align_up(o + b); return r; };
  const size_t K = 2 * (size_t)P - 1;
  L->off_meta = take(2 * sizeof(uint64_t));
  L->off_meta_all = take(2 * sizeof(uint64_t) * P);
  L->off_smp = take(S * sizeof(Key));
  L->off_smp_all = take(PS * sizeof(Key));
  L->off_smp_sorted = take(PS * sizeof(Key));
  L->off_smp_temp = take(L->smp_temp);
  L->off_spl = take((size_t)P * sizeof(Key));
  L->off_cnt = take(K * sizeof(uint64_t));
  L->off_cnt_all = take(K * P * sizeof(uint64_t));
  L->off_part_k = fused ? 0 : take(n_local * sizeof(Key));      // the fused path never writes the partition locally
  L->off_part_v = (KV && !fused) ? take(n_local * sizeof(Key)) : 0;
  L->off_part_temp = take(L->part_temp);
  L->off_sort_temp = take(L->sort_temp);
  L->off_peer = take(2 * (size_t)P * sizeof(void*));
  L->off_seg = take((size_t)P * 32);
  L->off_one = take(sizeof(uint64_t));
  L->total = o;
  return GSS_SUCCESS;
}

// Val = void: keys only; Val = Key: pairs (values have the key's width).
template <class Key, class Val>
gss_status dist_sort(gss_dist* d, const Key* kin, const Key* vin, size_t n_local, Key* kout, Key* vout, size_t cap,
                     size_t* n_out, void* temp, size_t* temp_bytes, void* stream, const gss_params* p) {
  constexpr bool KV = !std::is_same<Val, void>::value;
  using Ops = KeyOps<Key>;
  if (!d || !temp_bytes) return GSS_ERROR_INVALID_VALUE;
  const int P = d->P, r = d->rank;
  DistLayout<Key, Val> L;
  DTRY(dist_layout<Key, Val>(P, n_local, cap, p, &L));
  if (!temp) { *temp_bytes = L.total; return GSS_SUCCESS; }
  if (*temp_bytes < L.total) return GSS_ERROR_TEMP_TOO_SMALL;
  if (!n_out || (uintptr_t)temp % 256) return GSS_ERROR_INVALID_VALUE;
  if ((n_local && !kin) || (cap && !kout) || (KV && ((n_local && !vin) || (cap && !vout)))) return GSS_ERROR_INVALID_VALUE;
  if (cudaSetDevice(d->dev) != cudaSuccess) { cudaGetLastError(); return GSS_ERROR_CUDA; }
  cudaStream_t s = reinterpret_cast<cudaStream_t>(stream);
  unsigned char* base = reinterpret_cast<unsigned char*>(temp);
  auto at = [&](size_t off) { return reinterpret_cast<void*>(base + off); };
  const ncclDataType_t dt = Ops::nccl;
  const uint32_t S = kDistSamples;
  const size_t K = 2 * (size_t)P - 1;
  DTRY(host_buf(d, std::max<size_t>(2 * (size_t)P, K * P) + 4 * (size_t)P));
  const bool fused = fused_mode(p);
  uint64_t* h = d->h_buf;
  gss_params sp = sub_params(p, false);
  const uint64_t seed = (p && p->seed) ? p->seed : 5489;

  // 1. (n_local, capacity) of every rank
  uint64_t meta[2] = {n_local, cap};
  uint64_t* d_meta = reinterpret_cast<uint64_t*>(at(L.off_meta));
  uint64_t* d_meta_all = reinterpret_cast<uint64_t*>(at(L.off_meta_all));
  CTRY(cudaMemcpyAsync(d_meta, meta, sizeof(meta), cudaMemcpyHostToDevice, s));
  NTRY(ncclAllGather(d_meta, d_meta_all, 2, ncclUint64, d->comm, s));
  CTRY(cudaMemcpyAsync(h, d_meta_all, 2 * sizeof(uint64_t) * P, cudaMemcpyDeviceToHost, s));
  CTRY(cudaStreamSynchronize(s));
  std::vector<uint64_t> ns(P), caps(P);
  uint64_t N = 0, lo_r = 0;
  uint32_t V = 0;
  for (int q = 0; q < P; q++) {
    ns[q] = h[2 * q]; caps[q] = h[2 * q + 1];
    if (q < r) lo_r += ns[q];
    N += ns[q];
    V += ns[q] ? 1u : 0u;
  }
  d->send_cnt.assign(P, 0); d->recv_cnt.assign(P, 0); d->cuts.assign(P + 1, 0);
  if (N == 0) { *n_out = 0; return GSS_SUCCESS; }
  if (fused) {
    // windows sized for the largest capacity of any rank (same call on every rank)
    const uint64_t maxcap = *std::max_element(caps.begin(), caps.end());
    DTRY(ensure_windows(d, std::max<uint64_t>(maxcap, 1), sizeof(Key), KV, reinterpret_cast<void**>(at(L.off_peer)), s));
  }

  // 2-3. global sample, identical sorted sample and splitters on every rank
  Key* smp = reinterpret_cast<Key*>(at(L.off_smp));
  Key* smp_all = reinterpret_cast<Key*>(at(L.off_smp_all));
  Key* smp_sorted = reinterpret_cast<Key*>(at(L.off_smp_sorted));
  Key* spl = reinterpret_cast<Key*>(at(L.off_spl));
  if (n_local) DTRY(Ops::sample(kin, n_local, lo_r, seed, smp, S, s));
  else CTRY(cudaMemsetAsync(smp, 0, S * sizeof(Key), s));
  NTRY(ncclAllGather(smp, smp_all, S, dt, d->comm, s));
  // only the blocks of ranks that hold keys count (V of them), compacted in rank order
  uint32_t vpos = 0;
  for (int q = 0; q < P; q++) {
    if (!ns[q]) continue;
    if (vpos != (uint32_t)q)
      CTRY(cudaMemcpyAsync(smp_all + (size_t)vpos * S, smp_all + (size_t)q * S, S * sizeof(Key),
                           cudaMemcpyDeviceToDevice, s));
    vpos++;
  }
  const size_t VS = (size_t)V * S;
  size_t tb = L.smp_temp;
  DTRY(Ops::sort(smp_all, smp_sorted, VS, at(L.off_smp_temp), &tb, s, &sp));
  if (P > 1) {
    k_pick_splitters<Key><<<1, 256, 0, s>>>(smp_sorted, VS, (uint32_t)P, spl);
    CTRY(cudaGetLastError());
  }

  // 4. equality-mode partition of the shard into 2P-1 buckets (stable)
  Key* pk = reinterpret_cast<Key*>(at(L.off_part_k));
  Key* pv = KV ? reinterpret_cast<Key*>(at(L.off_part_v)) : nullptr;
  uint64_t* d_cnt = reinterpret_cast<uint64_t*>(at(L.off_cnt));
  uint64_t* d_cnt_all = reinterpret_cast<uint64_t*>(at(L.off_cnt_all));
  Key* wk = reinterpret_cast<Key*>(d->wk);
  Key* wv = reinterpret_cast<Key*>(d->wv);
  if (n_local && fused) {
    // phase 1: classify + counts only (the window is a stand-in output buffer, never written here)
    tb = L.part_temp;
    DTRY(Ops::level(kin, KV ? vin : nullptr, wk, KV ? wv : nullptr, n_local, spl, (uint32_t)(P - 1), d_cnt, nullptr, 0,
                    1, at(L.off_part_temp), &tb, s));
  } else if (n_local) {
    tb = L.part_temp;
    DTRY(Ops::part(kin, KV ? vin : nullptr, pk, pv, n_local, spl, (uint32_t)(P - 1), d_cnt, at(L.off_part_temp), &tb, s));
  } else {
    CTRY(cudaMemsetAsync(d_cnt, 0, K * sizeof(uint64_t), s));
  }

  // 5. counts of every rank, the exchange plan (same on every rank)
  NTRY(ncclAllGather(d_cnt, d_cnt_all, K, ncclUint64, d->comm, s));
  CTRY(cudaMemcpyAsync(h, d_cnt_all, K * P * sizeof(uint64_t), cudaMemcpyDeviceToHost, s));
  CTRY(cudaStreamSynchronize(s));
  std::vector<uint64_t> cuts(P + 1), soff(P), scnt(P), rcnt(P);
  // capacity: every rank checks every rank, so all of them stop together
  bool over = false;
  uint64_t need_me = 0;
  std::vector<uint64_t> my_off_in(P, 0);                 // where this rank's data starts in rank q's receive layout
  for (int q = 0; q < P; q++) {
    DTRY(gss_dist_plan((uint32_t)P, (uint32_t)q, (uint32_t)K, h, cuts.data(), soff.data(), scnt.data(), rcnt.data()));
    uint64_t need = 0;
    for (int x = 0; x < P; x++) {
      if (x == r) my_off_in[q] = need;
      need += rcnt[x];
    }
    if (need > caps[q]) over = true;
    if (q == r) need_me = need;
  }
  DTRY(gss_dist_plan((uint32_t)P, (uint32_t)r, (uint32_t)K, h, cuts.data(), soff.data(), scnt.data(), rcnt.data()));
  d->send_cnt = scnt; d->recv_cnt = rcnt; d->cuts = cuts;
  *n_out = need_me;
  if (over) return GSS_ERROR_CAPACITY;

  if (fused) {
    // 6'. phase 2: the scatter writes each run into the window of the rank that owns it, at
    //     (this rank's start in that rank's receive layout) + (partition index - segment start)
    uint64_t* hs = h + std::max<size_t>(2 * (size_t)P, K * P);
    for (int q = 0; q < P; q++) {
      uint32_t* seg = reinterpret_cast<uint32_t*>(hs + 4 * (size_t)q);
      seg[0] = (uint32_t)soff[q];
      seg[1] = (uint32_t)(soff[q] + scnt[q]);
      seg[2] = seg[3] = 0;
      const int64_t shift = (int64_t)my_off_in[q] - (int64_t)soff[q];
      Key* kd = reinterpret_cast<Key*>(d->peer_k[q]) + shift;
      Key* vd = KV ? reinterpret_cast<Key*>(d->peer_v[q]) + shift : nullptr;
      memcpy(hs + 4 * (size_t)q + 2, &kd, sizeof(void*));
      memcpy(hs + 4 * (size_t)q + 3, &vd, sizeof(void*));
    }
    void* d_seg = at(L.off_seg);
    CTRY(cudaMemcpyAsync(d_seg, hs, 32 * (size_t)P, cudaMemcpyHostToDevice, s));
    if (n_local) {
      tb = L.part_temp;
      DTRY(Ops::level(kin, KV ? vin : nullptr, wk, KV ? wv : nullptr, n_local, spl, (uint32_t)(P - 1), d_cnt, d_seg,
                      (uint32_t)P, 2, at(L.off_part_temp), &tb, s));
    }
    // every rank's stores into every window are complete before anyone reads its window
    uint64_t* d_one = reinterpret_cast<uint64_t*>(at(L.off_one));
    NTRY(ncclAllReduce(d_one, d_one, 1, ncclUint64, ncclSum, d->comm, s));
    // 7'. local sort: window -> keys_out
    gss_params lp = sub_params(p, true);
    tb = L.sort_temp;
    if constexpr (KV) DTRY(Ops::sort_pairs(wk, wv, kout, vout, need_me, at(L.off_sort_temp), &tb, s, &lp));
    else DTRY(Ops::sort(wk, kout, need_me, at(L.off_sort_temp), &tb, s, &lp));
    return GSS_SUCCESS;
  }

  // 6. all-to-all-v over NCCL: one message per peer and array, received source-major
  std::vector<uint64_t> roff(P);
  uint64_t acc = 0;
  for (int q = 0; q < P; q++) { roff[q] = acc; acc += rcnt[q]; }
  NTRY(ncclGroupStart());
  for (int q = 0; q < P; q++) {
    if (scnt[q]) {
      NTRY(ncclSend(pk + soff[q], scnt[q], dt, q, d->comm, s));
      if constexpr (KV) NTRY(ncclSend(pv + soff[q], scnt[q], dt, q, d->comm, s));
    }
    if (rcnt[q]) {
      NTRY(ncclRecv(kout + roff[q], rcnt[q], dt, q, d->comm, s));
      if constexpr (KV) NTRY(ncclRecv(vout + roff[q], rcnt[q], dt, q, d->comm, s));
    }
  }
  NTRY(ncclGroupEnd());

  // 7. local sort of the received range, in place
  gss_params lp = sub_params(p, true);
  tb = L.sort_temp;
  if constexpr (KV) DTRY(Ops::sort_pairs(kout, vout, kout, vout, need_me, at(L.off_sort_temp), &tb, s, &lp));
  else DTRY(Ops::sort(kout, kout, need_me, at(L.off_sort_temp), &tb, s, &lp));
  return GSS_SUCCESS;
}

}  // namespace

extern "C" {

gss_status gss_dist_plan(uint32_t P, uint32_t me, uint32_t K, const uint64_t* counts, uint64_t* cuts,
                         uint64_t* send_off, uint64_t* send_cnt, uint64_t* recv_cnt) {
  if (P == 0 || me >= P || K != 2 * P - 1 || !counts || !cuts || !send_off || !send_cnt || !recv_cnt)
    return GSS_ERROR_INVALID_VALUE;
  // global bucket sizes G[i] and starts GS[i]; O[q][i]: start of source q's slice of bucket i
  std::vector<uint64_t> G(K, 0), GS(K + 1, 0), O((size_t)P * K, 0);
  for (uint32_t i = 0; i < K; i++) {
    uint64_t run = 0;
    for (uint32_t q = 0; q < P; q++) { O[(size_t)q * K + i] = run; run += counts[(size_t)q * K + i]; }
    G[i] = run;
    GS[i + 1] = GS[i] + run;
  }
  const uint64_t N = GS[K];
  cuts[0] = 0;
  cuts[P] = N;
  for (uint32_t q = 1; q < P; q++) {
    const uint64_t t = (uint64_t)(((unsigned __int128)N * q) / P);   // balanced target
    uint32_t i = 0;
    while (i + 1 < K && GS[i + 1] <= t) i++;                          // bucket holding position t
    uint64_t c;
    if (i & 1) {
      c = t;                                                          // equality bucket: split anywhere
    } else {
      const uint64_t a = GS[i], b = GS[i + 1];                        // range bucket: stays whole
      c = (t - a < b - t) ? a : b;
    }
    cuts[q] = std::max(c, cuts[q - 1]);
  }
  // elements of source q with a global position < X form a prefix of its
  // local partition (bucket order, then slice order)
  auto below = [&](uint32_t q, uint64_t X) {
    uint64_t s = 0;
    for (uint32_t i = 0; i < K; i++) {
      const uint64_t st = GS[i] + O[(size_t)q * K + i], c = counts[(size_t)q * K + i];
      if (X > st) s += std::min<uint64_t>(X - st, c);
    }
    return s;
  };
  for (uint32_t q = 0; q < P; q++) {
    const uint64_t a = below(me, cuts[q]), b = below(me, cuts[q + 1]);
    send_off[q] = a;
    send_cnt[q] = b - a;
    recv_cnt[q] = below(q, cuts[me + 1]) - below(q, cuts[me]);
  }
  return GSS_SUCCESS;
}

gss_status gss_dist_unique_id(uint8_t id_out[128]) {
  if (!id_out) return GSS_ERROR_INVALID_VALUE;
  static_assert(sizeof(ncclUniqueId) == 128, "ncclUniqueId is 128 bytes");
  ncclUniqueId id;
  if (ncclGetUniqueId(&id) != ncclSuccess) return GSS_ERROR_NCCL;
  memcpy(id_out, &id, 128);
  return GSS_SUCCESS;
}

gss_status gss_dist_create(gss_dist** out, const uint8_t id[128], int rank, int nranks, int device) {
  if (!out || !id || nranks < 1 || rank < 0 || rank >= nranks || nranks > 64) return GSS_ERROR_INVALID_VALUE;
  if (cudaSetDevice(device) != cudaSuccess) { cudaGetLastError(); return GSS_ERROR_CUDA; }
  gss_dist* d = new (std::nothrow) gss_dist();
  if (!d) return GSS_ERROR_INVALID_VALUE;
  ncclUniqueId uid;
  memcpy(&uid, id, 128);
  if (ncclCommInitRank(&d->comm, nranks, uid, rank) != ncclSuccess) { delete d; return GSS_ERROR_NCCL; }
  d->rank = rank; d->P = nranks; d->dev = device;
  *out = d;
  return GSS_SUCCESS;
}

gss_status gss_dist_destroy(gss_dist* d) {
  if (!d) return GSS_ERROR_INVALID_VALUE;
  gss_status st = GSS_SUCCESS;
  cudaSetDevice(d->dev);
  if (d->win_k) ncclCommWindowDeregister(d->comm, d->win_k);
  if (d->win_v) ncclCommWindowDeregister(d->comm, d->win_v);
  if (d->wk) ncclMemFree(d->wk);
  if (d->wv) ncclMemFree(d->wv);
  if (d->comm && ncclCommDestroy(d->comm) != ncclSuccess) st = GSS_ERROR_NCCL;
  if (d->h_buf) cudaFreeHost(d->h_buf);
  delete d;
  return st;
}

gss_status gss_dist_last_exchange(const gss_dist* d, uint64_t* send_counts, uint64_t* recv_counts, uint64_t* cuts) {
  if (!d) return GSS_ERROR_INVALID_VALUE;
  for (int q = 0; q < d->P; q++) {
    if (send_counts) send_counts[q] = q < (int)d->send_cnt.size() ? d->send_cnt[q] : 0;
    if (recv_counts) recv_counts[q] = q < (int)d->recv_cnt.size() ? d->recv_cnt[q] : 0;
  }
  if (cuts)
    for (int q = 0; q <= d->P; q++) cuts[q] = q < (int)d->cuts.size() ? d->cuts[q] : 0;
  return GSS_SUCCESS;
}

gss_status gss_dist_sort_u32(gss_dist* d, const uint32_t* keys_in, size_t n_local, uint32_t* keys_out,
                             size_t out_capacity, size_t* n_out, void* temp, size_t* temp_bytes, void* stream,
                             const gss_params* p) {
  return dist_sort<uint32_t, void>(d, keys_in, nullptr, n_local, keys_out, nullptr, out_capacity, n_out, temp,
                                   temp_bytes, stream, p);
}
gss_status gss_dist_sort_u64(gss_dist* d, const uint64_t* keys_in, size_t n_local, uint64_t* keys_out,
                             size_t out_capacity, size_t* n_out, void* temp, size_t* temp_bytes, void* stream,
                             const gss_params* p) {
  return dist_sort<uint64_t, void>(d, keys_in, nullptr, n_local, keys_out, nullptr, out_capacity, n_out, temp,
                                   temp_bytes, stream, p);
}
gss_status gss_dist_sort_pairs_u32(gss_dist* d, const uint32_t* keys_in, const uint32_t* vals_in, size_t n_local,
                                   uint32_t* keys_out, uint32_t* vals_out, size_t out_capacity, size_t* n_out,
                                   void* temp, size_t* temp_bytes, void* stream, const gss_params* p) {
  return dist_sort<uint32_t, uint32_t>(d, keys_in, vals_in, n_local, keys_out, vals_out, out_capacity, n_out, temp,
                                       temp_bytes, stream, p);
}
gss_status gss_dist_sort_pairs_u64(gss_dist* d, const uint64_t* keys_in, const uint64_t* vals_in, size_t n_local,
                                   uint64_t* keys_out, uint64_t* vals_out, size_t out_capacity, size_t* n_out,
                                   void* temp, size_t* temp_bytes, void* stream, const gss_params* p) {
  return dist_sort<uint64_t, uint64_t>(d, keys_in, vals_in, n_local, keys_out, vals_out, out_capacity, n_out, temp,
                                       temp_bytes, stream, p);
}

}  // extern "C"
