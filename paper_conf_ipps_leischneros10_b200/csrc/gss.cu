// gss.cu -- the C ABI (include/gss.h) of the B200 GPU sample sort.  The sort
// engine (gss_impl.cuh) is instantiated in gss_inst_*.cu.
#include "gss_impl.cuh"

using namespace gss;
using namespace gssh;

// ============================================================================
// C ABI
// ============================================================================
extern "C" {

const char* gss_status_string(gss_status s) {
  switch (s) {
    case GSS_SUCCESS: return "GSS_SUCCESS";
    case GSS_ERROR_INVALID_VALUE: return "GSS_ERROR_INVALID_VALUE";
    case GSS_ERROR_TEMP_TOO_SMALL: return "GSS_ERROR_TEMP_TOO_SMALL";
    case GSS_ERROR_NOT_SUPPORTED: return "GSS_ERROR_NOT_SUPPORTED";
    case GSS_ERROR_CUDA: return "GSS_ERROR_CUDA";
    case GSS_ERROR_NCCL: return "GSS_ERROR_NCCL";
    case GSS_ERROR_CAPACITY: return "GSS_ERROR_CAPACITY";
  }
  return "GSS_UNKNOWN_STATUS";
}

uint32_t gss_version(void) { return kVersion; }

gss_status gss_default_params(uint32_t key_bytes, uint32_t val_bytes, gss_params* out) {
  if (!out || (key_bytes != 4 && key_bytes != 8) || (val_bytes != 0 && val_bytes != key_bytes))
    return GSS_ERROR_INVALID_VALUE;
  memset(out, 0, sizeof(*out));
  out->k = 0;                                   // n-dependent: 256, or 512 / 1024 for large n (see gss.h)
  out->oversample = 30;
  out->small_threshold = (val_bytes && key_bytes + val_bytes > 8) ? 8192 : 16384;
  out->tile = 0;                                // n-dependent: 65536, smaller for small n (see gss.h)
  out->k_policy = 1;
  out->fill_div = 4;
  out->seed = 5489;
  return GSS_SUCCESS;
}

gss_status gss_sort_u32(const uint32_t* ki, uint32_t* ko, size_t n, void* t, size_t* tb, void* s,
                        const gss_params* p) {
  return drive<uint32_t, NoVal, Less>(io_dev(ki, nullptr, ko, nullptr), n, t, tb, s, p, MODE_SORT, false);
}
gss_status gss_sort_u64(const uint64_t* ki, uint64_t* ko, size_t n, void* t, size_t* tb, void* s,
                        const gss_params* p) {
  return drive<uint64_t, NoVal, Less>(io_dev(ki, nullptr, ko, nullptr), n, t, tb, s, p, MODE_SORT, false);
}
gss_status gss_sort_pairs_u32(const uint32_t* ki, const uint32_t* vi, uint32_t* ko, uint32_t* vo, size_t n, void* t,
                              size_t* tb, void* s, const gss_params* p) {
  return drive<uint32_t, uint32_t, Less>(io_dev(ki, vi, ko, vo), n, t, tb, s, p, MODE_SORT, false);
}
gss_status gss_sort_pairs_u64(const uint64_t* ki, const uint64_t* vi, uint64_t* ko, uint64_t* vo, size_t n, void* t,
                              size_t* tb, void* s, const gss_params* p) {
  return drive<uint64_t, uint64_t, Less>(io_dev(ki, vi, ko, vo), n, t, tb, s, p, MODE_SORT, false);
}
gss_status gss_sort_u64_descending(const uint64_t* ki, uint64_t* ko, size_t n, void* t, size_t* tb, void* s,
                                   const gss_params* p) {
  return drive<uint64_t, NoVal, Greater>(io_dev(ki, nullptr, ko, nullptr), n, t, tb, s, p, MODE_SORT, false);
}
gss_status gss_sort_u32_descending(const uint32_t* ki, uint32_t* ko, size_t n, void* t, size_t* tb, void* s,
                                   const gss_params* p) {
  return drive<uint32_t, NoVal, Greater>(io_dev(ki, nullptr, ko, nullptr), n, t, tb, s, p, MODE_SORT, false);
}
gss_status gss_sort_pairs_u32_descending(const uint32_t* ki, const uint32_t* vi, uint32_t* ko, uint32_t* vo, size_t n,
                                         void* t, size_t* tb, void* s, const gss_params* p) {
  return drive<uint32_t, uint32_t, Greater>(io_dev(ki, vi, ko, vo), n, t, tb, s, p, MODE_SORT, false);
}
gss_status gss_sort_pairs_u64_descending(const uint64_t* ki, const uint64_t* vi, uint64_t* ko, uint64_t* vo, size_t n,
                                         void* t, size_t* tb, void* s, const gss_params* p) {
  return drive<uint64_t, uint64_t, Greater>(io_dev(ki, vi, ko, vo), n, t, tb, s, p, MODE_SORT, false);
}

gss_status gss_sort_f32(const float* ki, float* ko, size_t n, void* t, size_t* tb, void* s, const gss_params* p) {
  return drive<float, NoVal, TotalLess>(io_dev(ki, nullptr, ko, nullptr), n, t, tb, s, p, MODE_SORT, false);
}
gss_status gss_sort_f64(const double* ki, double* ko, size_t n, void* t, size_t* tb, void* s, const gss_params* p) {
  return drive<double, NoVal, TotalLess>(io_dev(ki, nullptr, ko, nullptr), n, t, tb, s, p, MODE_SORT, false);
}

gss_status gss_sort_host_u32(const uint32_t* ki, uint32_t* ko, size_t n, void* t, size_t* tb, void* s,
                             const gss_params* p) {
  return drive<uint32_t, NoVal, Less>(io_host(ki, nullptr, ko, nullptr), n, t, tb, s, p, MODE_SORT, true);
}
gss_status gss_sort_host_u64(const uint64_t* ki, uint64_t* ko, size_t n, void* t, size_t* tb, void* s,
                             const gss_params* p) {
  return drive<uint64_t, NoVal, Less>(io_host(ki, nullptr, ko, nullptr), n, t, tb, s, p, MODE_SORT, true);
}
gss_status gss_sort_host_pairs_u32(const uint32_t* ki, const uint32_t* vi, uint32_t* ko, uint32_t* vo, size_t n,
                                   void* t, size_t* tb, void* s, const gss_params* p) {
  return drive<uint32_t, uint32_t, Less>(io_host(ki, vi, ko, vo), n, t, tb, s, p, MODE_SORT, true);
}
gss_status gss_sort_host_pairs_u64(const uint64_t* ki, const uint64_t* vi, uint64_t* ko, uint64_t* vo, size_t n,
                                   void* t, size_t* tb, void* s, const gss_params* p) {
  return drive<uint64_t, uint64_t, Less>(io_host(ki, vi, ko, vo), n, t, tb, s, p, MODE_SORT, true);
}

// ---------------------------------------------------------------------------
// Pipelined host-buffer sorting: consecutive calls overlap the host->device
// copy of call i+1, the sort of call i and the device->host copy of call i-1
// on three internal streams (two device buffer sets in temp).
// ---------------------------------------------------------------------------
struct gss_host_pipeline {
  uint32_t kb, vb;
  size_t n;
  gss_params params;
  bool has_params;
  unsigned char* temp;
  size_t sort_off, sort_bytes;
  void* din[2]; void* dout[2]; void* dvin[2]; void* dvout[2];
  cudaStream_t s_in, s_cmp, s_out;
  cudaEvent_t ev_user, ev_in[2], ev_sorted[2], ev_out[2];
  uint64_t calls;
};

static gss_status pipeline_sort_query(uint32_t kb, uint32_t vb, size_t n, const gss_params* p, size_t* bytes) {
  if (kb == 4 && vb == 0) return gss_sort_u32(nullptr, nullptr, n, nullptr, bytes, nullptr, p);
  if (kb == 8 && vb == 0) return gss_sort_u64(nullptr, nullptr, n, nullptr, bytes, nullptr, p);
  if (kb == 4 && vb == 4) return gss_sort_pairs_u32(nullptr, nullptr, nullptr, nullptr, n, nullptr, bytes, nullptr, p);
  if (kb == 8 && vb == 8) return gss_sort_pairs_u64(nullptr, nullptr, nullptr, nullptr, n, nullptr, bytes, nullptr, p);
  return GSS_ERROR_INVALID_VALUE;
}

gss_status gss_host_pipeline_create(gss_host_pipeline** out, uint32_t key_bytes, uint32_t val_bytes, size_t n,
                                    const gss_params* p, void* temp, size_t* temp_bytes) {
  if (!temp_bytes) return GSS_ERROR_INVALID_VALUE;
  size_t sb = 0;
  GSS_TRY(pipeline_sort_query(key_bytes, val_bytes, n, p, &sb));
  const size_t kbuf = align_up(n * key_bytes), vbuf = val_bytes ? align_up(n * val_bytes) : 0;
  const size_t total = 4 * kbuf + 4 * vbuf + align_up(sb);
  if (!temp) { *temp_bytes = total; return GSS_SUCCESS; }
  if (!out || *temp_bytes < total) return !out ? GSS_ERROR_INVALID_VALUE : GSS_ERROR_TEMP_TOO_SMALL;
  if ((uintptr_t)temp % 256) return GSS_ERROR_INVALID_VALUE;
  gss_host_pipeline* h = new gss_host_pipeline();
  h->kb = key_bytes; h->vb = val_bytes; h->n = n; h->calls = 0;
  h->has_params = p != nullptr;
  if (p) { h->params = *p; h->params.stats = nullptr; h->params.profiler = nullptr; }
  h->temp = reinterpret_cast<unsigned char*>(temp);
  size_t o = 0;
  for (int i = 0; i < 2; i++) {
    h->din[i] = h->temp + o; o += kbuf;
    h->dout[i] = h->temp + o; o += kbuf;
    h->dvin[i] = vbuf ? h->temp + o : nullptr; o += vbuf;
    h->dvout[i] = vbuf ? h->temp + o : nullptr; o += vbuf;
  }
  h->sort_off = o; h->sort_bytes = align_up(sb);
  bool ok = cudaStreamCreateWithFlags(&h->s_in, cudaStreamNonBlocking) == cudaSuccess &&
            cudaStreamCreateWithFlags(&h->s_cmp, cudaStreamNonBlocking) == cudaSuccess &&
            cudaStreamCreateWithFlags(&h->s_out, cudaStreamNonBlocking) == cudaSuccess &&
            cudaEventCreateWithFlags(&h->ev_user, cudaEventDisableTiming) == cudaSuccess;
  for (int i = 0; i < 2 && ok; i++)
    ok = cudaEventCreateWithFlags(&h->ev_in[i], cudaEventDisableTiming) == cudaSuccess &&
         cudaEventCreateWithFlags(&h->ev_sorted[i], cudaEventDisableTiming) == cudaSuccess &&
         cudaEventCreateWithFlags(&h->ev_out[i], cudaEventDisableTiming) == cudaSuccess;
  if (!ok) { cudaGetLastError(); delete h; return GSS_ERROR_CUDA; }
  *out = h;
  return GSS_SUCCESS;
}

gss_status gss_host_pipeline_run(gss_host_pipeline* h, const void* h_keys_in, const void* h_vals_in, void* h_keys_out,
                                 void* h_vals_out, void* stream) {
  if (!h || !h_keys_in || !h_keys_out || (h->vb && (!h_vals_in || !h_vals_out))) return GSS_ERROR_INVALID_VALUE;
  if (h->n == 0) return GSS_SUCCESS;
  cudaStream_t us = reinterpret_cast<cudaStream_t>(stream);
  const int s = (int)(h->calls & 1);
  const size_t kbytes = h->n * h->kb, vbytes = h->n * h->vb;
  bool ok = cudaEventRecord(h->ev_user, us) == cudaSuccess && cudaStreamWaitEvent(h->s_in, h->ev_user, 0) == cudaSuccess;
  // host -> device (set s), once the sort two calls back has consumed it
  if (h->calls >= 2) ok = ok && cudaStreamWaitEvent(h->s_in, h->ev_sorted[s], 0) == cudaSuccess;
  ok = ok && cudaMemcpyAsync(h->din[s], h_keys_in, kbytes, cudaMemcpyHostToDevice, h->s_in) == cudaSuccess;
  if (h->vb) ok = ok && cudaMemcpyAsync(h->dvin[s], h_vals_in, vbytes, cudaMemcpyHostToDevice, h->s_in) == cudaSuccess;
  ok = ok && cudaEventRecord(h->ev_in[s], h->s_in) == cudaSuccess;
  // sort (after its input arrived and the copy-out two calls back drained dout[s])
  ok = ok && cudaStreamWaitEvent(h->s_cmp, h->ev_in[s], 0) == cudaSuccess;
  if (h->calls >= 2) ok = ok && cudaStreamWaitEvent(h->s_cmp, h->ev_out[s], 0) == cudaSuccess;
  if (!ok) { cudaGetLastError(); return GSS_ERROR_CUDA; }
  size_t tb = h->sort_bytes;
  void* t = h->temp + h->sort_off;
  const gss_params* p = h->has_params ? &h->params : nullptr;
  gss_status st;
  if (h->kb == 4 && h->vb == 0)
    st = gss_sort_u32((const uint32_t*)h->din[s], (uint32_t*)h->dout[s], h->n, t, &tb, h->s_cmp, p);
  else if (h->kb == 8 && h->vb == 0)
    st = gss_sort_u64((const uint64_t*)h->din[s], (uint64_t*)h->dout[s], h->n, t, &tb, h->s_cmp, p);
  else if (h->kb == 4)
    st = gss_sort_pairs_u32((const uint32_t*)h->din[s], (const uint32_t*)h->dvin[s], (uint32_t*)h->dout[s],
                            (uint32_t*)h->dvout[s], h->n, t, &tb, h->s_cmp, p);
  else
    st = gss_sort_pairs_u64((const uint64_t*)h->din[s], (const uint64_t*)h->dvin[s], (uint64_t*)h->dout[s],
                            (uint64_t*)h->dvout[s], h->n, t, &tb, h->s_cmp, p);
  if (st != GSS_SUCCESS) return st;
  ok = cudaEventRecord(h->ev_sorted[s], h->s_cmp) == cudaSuccess;
  // device -> host, then the caller's stream waits for this call's output
  ok = ok && cudaStreamWaitEvent(h->s_out, h->ev_sorted[s], 0) == cudaSuccess;
  ok = ok && cudaMemcpyAsync(h_keys_out, h->dout[s], kbytes, cudaMemcpyDeviceToHost, h->s_out) == cudaSuccess;
  if (h->vb) ok = ok && cudaMemcpyAsync(h_vals_out, h->dvout[s], vbytes, cudaMemcpyDeviceToHost, h->s_out) == cudaSuccess;
  ok = ok && cudaEventRecord(h->ev_out[s], h->s_out) == cudaSuccess;
  // the caller's stream waits for the PREVIOUS call's output (a one-call lag, so
  // that this call's copy-in can overlap the previous copy-out); flush() waits
  // for the last one
  if (h->calls >= 1) ok = ok && cudaStreamWaitEvent(us, h->ev_out[s ^ 1], 0) == cudaSuccess;
  if (!ok) { cudaGetLastError(); return GSS_ERROR_CUDA; }
  h->calls++;
  return GSS_SUCCESS;
}

gss_status gss_host_pipeline_flush(gss_host_pipeline* h, void* stream) {
  if (!h) return GSS_ERROR_INVALID_VALUE;
  if (h->calls == 0) return GSS_SUCCESS;
  const int last = (int)((h->calls - 1) & 1);
  if (cudaStreamWaitEvent(reinterpret_cast<cudaStream_t>(stream), h->ev_out[last], 0) != cudaSuccess) {
    cudaGetLastError();
    return GSS_ERROR_CUDA;
  }
  return GSS_SUCCESS;
}

gss_status gss_host_pipeline_destroy(gss_host_pipeline* h) {
  if (!h) return GSS_ERROR_INVALID_VALUE;
  cudaStreamSynchronize(h->s_out);
  cudaStreamDestroy(h->s_in); cudaStreamDestroy(h->s_cmp); cudaStreamDestroy(h->s_out);
  cudaEventDestroy(h->ev_user);
  for (int i = 0; i < 2; i++) { cudaEventDestroy(h->ev_in[i]); cudaEventDestroy(h->ev_sorted[i]); cudaEventDestroy(h->ev_out[i]); }
  delete h;
  return GSS_SUCCESS;
}

gss_status gss_partition_u32(const uint32_t* ki, const uint32_t* vi, uint32_t* ko, uint32_t* vo, size_t n,
                             uint32_t* spl_out, uint64_t* off_out, uint32_t* info_out, void* t, size_t* tb, void* s,
                             const gss_params* p) {
  IO io = io_dev(ki, vi, ko, vo);
  io.spl_out = spl_out; io.off_out = off_out; io.info_out = info_out;
  if (vi) return drive<uint32_t, uint32_t, Less>(io, n, t, tb, s, p, MODE_PARTITION, false);
  return drive<uint32_t, NoVal, Less>(io, n, t, tb, s, p, MODE_PARTITION, false);
}
gss_status gss_partition_u64(const uint64_t* ki, const uint64_t* vi, uint64_t* ko, uint64_t* vo, size_t n,
                             uint64_t* spl_out, uint64_t* off_out, uint32_t* info_out, void* t, size_t* tb, void* s,
                             const gss_params* p) {
  IO io = io_dev(ki, vi, ko, vo);
  io.spl_out = spl_out; io.off_out = off_out; io.info_out = info_out;
  if (vi) return drive<uint64_t, uint64_t, Less>(io, n, t, tb, s, p, MODE_PARTITION, false);
  return drive<uint64_t, NoVal, Less>(io, n, t, tb, s, p, MODE_PARTITION, false);
}

gss_status gss_partition_by_u32(const uint32_t* ki, const uint32_t* vi, uint32_t* ko, uint32_t* vo, size_t n,
                                const uint32_t* spl, uint32_t nspl, uint64_t* counts, void* t, size_t* tb, void* s) {
  IO io = io_dev(ki, vi, ko, vo);
  io.counts_out = counts; io.given_spl = spl; io.given_nspl = nspl;
  if (t && n && nspl && !spl) return GSS_ERROR_INVALID_VALUE;
  if (vi) return drive<uint32_t, uint32_t, Less>(io, n, t, tb, s, nullptr, MODE_PARTITION_BY, false);
  return drive<uint32_t, NoVal, Less>(io, n, t, tb, s, nullptr, MODE_PARTITION_BY, false);
}
gss_status gss_partition_by_u64(const uint64_t* ki, const uint64_t* vi, uint64_t* ko, uint64_t* vo, size_t n,
                                const uint64_t* spl, uint32_t nspl, uint64_t* counts, void* t, size_t* tb, void* s) {
  IO io = io_dev(ki, vi, ko, vo);
  io.counts_out = counts; io.given_spl = spl; io.given_nspl = nspl;
  if (t && n && nspl && !spl) return GSS_ERROR_INVALID_VALUE;
  if (vi) return drive<uint64_t, uint64_t, Less>(io, n, t, tb, s, nullptr, MODE_PARTITION_BY, false);
  return drive<uint64_t, NoVal, Less>(io, n, t, tb, s, nullptr, MODE_PARTITION_BY, false);
}

gss_status gss_partition_by_eq_u32(const uint32_t* ki, const uint32_t* vi, uint32_t* ko, uint32_t* vo, size_t n,
                                   const uint32_t* spl, uint32_t nspl, uint64_t* counts, void* t, size_t* tb,
                                   void* s) {
  IO io = io_dev(ki, vi, ko, vo);
  io.counts_out = counts; io.given_spl = spl; io.given_nspl = nspl; io.given_eq = 1;
  if (t && n && nspl && !spl) return GSS_ERROR_INVALID_VALUE;
  if (nspl > 127) return GSS_ERROR_INVALID_VALUE;
  if (vi) return drive<uint32_t, uint32_t, Less>(io, n, t, tb, s, nullptr, MODE_PARTITION_BY, false);
  return drive<uint32_t, NoVal, Less>(io, n, t, tb, s, nullptr, MODE_PARTITION_BY, false);
}
gss_status gss_partition_by_eq_u64(const uint64_t* ki, const uint64_t* vi, uint64_t* ko, uint64_t* vo, size_t n,
                                   const uint64_t* spl, uint32_t nspl, uint64_t* counts, void* t, size_t* tb,
                                   void* s) {
  IO io = io_dev(ki, vi, ko, vo);
  io.counts_out = counts; io.given_spl = spl; io.given_nspl = nspl; io.given_eq = 1;
  if (t && n && nspl && !spl) return GSS_ERROR_INVALID_VALUE;
  if (nspl > 127) return GSS_ERROR_INVALID_VALUE;
  if (vi) return drive<uint64_t, uint64_t, Less>(io, n, t, tb, s, nullptr, MODE_PARTITION_BY, false);
  return drive<uint64_t, NoVal, Less>(io, n, t, tb, s, nullptr, MODE_PARTITION_BY, false);
}

// Internal, not part of gss.h: the two phases of the fused global level of the
// distributed sort (gss_dist.cu).  Phase 1 = equality-mode classification of
// keys_in by the splitters, the per-tile histograms and their scan, and the
// 2*nspl+1 bucket counts; phase 2 (same temp, called after phase 1) = the
// scatter of that partition straight into the remote segments (peer windows).
// kbuf/vbuf: any device buffers of n elements disjoint from the inputs (the
// partition is never written locally).
}  // extern "C"
template <class Key>
static gss_status dist_level(const Key* ki, const Key* vi, Key* kbuf, Key* vbuf, size_t n, const Key* spl,
                             uint32_t nspl, uint64_t* counts, const void* remote, uint32_t nremote, uint32_t phase,
                             void* t, size_t* tb, void* s) {
  IO io = io_dev(ki, vi, kbuf, vbuf);
  io.counts_out = counts; io.given_spl = spl; io.given_nspl = nspl; io.given_eq = 1;
  io.unstable = 1; io.phase = phase; io.remote = remote; io.nremote = nremote;
  if (nspl > 127 || nremote > 64 || phase < 1 || phase > 2) return GSS_ERROR_INVALID_VALUE;
  if (t && phase == 2 && !remote) return GSS_ERROR_INVALID_VALUE;
  if (vi) return drive<Key, Key, Less>(io, n, t, tb, s, nullptr, MODE_PARTITION_BY, false);
  return drive<Key, NoVal, Less>(io, n, t, tb, s, nullptr, MODE_PARTITION_BY, false);
}
extern "C" {
gss_status gssi_dist_level_u32(const uint32_t* ki, const uint32_t* vi, uint32_t* kb, uint32_t* vb, size_t n,
                               const uint32_t* spl, uint32_t nspl, uint64_t* counts, const void* remote,
                               uint32_t nremote, uint32_t phase, void* t, size_t* tb, void* s) {
  return dist_level<uint32_t>(ki, vi, kb, vb, n, spl, nspl, counts, remote, nremote, phase, t, tb, s);
}
gss_status gssi_dist_level_u64(const uint64_t* ki, const uint64_t* vi, uint64_t* kb, uint64_t* vb, size_t n,
                               const uint64_t* spl, uint32_t nspl, uint64_t* counts, const void* remote,
                               uint32_t nremote, uint32_t phase, void* t, size_t* tb, void* s) {
  return dist_level<uint64_t>(ki, vi, kb, vb, n, spl, nspl, counts, remote, nremote, phase, t, tb, s);
}

gss_status gss_sample_u32(const uint32_t* keys, size_t n, uint64_t lo_global, uint32_t level_tag, uint64_t seed,
                          uint32_t* out, size_t s, void* stream) {
  if (s == 0) return GSS_SUCCESS;
  if (!keys || !out || n == 0) return GSS_ERROR_INVALID_VALUE;
  cudaStream_t st = reinterpret_cast<cudaStream_t>(stream);
  k_gather_sample<uint32_t><<<(unsigned)std::min<size_t>((s + 255) / 256, 4096), 256, 0, st>>>(keys, n, lo_global,
                                                                                              level_tag, seed, out, s);
  return cudaGetLastError() == cudaSuccess ? GSS_SUCCESS : GSS_ERROR_CUDA;
}
gss_status gss_sample_u64(const uint64_t* keys, size_t n, uint64_t lo_global, uint32_t level_tag, uint64_t seed,
                          uint64_t* out, size_t s, void* stream) {
  if (s == 0) return GSS_SUCCESS;
  if (!keys || !out || n == 0) return GSS_ERROR_INVALID_VALUE;
  cudaStream_t st = reinterpret_cast<cudaStream_t>(stream);
  k_gather_sample<uint64_t><<<(unsigned)std::min<size_t>((s + 255) / 256, 4096), 256, 0, st>>>(keys, n, lo_global,
                                                                                              level_tag, seed, out, s);
  return cudaGetLastError() == cudaSuccess ? GSS_SUCCESS : GSS_ERROR_CUDA;
}

gss_status gss_profiler_create(gss_profiler** out) {
  if (!out) return GSS_ERROR_INVALID_VALUE;
  *out = new gss_profiler();
  gss_profiler_reset(*out);
  return GSS_SUCCESS;
}
gss_status gss_profiler_destroy(gss_profiler* p) {
  if (!p) return GSS_ERROR_INVALID_VALUE;
  for (auto& r : p->recs) { cudaEventDestroy(r.a); cudaEventDestroy(r.b); }
  for (auto e : p->pool) cudaEventDestroy(e);
  delete p;
  return GSS_SUCCESS;
}
gss_status gss_profiler_reset(gss_profiler* p) {
  if (!p) return GSS_ERROR_INVALID_VALUE;
  for (auto& r : p->recs) { p->pool.push_back(r.a); p->pool.push_back(r.b); }
  p->recs.clear();
  for (int i = 0; i < GSS_KERNEL_KINDS; i++) { p->ms[i] = 0; p->launches[i] = 0; }
  return GSS_SUCCESS;
}
gss_status gss_profiler_read(gss_profiler* p, double* ms, uint64_t* launches) {
  if (!p) return GSS_ERROR_INVALID_VALUE;
  for (auto& r : p->recs) {
    float t = 0;
    if (cudaEventSynchronize(r.b) != cudaSuccess || cudaEventElapsedTime(&t, r.a, r.b) != cudaSuccess) {
      cudaGetLastError();
      return GSS_ERROR_CUDA;
    }
    p->ms[r.kind] += t;
    p->launches[r.kind] += 1;
    p->pool.push_back(r.a);
    p->pool.push_back(r.b);
  }
  p->recs.clear();
  for (int i = 0; i < GSS_KERNEL_KINDS; i++) {
    if (ms) ms[i] = p->ms[i];
    if (launches) launches[i] = p->launches[i];
  }
  return GSS_SUCCESS;
}

}  // extern "C"
