/*
 * gss.h -- C ABI of the B200 GPU sample sort (libgss.so).
 *
 * Implements the k-way distribution pass of Leischner, Osipov & Sanders,
 * "GPU Sample Sort" (IPDPS 2010; /root/reference/PAPER.md, cited P:<line>):
 * sample and sort splitters (Phase 1), classify every key
 * by a branch-free descent of the implicit splitter tree (Phase 2,
 * Algorithm 2), prefix-sum the per-tile bucket
 * histograms bucket-major (Phase 3), scatter keys and values into
 * their buckets (Phase 4), recurse until buckets hold at most M
 * keys (Algorithm 1), and finish those buckets with an
 * in-SM merge sort built on an odd-even merge network.
 *
 * Conventions (all entry points):
 *   - Keys are unsigned integers ordered by "<" (the comparator-only
 *     contract of P:52-54: the kernels only ever evaluate less(a, b)).
 *     Values are opaque payloads that move with their keys.
 *   - Pointers are DEVICE pointers unless the name or comment says host.
 *     The caller owns every buffer; the library never allocates device
 *     memory.  `temp` is caller-provided scratch: call once with
 *     temp == NULL to get *temp_bytes (no launch, no GPU access), then
 *     again with at least that many bytes (256-byte aligned).
 *   - `stream` is a cudaStream_t (NULL = the legacy default stream).  Every
 *     call only enqueues work on it (stream ordered, asynchronous) unless
 *     params->stats is set, in which case it synchronises the stream to
 *     fill the statistics.
 *   - keys_in may equal keys_out (in place); vals_in may equal vals_out.
 *     Partial overlap, or temp overlapping an I/O buffer, is
 *     GSS_ERROR_INVALID_VALUE.
 *   - n == 0 succeeds without a launch.  Offsets are u32: a call needs
 *     n + T < 2^32 (T = the tile) and n + 16*(n/(M+1) + 3) < 2^32 (per-bucket
 *     16-aligned id ranges); with the default T and M that is about
 *     n <= 2^32 - 2^19 - 2^16 for u64 keys.  Larger n returns
 *     GSS_ERROR_NOT_SUPPORTED.
 *   - Errors are reported only through the return code: nothing aborts,
 *     throws or prints.  Asynchronous device faults surface at the
 *     caller's next synchronisation as usual in CUDA.
 *   - Output keys are the unique non-decreasing permutation of the input.
 *     Values of equal keys may appear in any order (the sort is unstable,
 *     P:262) but the output is deterministic for a fixed input,
 *     parameter set and device.
 */
#ifndef GSS_H
#define GSS_H

#include <stddef.h>
#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

typedef enum gss_status {
  GSS_SUCCESS = 0,
  GSS_ERROR_INVALID_VALUE = 1,   /* NULL with n>0, bad k/a/M/tile, overlapping buffers   */
  GSS_ERROR_TEMP_TOO_SMALL = 2,  /* *temp_bytes smaller than the query returned         */
  GSS_ERROR_NOT_SUPPORTED = 3,   /* n >= 2^32, or device is not sm_100                   */
  GSS_ERROR_CUDA = 4,            /* a launch or runtime call failed                      */
  GSS_ERROR_NCCL = 5,            /* a collective of gss_dist_* failed                    */
  GSS_ERROR_CAPACITY = 6         /* an output capacity is smaller than the result        */
} gss_status;

/* Kernel kinds, for gss_profiler_read(). */
enum {
  GSS_K_INIT = 0, GSS_K_SAMPLE, GSS_K_CLASSIFY, GSS_K_SCAN, GSS_K_SCATTER, GSS_K_PLAN,
  GSS_K_SMALL_SORT, GSS_K_COPY, GSS_K_OVERFLOW, GSS_K_H2D, GSS_K_D2H, GSS_K_OTHER,
  GSS_KERNEL_KINDS
};

/* Statistics of one call (host struct, filled only when requested). */
typedef struct gss_stats {
  uint32_t levels;              /* distribution levels that split >= 1 bucket            */
  uint32_t launches;            /* kernels the call enqueued                             */
  uint32_t levels_launched;     /* distribution levels enqueued (max_levels resolved)     */
  uint32_t error_flags;         /* internal capacity checks; 0 means the result is valid */
  uint64_t split_elems[16];     /* keys distributed at level l (sum of m over its buckets) */
  uint64_t split_buckets[16];   /* buckets split at level l                              */
  uint64_t small_buckets;       /* buckets finished by the in-SM sort                   */
  uint64_t small_elems;         /* keys in those buckets                                 */
  uint64_t max_small;           /* largest bucket given to the in-SM sort                */
  uint64_t eq_buckets;          /* final equality buckets (all keys equal, R4)           */
  uint64_t eq_elems;
  uint64_t overflow_buckets;    /* buckets finished by the fallback after max_levels     */
  uint64_t overflow_elems;
  uint64_t cluster_buckets;     /* buckets sorted by a thread-block cluster (GSS_FLAG_CLUSTER_SORT) */
} gss_stats;

typedef struct gss_profiler gss_profiler;

/* Tuning and method parameters; pass NULL for the per-type defaults. A zero
 * field also selects its default. */
typedef struct gss_params {
  uint32_t k;               /* max buckets per split: power of 2 in [2,1024]; 0 ->
                               256, or 512 / 1024 when n > k*k*M/2 (two levels suffice)  */
  uint32_t oversample;      /* a; 0 -> 30                               */
  uint64_t small_threshold; /* M: buckets with m <= M go to the in-SM sort;       */
                            /* 0 -> the in-SM capacity of the type; at most that           */
  uint32_t tile;            /* keys per tile T = t*l; multiple of 2048; 0 ->
                               65536, halved while n < 296 tiles (min 2048)               */
  uint32_t max_levels;      /* distribution levels launched before the fallback; 0 -> auto */
  uint32_t k_policy;        /* 1 (default) adaptive k_b (R29), 2 = fixed k_b = k (paper)   */
  uint32_t fill_div;        /* adaptive rule divisor f (R29); 0 -> 4              */
  uint64_t seed;            /* sampling seed (R2); 0 -> 5489                               */
  uint32_t flags;           /* GSS_FLAG_* below                                            */
  uint32_t cls_arrays;      /* Phase-2 counter arrays per CTA of 8 warps: 1, 2, 4 or 8; 0 ->
                               8, one per warp (the paper splits counter contention over 8
                               arrays; ablation SURVEY NEXT-4 iii)               */
  gss_stats* stats;         /* optional host pointer: the call syncs and fills it          */
  gss_profiler* profiler;   /* optional: CUDA-event time of every launch                   */
  uint32_t* error_out;      /* optional DEVICE pointer: a sort copies its internal
                               capacity-check flags there, stream ordered, without a host
                               sync (0 = the result is valid; also captured by
                               GSS_FLAG_GRAPH)                                              */
} gss_params;

#define GSS_FLAG_RECOMPUTE_IDS 1u  /* Phase 4 re-descends the splitter tree instead of reading
                                      bucket ids stored by Phase 2 (the paper's choice,
                                      P:264-267; ablation: slower on B200); sorts only       */
#define GSS_FLAG_STABLE 4u         /* Phase 4 ranks keys stably (R7: each level is a stable
                                      partition); default: one shared atomic per key, which
                                      partitions correctly but orders keys within a bucket in
                                      the hardware's atomic order                             */
#define GSS_FLAG_DIRECT_SCATTER 8u /* Phase 4 as in the paper: keys written straight from
                                      registers at atomic-cursor positions, no smem reorder
                                      (ablation, slower on B200)                  */
#define GSS_FLAG_GRAPH 16u         /* capture the launch sequence of a device-buffer sort as a
                                      CUDA graph on first use and replay it on later calls
                                      with identical buffers, n and parameters (launch-bound
                                      sizes); ignored with stats or a profiler              */
#define GSS_FLAG_SCATTER_REGS 32u  /* 8-byte keys without values: Phase 4 writes bucket runs
                                      with per-key shared loads and coalesced global stores
                                      (the round-1 scatter; ablation) instead of one bulk copy
                                      (cp.async.bulk) per run; every other kind always does  */
#define GSS_FLAG_DIST_FUSED 64u    /* gss_dist_sort_*: fuse the global scatter with the exchange
                                      (SURVEY NEXT-1): the partition's bucket runs are stored
                                      by the scatter kernel straight into the receiving GPU's
                                      NCCL symmetric window over NVLink instead of a local
                                      partition + ncclSend/ncclRecv.  The first call (and any
                                      call needing larger windows) allocates and registers the
                                      windows collectively (ncclMemAlloc +
                                      ncclCommWindowRegister)                                 */
#define GSS_FLAG_BITONIC_NET 128u  /* u64 keys: each thread of the in-SM sort sorts its 16 keys
                                      with a bitonic network instead of Batcher's odd-even
                                      merge network (the paper's comparison, P:339-341;
                                      ablation SURVEY NEXT-4 iv); ignored for other kinds    */
#define GSS_FLAG_CLUSTER_SORT 256u /* buckets above one CTA's shared-memory capacity (up to M)
                                      are sorted by a cluster of 8 CTAs through distributed
                                      shared memory (the on-chip answer to the
                                      paper's quicksort tier below M = 2^17); the
                                      default M becomes the cluster capacity (8x the CTA's)  */
#define GSS_FLAG_TREE_CLASSIFY 512u /* unsigned keys under operator<: Phase 2 classifies every key
                                      by the paper's branch-free descent of the splitter tree
                                      (Algorithm 2) instead of the default
                                      radix-indexed lookup (a table of 4096 key-value bins per
                                      bucket, one shared load per key, the descent only inside
                                      bins that hold a splitter); both give identical ids
                                      (ablation)                                             */
#define GSS_FLAG_SPLIT_SORT 2u     /* finish buckets of two or more warps with one more
                                      sample-sort split inside the SM + warp merge sorts of
                                      packed segments; ablation: on B200 its
                                      serial sample/segment phases and partial warps cost
                                      more than the CTA-wide merge rounds they remove       */

/* Human-readable name of a status code (static storage). */
const char* gss_status_string(gss_status s);

/* Library version and the per-type default parameters (host-only, no GPU). */
uint32_t gss_version(void);
gss_status gss_default_params(uint32_t key_bytes, uint32_t val_bytes, gss_params* out);

/* ---------------------------------------------------------------------- */
/* Sorting (Algorithm 1).  Device buffers of n elements.        */
/* ---------------------------------------------------------------------- */
gss_status gss_sort_u32(const uint32_t* keys_in, uint32_t* keys_out, size_t n,
                        void* temp, size_t* temp_bytes, void* stream, const gss_params* p);
gss_status gss_sort_u64(const uint64_t* keys_in, uint64_t* keys_out, size_t n,
                        void* temp, size_t* temp_bytes, void* stream, const gss_params* p);
gss_status gss_sort_pairs_u32(const uint32_t* keys_in, const uint32_t* vals_in,
                              uint32_t* keys_out, uint32_t* vals_out, size_t n,
                              void* temp, size_t* temp_bytes, void* stream, const gss_params* p);
gss_status gss_sort_pairs_u64(const uint64_t* keys_in, const uint64_t* vals_in,
                              uint64_t* keys_out, uint64_t* vals_out, size_t n,
                              void* temp, size_t* temp_bytes, void* stream, const gss_params* p);

/* Descending order (every integer kind): the same kernels instantiated with
 * less(a,b) = a > b, exercising the comparator-only contract. */
gss_status gss_sort_u64_descending(const uint64_t* keys_in, uint64_t* keys_out, size_t n,
                                   void* temp, size_t* temp_bytes, void* stream,
                                   const gss_params* p);
gss_status gss_sort_u32_descending(const uint32_t* keys_in, uint32_t* keys_out, size_t n,
                                   void* temp, size_t* temp_bytes, void* stream,
                                   const gss_params* p);
gss_status gss_sort_pairs_u32_descending(const uint32_t* keys_in, const uint32_t* vals_in,
                                         uint32_t* keys_out, uint32_t* vals_out, size_t n,
                                         void* temp, size_t* temp_bytes, void* stream,
                                         const gss_params* p);
gss_status gss_sort_pairs_u64_descending(const uint64_t* keys_in, const uint64_t* vals_in,
                                         uint64_t* keys_out, uint64_t* vals_out, size_t n,
                                         void* temp, size_t* temp_bytes, void* stream,
                                         const gss_params* p);
/* Any other key type or strict weak order: include/gss.hpp (gss::sort<Key, Less>,
 * gss::sort_pairs<Key, Val, Less>), compiled into the caller's own nvcc translation unit. */

/* Floating-point keys under the IEEE-754 total order (-NaN < -inf < ... < -0 <
 * +0 < ... < +inf < +NaN): the same kernels with a different comparator
 * (the paper sorts floats). */
gss_status gss_sort_f32(const float* keys_in, float* keys_out, size_t n,
                        void* temp, size_t* temp_bytes, void* stream, const gss_params* p);
gss_status gss_sort_f64(const double* keys_in, double* keys_out, size_t n,
                        void* temp, size_t* temp_bytes, void* stream, const gss_params* p);

/* End-to-end variants: keys (and values) are HOST buffers (pinned for full
 * speed); the call enqueues the host->device copy, the sort and the
 * device->host copy on `stream`.  temp must also hold the device copies
 * (the query includes them).  The output is valid after the stream is
 * synchronised. */
gss_status gss_sort_host_u32(const uint32_t* h_keys_in, uint32_t* h_keys_out, size_t n,
                             void* temp, size_t* temp_bytes, void* stream, const gss_params* p);
gss_status gss_sort_host_u64(const uint64_t* h_keys_in, uint64_t* h_keys_out, size_t n,
                             void* temp, size_t* temp_bytes, void* stream, const gss_params* p);
gss_status gss_sort_host_pairs_u32(const uint32_t* h_keys_in, const uint32_t* h_vals_in,
                                   uint32_t* h_keys_out, uint32_t* h_vals_out, size_t n,
                                   void* temp, size_t* temp_bytes, void* stream,
                                   const gss_params* p);
gss_status gss_sort_host_pairs_u64(const uint64_t* h_keys_in, const uint64_t* h_vals_in,
                                   uint64_t* h_keys_out, uint64_t* h_vals_out, size_t n,
                                   void* temp, size_t* temp_bytes, void* stream,
                                   const gss_params* p);

/* Pipelined end-to-end sorting of a stream of host arrays of n elements:
 * call i's host->device copy, the sort of call i-1 and the device->host copy
 * of call i-2 overlap on three internal streams (two device buffer sets kept
 * in temp).  Each run() is ordered after earlier work on `stream`; `stream`
 * then waits for the PREVIOUS run's output (one-call lag), and flush() makes
 * it wait for the last one, so after flush() + synchronising `stream` every
 * output is valid.  key_bytes 4|8, val_bytes 0 or key_bytes.  temp == NULL
 * queries *temp_bytes (no GPU access, *out untouched). */
typedef struct gss_host_pipeline gss_host_pipeline;
gss_status gss_host_pipeline_create(gss_host_pipeline** out, uint32_t key_bytes, uint32_t val_bytes, size_t n,
                                    const gss_params* p, void* temp, size_t* temp_bytes);
gss_status gss_host_pipeline_run(gss_host_pipeline* h, const void* h_keys_in, const void* h_vals_in,
                                 void* h_keys_out, void* h_vals_out, void* stream);
gss_status gss_host_pipeline_flush(gss_host_pipeline* h, void* stream);
gss_status gss_host_pipeline_destroy(gss_host_pipeline* h);

/* ---------------------------------------------------------------------- */
/* One k-way distribution step over the whole input (Phases 1-4,           */
/* P:251-263), regardless of M.  The partition is stable (R7).   */
/*   vals_in/vals_out: NULL for keys only; values have the key's width.     */
/*   splitters_out: device, capacity k-1 keys: the k_s - 1 sorted splitters */
/*   bucket_offsets_out: device u64, capacity 2k: K+1 bucket boundaries      */
/*   info_out: device u32[4] = { k_b, k_s, eq, K }                           */
/* ---------------------------------------------------------------------- */
gss_status gss_partition_u32(const uint32_t* keys_in, const uint32_t* vals_in,
                             uint32_t* keys_out, uint32_t* vals_out, size_t n,
                             uint32_t* splitters_out, uint64_t* bucket_offsets_out,
                             uint32_t* info_out, void* temp, size_t* temp_bytes, void* stream,
                             const gss_params* p);
gss_status gss_partition_u64(const uint64_t* keys_in, const uint64_t* vals_in,
                             uint64_t* keys_out, uint64_t* vals_out, size_t n,
                             uint64_t* splitters_out, uint64_t* bucket_offsets_out,
                             uint32_t* info_out, void* temp, size_t* temp_bytes, void* stream,
                             const gss_params* p);

/* ---------------------------------------------------------------------- */
/* Building blocks of the distributed sample sort. */
/* ---------------------------------------------------------------------- */
/* Gather s keys of keys[0..n) at positions lo_global-keyed hashed indices:
 * out[j] = keys[mulhi64(H(seed, level_tag, lo_global, j), n)] (R2). */
gss_status gss_sample_u32(const uint32_t* keys, size_t n, uint64_t lo_global, uint32_t level_tag,
                          uint64_t seed, uint32_t* out, size_t s, void* stream);
gss_status gss_sample_u64(const uint64_t* keys, size_t n, uint64_t lo_global, uint32_t level_tag,
                          uint64_t seed, uint64_t* out, size_t s, void* stream);

/* Partition keys_in[0..n) (and values) into nspl+1 buckets by the given
 * sorted device splitters (ties go left, R3; no equality buckets), writing
 * the stable partition to keys_out/vals_out and the nspl+1 bucket sizes to
 * counts_out (device u64). */
gss_status gss_partition_by_u32(const uint32_t* keys_in, const uint32_t* vals_in,
                                uint32_t* keys_out, uint32_t* vals_out, size_t n,
                                const uint32_t* splitters, uint32_t nspl, uint64_t* counts_out,
                                void* temp, size_t* temp_bytes, void* stream);
gss_status gss_partition_by_u64(const uint64_t* keys_in, const uint64_t* vals_in,
                                uint64_t* keys_out, uint64_t* vals_out, size_t n,
                                const uint64_t* splitters, uint32_t nspl, uint64_t* counts_out,
                                void* temp, size_t* temp_bytes, void* stream);

/* The same in equality mode (R4 applied to given splitters; the global level
 * of gss_dist_sort_*): key e gets id 2b (range: spl[b-1] < e < spl[b]) or
 * 2b+1 (e == spl[b]) with b = #{spl < e}; counts_out holds 2*nspl+1 sizes.
 * Duplicate splitters are allowed (every copy of a key lands in one
 * equality bucket).  nspl <= 127. */
gss_status gss_partition_by_eq_u32(const uint32_t* keys_in, const uint32_t* vals_in,
                                   uint32_t* keys_out, uint32_t* vals_out, size_t n,
                                   const uint32_t* splitters, uint32_t nspl, uint64_t* counts_out,
                                   void* temp, size_t* temp_bytes, void* stream);
gss_status gss_partition_by_eq_u64(const uint64_t* keys_in, const uint64_t* vals_in,
                                   uint64_t* keys_out, uint64_t* vals_out, size_t n,
                                   const uint64_t* splitters, uint32_t nspl, uint64_t* counts_out,
                                   void* temp, size_t* temp_bytes, void* stream);

/* ---------------------------------------------------------------------- */
/* Distributed sample sort across GPUs: one process per GPU, NCCL over     */
/* NVLink (sample sort's home is distributed memory, */
/* P:195-196; large random samples balance the parts).          */
/* Each rank passes its shard keys_in[0..n_local); on return rank r holds  */
/* the r-th contiguous range of the global sorted order in                 */
/* keys_out[0..*n_out) (values with their keys).  Steps: all-gather of      */
/* (n_local, out_capacity); 16384 hashed samples per rank (level tag 255,  */
/* lo = the shard's global start, R2), all-gathered and sorted identically */
/* on every rank; P-1 splitters S[(i+1)VS/P - 1] (R1); equality-mode       */
/* partition (gss_partition_by_eq); all-gather of the 2P-1 counts; the      */
/* exchange plan gss_dist_plan; grouped ncclSend/ncclRecv (all-to-all-v);   */
/* in-place gss_sort of the received range.  Two host synchronisations per */
/* call (the two small all-gathers).  temp == NULL queries *temp_bytes     */
/* (depends on n_local and out_capacity; no GPU or NCCL access).            */
/* Errors: GSS_ERROR_NCCL (a collective failed), GSS_ERROR_CAPACITY (some  */
/* rank's out_capacity is below what it would receive: every rank returns  */
/* it, nothing is exchanged, *n_out = this rank's required count).  A      */
/* handle is not thread-safe; all ranks must call collectively.            */
/* ---------------------------------------------------------------------- */
typedef struct gss_dist gss_dist;
/* rank 0 creates the id and shares it (e.g. torch.distributed broadcast) */
gss_status gss_dist_unique_id(uint8_t id_out[128]);
gss_status gss_dist_create(gss_dist** d, const uint8_t id[128], int rank, int nranks, int device);
gss_status gss_dist_destroy(gss_dist* d);
gss_status gss_dist_sort_u32(gss_dist* d, const uint32_t* keys_in, size_t n_local, uint32_t* keys_out,
                             size_t out_capacity, size_t* n_out /* host */, void* temp, size_t* temp_bytes,
                             void* stream, const gss_params* p);
gss_status gss_dist_sort_u64(gss_dist* d, const uint64_t* keys_in, size_t n_local, uint64_t* keys_out,
                             size_t out_capacity, size_t* n_out, void* temp, size_t* temp_bytes,
                             void* stream, const gss_params* p);
gss_status gss_dist_sort_pairs_u32(gss_dist* d, const uint32_t* keys_in, const uint32_t* vals_in, size_t n_local,
                                   uint32_t* keys_out, uint32_t* vals_out, size_t out_capacity, size_t* n_out,
                                   void* temp, size_t* temp_bytes, void* stream, const gss_params* p);
gss_status gss_dist_sort_pairs_u64(gss_dist* d, const uint64_t* keys_in, const uint64_t* vals_in, size_t n_local,
                                   uint64_t* keys_out, uint64_t* vals_out, size_t out_capacity, size_t* n_out,
                                   void* temp, size_t* temp_bytes, void* stream, const gss_params* p);
/* The last call's plan on this rank: P send counts, P receive counts, P+1 cuts (host arrays, may be NULL). */
gss_status gss_dist_last_exchange(const gss_dist* d, uint64_t* send_counts, uint64_t* recv_counts, uint64_t* cuts);

/* The exchange plan (host only, no GPU): counts[q*K + i] = rank q's number of
 * keys with global-level id i (K = 2P-1; even ids are range buckets, which
 * stay whole, odd ids equality buckets, whose keys are all equal and may be
 * split).  Rank q owns global positions [cuts[q], cuts[q+1]) of the order
 * (bucket, source rank, position): each cut is the balanced target q*N/P,
 * moved to the nearer boundary when it falls inside a range bucket.  For
 * rank `me`: send_off/send_cnt[q] = the range of its partitioned shard that
 * goes to rank q; recv_cnt[q] = what it receives from rank q. */
gss_status gss_dist_plan(uint32_t P, uint32_t me, uint32_t K, const uint64_t* counts, uint64_t* cuts,
                         uint64_t* send_off, uint64_t* send_cnt, uint64_t* recv_cnt);

/* ---------------------------------------------------------------------- */
/* Profiling: CUDA events around every launch of the calls that carry the */
/* profiler in their params.  Read after the stream has been synchronised. */
/* ---------------------------------------------------------------------- */
gss_status gss_profiler_create(gss_profiler** out);
gss_status gss_profiler_destroy(gss_profiler* p);
gss_status gss_profiler_reset(gss_profiler* p);
/* ms[GSS_KERNEL_KINDS] and launches[GSS_KERNEL_KINDS]: host arrays */
gss_status gss_profiler_read(gss_profiler* p, double* ms, uint64_t* launches);

#ifdef __cplusplus
}
#endif
#endif /* GSS_H */
