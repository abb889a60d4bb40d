/*
 * oracle/oracle.c -- TEST INFRASTRUCTURE ONLY.
 *
 * A plain, slow, sequential CPU implementation of sample sort exactly as
 * Leischner, Osipov & Sanders, "GPU Sample Sort" (IPDPS 2010) defines it,
 * written from /root/reference/PAPER.md (cited as P:<line>) and the readings
 * R1..R29 of SURVEY.md section 8(c) as adopted in DESIGN.md ("Readings").
 *
 * Only tests/, __graft_entry__.smoke() and bench.py (cpu_baseline leg and
 * --impl reference) may load this library.  It shares no code, header,
 * table or constant generator with the CUDA path under
 * paper_conf_ipps_leischneros10_b200/; neither side includes the other.
 *
 * Everything is integer arithmetic.  Keys are handled as uint64_t (a u32 key
 * zero-extends, which preserves order and equality); values, when present,
 * are uint64_t payloads that travel with their keys.
 *
 * Threads (timing only): with params.threads > 1 the
 * child buckets of a level are sorted as independent OpenMP tasks, and a
 * large bucket's Phases 2-4 run over chunks (per-chunk counts, the
 * bucket-major exclusive scan over (bucket, chunk), then a stable
 * per-chunk placement -- the CPU analogue of P:256-263).  Each step is the
 * same plain computation; the output and the level records (sorted by
 * (level, lo)) are identical for any thread count (test_oracle.py).
 *
 * Parity pins (tests/test_oracle.py): brute force / library sort on every
 * input of length <= 6 over {0,1,2}; the paper's k=8 tree layout (P:295-304,
 * tests/golden/tree_k8.txt); Algorithm 2 == lower_bound; SplitMix64 known
 * answers; stable-partition and bucket-range invariants per level record;
 * all-equal / sorted / n<=M special cases; KV permutation checks.
 */
#include <stdint.h>
#include <stdlib.h>
#include <string.h>
#include <omp.h>

/* ------------------------------------------------------------------ */
/* Parameters (paper defaults)          */
/* ------------------------------------------------------------------ */
typedef struct oracle_params {
  uint32_t k;          /* maximum buckets per split, power of 2 in [2,1024] (R11) */
  uint32_t a;          /* oversampling factor                         */
  uint64_t M;          /* small-bucket threshold: m <= M -> SmallSort (R5)        */
  uint32_t k_policy;   /* 0 = fixed k_b = k (the paper); 1 = adaptive (R29)             */
  uint32_t fill_div;   /* adaptive rule: k_b = min(k, max(4, pow2ceil(ceil(f*m/M))))    */
  uint32_t sample_cap; /* a_eff = min(a, sample_cap / k_b), at least 1 (smem bound, R9) */
  uint32_t threads;    /* 0/1 sequential; > 1: OpenMP tasks over child buckets (timing)  */
  uint64_t seed;       /* sampling seed (R2)                                             */
} oracle_params;

/* One k-way distribution step of Algorithm 1 on A[lo, lo+m). */
typedef struct oracle_record {
  uint32_t level, kb, ks, eq, K, a_eff;
  uint64_t lo, m;
  uint64_t* spl;       /* ks-1 sorted splitters                         */
  uint64_t* child;     /* K child-bucket sizes (id order)               */
} oracle_record;

typedef struct oracle_log {
  oracle_record* r;
  size_t n, cap;
} oracle_log;

/* ------------------------------------------------------------------ */
/* Counter-based RNG for the sample positions (R2 replaces the paper's  */
/* "simple GPU LCG ... seed from the CPU Mersenne Twister"). */
/* sm(x) = SplitMix64 finaliser of x + golden gamma.                    */
/* ------------------------------------------------------------------ */
uint64_t oracle_splitmix64(uint64_t x) {
  uint64_t z = x + 0x9E3779B97F4A7C15ull;
  z = (z ^ (z >> 30)) * 0xBF58476D1CE4E5B9ull;
  z = (z ^ (z >> 27)) * 0x94D049BB133111EBull;
  return z ^ (z >> 31);
}

/* H(seed, level, lo, j) = sm(sm(sm(seed ^ (level << 56)) ^ lo) ^ j)  (R2) */
uint64_t oracle_sample_hash(uint64_t seed, uint32_t level, uint64_t lo, uint64_t j) {
  uint64_t h = oracle_splitmix64(seed ^ ((uint64_t)level << 56));
  h = oracle_splitmix64(h ^ lo);
  return oracle_splitmix64(h ^ j);
}

/* floor(h * m / 2^64): a position in [0, m) without modulo (R2). */
static uint64_t mulhi64(uint64_t h, uint64_t m) {
  return (uint64_t)(((unsigned __int128)h * (unsigned __int128)m) >> 64);
}

/* ------------------------------------------------------------------ */
/* Bucket-count rule                                                   */
/* ------------------------------------------------------------------ */
static uint64_t pow2ceil(uint64_t x) {
  uint64_t p = 1;
  while (p < x) p <<= 1;
  return p;
}

/* k_b for a bucket of m keys: the paper's fixed k or R29. */
uint32_t oracle_choose_kb(const oracle_params* p, uint64_t m) {
  if (p->k_policy == 0) return p->k;
  uint64_t f = p->fill_div ? p->fill_div : 1;
  uint64_t want = (f * m + p->M - 1) / p->M;        /* ceil(f*m/M) */
  uint64_t kb = pow2ceil(want);
  if (kb < 4) kb = 4;
  if (kb > p->k) kb = p->k;
  return (uint32_t)kb;
}

uint32_t oracle_a_eff(const oracle_params* p, uint32_t kb) {
  uint32_t a = p->a;
  uint32_t cap = p->sample_cap / kb;
  if (cap < a) a = cap;
  if (a < 1) a = 1;
  return a;
}

/* ------------------------------------------------------------------ */
/* Classification                                                      */
/* ------------------------------------------------------------------ */

/* b = #{ i : spl[i] < e } for sorted spl[0..ns) -- the bucket of e under
 * "ties go left" (Algorithm 2 compares e > bt[j]; R3).  Computed
 * as a lower bound by bisection, which equals the count because spl is
 * sorted. */
uint32_t oracle_count_less(const uint64_t* spl, uint32_t ns, uint64_t e) {
  uint32_t lo = 0, hi = ns;
  while (lo < hi) {
    uint32_t mid = lo + (hi - lo) / 2;
    if (spl[mid] < e) lo = mid + 1; else hi = mid;
  }
  return lo;
}

/* Bucket id of e (R4): range bucket b, or in equality mode 2b (range) /
 * 2b+1 (e equals splitter b). */
uint32_t oracle_classify(const uint64_t* spl, uint32_t ns, uint32_t eq, uint64_t e) {
  uint32_t b = oracle_count_less(spl, ns, e);
  if (!eq) return b;
  return 2 * b + ((b < ns && e == spl[b]) ? 1u : 0u);
}

/* Implicit search tree bt[1..k-1] (figure):
 * bt[1] = s_{k/2}; children of bt[j] at 2j and 2j+1.  Closed form
 * bt[j] = s_{(2q+1) k / 2^(d+1)}, d = floor(log2 j), q = j - 2^d, with
 * s_i (1-based) = spl[i-1].  bt[0] is unused and set to 0. */
void oracle_tree(const uint64_t* spl, uint32_t k, uint64_t* bt) {
  bt[0] = 0;
  for (uint32_t j = 1; j < k; j++) {
    uint32_t d = 0;
    while ((2u << d) <= j) d++;
    uint32_t q = j - (1u << d);
    uint64_t idx1 = ((uint64_t)(2 * q + 1) * k) >> (d + 1);   /* 1-based splitter index */
    bt[j] = spl[idx1 - 1];
  }
}

/* Algorithm 2 TraverseTree, literally: j := 1; repeat log k
 * times j := 2j + (e > bt[j]); return j - k + 1 (a 1-based bucket). */
uint32_t oracle_traverse_tree(const uint64_t* bt, uint32_t k, uint64_t e) {
  uint32_t j = 1;
  for (uint32_t s = 1; s < k; s <<= 1) j = 2 * j + (e > bt[j] ? 1u : 0u);
  return j - k + 1;
}

/* ------------------------------------------------------------------ */
/* SmallSort ("any GPU sorting algorithm"): the C library qsort */
/* on (key, value) pairs, ordered by key.                              */
/* ------------------------------------------------------------------ */
typedef struct kv { uint64_t k, v; } kv;

static int cmp_u64(const void* a, const void* b) {
  uint64_t x = *(const uint64_t*)a, y = *(const uint64_t*)b;
  return (x > y) - (x < y);
}
static int cmp_kv(const void* a, const void* b) {
  uint64_t x = ((const kv*)a)->k, y = ((const kv*)b)->k;
  return (x > y) - (x < y);
}

static void small_sort(uint64_t* A, uint64_t* V, uint64_t m) {
  if (m < 2) return;
  if (!V) { qsort(A, m, sizeof(uint64_t), cmp_u64); return; }
  kv* t = (kv*)malloc(m * sizeof(kv));
  for (uint64_t i = 0; i < m; i++) { t[i].k = A[i]; t[i].v = V[i]; }
  qsort(t, m, sizeof(kv), cmp_kv);
  for (uint64_t i = 0; i < m; i++) { A[i] = t[i].k; V[i] = t[i].v; }
  free(t);
}

/* ------------------------------------------------------------------ */
/* Level log                                                           */
/* ------------------------------------------------------------------ */
static void log_push(oracle_log* lg, const oracle_record* r) {
  if (!lg) return;
#pragma omp critical(oracle_log)
  {
    if (lg->n == lg->cap) {
      lg->cap = lg->cap ? 2 * lg->cap : 64;
      lg->r = (oracle_record*)realloc(lg->r, lg->cap * sizeof(oracle_record));
    }
    lg->r[lg->n++] = *r;
  }
}

/* Records in (level, lo) order: the sequential recursion's order does not
 * survive tasks, this one is the same for any thread count. */
static int cmp_rec(const void* a, const void* b) {
  const oracle_record* x = (const oracle_record*)a;
  const oracle_record* y = (const oracle_record*)b;
  if (x->level != y->level) return (x->level > y->level) - (x->level < y->level);
  return (x->lo > y->lo) - (x->lo < y->lo);
}

/* ------------------------------------------------------------------ */
/* One k-way distribution step on A[lo, lo+m) (Phases 1-4)  */
/* ------------------------------------------------------------------ */
typedef struct step_out {
  uint32_t kb, ks, eq, K, a_eff;
  uint64_t* spl;      /* ks-1 */
  uint64_t* child;    /* K    */
} step_out;

/* Phases 2-4 of one bucket over fixed chunks of PAR_CHUNK elements (used
 * with threads > 1 only): ids and per-chunk counts, then the exclusive scan
 * in bucket-major order over (bucket, chunk) -- the paper's k x p table
 * (R6) -- then every chunk places its elements in input order.
 * The result is the same stable partition as the sequential loops. */
#define PAR_CHUNK ((uint64_t)1 << 16)
#define PAR_MIN_ELEMS ((uint64_t)1 << 18)
static void distribute_chunks(uint64_t* A, uint64_t* V, uint64_t lo, uint64_t m, const uint64_t* spl,
                              uint32_t ks, uint32_t eq, uint32_t K, uint64_t** cnt_out) {
  const uint64_t nch = (m + PAR_CHUNK - 1) / PAR_CHUNK;
  uint32_t* id = (uint32_t*)malloc(m * sizeof(uint32_t));
  uint64_t* h = (uint64_t*)calloc(nch * K, sizeof(uint64_t));      /* h[c*K + b] */
#pragma omp taskloop grainsize(1)
  for (uint64_t c = 0; c < nch; c++) {
    const uint64_t e = (c + 1) * PAR_CHUNK < m ? (c + 1) * PAR_CHUNK : m;
    for (uint64_t i = c * PAR_CHUNK; i < e; i++) {
      id[i] = oracle_classify(spl, ks - 1, eq, A[lo + i]);
      h[c * K + id[i]]++;
    }
  }
  uint64_t* cnt = (uint64_t*)calloc(K, sizeof(uint64_t));
  uint64_t run = 0;
  for (uint32_t b = 0; b < K; b++)
    for (uint64_t c = 0; c < nch; c++) {
      const uint64_t x = h[c * K + b];
      h[c * K + b] = run;
      run += x;
      cnt[b] += x;
    }
  uint64_t* TA = (uint64_t*)malloc(m * sizeof(uint64_t));
  uint64_t* TV = V ? (uint64_t*)malloc(m * sizeof(uint64_t)) : NULL;
#pragma omp taskloop grainsize(1)
  for (uint64_t c = 0; c < nch; c++) {
    const uint64_t e = (c + 1) * PAR_CHUNK < m ? (c + 1) * PAR_CHUNK : m;
    for (uint64_t i = c * PAR_CHUNK; i < e; i++) {
      uint64_t d = h[c * K + id[i]]++;
      TA[d] = A[lo + i];
      if (V) TV[d] = V[lo + i];
    }
  }
  memcpy(A + lo, TA, m * sizeof(uint64_t));
  if (V) memcpy(V + lo, TV, m * sizeof(uint64_t));
  free(TA); free(TV); free(h); free(id);
  *cnt_out = cnt;
}

static void distribute(uint64_t* A, uint64_t* V, uint64_t lo, uint64_t m, uint32_t level,
                       const oracle_params* p, step_out* o, int par) {
  /* Phase 1: random sample S of a*k elements (R1, R2), sorted. */
  uint32_t kb = oracle_choose_kb(p, m);
  uint32_t a = oracle_a_eff(p, kb);
  uint64_t s = (uint64_t)a * kb;
  uint64_t* S = (uint64_t*)malloc(s * sizeof(uint64_t));
  for (uint64_t j = 0; j < s; j++)
    S[j] = A[lo + mulhi64(oracle_sample_hash(p->seed, level, lo, j), m)];
  qsort(S, s, sizeof(uint64_t), cmp_u64);

  /* Splitters <S_a, S_2a, ..., S_a(k-1)>: spl[i] = S[a(i+1)-1]. */
  uint32_t ks = kb, eq = 0;
  uint64_t* spl = (uint64_t*)malloc((kb > 1 ? kb - 1 : 1) * sizeof(uint64_t));
  for (uint32_t i = 0; i + 1 < kb; i++) spl[i] = S[(uint64_t)a * (i + 1) - 1];
  /* Equality mode (R4): duplicate splitters, or a single splitter. */
  if (kb == 2) eq = 1;
  for (uint32_t i = 0; i + 2 < kb; i++) if (spl[i] == spl[i + 1]) eq = 1;
  if (eq) {
    ks = kb / 2 < 2 ? 2 : kb / 2;
    uint64_t stride = s / ks;
    for (uint32_t i = 0; i + 1 < ks; i++) spl[i] = S[stride * (i + 1) - 1];
  }
  uint32_t K = eq ? 2 * ks - 1 : ks;
  free(S);
  uint64_t* cnt;

  if (par && m >= PAR_MIN_ELEMS) {
    distribute_chunks(A, V, lo, m, spl, ks, eq, K, &cnt);
  } else {
    /* Phase 2: bucket index of every element and the bucket sizes. */
    uint32_t* id = (uint32_t*)malloc(m * sizeof(uint32_t));
    cnt = (uint64_t*)calloc(K, sizeof(uint64_t));
    for (uint64_t i = 0; i < m; i++) {
      id[i] = oracle_classify(spl, ks - 1, eq, A[lo + i]);
      cnt[id[i]]++;
    }
    /* Phase 3: exclusive prefix sum over the bucket sizes. */
    uint64_t* off = (uint64_t*)malloc(K * sizeof(uint64_t));
    uint64_t run = 0;
    for (uint32_t b = 0; b < K; b++) { off[b] = run; run += cnt[b]; }
    /* Phase 4: place every element at its bucket's next free slot, in input
     * order -- a stable partition (R7). */
    uint64_t* TA = (uint64_t*)malloc(m * sizeof(uint64_t));
    uint64_t* TV = V ? (uint64_t*)malloc(m * sizeof(uint64_t)) : NULL;
    for (uint64_t i = 0; i < m; i++) {
      uint64_t d = off[id[i]]++;
      TA[d] = A[lo + i];
      if (V) TV[d] = V[lo + i];
    }
    memcpy(A + lo, TA, m * sizeof(uint64_t));
    if (V) memcpy(V + lo, TV, m * sizeof(uint64_t));
    free(TA); free(TV); free(off); free(id);
  }

  o->kb = kb; o->ks = ks; o->eq = eq; o->K = K; o->a_eff = a;
  o->spl = spl; o->child = cnt;
}

/* ------------------------------------------------------------------ */
/* Algorithm 1 SampleSort, with delayed small sorts */
/* ------------------------------------------------------------------ */
#define TASK_MIN_ELEMS 4096
static void sort_range(uint64_t* A, uint64_t* V, uint64_t lo, uint64_t m, uint32_t level,
                       const oracle_params* p, oracle_log* lg, int par) {
  if (m <= p->M) {                              /* "if n < M then SmallSort" (R5) */
    small_sort(A + lo, V ? V + lo : NULL, m);
    return;
  }
  step_out o;
  distribute(A, V, lo, m, level, p, &o, par);
  oracle_record r;
  r.level = level; r.kb = o.kb; r.ks = o.ks; r.eq = o.eq; r.K = o.K; r.a_eff = o.a_eff;
  r.lo = lo; r.m = m; r.spl = o.spl; r.child = o.child;
  /* Concatenate(SampleSort(b1), ..., SampleSort(bk)). */
  if (lg) log_push(lg, &r);                     /* the log owns spl/child from here */
  uint64_t c = lo;
  for (uint32_t b = 0; b < o.K; b++) {
    uint64_t cm = o.child[b];
    if (!(o.eq && (b & 1))) {                   /* equality buckets hold one key value: final (R4) */
      if (par && cm >= TASK_MIN_ELEMS) {
#pragma omp task firstprivate(c, cm)
        sort_range(A, V, c, cm, level + 1, p, lg, par);
      } else {
        sort_range(A, V, c, cm, level + 1, p, lg, par);
      }
    }
    c += cm;
  }
  if (par) {
#pragma omp taskwait
  }
  if (!lg) { free(o.spl); free(o.child); }
}

/* ------------------------------------------------------------------ */
/* Exported API                                                        */
/* ------------------------------------------------------------------ */

/* Sorts keys[0..n) in place (values, if non-NULL, travel with keys).
 * If want_log is non-zero, returns a log handle of every distribution
 * step (free with oracle_log_free); otherwise returns NULL. */
void* oracle_sort(uint64_t* keys, uint64_t* vals, uint64_t n, const oracle_params* p, int want_log) {
  oracle_log* lg = want_log ? (oracle_log*)calloc(1, sizeof(oracle_log)) : NULL;
  if (p->threads > 1) {
#pragma omp parallel num_threads(p->threads)
#pragma omp single
    sort_range(keys, vals, 0, n, 0, p, lg, 1);
  } else {
    sort_range(keys, vals, 0, n, 0, p, lg, 0);
  }
  if (lg && lg->n > 1) qsort(lg->r, lg->n, sizeof(oracle_record), cmp_rec);
  return lg;
}

/* One distribution step on keys[0..n) at level 0, regardless of M: the
 * partition written in place, splitters and child sizes returned
 * through the log (one record). */
void* oracle_distribute(uint64_t* keys, uint64_t* vals, uint64_t n, const oracle_params* p) {
  oracle_log* lg = (oracle_log*)calloc(1, sizeof(oracle_log));
  step_out o;
  distribute(keys, vals, 0, n, 0, p, &o, 0);
  oracle_record r;
  r.level = 0; r.kb = o.kb; r.ks = o.ks; r.eq = o.eq; r.K = o.K; r.a_eff = o.a_eff;
  r.lo = 0; r.m = n; r.spl = o.spl; r.child = o.child;
  log_push(lg, &r);
  return lg;
}

size_t oracle_log_count(const void* h) { return h ? ((const oracle_log*)h)->n : 0; }

/* info[0..8) = level, kb, ks, eq, K, a_eff, lo, m */
void oracle_log_info(const void* h, size_t i, uint64_t* info) {
  const oracle_record* r = &((const oracle_log*)h)->r[i];
  info[0] = r->level; info[1] = r->kb; info[2] = r->ks; info[3] = r->eq;
  info[4] = r->K; info[5] = r->a_eff; info[6] = r->lo; info[7] = r->m;
}
void oracle_log_splitters(const void* h, size_t i, uint64_t* out) {
  const oracle_record* r = &((const oracle_log*)h)->r[i];
  if (r->ks > 1) memcpy(out, r->spl, (size_t)(r->ks - 1) * sizeof(uint64_t));
}
void oracle_log_children(const void* h, size_t i, uint64_t* out) {
  const oracle_record* r = &((const oracle_log*)h)->r[i];
  memcpy(out, r->child, (size_t)r->K * sizeof(uint64_t));
}
void oracle_log_free(void* h) {
  oracle_log* lg = (oracle_log*)h;
  if (!lg) return;
  for (size_t i = 0; i < lg->n; i++) { free(lg->r[i].spl); free(lg->r[i].child); }
  free(lg->r);
  free(lg);
}

/* The element of rank r (0-based) of keys[0..n): by definition the r-th
 * entry of the sorted output.  Hoare quickselect on a private copy, so
 * single sorted outputs can be checked at sizes where a full oracle sort
 * is too slow. */
uint64_t oracle_select(const uint64_t* keys, uint64_t n, uint64_t r) {
  uint64_t* a = (uint64_t*)malloc(n * sizeof(uint64_t));
  memcpy(a, keys, n * sizeof(uint64_t));
  int64_t lo = 0, hi = (int64_t)n - 1, rr = (int64_t)r;
  uint64_t state = 0x12345678ull;
  while (lo < hi) {
    state = oracle_splitmix64(state);
    uint64_t pivot = a[lo + (int64_t)mulhi64(state, (uint64_t)(hi - lo + 1))];
    int64_t i = lo, j = hi;
    while (i <= j) {
      while (a[i] < pivot) i++;
      while (a[j] > pivot) j--;
      if (i <= j) { uint64_t t = a[i]; a[i] = a[j]; a[j] = t; i++; j--; }
    }
    /* a[lo..j] <= pivot <= a[i..hi]; everything strictly between equals pivot */
    if (rr <= j) hi = j;
    else if (rr >= i) lo = i;
    else break;
  }
  uint64_t v = a[r];
  free(a);
  return v;
}
