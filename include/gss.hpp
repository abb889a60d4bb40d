/*
 * gss.hpp -- the comparator-only C++ interface of the B200 GPU sample sort.
 *
 * The paper sorts keys given only a comparison function (PAPER.md P:52-54,
 * section 1): every kernel of the path (Phase 1 sample sort, Phase 2 tree
 * descent -- Algorithm 2's e > bt[j] becomes less(bt[j], e) --, the
 * equality-bucket test !less(a,b) && !less(b,a), the in-SM merge sort)
 * evaluates keys only through Less.  libgss.so exports the std::less and
 * greater instantiations for u32/u64 keys and pairs (include/gss.h); this
 * header instantiates the same kernels for any other Key / Val / Less in the
 * caller's own translation unit:
 *
 *   #include "gss.hpp"       // nvcc -gencode arch=compute_100a,code=sm_100a -std=c++17
 *                            //      --expt-relaxed-constexpr -I <repo>/include
 *   struct ByResidue { __device__ bool operator()(uint64_t a, uint64_t b) const { return a % 97 < b % 97; } };
 *   gss::sort<uint64_t, ByResidue>(d_in, d_out, n, nullptr, &bytes);   // size query
 *   gss::sort<uint64_t, ByResidue>(d_in, d_out, n, d_temp, &bytes, stream);
 *
 * Requirements: Key and Val trivially copyable, 4 or 8 bytes; Less a
 * default-constructible, trivially copyable strict weak ordering with a
 * __device__ operator()(const Key&, const Key&) const.  Keys that are
 * equivalent under Less may appear in any order (the sort is unstable,
 * P:262).  Arguments, temp-size queries, aliasing, streams and
 * status codes follow include/gss.h.
 */
#ifndef GSS_HPP
#define GSS_HPP

#include "gss.h"
#include "../paper_conf_ipps_leischneros10_b200/csrc/gss_impl.cuh"

namespace gss {

template <class Key, class Less>
inline gss_status sort(const Key* keys_in, Key* keys_out, size_t n, void* temp, size_t* temp_bytes,
                       cudaStream_t stream = nullptr, const gss_params* p = nullptr) {
  static_assert(sizeof(Key) == 4 || sizeof(Key) == 8, "keys of 4 or 8 bytes");
  return gssh::drive<Key, NoVal, Less>(gssh::io_dev(keys_in, nullptr, keys_out, nullptr), n, temp, temp_bytes,
                                       stream, p, MODE_SORT, false);
}

template <class Key, class Val, class Less>
inline gss_status sort_pairs(const Key* keys_in, const Val* vals_in, Key* keys_out, Val* vals_out, size_t n,
                             void* temp, size_t* temp_bytes, cudaStream_t stream = nullptr,
                             const gss_params* p = nullptr) {
  static_assert(sizeof(Key) == 4 || sizeof(Key) == 8, "keys of 4 or 8 bytes");
  static_assert(sizeof(Val) == 4 || sizeof(Val) == 8, "values of 4 or 8 bytes");
  return gssh::drive<Key, Val, Less>(gssh::io_dev(keys_in, vals_in, keys_out, vals_out), n, temp, temp_bytes, stream,
                                     p, MODE_SORT, false);
}

}  // namespace gss

#endif  // GSS_HPP
