// tests/cxx/custom_less.cu -- instantiates include/gss.hpp with comparators and
// types libgss.so does not export (comparator-only contract):
//  * u64 keys ordered by their residue modulo 1000003 (a strict weak order with
//    large equivalence classes: the equality-bucket path runs on equivalent,
//    not equal, keys);
//  * u32 keys with u64 values in descending order (a key/value width pair the
//    library does not export).
// Built by paper_conf_ipps_leischneros10_b200._build.build_cxx_test() into
// tests/cxx/libgss_cxx_test.so; exercised by tests/test_gpu_sort.py.
#include "../../include/gss.hpp"

struct ResidueLess {
  __device__ __forceinline__ bool operator()(const uint64_t& a, const uint64_t& b) const {
    return a % 1000003ull < b % 1000003ull;
  }
};
struct Desc {
  template <class T> __device__ __forceinline__ bool operator()(const T& a, const T& b) const { return b < a; }
};

extern "C" gss_status cxx_sort_residue_u64(const uint64_t* in, uint64_t* out, size_t n, void* t, size_t* tb, void* s) {
  return gss::sort<uint64_t, ResidueLess>(in, out, n, t, tb, reinterpret_cast<cudaStream_t>(s));
}
extern "C" gss_status cxx_sort_pairs_desc_u32_u64(const uint32_t* ki, const uint64_t* vi, uint32_t* ko, uint64_t* vo,
                                                  size_t n, void* t, size_t* tb, void* s) {
  return gss::sort_pairs<uint32_t, uint64_t, Desc>(ki, vi, ko, vo, n, t, tb, reinterpret_cast<cudaStream_t>(s));
}
