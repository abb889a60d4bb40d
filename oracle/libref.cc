// oracle/libref.cc -- TEST INFRASTRUCTURE ONLY (bench.py cpu_baseline leg).
//
// Library sorts timed beside the oracle as CPU references:
// std::sort on one thread and libstdc++'s __gnu_parallel::sort on `threads`
// threads.  They are not the oracle (the oracle is oracle.c, written from the
// paper); they only put the oracle's CPU time in context.  No code here is
// shared with the CUDA path.
#include <algorithm>
#include <cstdint>
#include <parallel/algorithm>
#include <omp.h>

extern "C" {

void libref_std_sort_u64(uint64_t* a, uint64_t n) { std::sort(a, a + n); }
void libref_std_sort_u32(uint32_t* a, uint64_t n) { std::sort(a, a + n); }

void libref_parallel_sort_u64(uint64_t* a, uint64_t n, int threads) {
  omp_set_num_threads(threads > 0 ? threads : 1);
  __gnu_parallel::sort(a, a + n);
}
void libref_parallel_sort_u32(uint32_t* a, uint64_t n, int threads) {
  omp_set_num_threads(threads > 0 ? threads : 1);
  __gnu_parallel::sort(a, a + n);
}

}  // extern "C"
