// gss_inst_pairs_u64_desc.cu -- the sort engine instantiated for (uint64_t, uint64_t, Greater).
#define GSS_INSTANTIATING 1
#include "gss_impl.cuh"

namespace gssh {
using namespace gss;
template GSS_DRIVE_SIG(uint64_t, uint64_t, Greater);
}  // namespace gssh
