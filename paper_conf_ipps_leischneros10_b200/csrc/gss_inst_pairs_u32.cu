// gss_inst_pairs_u32.cu -- the sort engine instantiated for (uint32_t, uint32_t, Less).
#define GSS_INSTANTIATING 1
#include "gss_impl.cuh"

namespace gssh {
using namespace gss;
template GSS_DRIVE_SIG(uint32_t, uint32_t, Less);
}  // namespace gssh
