// gss_inst_u32.cu -- the sort engine instantiated for (uint32_t, NoVal, Less).
#define GSS_INSTANTIATING 1
#include "gss_impl.cuh"

namespace gssh {
using namespace gss;
template GSS_DRIVE_SIG(uint32_t, NoVal, Less);
}  // namespace gssh
