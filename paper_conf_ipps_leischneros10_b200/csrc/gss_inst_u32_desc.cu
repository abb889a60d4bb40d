// gss_inst_u32_desc.cu -- the sort engine instantiated for (uint32_t, NoVal, Greater).
#define GSS_INSTANTIATING 1
#include "gss_impl.cuh"

namespace gssh {
using namespace gss;
template GSS_DRIVE_SIG(uint32_t, NoVal, Greater);
}  // namespace gssh
