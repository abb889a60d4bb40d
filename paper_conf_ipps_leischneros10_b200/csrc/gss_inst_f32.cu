// gss_inst_f32.cu -- the sort engine instantiated for (float, NoVal, TotalLess).
#define GSS_INSTANTIATING 1
#include "gss_impl.cuh"

namespace gssh {
using namespace gss;
template GSS_DRIVE_SIG(float, NoVal, TotalLess);
}  // namespace gssh
