// gss_inst_f64.cu -- the sort engine instantiated for (double, NoVal, TotalLess).
#define GSS_INSTANTIATING 1
#include "gss_impl.cuh"

namespace gssh {
using namespace gss;
template GSS_DRIVE_SIG(double, NoVal, TotalLess);
}  // namespace gssh
