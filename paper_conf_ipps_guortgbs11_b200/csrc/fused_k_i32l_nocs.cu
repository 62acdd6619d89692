// Explicit instantiations of fused_tma_kernel<int32_t in, int32_t out, kR=1, kSwz=0 (linear rows, 1-D bulk copies), checksum=false>
// (split for parallel builds).
#include "fused_kernel.cuh"

namespace aol {
namespace fused {
KernelFn tma_kernel_i32l_nocs(int block, int cps) {
    return pick_tma_kernel<int32_t, int32_t, 1, 0, false>(block, cps);
}
}  // namespace fused
}  // namespace aol
