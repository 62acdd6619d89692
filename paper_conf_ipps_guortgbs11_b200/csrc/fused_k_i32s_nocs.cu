// Explicit instantiations of fused_tma_kernel<int32_t in, int32_t out, kR=1, kSwz=1 (column strips, linear rows), checksum=false>
// (split for parallel builds).
#include "fused_kernel.cuh"

namespace aol {
namespace fused {
KernelFn tma_kernel_i32s_nocs(int block, int cps) {
    return pick_tma_kernel<int32_t, int32_t, 1, 1, false>(block, cps);
}
}  // namespace fused
}  // namespace aol
