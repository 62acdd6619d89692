// Explicit instantiations of fused_tma_kernel<uint8_t in, int32_t out, kR=1, kSwz=0, checksum=false>
// (split for parallel builds).
#include "fused_kernel.cuh"

namespace aol {
namespace fused {
KernelFn tma_kernel_u8_nocs(int block, int cps) {
    return pick_tma_kernel<uint8_t, int32_t, 1, 0, false>(block, cps);
}
}  // namespace fused
}  // namespace aol
