// Explicit instantiations of fused_tma_kernel<uint8_t in, int32_t out, kR=2, kSwz=0, checksum=true>
// (split for parallel builds).
#include "fused_kernel.cuh"

namespace aol {
namespace fused {
KernelFn tma_kernel_u8r2_cs(int block, int cps) {
    return pick_tma_kernel<uint8_t, int32_t, 2, 0, true>(block, cps);
}
}  // namespace fused
}  // namespace aol
