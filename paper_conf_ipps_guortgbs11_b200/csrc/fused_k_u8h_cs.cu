// Explicit instantiations of fused_tma_kernel<uint8_t in, int16_t out, kR=1, kSwz=0, checksum=true>
// (split for parallel builds).
#include "fused_kernel.cuh"

namespace aol {
namespace fused {
KernelFn tma_kernel_u8h_cs(int block, int cps) {
    return pick_tma_kernel<uint8_t, int16_t, 1, 0, true>(block, cps);
}
}  // namespace fused
}  // namespace aol
