// Explicit instantiations of fused_tma_kernel<uint8_t packed 24-bit pixels in, int32_t out, kR=3 channels,
// kSwz=3 (packed marker), checksum=true> (split for parallel builds).
#include "fused_kernel.cuh"

namespace aol {
namespace fused {
KernelFn tma_kernel_rgb_cs(int block, int cps) {
    return pick_tma_kernel<uint8_t, int32_t, 3, 3, true>(block, cps);
}
}  // namespace fused
}  // namespace aol
