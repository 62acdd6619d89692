// Explicit instantiations of fused_tma_kernel<uint8_t packed 24-bit pixels in, int16_t out, kR=3 channels,
// kSwz=3 (packed marker), checksum=false> (split for parallel builds).
#include "fused_kernel.cuh"

namespace aol {
namespace fused {
KernelFn tma_kernel_rgbh_nocs(int block, int cps) {
    return pick_tma_kernel<uint8_t, int16_t, 3, 3, false>(block, cps);
}
}  // namespace fused
}  // namespace aol
