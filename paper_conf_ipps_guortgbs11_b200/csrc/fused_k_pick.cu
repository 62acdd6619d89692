// Dispatch between the separately compiled fused_tma_kernel instantiations.
#include "fused_kernel.cuh"

namespace aol {
namespace fused {
KernelFn tma_kernel_i32_cs(int block, int cps);
KernelFn tma_kernel_i32_nocs(int block, int cps);
KernelFn tma_kernel_i32l_cs(int block, int cps);
KernelFn tma_kernel_i32l_nocs(int block, int cps);
KernelFn tma_kernel_i32s_cs(int block, int cps);
KernelFn tma_kernel_i32s_nocs(int block, int cps);
KernelFn tma_kernel_u8_cs(int block, int cps);
KernelFn tma_kernel_u8_nocs(int block, int cps);
KernelFn tma_kernel_u8r2_cs(int block, int cps);
KernelFn tma_kernel_u8r2_nocs(int block, int cps);
KernelFn tma_kernel_u8h_cs(int block, int cps);
KernelFn tma_kernel_u8h_nocs(int block, int cps);
KernelFn tma_kernel_u8r2h_cs(int block, int cps);
KernelFn tma_kernel_u8r2h_nocs(int block, int cps);

KernelFn tma_kernel_rgb_cs(int block, int cps);
KernelFn tma_kernel_rgb_nocs(int block, int cps);
KernelFn tma_kernel_rgbh_cs(int block, int cps);
KernelFn tma_kernel_rgbh_nocs(int block, int cps);

KernelFn tma_kernel_rgb8(bool checksum, bool out16, int block, int cps) {
    if (out16) return checksum ? tma_kernel_rgbh_cs(block, cps) : tma_kernel_rgbh_nocs(block, cps);
    return checksum ? tma_kernel_rgb_cs(block, cps) : tma_kernel_rgb_nocs(block, cps);
}

KernelFn tma_kernel_i32(bool checksum, int layout, int block, int cps) {
    if (layout == 0) return checksum ? tma_kernel_i32l_cs(block, cps) : tma_kernel_i32l_nocs(block, cps);
    if (layout == 1) return checksum ? tma_kernel_i32s_cs(block, cps) : tma_kernel_i32s_nocs(block, cps);
    return checksum ? tma_kernel_i32_cs(block, cps) : tma_kernel_i32_nocs(block, cps);
}
KernelFn tma_kernel_u8(bool checksum, bool out16, int reps_per_thread, int block, int cps) {
    if (out16) {
        if (reps_per_thread == 2) return checksum ? tma_kernel_u8r2h_cs(block, cps) : tma_kernel_u8r2h_nocs(block, cps);
        return checksum ? tma_kernel_u8h_cs(block, cps) : tma_kernel_u8h_nocs(block, cps);
    }
    if (reps_per_thread == 2) return checksum ? tma_kernel_u8r2_cs(block, cps) : tma_kernel_u8r2_nocs(block, cps);
    return checksum ? tma_kernel_u8_cs(block, cps) : tma_kernel_u8_nocs(block, cps);
}
}  // namespace fused
}  // namespace aol
