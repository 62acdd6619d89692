// tiler_es1.cu -- generic tiler kernels instantiated for 1-byte elements (see tiler_kernels.cuh).
#include "tiler_kernels.cuh"

namespace aol {

aol_status_t tiler_launch_es1(int mode, const TilerDev& td, int vec, const void* src, void* dst,
                                unsigned long long* ws, int num_sms, cudaStream_t s) {
    switch (mode) {
        case 0: return launch_es<1, 0>(td, vec, src, dst, ws, num_sms, s);
        case 1: return launch_es<1, 1>(td, vec, src, dst, ws, num_sms, s);
        case 2: return launch_es<1, 2>(td, vec, src, dst, ws, num_sms, s);
        case 3: return launch_es<1, 3>(td, vec, src, dst, ws, num_sms, s);
        case 4: return launch_es<1, 4>(td, vec, src, dst, ws, num_sms, s);
        default: return launch_es<1, 5>(td, vec, src, dst, ws, num_sms, s);
    }
}

}  // namespace aol
