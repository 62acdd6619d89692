// synth.cu -- K-6: counter-based synthetic frame generator (test/bench input
// support, not part of the method).  Same definition as synth/__init__.py,
// implemented independently here; a GPU test checks the two agree bit-exactly.
#include <cuda_runtime.h>

#include <algorithm>
#include <cstdint>

#include "common.h"

namespace aol {

namespace {

__device__ __forceinline__ uint64_t splitmix64(uint64_t z) {
    z += 0x9E3779B97F4A7C15ull;
    z = (z ^ (z >> 30)) * 0xBF58476D1CE4E5B9ull;
    z = (z ^ (z >> 27)) * 0x94D049BB133111EBull;
    return z ^ (z >> 31);
}

template <typename T>
__global__ void __launch_bounds__(256) synth_kernel(T* __restrict__ out, uint64_t seedphi, uint64_t start,
                                                    int64_t total, int32_t W, int32_t kind, int32_t value) {
    for (int64_t i = int64_t(blockIdx.x) * blockDim.x + threadIdx.x; i < total; i += int64_t(gridDim.x) * blockDim.x) {
        int32_t v;
        if (kind == 3) {
            v = int32_t(i % W);
        } else if (kind == 4) {
            v = value;
        } else {
            const uint64_t u = splitmix64(seedphi + start + uint64_t(i));
            v = kind == 0 ? int32_t(u >> 56) : kind == 1 ? int32_t(u >> 61) : int32_t(int64_t(u >> 37) - (1ll << 26));
        }
        out[i] = T(v);
    }
}

}  // namespace

aol_status_t launch_synth(uint64_t seed, int64_t frame0, int64_t nframes, int64_t channels, int64_t H, int64_t W,
                          int32_t kind, int32_t value, int out_u8, void* d_out, cudaStream_t s) {
    const int64_t total = nframes * channels * H * W;
    if (total == 0) return AOL_OK;
    DeviceInfo dev;
    aol_status_t st = device_info(&dev);
    if (st != AOL_OK) return st;
    const uint64_t seedphi = seed * 0x9E3779B97F4A7C15ull;
    const uint64_t start = uint64_t(frame0) * uint64_t(channels) * uint64_t(H) * uint64_t(W);
    const int grid = int(std::max<int64_t>(1, std::min<int64_t>((total + 255) / 256, int64_t(dev.num_sms) * 32)));
    if (out_u8)
        synth_kernel<uint8_t><<<grid, 256, 0, s>>>(static_cast<uint8_t*>(d_out), seedphi, start, total, int32_t(W),
                                                   kind, value);
    else
        synth_kernel<int32_t><<<grid, 256, 0, s>>>(static_cast<int32_t*>(d_out), seedphi, start, total, int32_t(W),
                                                   kind, value);
    AOL_LAUNCH_CHECK("synth_kernel");
    return AOL_OK;
}

}  // namespace aol
