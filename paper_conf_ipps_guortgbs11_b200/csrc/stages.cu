// stages.cu -- K-3 (horizontal filter alone), K-4 (vertical filter alone) and
// the per-frame checksum kernel used by the unfused paths.
//
//  K-3: Y[y][3r+k] = T( sum_{t<6} X[y][(8r + s_k + t) mod W] ), s = (0,2,5)
//       (Fig. 10 tilers P:L681-694, Fig. 5 task P:L435-446, Fig. 7 scatter P:L476-478)
//  K-4: Z[4b+k][x] = T( sum_{t<6} Y[(9b + 2k + t) mod H][x] )   (reading Z1/Z2)
//  T(S) = S/6 - S%6 == 7*(S/6) - S.
#include <cuda_runtime.h>

#include <algorithm>
#include <cstdint>

#include "common.h"

namespace aol {

namespace {

__device__ __forceinline__ int32_t task_T(int32_t S) { return 7 * (S / 6) - S; }

// One CTA walks rows; thread t owns repetition t (+ k*blockDim).  Two 128-bit
// loads per repetition, the 3-column pattern overlap comes from lane+1 by
// shuffle (lane 31 / the wrapping repetition reload it).
__global__ void __launch_bounds__(256) downscale_h_kernel(const int32_t* __restrict__ X, int32_t* __restrict__ Y,
                                                          int64_t rows, int32_t W, int32_t reps) {
    const int32_t Wo = 3 * reps;
    const int lane = threadIdx.x & 31;
    for (int64_t row = blockIdx.x; row < rows; row += gridDim.x) {
        const int32_t* xr = X + size_t(row) * W;
        int32_t* yr = Y + size_t(row) * Wo;
        for (int32_t rbase = 0; rbase < reps; rbase += blockDim.x) {
            const int32_t rt = rbase + int32_t(threadIdx.x);
            const bool active = rt < reps;
            const int32_t r = active ? rt : reps - 1;
            const int4 q0 = __ldg(reinterpret_cast<const int4*>(xr + 8 * r));
            const int4 q1 = __ldg(reinterpret_cast<const int4*>(xr + 8 * r + 4));
            const int32_t e = q0.x + q0.y, d = e + q0.z, q = q0.z + q0.w, p = q1.x + q1.y, f = q1.z + q1.w;
            int32_t dn = __shfl_down_sync(0xffffffffu, d, 1);
            if (lane == 31 || r + 1 == reps) {
                const int32_t rn = (r + 1 == reps) ? 0 : r + 1;
                const int4 qn = __ldg(reinterpret_cast<const int4*>(xr + 8 * rn));
                dn = qn.x + qn.y + qn.z;
            }
            if (active) {
                yr[3 * r + 0] = task_T(e + q + p);
                yr[3 * r + 1] = task_T(q + p + f);
                yr[3 * r + 2] = task_T(q1.y + f + dn);
            }
        }
    }
}

// Scalar fallback for W % 8 == 0 but rows not 16-byte aligned (W % 4 != 0 cannot
// happen; kept for pointer misalignment).
__global__ void __launch_bounds__(256) downscale_h_scalar_kernel(const int32_t* __restrict__ X,
                                                                 int32_t* __restrict__ Y, int64_t rows, int32_t W,
                                                                 int32_t reps) {
    const int32_t Wo = 3 * reps;
    const int64_t total = rows * Wo;
    for (int64_t i = int64_t(blockIdx.x) * blockDim.x + threadIdx.x; i < total; i += int64_t(gridDim.x) * blockDim.x) {
        const int64_t row = i / Wo;
        const int32_t xo = int32_t(i - row * Wo);
        const int32_t r = xo / 3, k = xo - 3 * (xo / 3);
        const int32_t s0 = k == 0 ? 0 : (k == 1 ? 2 : 5);
        const int32_t* xr = X + size_t(row) * W;
        int32_t S = 0;
        for (int t = 0; t < 6; ++t) {
            int32_t c = 8 * r + s0 + t;
            if (c >= W) c -= W;
            S += xr[c];
        }
        Y[i] = task_T(S);
    }
}

// Thread per (plane, band, column): 12 coalesced row reads, 4 outputs.
__global__ void __launch_bounds__(256) downscale_v_kernel(const int32_t* __restrict__ Y, int32_t* __restrict__ Z,
                                                          int64_t planes, int32_t H, int32_t W) {
    const int32_t nb = H / 9;
    const int64_t per_plane = int64_t(nb) * W;
    const int64_t total = planes * per_plane;
    for (int64_t i = int64_t(blockIdx.x) * blockDim.x + threadIdx.x; i < total; i += int64_t(gridDim.x) * blockDim.x) {
        const int64_t plane = i / per_plane;
        const int64_t rem = i - plane * per_plane;
        const int32_t b = int32_t(rem / W);
        const int32_t x = int32_t(rem - int64_t(b) * W);
        const int32_t* yp = Y + size_t(plane) * H * W + x;
        int32_t v[12];
#pragma unroll
        for (int j = 0; j < 12; ++j) {
            int32_t row = 9 * b + j;
            if (row >= H) row -= H;
            v[j] = __ldg(yp + size_t(row) * W);
        }
        int32_t* zp = Z + (size_t(plane) * (4 * nb) + size_t(4 * b)) * W + x;
#pragma unroll
        for (int k = 0; k < 4; ++k) {
            const int32_t S = v[2 * k] + v[2 * k + 1] + v[2 * k + 2] + v[2 * k + 3] + v[2 * k + 4] + v[2 * k + 5];
            zp[size_t(k) * W] = task_T(S);
        }
    }
}

// Vectorised K-4 (W % 4 == 0, 16-byte aligned): thread per (plane, run of kVBands bands, 4 adjacent
// columns).  It walks its bands top to bottom with 128-bit loads, carrying rows 9..11 of band b over as
// rows 0..2 of band b+1, so every Y row is loaded once per thread (plus the 3 halo rows of the run).
constexpr int kVBands = 8;

__global__ void __launch_bounds__(256) downscale_v_vec_kernel(const int32_t* __restrict__ Y, int32_t* __restrict__ Z,
                                                              int64_t planes, int32_t H, int32_t W) {
    const int32_t nb = H / 9, Q = W / 4, nchunks = (nb + kVBands - 1) / kVBands;
    const int64_t total = planes * nchunks * Q;
    for (int64_t i = int64_t(blockIdx.x) * blockDim.x + threadIdx.x; i < total; i += int64_t(gridDim.x) * blockDim.x) {
        const int32_t q = int32_t(i % Q);
        const int64_t rest = i / Q;
        const int32_t c = int32_t(rest % nchunks);
        const int64_t plane = rest / nchunks;
        const int4* yp = reinterpret_cast<const int4*>(Y + size_t(plane) * H * W) + q;
        int4* zp = reinterpret_cast<int4*>(Z + size_t(plane) * (4 * nb) * W) + q;
        const int32_t b0 = c * kVBands, b1 = min(b0 + kVBands, nb);
        int4 v[12];
#pragma unroll
        for (int j = 0; j < 3; ++j) v[j] = __ldg(yp + size_t(9 * b0 + j) * Q);
        for (int32_t b = b0; b < b1; ++b) {
#pragma unroll
            for (int j = 3; j < 12; ++j) {
                int32_t row = 9 * b + j;
                if (row >= H) row -= H;   // the last band's halo wraps to rows 0..2 (reading Z1)
                v[j] = __ldg(yp + size_t(row) * Q);
            }
#pragma unroll
            for (int k = 0; k < 4; ++k) {
                int4 S = v[2 * k];
#pragma unroll
                for (int t = 1; t < 6; ++t) {
                    S.x += v[2 * k + t].x;
                    S.y += v[2 * k + t].y;
                    S.z += v[2 * k + t].z;
                    S.w += v[2 * k + t].w;
                }
                zp[size_t(4 * b + k) * Q] = make_int4(task_T(S.x), task_T(S.y), task_T(S.z), task_T(S.w));
            }
#pragma unroll
            for (int j = 0; j < 3; ++j) v[j] = v[9 + j];
        }
    }
}

// cs[f] += sum_e (u64)(u32)Z[f][e] * (e + 1)   (e = flat index within the frame)
__global__ void __launch_bounds__(256) checksum_kernel(const int32_t* __restrict__ Z, int64_t frames,
                                                       int64_t per_frame, uint64_t* __restrict__ cs) {
    for (int64_t f = blockIdx.y; f < frames; f += gridDim.y) {
        const int32_t* zf = Z + size_t(f) * per_frame;
        uint64_t acc = 0;
        for (int64_t e = int64_t(blockIdx.x) * blockDim.x + threadIdx.x; e < per_frame;
             e += int64_t(gridDim.x) * blockDim.x)
            acc += uint64_t(uint32_t(zf[e])) * uint64_t(e + 1);
#pragma unroll
        for (int off = 16; off > 0; off >>= 1) acc += __shfl_xor_sync(0xffffffffu, acc, off);
        if ((threadIdx.x & 31) == 0 && acc)
            atomicAdd(reinterpret_cast<unsigned long long*>(cs + f), (unsigned long long)acc);
    }
}

}  // namespace

aol_status_t launch_downscale_h(const int32_t* d_in, int32_t* d_out, int64_t planes, int64_t H, int64_t W,
                                cudaStream_t s) {
    DeviceInfo dev;
    aol_status_t st = device_info(&dev);
    if (st != AOL_OK) return st;
    const int64_t rows = planes * H;
    const int32_t reps = int32_t(W / 8);
    if (aligned16(d_in)) {
        const int block = std::min(256, (reps + 31) / 32 * 32);
        const int grid = int(std::min<int64_t>(rows, int64_t(dev.num_sms) * 16));
        downscale_h_kernel<<<grid, block, 0, s>>>(d_in, d_out, rows, int32_t(W), reps);
        AOL_LAUNCH_CHECK("downscale_h_kernel");
    } else {
        const int64_t total = rows * 3 * reps;
        const int grid = int(std::max<int64_t>(1, std::min<int64_t>((total + 255) / 256, int64_t(dev.num_sms) * 16)));
        downscale_h_scalar_kernel<<<grid, 256, 0, s>>>(d_in, d_out, rows, int32_t(W), reps);
        AOL_LAUNCH_CHECK("downscale_h_scalar_kernel");
    }
    return AOL_OK;
}

aol_status_t launch_downscale_v(const int32_t* d_in, int32_t* d_out, int64_t planes, int64_t H, int64_t W,
                                cudaStream_t s) {
    DeviceInfo dev;
    aol_status_t st = device_info(&dev);
    if (st != AOL_OK) return st;
    if (W % 4 == 0 && aligned16(d_in) && aligned16(d_out)) {
        const int64_t total = planes * ((H / 9 + kVBands - 1) / kVBands) * (W / 4);
        const int grid = int(std::max<int64_t>(1, std::min<int64_t>((total + 255) / 256, int64_t(dev.num_sms) * 16)));
        downscale_v_vec_kernel<<<grid, 256, 0, s>>>(d_in, d_out, planes, int32_t(H), int32_t(W));
        AOL_LAUNCH_CHECK("downscale_v_vec_kernel");
        return AOL_OK;
    }
    const int64_t total = planes * (H / 9) * W;
    const int grid = int(std::max<int64_t>(1, std::min<int64_t>((total + 255) / 256, int64_t(dev.num_sms) * 16)));
    downscale_v_kernel<<<grid, 256, 0, s>>>(d_in, d_out, planes, int32_t(H), int32_t(W));
    AOL_LAUNCH_CHECK("downscale_v_kernel");
    return AOL_OK;
}

aol_status_t launch_checksum(const int32_t* d_out, int64_t frames, int64_t per_frame, uint64_t* d_cs,
                             cudaStream_t s) {
    AOL_CUDA_TRY(cudaMemsetAsync(d_cs, 0, size_t(frames) * sizeof(uint64_t), s));
    if (frames == 0) return AOL_OK;
    DeviceInfo dev;
    aol_status_t st = device_info(&dev);
    if (st != AOL_OK) return st;
    const int64_t bx = std::max<int64_t>(1, std::min<int64_t>((per_frame + 255) / 256, 64));
    const int64_t by = std::min<int64_t>(frames, 65535);
    const dim3 grid{unsigned(bx), unsigned(by), 1u};
    checksum_kernel<<<grid, 256, 0, s>>>(d_out, frames, per_frame, d_cs);
    AOL_LAUNCH_CHECK("checksum_kernel");
    return AOL_OK;
}

}  // namespace aol
