// tiler.cu -- K-1 generic ArrayOL tiler gather and K-2 scatter (any rank <= 8,
// element size 1/2/4/8 bytes, Euclidean modulo).
//
//   gather : tiles[r][i]  = array[(o + P.r + F.i) mod s]     (Section IV, Fig. 4)
//   scatter: array[(o + P.r + F.i) mod s] = tiles[r][i]      (Fig. 6, modarray P:L479)
//
// The host reduces o, P and F modulo the array extents once (so every partial
// sum is non-negative) and validates that no sum can overflow int64.  Each
// thread handles a run of kRun consecutive tile elements: it decomposes the
// run's first flat index once, then walks the innermost pattern dimension
// with an incremental (add, conditional subtract) update of every array
// coordinate -- the tiler analogue of Fig. 11's inner `tl[0]` loop, without a
// modulo per element.  Tile-side accesses are contiguous per thread.
#include <cuda_runtime.h>

#include <algorithm>
#include <cstdint>

#include "common.h"

namespace aol {

namespace {

constexpr int kRun = 8;

template <int ES>
struct Elem;
template <>
struct Elem<1> {
    using T = uint8_t;
};
template <>
struct Elem<2> {
    using T = uint16_t;
};
template <>
struct Elem<4> {
    using T = uint32_t;
};
template <>
struct Elem<8> {
    using T = unsigned long long;
};

struct Walker {
    int64_t idx[2 * AOL_MAX_RANK];
    int64_t c[AOL_MAX_RANK];

    __device__ __forceinline__ void seek(const TilerDev& td, int64_t g) {
        for (int d = td.nd - 1; d >= 0; --d) {
            const int64_t e = td.ext[d];
            const int64_t q = g / e;
            idx[d] = g - q * e;
            g = q;
        }
        recompute(td);
    }
    __device__ __forceinline__ void recompute(const TilerDev& td) {
        for (int a = 0; a < td.ra; ++a) {
            int64_t v = td.org[a];
            for (int d = 0; d < td.nd; ++d) v += td.coef[a][d] * idx[d];
            c[a] = v % td.ashape[a];  // all terms non-negative: plain modulo == Euclidean
        }
    }
    __device__ __forceinline__ int64_t offset(const TilerDev& td) const {
        int64_t off = 0;
        for (int a = 0; a < td.ra; ++a) off += c[a] * td.astride[a];
        return off;
    }
    __device__ __forceinline__ void advance(const TilerDev& td) {
        if (td.nd == 0) return;
        const int last = td.nd - 1;
        if (++idx[last] < td.ext[last]) {
            for (int a = 0; a < td.ra; ++a) {
                int64_t v = c[a] + td.coef[a][last];
                if (v >= td.ashape[a]) v -= td.ashape[a];
                c[a] = v;
            }
            return;
        }
        idx[last] = 0;
        int d = last - 1;
        while (d >= 0 && ++idx[d] == td.ext[d]) {
            idx[d] = 0;
            --d;
        }
        recompute(td);
    }
};

template <int ES>
__global__ void __launch_bounds__(256) gather_kernel(const TilerDev td, const void* __restrict__ array,
                                                     void* __restrict__ tiles) {
    using T = typename Elem<ES>::T;
    const T* A = static_cast<const T*>(array);
    T* G = static_cast<T*>(tiles);
    const int64_t nruns = (td.total + kRun - 1) / kRun;
    for (int64_t run = int64_t(blockIdx.x) * blockDim.x + threadIdx.x; run < nruns;
         run += int64_t(gridDim.x) * blockDim.x) {
        const int64_t g0 = run * kRun;
        const int n = (td.total - g0 < kRun) ? int(td.total - g0) : kRun;
        Walker w;
        w.seek(td, g0);
        T v[kRun];
#pragma unroll
        for (int k = 0; k < kRun; ++k) {
            if (k < n) {
                v[k] = A[w.offset(td)];
                if (k + 1 < n) w.advance(td);
            }
        }
#pragma unroll
        for (int k = 0; k < kRun; ++k)
            if (k < n) G[g0 + k] = v[k];
    }
}

// mode 0: FAST (injective, plain stores); mode 1: SEQUENTIAL pass 1 (claim: max
// flat index + 1 per target); mode 2: SEQUENTIAL pass 2 (write if we are the claim).
template <int ES, int MODE>
__global__ void __launch_bounds__(256) scatter_kernel(const TilerDev td, const void* __restrict__ tiles,
                                                      void* __restrict__ array, unsigned long long* __restrict__ ws) {
    using T = typename Elem<ES>::T;
    const T* G = static_cast<const T*>(tiles);
    T* A = static_cast<T*>(array);
    const int64_t nruns = (td.total + kRun - 1) / kRun;
    for (int64_t run = int64_t(blockIdx.x) * blockDim.x + threadIdx.x; run < nruns;
         run += int64_t(gridDim.x) * blockDim.x) {
        const int64_t g0 = run * kRun;
        const int n = (td.total - g0 < kRun) ? int(td.total - g0) : kRun;
        Walker w;
        w.seek(td, g0);
#pragma unroll
        for (int k = 0; k < kRun; ++k) {
            if (k < n) {
                const int64_t off = w.offset(td);
                const unsigned long long tag = (unsigned long long)(g0 + k) + 1ull;
                if (MODE == 0) {
                    A[off] = G[g0 + k];
                } else if (MODE == 1) {
                    atomicMax(ws + off, tag);
                } else {
                    if (ws[off] == tag) A[off] = G[g0 + k];
                }
                if (k + 1 < n) w.advance(td);
            }
        }
    }
}

int grid_for(int64_t total, int num_sms) {
    const int64_t runs = (total + kRun - 1) / kRun;
    return int(std::max<int64_t>(1, std::min<int64_t>((runs + 255) / 256, int64_t(num_sms) * 16)));
}

template <int ES>
aol_status_t gather_es(const TilerDev& td, const void* a, void* t, int grid, cudaStream_t s) {
    gather_kernel<ES><<<grid, 256, 0, s>>>(td, a, t);
    AOL_LAUNCH_CHECK("gather_kernel");
    return AOL_OK;
}

template <int ES>
aol_status_t scatter_es(const TilerDev& td, const void* t, void* a, int seq, void* ws, int grid, cudaStream_t s) {
    auto* w = static_cast<unsigned long long*>(ws);
    if (!seq) {
        scatter_kernel<ES, 0><<<grid, 256, 0, s>>>(td, t, a, w);
        AOL_LAUNCH_CHECK("scatter_kernel");
        return AOL_OK;
    }
    AOL_CUDA_TRY(cudaMemsetAsync(ws, 0, size_t(td.array_elems) * 8, s));
    scatter_kernel<ES, 1><<<grid, 256, 0, s>>>(td, t, a, w);
    AOL_LAUNCH_CHECK("scatter_kernel(claim)");
    scatter_kernel<ES, 2><<<grid, 256, 0, s>>>(td, t, a, w);
    AOL_LAUNCH_CHECK("scatter_kernel(write)");
    return AOL_OK;
}

}  // namespace

aol_status_t launch_gather(const TilerDev& td, int elsize, const void* d_array, void* d_tiles, cudaStream_t s) {
    if (td.total == 0) return AOL_OK;
    DeviceInfo dev;
    aol_status_t st = device_info(&dev);
    if (st != AOL_OK) return st;
    const int grid = grid_for(td.total, dev.num_sms);
    switch (elsize) {
        case 1: return gather_es<1>(td, d_array, d_tiles, grid, s);
        case 2: return gather_es<2>(td, d_array, d_tiles, grid, s);
        case 4: return gather_es<4>(td, d_array, d_tiles, grid, s);
        case 8: return gather_es<8>(td, d_array, d_tiles, grid, s);
    }
    return fail(AOL_E_DTYPE, "element size must be 1, 2, 4 or 8 bytes");
}

aol_status_t launch_scatter(const TilerDev& td, int elsize, const void* d_tiles, void* d_array, int sequential,
                            void* d_ws, cudaStream_t s) {
    if (td.total == 0) return AOL_OK;
    DeviceInfo dev;
    aol_status_t st = device_info(&dev);
    if (st != AOL_OK) return st;
    const int grid = grid_for(td.total, dev.num_sms);
    switch (elsize) {
        case 1: return scatter_es<1>(td, d_tiles, d_array, sequential, d_ws, grid, s);
        case 2: return scatter_es<2>(td, d_tiles, d_array, sequential, d_ws, grid, s);
        case 4: return scatter_es<4>(td, d_tiles, d_array, sequential, d_ws, grid, s);
        case 8: return scatter_es<8>(td, d_tiles, d_array, sequential, d_ws, grid, s);
    }
    return fail(AOL_E_DTYPE, "element size must be 1, 2, 4 or 8 bytes");
}

}  // namespace aol
