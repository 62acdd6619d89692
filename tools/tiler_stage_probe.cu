// tiler_stage_probe.cu -- measurement tool (not part of libaol.so): is the d3 tiler gather bound by its
// access pattern or by the generic kernel?  Hard-coded d3 instance: array {64,1024,1024}
// int32, tiles[b][ty][tx][i][j] = A[b][8ty+i][8tx+j].
//   copy    : plain uint4 grid-stride copy of the same bytes (the roofline for this traffic)
//   direct  : uint4 per thread in array order, scattered 16-byte tile stores (what the generic kernel does)
//   staged  : one CTA per (b, ty) block of 32 KB: coalesced loads in array order into swizzled smem,
//             coalesced stores in tile order
// build: nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o build/tiler_stage_probe tools/tiler_stage_probe.cu
#include <cuda_runtime.h>

#include <cstdint>
#include <algorithm>
#include <cstdio>
#include <vector>

constexpr int B = 64, Y = 1024, X = 1024;
constexpr size_t N = size_t(B) * Y * X;   // elements
constexpr size_t NV = N / 4;              // uint4 vectors

__global__ void copy_kernel(const uint4* __restrict__ a, uint4* __restrict__ t) {
    for (size_t v = blockIdx.x * size_t(blockDim.x) + threadIdx.x; v < NV; v += size_t(gridDim.x) * blockDim.x)
        t[v] = a[v];
}

__global__ void direct_kernel(const uint4* __restrict__ a, uint4* __restrict__ t) {
    for (size_t v = blockIdx.x * size_t(blockDim.x) + threadIdx.x; v < NV; v += size_t(gridDim.x) * blockDim.x) {
        // array-order vector v: b, y, x/4
        const uint32_t xv = uint32_t(v % (X / 4)), y = uint32_t((v / (X / 4)) % Y), b = uint32_t(v / (size_t(Y) * X / 4));
        const uint32_t tx = xv >> 1, jh = xv & 1, ty = y >> 3, i = y & 7;
        const size_t o = ((((size_t(b) * 128 + ty) * 128 + tx) * 8 + i) * 2 + jh);
        t[o] = a[v];
    }
}

// One CTA iteration = one (b, ty) block: 8 array rows x 1024 = 2048 uint4, contiguous on both sides.
template <int kThreads>
__global__ void __launch_bounds__(kThreads) staged_kernel(const uint4* __restrict__ a, uint4* __restrict__ t) {
    __shared__ uint4 s[2048];
    constexpr int kPer = 2048 / kThreads;
    for (int blk = blockIdx.x; blk < B * 128; blk += gridDim.x) {
        const uint4* src = a + size_t(blk) * 2048;
        uint4* dst = t + size_t(blk) * 2048;
        uint4 v[kPer];
#pragma unroll
        for (int k = 0; k < kPer; ++k) v[k] = src[threadIdx.x + k * kThreads];
#pragma unroll
        for (int k = 0; k < kPer; ++k) {
            const int e = threadIdx.x + k * kThreads;   // array order: i = e / 256, c = e % 256 (c = 2 tx + jh)
            const int i = e >> 8, c = e & 255;
            s[(i << 8) | (c ^ (i << 1))] = v[k];
        }
        __syncthreads();
#pragma unroll
        for (int k = 0; k < kPer; ++k) {
            const int o = threadIdx.x + k * kThreads;   // tile order: tx = o / 16, i = (o / 2) % 8, jh = o % 2
            const int tx = o >> 4, i = (o >> 1) & 7, jh = o & 1;
            const int c = 2 * tx + jh;
            v[k] = s[(i << 8) | (c ^ (i << 1))];
        }
#pragma unroll
        for (int k = 0; k < kPer; ++k) dst[threadIdx.x + k * kThreads] = v[k];
        __syncthreads();
    }
}

int main() {
    uint4 *a, *t, *ref;
    cudaMalloc(&a, N * 4);
    cudaMalloc(&t, N * 4);
    cudaMalloc(&ref, N * 4);
    std::vector<int32_t> h(N);
    for (size_t k = 0; k < N; ++k) h[k] = int32_t(k * 2654435761u);
    cudaMemcpy(a, h.data(), N * 4, cudaMemcpyHostToDevice);
    int sms = 0;
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
    cudaEvent_t e0, e1;
    cudaEventCreate(&e0);
    cudaEventCreate(&e1);
    auto timeit = [&](const char* name, auto launch) {
        for (int w = 0; w < 3; ++w) launch();
        std::vector<float> ts;
        for (int r = 0; r < 20; ++r) {
            cudaEventRecord(e0);
            launch();
            cudaEventRecord(e1);
            cudaEventSynchronize(e1);
            float ms = 0;
            cudaEventElapsedTime(&ms, e0, e1);
            ts.push_back(ms);
        }
        std::sort(ts.begin(), ts.end());
        const float ms = ts[ts.size() / 2];
        printf("{\"case\": \"%s\", \"ms\": %.5f, \"GBps\": %.1f, \"err\": \"%s\"}\n", name, ms, 2.0 * N * 4 / (ms * 1e-3) / 1e9,
               cudaGetErrorString(cudaGetLastError()));
    };
    timeit("copy grid x8", [&] { copy_kernel<<<sms * 8, 256>>>(a, t); });
    timeit("copy grid x32", [&] { copy_kernel<<<sms * 32, 256>>>(a, t); });
    timeit("direct grid x32", [&] { direct_kernel<<<sms * 32, 256>>>(a, ref); });
    timeit("direct grid x128", [&] { direct_kernel<<<sms * 128, 256>>>(a, ref); });
    for (int mult : {4, 6, 8, 16, 56}) {
        char name[64];
        snprintf(name, sizeof name, "staged256 grid x%d", mult);
        timeit(name, [&] { staged_kernel<256><<<sms * mult, 256>>>(a, t); });
        snprintf(name, sizeof name, "staged512 grid x%d", mult);
        timeit(name, [&] { staged_kernel<512><<<sms * mult, 512>>>(a, t); });
    }
    std::vector<int32_t> h1(N), h2(N);
    cudaMemcpy(h1.data(), t, N * 4, cudaMemcpyDeviceToHost);
    cudaMemcpy(h2.data(), ref, N * 4, cudaMemcpyDeviceToHost);
    printf("{\"staged_equals_direct\": %s}\n", h1 == h2 ? "true" : "false");
    return 0;
}
