// hbm_probe.cu -- measurement tool (not part of libaol.so): the best HBM rate this B200 reaches for the
// downscaler's traffic mix with an idealised TMA streamer, to put the fused kernel's number in context.
//
// Each persistent CTA streams its share of a read buffer through an S-stage ring of 1-D bulk copies
// (one thread issues and waits -- no compute), and for every `ratio` bytes read it bulk-stores one byte's
// worth from smem to a write buffer.  ratio = 6 reproduces the fused kernel's 7.465 GB : 1.244 GB mix.
//
// build: nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o build/hbm_probe tools/hbm_probe.cu
// run:   build/hbm_probe   (prints one JSON line per configuration)
#include <cuda_runtime.h>

#include <cstdint>
#include <cstdio>
#include <vector>

__device__ __forceinline__ uint32_t sa(const void* p) { return uint32_t(__cvta_generic_to_shared(p)); }

__global__ void __launch_bounds__(32) stream_kernel(const uint8_t* __restrict__ src, uint8_t* __restrict__ dst,
                                                    size_t read_bytes, size_t chunk, int stages, int ratio) {
    extern __shared__ __align__(1024) uint8_t smem[];
    uint64_t* bar = reinterpret_cast<uint64_t*>(smem + size_t(stages) * chunk);
    if (threadIdx.x != 0) return;
    for (int s = 0; s < stages; ++s)
        asm volatile("mbarrier.init.shared::cta.b64 [%0], 1;" ::"r"(sa(&bar[s])));
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
    const size_t nchunks = read_bytes / chunk;
    const size_t per = (nchunks + gridDim.x - 1) / gridDim.x;
    const size_t c0 = blockIdx.x * per, c1 = c0 + per < nchunks ? c0 + per : nchunks;
    uint32_t phase[64] = {0};
    size_t wr = ratio ? (c0 * chunk / ratio) & ~size_t(15) : 0;   // this CTA slice of the write buffer (16 B aligned)
    size_t issued = c0;
    // prologue: fill the ring
    for (int s = 0; s < stages && issued < c1; ++s, ++issued) {
        asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(sa(&bar[s])), "r"(uint32_t(chunk))
                     : "memory");
        asm volatile("cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];" ::"r"(
                         sa(smem + size_t(s) * chunk)),
                     "l"(src + issued * chunk), "r"(uint32_t(chunk)), "r"(sa(&bar[s]))
                     : "memory");
    }
    int s = 0;
    for (size_t c = c0; c < c1; ++c) {
        uint32_t ok = 0;
        while (!ok)
            asm volatile("{ .reg .pred p; mbarrier.try_wait.parity.shared::cta.b64 p, [%1], %2; selp.u32 %0, 1, 0, p; }"
                         : "=r"(ok)
                         : "r"(sa(&bar[s])), "r"(phase[s])
                         : "memory");
        phase[s] ^= 1u;
        if (ratio > 0) {   // write chunk/ratio bytes of what just arrived
            const uint32_t wb = uint32_t(chunk / ratio) & ~15u;
            asm volatile("cp.async.bulk.global.shared::cta.bulk_group [%0], [%1], %2;" ::"l"(dst + wr),
                         "r"(sa(smem + size_t(s) * chunk)), "r"(wb)
                         : "memory");
            asm volatile("cp.async.bulk.commit_group;" ::: "memory");
            asm volatile("cp.async.bulk.wait_group.read 0;" ::: "memory");
            wr += wb;
        }
        if (issued < c1) {
            asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(sa(&bar[s])),
                         "r"(uint32_t(chunk))
                         : "memory");
            asm volatile(
                "cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];" ::"r"(
                    sa(smem + size_t(s) * chunk)),
                "l"(src + issued * chunk), "r"(uint32_t(chunk)), "r"(sa(&bar[s]))
                : "memory");
            ++issued;
        }
        if (++s == stages) s = 0;
    }
    asm volatile("cp.async.bulk.wait_group 0;" ::: "memory");
}

int main() {
    const size_t read_bytes = size_t(7464960000ull) / 1024 * 1024;   // the 300-frame HD int32 input
    uint8_t *src, *dst;
    cudaMalloc(&src, read_bytes);
    cudaMalloc(&dst, read_bytes / 4);
    cudaMemset(src, 1, read_bytes);
    int sms = 0;
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
    cudaFuncSetAttribute(stream_kernel, cudaFuncAttributeMaxDynamicSharedMemorySize, 200 * 1024);
    cudaEvent_t a, b;
    cudaEventCreate(&a);
    cudaEventCreate(&b);
    struct Cfg { size_t chunk; int stages, ratio, cps; };
    std::vector<Cfg> cfgs;
    for (int ratio : {6, 0})
        for (size_t chunk : {size_t(16384), size_t(23040), size_t(32768)})
            for (int stages : {2, 4, 6, 8})
                for (int cps : {1, 2})
                    if (chunk * stages * cps + 1024 * cps <= 220 * 1024) cfgs.push_back({chunk, stages, ratio, cps});
    for (const Cfg& c : cfgs) {
        const int smem = int(c.chunk * c.stages + 64 * 8);
        cudaFuncSetAttribute(stream_kernel, cudaFuncAttributeMaxDynamicSharedMemorySize, smem);
        const int grid = sms * c.cps;
        for (int w = 0; w < 2; ++w) stream_kernel<<<grid, 32, smem>>>(src, dst, read_bytes, c.chunk, c.stages, c.ratio);
        cudaEventRecord(a);
        const int reps = 10;
        for (int r = 0; r < reps; ++r) stream_kernel<<<grid, 32, smem>>>(src, dst, read_bytes, c.chunk, c.stages, c.ratio);
        cudaEventRecord(b);
        cudaEventSynchronize(b);
        float ms = 0;
        cudaEventElapsedTime(&ms, a, b);
        ms /= reps;
        const double bytes = double(read_bytes) + (c.ratio ? double(read_bytes / c.ratio) : 0.0);
        printf("{\"chunk\": %zu, \"stages\": %d, \"ctas_per_sm\": %d, \"write_ratio\": %d, \"ms\": %.4f, \"GBps\": %.1f, "
               "\"err\": \"%s\"}\n",
               c.chunk, c.stages, c.cps, c.ratio, ms, bytes / (ms * 1e-3) / 1e9, cudaGetErrorString(cudaGetLastError()));
    }
    return 0;
}
