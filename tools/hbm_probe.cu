// hbm_probe.cu -- measurement tool (not part of libaol.so): the best HBM rate this B200 reaches for the
// downscaler's traffic mix with an idealised TMA streamer, to put the fused kernel's number in context.
//
// Each persistent CTA streams its share of a read buffer through an S-stage ring of 1-D bulk copies
// (one thread issues and waits -- no compute), and for every 1000 bytes read it bulk-stores `wpm` bytes
// from smem to a write buffer.  wpm = 166 reproduces the int32 kernel's 7.465 GB : 1.244 GB mix; the uint8
// kernel reads 1.866 GB and writes 1.244 GB (wpm = 666) or 0.622 GB with int16 outputs (wpm = 333).
//
// build: nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o build/hbm_probe tools/hbm_probe.cu
// run:   build/hbm_probe [i32|u8]   (prints one JSON line per configuration)
#include <cuda_runtime.h>

#include <cstdint>
#include <cstdio>
#include <string>
#include <vector>

__device__ __forceinline__ uint32_t sa(const void* p) { return uint32_t(__cvta_generic_to_shared(p)); }

__global__ void __launch_bounds__(32) stream_kernel(const uint8_t* __restrict__ src, uint8_t* __restrict__ dst,
                                                    size_t read_bytes, size_t chunk, int stages, int wpm,
                                                    int inter) {
    extern __shared__ __align__(1024) uint8_t smem[];
    uint64_t* bar = reinterpret_cast<uint64_t*>(smem + size_t(stages) * chunk);
    if (threadIdx.x != 0) return;
    for (int s = 0; s < stages; ++s)
        asm volatile("mbarrier.init.shared::cta.b64 [%0], 1;" ::"r"(sa(&bar[s])));
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
    const size_t nchunks = read_bytes / chunk;
    const size_t per = (nchunks + gridDim.x - 1) / gridDim.x;
    const size_t b0 = blockIdx.x * per, b1 = b0 + per < nchunks ? b0 + per : nchunks;
    // inter = 0: a contiguous block of chunks per CTA; 1: chunk k of this CTA is blockIdx.x + k * gridDim.x
    // (round-robin, like the fused kernel's work units: concurrently running CTAs read adjacent chunks)
    const size_t c0 = 0;
    const size_t c1 = inter ? (blockIdx.x < nchunks ? (nchunks - blockIdx.x + gridDim.x - 1) / gridDim.x : 0)
                            : (b1 > b0 ? b1 - b0 : 0);
    auto at = [&](size_t k) { return inter ? blockIdx.x + k * gridDim.x : b0 + k; };
    const uint32_t wb = uint32_t(chunk * wpm / 1000) & ~15u;
    uint32_t phase[64] = {0};
    size_t issued = c0;
    // prologue: fill the ring
    for (int s = 0; s < stages && issued < c1; ++s, ++issued) {
        asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(sa(&bar[s])), "r"(uint32_t(chunk))
                     : "memory");
        asm volatile("cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];" ::"r"(
                         sa(smem + size_t(s) * chunk)),
                     "l"(src + at(issued) * chunk), "r"(uint32_t(chunk)), "r"(sa(&bar[s]))
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
        if (wpm > 0) {   // write chunk*wpm/1000 bytes of what just arrived
            asm volatile("cp.async.bulk.global.shared::cta.bulk_group [%0], [%1], %2;" ::"l"(dst + at(c) * wb),
                         "r"(sa(smem + size_t(s) * chunk)), "r"(wb)
                         : "memory");
            asm volatile("cp.async.bulk.commit_group;" ::: "memory");
            asm volatile("cp.async.bulk.wait_group.read 0;" ::: "memory");
        }
        if (issued < c1) {
            asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(sa(&bar[s])),
                         "r"(uint32_t(chunk))
                         : "memory");
            asm volatile(
                "cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];" ::"r"(
                    sa(smem + size_t(s) * chunk)),
                "l"(src + at(issued) * chunk), "r"(uint32_t(chunk)), "r"(sa(&bar[s]))
                : "memory");
            ++issued;
        }
        if (++s == stages) s = 0;
    }
    asm volatile("cp.async.bulk.wait_group 0;" ::: "memory");
}

int main(int argc, char** argv) {
    const bool u8 = argc > 1 && std::string(argv[1]) == "u8";
    // the 300-frame HD input: int32 7.465 GB, uint8 1.866 GB
    const size_t read_bytes = size_t(u8 ? 1866240000ull : 7464960000ull) / 1024 * 1024;
    uint8_t *src, *dst;
    cudaMalloc(&src, read_bytes);
    cudaMalloc(&dst, read_bytes);
    cudaMemset(src, 1, read_bytes);
    int sms = 0;
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
    cudaFuncSetAttribute(stream_kernel, cudaFuncAttributeMaxDynamicSharedMemorySize, 200 * 1024);
    cudaEvent_t a, b;
    cudaEventCreate(&a);
    cudaEventCreate(&b);
    struct Cfg { size_t chunk; int stages, wpm, cps, inter = 0; };
    std::vector<Cfg> cfgs;
    if (argc > 1 && std::string(argv[1]) == "inter") {
        // blocked vs round-robin chunk order, int32 mix (166) and read-only, around the fused kernel's point
        for (int inter : {0, 1})
            for (int wpm : {166, 0})
                for (size_t chunk : {size_t(16384), size_t(23040)})
                    for (int stages : {4, 5, 6})
                        for (int cps : {1, 2})
                            if (chunk * stages * cps + 1024 * cps <= 220 * 1024) cfgs.push_back({chunk, stages, wpm, cps, inter});
    } else if (!u8) {
        for (int wpm : {166, 0})
            for (size_t chunk : {size_t(16384), size_t(23040), size_t(32768)})
                for (int stages : {2, 4, 6, 8})
                    for (int cps : {1, 2})
                        if (chunk * stages * cps + 1024 * cps <= 220 * 1024) cfgs.push_back({chunk, stages, wpm, cps});
    } else {
        // uint8 triples are 5760 B (HD); 2 or 3 triples per copy model a wider per-stage footprint
        for (int wpm : {666, 333})
            for (size_t chunk : {size_t(5760), size_t(11520), size_t(17280)})
                for (int inflight_kb : {48, 96, 144})
                    for (int cps : {1, 2, 3, 4}) {
                        const int stages = int(inflight_kb * 1024 / cps / chunk);
                        if (stages >= 2 && stages <= 64 && chunk * stages * cps + 1024 * cps <= 220 * 1024)
                            cfgs.push_back({chunk, stages, wpm, cps});
                    }
    }
    for (const Cfg& c : cfgs) {
        const int smem = int(c.chunk * c.stages + 64 * 8);
        cudaFuncSetAttribute(stream_kernel, cudaFuncAttributeMaxDynamicSharedMemorySize, smem);
        const int grid = sms * c.cps;
        for (int w = 0; w < 2; ++w) stream_kernel<<<grid, 32, smem>>>(src, dst, read_bytes, c.chunk, c.stages, c.wpm, c.inter);
        cudaEventRecord(a);
        const int reps = 10;
        for (int r = 0; r < reps; ++r) stream_kernel<<<grid, 32, smem>>>(src, dst, read_bytes, c.chunk, c.stages, c.wpm, c.inter);
        cudaEventRecord(b);
        cudaEventSynchronize(b);
        float ms = 0;
        cudaEventElapsedTime(&ms, a, b);
        ms /= reps;
        const double bytes = double(read_bytes) + double(read_bytes) * c.wpm / 1000.0;
        printf("{\"chunk\": %zu, \"stages\": %d, \"ctas_per_sm\": %d, \"write_permille\": %d, \"interleaved\": %d, "
               "\"ms\": %.4f, \"GBps\": %.1f, \"err\": \"%s\"}\n",
               c.chunk, c.stages, c.cps, c.wpm, c.inter, ms, bytes / (ms * 1e-3) / 1e9, cudaGetErrorString(cudaGetLastError()));
    }
    return 0;
}
