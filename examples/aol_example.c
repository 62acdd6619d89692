/*
 * aol_example.c -- using libaol.so from plain C through include/aol.h (no Python, no PyTorch).
 *
 * Generates N synthetic HD frames on the device, downscales them with the fused kernel
 * (aol_downscale_frame), the unfused H -> V route and the run-time generic filters, checks the
 * three agree, and prints the per-frame checksums (compared against the CPU oracle by
 * tests/test_gpu_example.py).
 *
 * build: gcc -std=c11 -O2 -I include -I /usr/local/cuda/include examples/aol_example.c \
 *            -L paper_conf_ipps_guortgbs11_b200 -laol -L /usr/local/cuda/lib64 -lcudart \
 *            -Wl,-rpath,$PWD/paper_conf_ipps_guortgbs11_b200 -o build/aol_example
 * run:   build/aol_example [frames=4] [seed=7]
 */
#include <stdint.h>
#include <stdio.h>
#include <stdlib.h>
#include <string.h>

#include <cuda_runtime_api.h>

#include "aol.h"

#define CHECK_AOL(call)                                                                      \
    do {                                                                                     \
        aol_status_t st__ = (call);                                                          \
        if (st__ != AOL_OK) {                                                                \
            fprintf(stderr, "%s failed: %d %s\n", #call, (int)st__, aol_last_error());     \
            return 1;                                                                        \
        }                                                                                    \
    } while (0)

#define CHECK_CUDA(call)                                                                     \
    do {                                                                                     \
        cudaError_t e__ = (call);                                                            \
        if (e__ != cudaSuccess) {                                                            \
            fprintf(stderr, "%s failed: %s\n", #call, cudaGetErrorString(e__));             \
            return 1;                                                                        \
        }                                                                                    \
    } while (0)

int main(int argc, char** argv) {
    const int64_t N = argc > 1 ? atoll(argv[1]) : 4, C = 3, H = 1080, W = 1920;
    const uint64_t seed = argc > 2 ? strtoull(argv[2], NULL, 10) : 7;
    const int64_t Ho = 4 * (H / 9), Wo = 3 * (W / 8);
    const size_t in_elems = (size_t)(N * C * H * W), out_elems = (size_t)(N * C * Ho * Wo);
    const size_t y_elems = (size_t)(N * C * H * Wo);

    int32_t *x, *z, *y, *z2, *z3;
    uint64_t *cs, *cs2;
    CHECK_CUDA(cudaMalloc((void**)&x, in_elems * 4));
    CHECK_CUDA(cudaMalloc((void**)&z, out_elems * 4));
    CHECK_CUDA(cudaMalloc((void**)&z2, out_elems * 4));
    CHECK_CUDA(cudaMalloc((void**)&z3, out_elems * 4));
    CHECK_CUDA(cudaMalloc((void**)&y, y_elems * 4));
    CHECK_CUDA(cudaMalloc((void**)&cs, (size_t)N * 8));
    CHECK_CUDA(cudaMalloc((void**)&cs2, (size_t)N * 8));
    cudaStream_t s;
    CHECK_CUDA(cudaStreamCreate(&s));

    /* frames 0..N-1 of the seeded synthetic stream (uniform [0,255]) */
    CHECK_AOL(aol_synth_frames(seed, 0, N, C, H, W, 0, 0, AOL_I32, x, s));

    /* fused: hf -> vf of Fig. 3 in one kernel, checksums fused */
    CHECK_AOL(aol_downscale_frame(x, AOL_I32, z, N, C, H, W, cs, s));

    /* unfused: the two filters alone, then the stand-alone checksum */
    CHECK_AOL(aol_downscale_h(x, y, N * C, H, W, s));
    CHECK_AOL(aol_downscale_v(y, z2, N * C, H, Wo, s));
    CHECK_AOL(aol_frame_checksum(z2, N, C, Ho, Wo, cs2, s));

    /* run-time generic repetitions with the paper's filter descriptions */
    aol_filter_t fh, fv;
    CHECK_AOL(aol_filter_preset(AOL_FILTER_H, N * C, H, W, &fh));
    CHECK_AOL(aol_filter_preset(AOL_FILTER_V, N * C, H, Wo, &fv));
    CHECK_AOL(aol_filter_apply(&fh, x, y, s));
    CHECK_AOL(aol_filter_apply(&fv, y, z3, s));
    CHECK_CUDA(cudaStreamSynchronize(s));

    int32_t* hz = (int32_t*)malloc(out_elems * 4);
    int32_t* hz2 = (int32_t*)malloc(out_elems * 4);
    int32_t* hz3 = (int32_t*)malloc(out_elems * 4);
    uint64_t* hcs = (uint64_t*)malloc((size_t)N * 8);
    uint64_t* hcs2 = (uint64_t*)malloc((size_t)N * 8);
    CHECK_CUDA(cudaMemcpy(hz, z, out_elems * 4, cudaMemcpyDeviceToHost));
    CHECK_CUDA(cudaMemcpy(hz2, z2, out_elems * 4, cudaMemcpyDeviceToHost));
    CHECK_CUDA(cudaMemcpy(hz3, z3, out_elems * 4, cudaMemcpyDeviceToHost));
    CHECK_CUDA(cudaMemcpy(hcs, cs, (size_t)N * 8, cudaMemcpyDeviceToHost));
    CHECK_CUDA(cudaMemcpy(hcs2, cs2, (size_t)N * 8, cudaMemcpyDeviceToHost));
    const int same = memcmp(hz, hz2, out_elems * 4) == 0 && memcmp(hz, hz3, out_elems * 4) == 0 &&
                     memcmp(hcs, hcs2, (size_t)N * 8) == 0;
    printf("aol %d: %lld frames %lldx%lld -> %lldx%lld, fused == unfused == generic: %s\n", aol_version(),
           (long long)N, (long long)W, (long long)H, (long long)Wo, (long long)Ho, same ? "yes" : "NO");
    for (int64_t n = 0; n < N; ++n) printf("checksum %lld %llu\n", (long long)n, (unsigned long long)hcs[n]);

    /* an invalid call fails synchronously with a message and enqueues nothing */
    aol_status_t st = aol_downscale_frame(x, AOL_I32, z, N, C, H, W + 4, NULL, s);
    printf("invalid width -> status %d (%s)\n", (int)st, aol_last_error());

    free(hz); free(hz2); free(hz3); free(hcs); free(hcs2);
    cudaFree(x); cudaFree(z); cudaFree(z2); cudaFree(z3); cudaFree(y); cudaFree(cs); cudaFree(cs2);
    cudaStreamDestroy(s);
    return same && st == AOL_E_SHAPE ? 0 : 2;
}
