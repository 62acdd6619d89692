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
 *        build/aol_example --enqueue-us [iters=2000]   (d1: host enqueue time of one single-HD-frame call,
 *                                                      plan launch vs aol_downscale_frame; one JSON line)
 */
#define _POSIX_C_SOURCE 199309L
#include <stdint.h>
#include <stdio.h>
#include <stdlib.h>
#include <string.h>
#include <time.h>

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

static double now_us(void) {
    struct timespec ts;
    clock_gettime(CLOCK_MONOTONIC, &ts);
    return ts.tv_sec * 1e6 + ts.tv_nsec * 1e-3;
}

/* SURVEY 8(d) d1's host side: microseconds the CPU spends enqueueing one single-HD-frame downscale, through a
 * persistent plan (one launch) and through aol_downscale_frame (planning + two launches).  The device is kept
 * busy by the stream itself; every 200 calls the stream is drained so the launch queue never fills. */
static int enqueue_us(int iters) {
    const int64_t N = 1, C = 3, H = 1080, W = 1920, Ho = 480, Wo = 720;
    int32_t *x, *z;
    uint64_t* cs;
    CHECK_CUDA(cudaMalloc((void**)&x, (size_t)(N * C * H * W) * 4));
    CHECK_CUDA(cudaMalloc((void**)&z, (size_t)(N * C * Ho * Wo) * 4));
    CHECK_CUDA(cudaMalloc((void**)&cs, 8));
    cudaStream_t s;
    CHECK_CUDA(cudaStreamCreate(&s));
    CHECK_AOL(aol_synth_frames(0, 0, N, C, H, W, 0, 0, AOL_I32, x, s));
    aol_frame_plan_t plan;
    CHECK_AOL(aol_frame_plan_create(x, AOL_I32, z, AOL_I32, N, C, H, W, NULL, &plan));
    double t_plan = 0, t_call = 0;
    for (int pass = 0; pass < 2; ++pass) {   /* pass 0 warms up */
        double tp = 0, tc = 0;
        for (int i = 0; i < iters; i += 200) {
            CHECK_CUDA(cudaStreamSynchronize(s));
            double t0 = now_us();
            for (int j = 0; j < 200; ++j) CHECK_AOL(aol_frame_plan_launch(plan, cs, s));
            tp += now_us() - t0;
            CHECK_CUDA(cudaStreamSynchronize(s));
            t0 = now_us();
            for (int j = 0; j < 200; ++j) CHECK_AOL(aol_downscale_frame(x, AOL_I32, z, N, C, H, W, cs, s));
            tc += now_us() - t0;
        }
        t_plan = tp / iters;
        t_call = tc / iters;
    }
    CHECK_CUDA(cudaStreamSynchronize(s));
    printf("{\"plan_launch_us\": %.3f, \"downscale_frame_us\": %.3f, \"iters\": %d}\n", t_plan, t_call, iters);
    CHECK_AOL(aol_frame_plan_destroy(plan));
    cudaFree(x); cudaFree(z); cudaFree(cs);
    cudaStreamDestroy(s);
    return 0;
}

int main(int argc, char** argv) {
    if (argc > 1 && strcmp(argv[1], "--enqueue-us") == 0) return enqueue_us(argc > 2 ? atoi(argv[2]) : 2000);
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

    /* a persistent plan of the same call: one launch per call; same outputs and checksums */
    uint64_t* cs3;
    CHECK_CUDA(cudaMalloc((void**)&cs3, (size_t)N * 8));
    aol_frame_plan_t plan;
    CHECK_AOL(aol_frame_plan_create(x, AOL_I32, z2, AOL_I32, N, C, H, W, NULL, &plan));
    CHECK_AOL(aol_frame_plan_launch(plan, cs3, s));
    CHECK_AOL(aol_frame_plan_launch(plan, cs3, s));
    CHECK_CUDA(cudaStreamSynchronize(s));
    CHECK_AOL(aol_frame_plan_destroy(plan));

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
    uint64_t* hcs3 = (uint64_t*)malloc((size_t)N * 8);
    CHECK_CUDA(cudaMemcpy(hcs3, cs3, (size_t)N * 8, cudaMemcpyDeviceToHost));
    const int same = memcmp(hz, hz2, out_elems * 4) == 0 && memcmp(hz, hz3, out_elems * 4) == 0 &&
                     memcmp(hcs, hcs2, (size_t)N * 8) == 0 && memcmp(hcs, hcs3, (size_t)N * 8) == 0;
    printf("aol %d: %lld frames %lldx%lld -> %lldx%lld, fused == unfused == generic == plan: %s\n", aol_version(),
           (long long)N, (long long)W, (long long)H, (long long)Wo, (long long)Ho, same ? "yes" : "NO");
    for (int64_t n = 0; n < N; ++n) printf("checksum %lld %llu\n", (long long)n, (unsigned long long)hcs[n]);

    /* an invalid call fails synchronously with a message and enqueues nothing */
    aol_status_t st = aol_downscale_frame(x, AOL_I32, z, N, C, H, W + 4, NULL, s);
    printf("invalid width -> status %d (%s)\n", (int)st, aol_last_error());

    free(hz); free(hz2); free(hz3); free(hcs); free(hcs2); free(hcs3);
    cudaFree(x); cudaFree(z); cudaFree(z2); cudaFree(z3); cudaFree(y); cudaFree(cs); cudaFree(cs2); cudaFree(cs3);
    cudaStreamDestroy(s);
    return same && st == AOL_E_SHAPE ? 0 : 2;
}
