/*
 * synth.c -- the seeded synthetic frame generator of synth/__init__.py, in plain C
 * with OpenMP, so that host-side inputs for the oracle at bench size (300 HD frames,
 * 1.87 G samples) take a fraction of a second instead of numpy's minutes.
 *
 * Holds NO arithmetic of the method: it only produces input samples.  It stands in for
 * the paper's FrameGenerator IP, which reads real video through OpenCV (PAPER.md
 * P:L657-659; the videos are unnamed, so synthetic frames replace them).
 *
 *   counter(seed, n, c, y, x) = seed * PHI + ((n*C + c)*H + y)*W + x      (mod 2^64)
 *   u = splitmix64(counter)
 *   kind 0 uniform u >> 56 | 1 dark u >> 61 | 2 signed (u >> 37) - 2^26 | 3 ramp x | 4 constant value
 *
 * Frame n of the output holds the content of global frame index[n] (index == NULL:
 * frame0 + n), so a device-pool slot or a sampled frame regenerates exactly the frame
 * the stream holds.  tests/test_synth.py checks this against the numpy generator.
 */
#include <stdint.h>

#ifdef _OPENMP
#include <omp.h>
#endif

#define PHI 0x9E3779B97F4A7C15ull

static inline uint64_t splitmix64(uint64_t z) {
    z += PHI;
    z = (z ^ (z >> 30)) * 0xBF58476D1CE4E5B9ull;
    z = (z ^ (z >> 27)) * 0x94D049BB133111EBull;
    return z ^ (z >> 31);
}

/* out: int32 (elsize 4) or uint8 (elsize 1) [nframes][channels][H][W].  Returns 0, or -1 on bad input. */
int synth_frames_c(uint64_t seed, int64_t frame0, const int64_t* index, int64_t nframes, int64_t channels,
                   int64_t H, int64_t W, int kind, int32_t value, int elsize, void* out, int nthreads) {
    if (!out || nframes < 0 || channels <= 0 || H <= 0 || W <= 0 || kind < 0 || kind > 4) return -1;
    if (elsize != 4 && elsize != 1) return -1;
    const int64_t rows = nframes * channels * H;
    const uint64_t base = seed * PHI;
    (void)nthreads;
#ifdef _OPENMP
#pragma omp parallel for schedule(static) num_threads(nthreads > 0 ? nthreads : 1)
#endif
    for (int64_t row = 0; row < rows; ++row) {
        const int64_t y = row % H, pc = row / H, c = pc % channels, n = pc / channels;
        const int64_t g = index ? index[n] : frame0 + n;
        const uint64_t ctr0 = base + (uint64_t)(((g * channels + c) * H + y) * W);
        int32_t* o32 = (int32_t*)out + row * W;
        uint8_t* o8 = (uint8_t*)out + row * W;
        for (int64_t x = 0; x < W; ++x) {
            int32_t v;
            switch (kind) {
            case 0: v = (int32_t)(splitmix64(ctr0 + (uint64_t)x) >> 56); break;
            case 1: v = (int32_t)(splitmix64(ctr0 + (uint64_t)x) >> 61); break;
            case 2: v = (int32_t)((int64_t)(splitmix64(ctr0 + (uint64_t)x) >> 37) - ((int64_t)1 << 26)); break;
            case 3: v = (int32_t)x; break;
            default: v = value; break;
            }
            if (elsize == 4) o32[x] = v;
            else o8[x] = (uint8_t)v;
        }
    }
    return 0;
}

int synth_max_threads(void) {
#ifdef _OPENMP
    return omp_get_max_threads();
#else
    return 1;
#endif
}
