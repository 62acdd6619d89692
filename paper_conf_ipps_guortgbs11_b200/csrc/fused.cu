// fused.cu -- K-5: the fused HD->SD downscaler (hf -> vf of Fig. 3 in one kernel).
//
// What it computes: per plane X[H][W] (one colour channel)
//   H stage  (Fig. 10 tilers P:L681-694, Fig. 5 task P:L435-446):
//     Y[y][3r+k] = T( sum_{t<6} X[y][(8r + s_k + t) mod W] ),  s = (0,2,5)
//   V stage  (reading Z1/Z2):
//     Z[4b+k][x] = T( sum_{t<6} Y[(9b + 2k + t) mod H][x] )
//   T(S) = S/6 - S%6 (C int semantics)  ==  7*(S/6) - S.
// Y never touches HBM: the hand-written analogue of SaC's WITH-loop folding
// (P:L528-546), in one launch instead of the 5 + 7 generator kernels
// SaC-CUDA produced.
//
// Design (B200, sm_100a):
//  * Work unit = (plane, run of `bands_per_unit` 9-row bands).  A unit streams
//    3*nb + 1 "triples" of full-width rows: first the 3 halo rows (the next
//    unit's first rows, or rows 0..2 for the plane's last band -- the toroidal
//    wrap of the V tiler), then its own 9*nb rows.  Loading the halo first
//    makes it coincide with the neighbouring CTA's read of the same rows (an
//    L2 hit instead of a second HBM read).  Persistent CTAs walk units
//    round-robin.
//  * One producer warp issues 3-D TMA tile loads (box = 3 rows x W int32,
//    SWIZZLE_128B) into an S-stage smem ring guarded by full/empty mbarriers.
//  * Consumer thread r owns repetition r (8 input columns -> 3 Y columns): two
//    conflict-free 128-bit LDS per row (the 128B swizzle spreads the 32-byte
//    per-thread stride over all banks) and ONE warp shuffle for the 3-column
//    pattern overlap (Fig. 10 pattern {11} vs paving step 8); lane 31 and the
//    row-wrapping repetition read the neighbour chunk from smem instead.
//  * The V stage is a running register accumulation over the band's rows
//    (4 outputs x 3 columns per thread), so every input row is read once.
//  * Each finished band (4 output rows, contiguous in Z) is staged in smem and
//    written by one 1-D TMA bulk store; the per-frame checksum is folded in
//    registers and added with one atomic per warp per unit.
#include <cuda.h>
#include <cuda_runtime.h>

#include <algorithm>
#include <cstdint>

#include "common.h"
#include "ptx.cuh"

namespace aol {

namespace {

constexpr int kMaxStages = 16;
constexpr int kMaxConsumers = 992;  // + 1 producer warp = 1024 threads
// Output staging buffers (4 output rows each).  One suffices: the bulk store of a
// band has long finished reading smem by the time the next band (3 triples
// later) is emitted, and the saved space buys one more ring stage.
constexpr int kOutBufs = 1;
// Bytes of TMA loads to keep in flight per SM (see plan_fused).
constexpr int kInflightBytesPerSM = 6 * 23552;

__device__ __forceinline__ int32_t task_T(int32_t S) {
    // Fig. 5: tmp/6 - tmp%6 == 7*(tmp/6) - tmp for C truncating division.
    return 7 * (S / 6) - S;
}

struct FusedArgs {
    int32_t* Z;
    uint64_t* cs;
    int64_t nunits;
    int32_t H, W, Ho, Wo;
    int32_t channels;
    int32_t reps;               // W/8  repetitions of the H tiler per row
    int32_t segs;               // W/32 128-byte segments per row
    int32_t triples_per_plane;  // H/3
    int32_t nbands;             // H/9
    int32_t bands_per_unit;
    int32_t units_per_plane;
    int32_t stages;
    uint32_t stage_bytes;   // 12*W
    uint32_t stage_stride;  // stage_bytes rounded up to 1024 (swizzle atom)
    uint32_t out_bytes;     // 16*Wo  (4 output rows)
    int32_t n_consumer;     // consumer threads, multiple of 32
    int32_t halo_last;      // 1: stream the halo triple after the unit's own rows
};

// Byte offset of 16-byte chunk `chunk` (0..7) of 128-byte line `line` under SWIZZLE_128B
// (chunk index XOR line index mod 8; stage buffers are 1024-byte aligned).
__device__ __forceinline__ uint32_t swz(uint32_t line, uint32_t chunk) {
    return (line << 7) | (((chunk ^ line) & 7u) << 4);
}

template <bool kChecksum, int kMaxThreads, int kMinBlocks>
__global__ void __launch_bounds__(kMaxThreads, kMinBlocks)
    fused_tma_kernel(const __grid_constant__ CUtensorMap tmap, const FusedArgs a) {
    extern __shared__ uint8_t smem_raw[];
    uint8_t* smem = reinterpret_cast<uint8_t*>((reinterpret_cast<uintptr_t>(smem_raw) + 1023) & ~uintptr_t(1023));
    uint8_t* stage_base = smem;
    int32_t* outbuf = reinterpret_cast<int32_t*>(smem + size_t(a.stages) * a.stage_stride);
    uint64_t* full = reinterpret_cast<uint64_t*>(smem + size_t(a.stages) * a.stage_stride + kOutBufs * a.out_bytes);
    uint64_t* empty = full + a.stages;

    const int tid = threadIdx.x;
    const int NC = a.n_consumer;
    if (tid == 0) {
        for (int s = 0; s < a.stages; ++s) {
            ptx::mbar_init(&full[s], 1);
            ptx::mbar_init(&empty[s], NC / 32);
        }
        ptx::fence_mbar_init();
    }
    __syncthreads();

    if (tid >= NC) {
        // ------------------------------------------------ producer warp (TMA)
        if (tid == NC) {
            ptx::prefetch_tensormap(&tmap);
            int s = 0;
            uint32_t ph = 0;
            for (int64_t u = blockIdx.x; u < a.nunits; u += gridDim.x) {
                const int64_t plane = u / a.units_per_plane;
                const int32_t b0 = int32_t(u - plane * a.units_per_plane) * a.bands_per_unit;
                const int32_t b1 = min(b0 + a.bands_per_unit, a.nbands);
                const int32_t ntrip = 3 * (b1 - b0) + 1;
                const int32_t row0 = int32_t(plane) * a.H;
                // halo triple first: rows 9*b1 .. 9*b1+2 (mod H -- the V tiler's toroidal wrap for the
                // last band).  They are the first rows of the NEXT unit, which a neighbouring CTA
                // streams at the same moment, so the second read hits L2 instead of HBM.
                const int32_t halo = (3 * b1 == a.triples_per_plane) ? 0 : 3 * b1;
                for (int32_t t = 0; t < ntrip; ++t) {
                    const int32_t trip = a.halo_last ? (t == ntrip - 1 ? halo : 3 * b0 + t)
                                                     : (t == 0 ? halo : 3 * b0 + t - 1);
                    ptx::mbar_wait(&empty[s], ph ^ 1u);
                    ptx::mbar_arrive_expect_tx(&full[s], a.stage_bytes);
                    ptx::tma_load_3d(stage_base + size_t(s) * a.stage_stride, &tmap, &full[s], 0, 0,
                                     row0 + 3 * trip);
                    if (++s == a.stages) {
                        s = 0;
                        ph ^= 1u;
                    }
                }
            }
        }
        return;
    }

    // ---------------------------------------------------- consumer threads
    const int lane = tid & 31;
    const bool active = tid < a.reps;
    const int r = active ? tid : a.reps - 1;        // repetition owned (clamped for idle lanes)
    const int rn = (r + 1 == a.reps) ? 0 : r + 1;  // neighbour repetition (toroidal, Fig. 11 '% 1920')
    const bool fix = (lane == 31) || (r + 1 == a.reps);
    const uint32_t seg = uint32_t(r) >> 2, ch0 = (uint32_t(r) & 3u) << 1;
    const uint32_t segn = uint32_t(rn) >> 2, chn = (uint32_t(rn) & 3u) << 1;
    const uint32_t segs = uint32_t(a.segs);
    const int Wo = a.Wo;
    const uint32_t stage_s32 = ptx::smem_u32(stage_base);

    int s = 0;
    uint32_t ph = 0;
    uint32_t emit_idx = 0;

    for (int64_t u = blockIdx.x; u < a.nunits; u += gridDim.x) {
        const int64_t plane = u / a.units_per_plane;
        const int32_t b0 = int32_t(u - plane * a.units_per_plane) * a.bands_per_unit;
        const int32_t b1 = min(b0 + a.bands_per_unit, a.nbands);
        const int32_t ntrip = 3 * (b1 - b0) + 1;
        const int32_t chan = int32_t(plane % a.channels);
        uint64_t csacc = 0;

        int32_t A0[3], A1[3], A2[3], A3[3];   // running V window sums of the current band
        int32_t Hr9[3], Hr911[3];             // halo: Y row 9 and rows 9..11 of the unit's last band
#pragma unroll
        for (int m = 0; m < 3; ++m) A0[m] = A1[m] = A2[m] = A3[m] = Hr9[m] = Hr911[m] = 0;

        // Band `band` is complete once rows 9..11 of its pattern are known: z = T(window sums).
        auto emit = [&](int32_t band, const int32_t* add9, const int32_t* add911) {
            int32_t z[4][3];
#pragma unroll
            for (int m = 0; m < 3; ++m) {
                z[0][m] = task_T(A0[m]);
                z[1][m] = task_T(A1[m]);
                z[2][m] = task_T(A2[m] + add9[m]);
                z[3][m] = task_T(A3[m] + add911[m]);
            }
            if (tid == 0) ptx::bulk_wait_read<kOutBufs - 1>();   // the out buffer we reuse is free again
            ptx::named_bar_sync(1, NC);
            int32_t* ob = outbuf + (emit_idx % kOutBufs) * (a.out_bytes / 4);
            if (active) {
#pragma unroll
                for (int k = 0; k < 4; ++k)
#pragma unroll
                    for (int m = 0; m < 3; ++m) ob[k * Wo + 3 * r + m] = z[k][m];
            }
            ptx::fence_proxy_async_smem();
            ptx::named_bar_sync(1, NC);
            if (tid == 0) {
                int32_t* gz = a.Z + (size_t(plane) * a.Ho + size_t(4 * band)) * size_t(Wo);
                ptx::bulk_store(gz, ob, a.out_bytes);   // 4 contiguous output rows
                ptx::bulk_commit();
            }
            ++emit_idx;
            if (kChecksum && active) {
                const uint64_t w0 =
                    1u + (uint64_t(chan) * a.Ho + uint64_t(4 * band)) * uint64_t(Wo) + uint64_t(3 * r);
#pragma unroll
                for (int k = 0; k < 4; ++k)
#pragma unroll
                    for (int m = 0; m < 3; ++m)
                        csacc += uint64_t(uint32_t(z[k][m])) * (w0 + uint64_t(k) * Wo + uint64_t(m));
            }
        };

        int tau = 0;
        for (int32_t ti = 0; ti < ntrip; ++ti) {
            // logical triple index: 0 = halo, 1.. = the unit's own triples in order
            const int32_t t = a.halo_last ? (ti == ntrip - 1 ? 0 : ti + 1) : ti;
            ptx::mbar_wait(&full[s], ph);
            const uint32_t sb = stage_s32 + uint32_t(s) * a.stage_stride;   // 32-bit shared address

            // ---- H stage on the 3 rows of this triple: y[row][col]
            int32_t y[3][3];
#pragma unroll
            for (int rr = 0; rr < 3; ++rr) {
                const uint32_t line = uint32_t(rr) * segs + seg;
                const int4 q0 = ptx::lds128(sb + swz(line, ch0));
                const int4 q1 = ptx::lds128(sb + swz(line, ch0 + 1));
                const int32_t e = q0.x + q0.y;
                const int32_t d = e + q0.z;                 // cols 8r..8r+2, the neighbour's halo
                const int32_t q = q0.z + q0.w;
                const int32_t p = q1.x + q1.y;
                const int32_t f = q1.z + q1.w;
                const int32_t qp = q + p;
                int32_t dn = __shfl_down_sync(0xffffffffu, d, 1);
                if (fix) {
                    const uint32_t ln = uint32_t(rr) * segs + segn;
                    const int4 qn = ptx::lds128(sb + swz(ln, chn));
                    dn = qn.x + qn.y + qn.z;
                }
                y[rr][0] = task_T(e + qp);                  // window cols 0..5
                y[rr][1] = task_T(qp + f);                  // window cols 2..7
                y[rr][2] = task_T(q1.y + f + dn);           // window cols 5..10
            }
            __syncwarp();
            if (lane == 0) ptx::mbar_arrive(&empty[s]);
            if (++s == a.stages) {
                s = 0;
                ph ^= 1u;
            }

            if (t == 0) {   // the halo triple: keep what the last band needs from it
#pragma unroll
                for (int m = 0; m < 3; ++m) {
                    Hr9[m] = y[0][m];
                    Hr911[m] = y[0][m] + y[1][m] + y[2][m];
                }
                continue;
            }

            // ---- V stage: running sums of the 12-row pattern (windows start at rows 0,2,4,6)
            if (tau == 0) {
                if (t > 1) {
                    // rows 0..2 of this band are rows 9..11 of the previous one: emit it
                    int32_t r9[3], r911[3];
#pragma unroll
                    for (int m = 0; m < 3; ++m) {
                        r9[m] = y[0][m];
                        r911[m] = y[0][m] + y[1][m] + y[2][m];
                    }
                    emit(b0 + (t - 1) / 3 - 1, r9, r911);
                }
#pragma unroll
                for (int m = 0; m < 3; ++m) {
                    A0[m] = y[0][m] + y[1][m] + y[2][m];   // rows 0..2 of window 0..5
                    A1[m] = y[2][m];                        // row 2 of window 2..7
                }
            } else if (tau == 1) {
#pragma unroll
                for (int m = 0; m < 3; ++m) {
                    const int32_t s3 = y[0][m] + y[1][m] + y[2][m];   // rows 3..5
                    A0[m] += s3;
                    A1[m] += s3;
                    A2[m] = y[1][m] + y[2][m];                        // rows 4,5 of window 4..9
                }
            } else {
#pragma unroll
                for (int m = 0; m < 3; ++m) {
                    const int32_t s2 = y[0][m] + y[1][m];             // rows 6,7
                    A1[m] += s2;
                    A2[m] += s2 + y[2][m];
                    A3[m] = s2 + y[2][m];                             // rows 6..8 of window 6..11
                }
            }
            if (++tau == 3) tau = 0;
        }
        emit(b1 - 1, Hr9, Hr911);   // the unit's last band, completed by the halo rows

        if (kChecksum) {
#pragma unroll
            for (int off = 16; off > 0; off >>= 1) csacc += __shfl_xor_sync(0xffffffffu, csacc, off);
            if (lane == 0 && csacc != 0)
                atomicAdd(reinterpret_cast<unsigned long long*>(a.cs + plane / a.channels),
                          static_cast<unsigned long long>(csacc));
        }
    }
    if (tid == 0) ptx::bulk_wait<0>();
}

// -------------------------------------------------------------------------
// Generic fused kernel: any W % 8 == 0, H % 9 == 0, int32 or uint8 input.
// One thread per (plane, band, output column): recomputes the 12 Y values it
// needs straight from global memory (L1/L2 absorb the overlap).  Correct for
// every shape; used when the TMA kernel's geometry constraints do not hold.
template <typename Tin, bool kChecksum>
__global__ void __launch_bounds__(256)
    fused_generic_kernel(const Tin* __restrict__ X, int32_t* __restrict__ Z, uint64_t* __restrict__ cs,
                         int64_t planes, int32_t H, int32_t W, int32_t Ho, int32_t Wo, int32_t channels) {
    const int32_t nb = H / 9;
    const int64_t total = planes * nb * int64_t(Wo);
    const int64_t stride = int64_t(gridDim.x) * blockDim.x;
    const int64_t start = int64_t(blockIdx.x) * blockDim.x + threadIdx.x;
    // warp-uniform trip count so the warp-level checksum reduction is safe
    const int64_t warp_base = start - (threadIdx.x & 31);
    for (int64_t base = warp_base; base < total; base += stride) {
        const int64_t idx = base + (threadIdx.x & 31);
        const bool live = idx < total;
        uint64_t contrib = 0;
        int64_t frame = -1;
        if (live) {
            const int32_t xo = int32_t(idx % Wo);
            const int64_t rest = idx / Wo;
            const int32_t b = int32_t(rest % nb);
            const int64_t plane = rest / nb;
            const int32_t rep = xo / 3, k = xo % 3;
            const int32_t s0 = (k == 0) ? 0 : (k == 1 ? 2 : 5);
            int32_t col[6];
#pragma unroll
            for (int t = 0; t < 6; ++t) {
                int32_t c = 8 * rep + s0 + t;
                col[t] = c >= W ? c - W : c;
            }
            const Tin* Xp = X + size_t(plane) * H * W;
            int32_t yv[12];
#pragma unroll
            for (int j = 0; j < 12; ++j) {
                int32_t row = 9 * b + j;
                if (row >= H) row -= H;
                const Tin* xr = Xp + size_t(row) * W;
                int32_t S = 0;
#pragma unroll
                for (int t = 0; t < 6; ++t) S += int32_t(xr[col[t]]);
                yv[j] = task_T(S);
            }
            int32_t* Zp = Z + size_t(plane) * Ho * Wo;
            const int32_t chan = int32_t(plane % channels);
#pragma unroll
            for (int kk = 0; kk < 4; ++kk) {
                int32_t S = 0;
#pragma unroll
                for (int t = 0; t < 6; ++t) S += yv[2 * kk + t];
                const int32_t z = task_T(S);
                const int32_t yo = 4 * b + kk;
                Zp[size_t(yo) * Wo + xo] = z;
                if (kChecksum)
                    contrib += uint64_t(uint32_t(z)) * (1u + (uint64_t(chan) * Ho + yo) * uint64_t(Wo) + xo);
            }
            frame = plane / channels;
        }
        if (kChecksum) {
            const int64_t f0 = __shfl_sync(0xffffffffu, frame, 0);
            const bool uniform = __all_sync(0xffffffffu, frame == f0 || frame < 0);
            if (uniform) {
#pragma unroll
                for (int off = 16; off > 0; off >>= 1) contrib += __shfl_xor_sync(0xffffffffu, contrib, off);
                if ((threadIdx.x & 31) == 0 && f0 >= 0)
                    atomicAdd(reinterpret_cast<unsigned long long*>(cs + f0), (unsigned long long)contrib);
            } else if (live) {
                atomicAdd(reinterpret_cast<unsigned long long*>(cs + frame), (unsigned long long)contrib);
            }
        }
    }
}

// ------------------------------------------------------------ TMA descriptor
using EncodeTiledFn = CUresult (*)(CUtensorMap*, CUtensorMapDataType, cuuint32_t, void*, const cuuint64_t*,
                                   const cuuint64_t*, const cuuint32_t*, const cuuint32_t*, CUtensorMapInterleave,
                                   CUtensorMapSwizzle, CUtensorMapL2promotion, CUtensorMapFloatOOBfill);

aol_status_t get_encode_fn(EncodeTiledFn* fn) {
    void* p = nullptr;
    cudaDriverEntryPointQueryResult q;
    cudaError_t e = cudaGetDriverEntryPoint("cuTensorMapEncodeTiled", &p, cudaEnableDefault, &q);
    if (e != cudaSuccess || q != cudaDriverEntryPointSuccess || p == nullptr) {
        set_error("cuTensorMapEncodeTiled unavailable (%s)", cudaGetErrorString(e));
        return AOL_E_CUDA;
    }
    *fn = reinterpret_cast<EncodeTiledFn>(p);
    return AOL_OK;
}

bool tma_shape_ok(int64_t planes, int64_t H, int64_t W) {
    return W % 32 == 0 && W / 32 <= 256 && W / 8 <= kMaxConsumers && planes * H < (int64_t(1) << 31) &&
           H >= 9;
}

}  // namespace

aol_status_t plan_fused(aol_dtype_t in_dtype, const void* d_in, const int32_t* d_out, int64_t frames,
                        int64_t channels, int64_t H, int64_t W, const aol_launch_opts_t* opts, FusedPlan* plan) {
    DeviceInfo dev;
    aol_status_t st = device_info(&dev);
    if (st != AOL_OK) return st;
    const aol_launch_opts_t o = opts ? *opts : aol_launch_opts_t{0, 0, 0, 0, 0};
    const int64_t planes = frames * channels;
    const int64_t Wo = 3 * (W / 8);
    *plan = FusedPlan{};
    plan->num_sms = dev.num_sms;

    bool tma_ok = in_dtype == AOL_I32 && tma_shape_ok(planes, H, W) && (d_in == nullptr || aligned16(d_in)) &&
                  (d_out == nullptr || aligned16(d_out));
    int ctas_per_sm = o.ctas_per_sm > 0 ? o.ctas_per_sm : 1;
    int stages = 0;
    const uint32_t stage_bytes = uint32_t(12 * W);
    const uint32_t stage_stride = (stage_bytes + 1023u) & ~1023u;
    const uint32_t out_bytes = uint32_t(16 * Wo);
    if (tma_ok) {
        // per-CTA budget: share of the SM's smem, minus the 1 KB the runtime reserves per CTA
        int budget = std::min(dev.smem_optin, dev.smem_per_sm / ctas_per_sm - 1024);
        int fixed = kOutBufs * int(out_bytes) + 2 * kMaxStages * 8 + 1024;  // out buffers, barriers, align slack
        stages = (budget - fixed) / int(stage_stride);
        stages = std::min(stages, kMaxStages);
        if (o.stages > 0) {
            stages = std::min(stages, o.stages);
        } else {
            // Measured on B200 (profiles/r01_*): throughput peaks at ~138 KB of TMA loads in flight per
            // SM (6 HD row-triples); deeper rings are SLOWER (9 stages: -5%), shallower starve HBM.
            const int target = (kInflightBytesPerSM / ctas_per_sm + int(stage_stride) / 2) / int(stage_stride);
            stages = std::min(stages, std::max(2, target));
        }
        if (stages < 2) tma_ok = false;
    }
    if (o.kernel == 1 && !tma_ok) {
        set_error("TMA fused kernel requested but unsupported for this shape/dtype/alignment "
                  "(needs int32, W %% 32 == 0, W <= 7936, 16-byte aligned buffers)");
        return AOL_E_SHAPE;
    }
    if (o.kernel == 2) tma_ok = false;

    if (tma_ok) {
        const int nbands = int(H / 9);
        const int64_t max_ctas = int64_t(dev.num_sms) * ctas_per_sm;
        int nb = o.bands_per_unit;
        if (nb <= 0) {
            // minimise (waves of units) x (triples per unit); prefer larger units on ties
            int64_t best_cost = INT64_MAX;
            for (int cand = 1; cand <= std::min(nbands, 40); ++cand) {
                const int64_t upp = (nbands + cand - 1) / cand;
                const int64_t units = planes * upp;
                const int64_t waves = (units + max_ctas - 1) / max_ctas;
                const int64_t cost = waves * (3 * cand + 1);
                if (cost <= best_cost) {
                    best_cost = cost;
                    nb = cand;
                }
            }
        }
        nb = std::max(1, std::min(nb, nbands));
        plan->kernel = 1;
        plan->bands_per_unit = nb;
        plan->units_per_plane = (nbands + nb - 1) / nb;
        plan->units = planes * plan->units_per_plane;
        plan->grid = int(std::min<int64_t>(plan->units, max_ctas));
        const int nc = int(((W / 8) + 31) / 32 * 32);
        plan->block = nc + 32;
        plan->stages = stages;
        plan->smem = stages * int(stage_stride) + kOutBufs * int(out_bytes) + 2 * stages * 8 + 1024;
        plan->ctas_per_sm = ctas_per_sm;
        plan->flags = o.flags;
    } else {
        plan->kernel = 2;
        plan->block = 256;
        const int64_t total = planes * (H / 9) * Wo;
        const int64_t blocks = (total + 255) / 256;
        plan->grid = int(std::max<int64_t>(1, std::min<int64_t>(blocks, int64_t(dev.num_sms) * 8)));
        plan->units = total;
    }
    return AOL_OK;
}

aol_status_t launch_fused(const FusedPlan& plan, const void* d_in, aol_dtype_t in_dtype, int32_t* d_out,
                          int64_t frames, int64_t channels, int64_t H, int64_t W, uint64_t* d_cs, cudaStream_t s) {
    const int64_t planes = frames * channels;
    const int32_t Ho = int32_t(4 * (H / 9)), Wo = int32_t(3 * (W / 8));
    if (d_cs) AOL_CUDA_TRY(cudaMemsetAsync(d_cs, 0, size_t(frames) * sizeof(uint64_t), s));

    if (plan.kernel == 2) {
        if (in_dtype == AOL_U8) {
            auto k = d_cs ? fused_generic_kernel<uint8_t, true> : fused_generic_kernel<uint8_t, false>;
            k<<<plan.grid, plan.block, 0, s>>>(static_cast<const uint8_t*>(d_in), d_out, d_cs, planes, int32_t(H),
                                               int32_t(W), Ho, Wo, int32_t(channels));
        } else {
            auto k = d_cs ? fused_generic_kernel<int32_t, true> : fused_generic_kernel<int32_t, false>;
            k<<<plan.grid, plan.block, 0, s>>>(static_cast<const int32_t*>(d_in), d_out, d_cs, planes, int32_t(H),
                                               int32_t(W), Ho, Wo, int32_t(channels));
        }
        AOL_LAUNCH_CHECK("fused_generic_kernel");
        return AOL_OK;
    }

    EncodeTiledFn encode;
    aol_status_t st = get_encode_fn(&encode);
    if (st != AOL_OK) return st;
    CUtensorMap map;
    const cuuint64_t gdim[3] = {32, cuuint64_t(W / 32), cuuint64_t(planes * H)};
    const cuuint64_t gstride[2] = {128, cuuint64_t(W) * 4};
    const cuuint32_t box[3] = {32, cuuint32_t(W / 32), 3};
    const cuuint32_t estr[3] = {1, 1, 1};
    CUresult cr = encode(&map, CU_TENSOR_MAP_DATA_TYPE_INT32, 3, const_cast<void*>(d_in), gdim, gstride, box, estr,
                         CU_TENSOR_MAP_INTERLEAVE_NONE, CU_TENSOR_MAP_SWIZZLE_128B,
                         CU_TENSOR_MAP_L2_PROMOTION_L2_256B, CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
    if (cr != CUDA_SUCCESS) {
        set_error("cuTensorMapEncodeTiled failed (CUresult %d)", int(cr));
        return AOL_E_CUDA;
    }
    FusedArgs a;
    a.Z = d_out;
    a.cs = d_cs;
    a.nunits = plan.units;
    a.H = int32_t(H);
    a.W = int32_t(W);
    a.Ho = Ho;
    a.Wo = Wo;
    a.channels = int32_t(channels);
    a.reps = int32_t(W / 8);
    a.segs = int32_t(W / 32);
    a.triples_per_plane = int32_t(H / 3);
    a.nbands = int32_t(H / 9);
    a.bands_per_unit = plan.bands_per_unit;
    a.units_per_plane = plan.units_per_plane;
    a.stages = plan.stages;
    a.stage_bytes = uint32_t(12 * W);
    a.stage_stride = (a.stage_bytes + 1023u) & ~1023u;
    a.out_bytes = uint32_t(16 * Wo);
    a.n_consumer = plan.block - 32;
    a.halo_last = (plan.flags & AOL_FLAG_HALO_LAST) ? 1 : 0;

    // <=512 threads (W <= 3840): register budget for 1-2 CTAs/SM; wider rows need the 1024-thread build
    // register budget per residency: <=320 threads x 2 CTAs/SM, <=512 x 1, <=1024 x 1
    auto k = (plan.block <= 320 && plan.ctas_per_sm >= 2)
                 ? (d_cs ? fused_tma_kernel<true, 320, 2> : fused_tma_kernel<false, 320, 2>)
             : plan.block <= 512 ? (d_cs ? fused_tma_kernel<true, 512, 1> : fused_tma_kernel<false, 512, 1>)
                                 : (d_cs ? fused_tma_kernel<true, 1024, 1> : fused_tma_kernel<false, 1024, 1>);
    AOL_CUDA_TRY(cudaFuncSetAttribute(k, cudaFuncAttributeMaxDynamicSharedMemorySize, plan.smem));
    k<<<plan.grid, plan.block, plan.smem, s>>>(map, a);
    AOL_LAUNCH_CHECK("fused_tma_kernel");
    return AOL_OK;
}

}  // namespace aol
