// fused_kernel.cuh -- K-5: the fused HD->SD downscaler (hf -> vf of Fig. 3 in one kernel).
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
//  * One producer warp fills an S-stage smem ring guarded by full/empty
//    mbarriers.  int32 input: 3-D TMA tensor loads (box = 3 rows x W,
//    SWIZZLE_128B) when W % 32 == 0, else 1-D TMA bulk copies of the contiguous
//    3-row triple into a linear layout read conflict-free by lane-rotated
//    LDS.128 (kSwz = 0).  uint8 input ("24-bit RGB"): 3-D TMA tensor loads of
//    {128 B, W/128, 3 rows} without swizzle when W % 128 == 0, else 1-D TMA bulk
//    copies of the contiguous 3-row triple (same smem layout either way).
//  * Consumer thread r owns repetition r (8 input columns -> 3 Y columns).
//    int32: two conflict-free LDS.128 per row (the 128B swizzle spreads the
//    32-byte per-thread stride over all banks); ONE warp shuffle supplies the
//    3-column pattern overlap (pattern {11} vs paving step 8), lane 31 and the
//    row-wrapping repetition read it from smem.  uint8: one LDS.64 per row plus
//    one LDS.32 of the neighbour's first word (cheaper than shuffle + predicated
//    load in this issue-bound variant); six DP4A byte-dot-products form the
//    three 6-tap sums.
//  * The V stage is a running register accumulation over the band's rows
//    (4 outputs x 3 columns per thread), so every input row is read once.
//  * Each finished band (4 output rows, contiguous in Z) is staged in smem and
//    written by one 1-D TMA bulk store; the per-frame checksum is folded in
//    registers, reduced across the CTA and added with one atomic per unit.
#pragma once
#include <cuda.h>
#include <cuda_runtime.h>

#include <cstdint>
#include <type_traits>

#include "common.h"
#include "ptx.cuh"

namespace aol {
namespace fused {


constexpr int kMaxStages = 32;
constexpr int kMaxConsumers = 992;  // + 1 producer warp = 1024 threads
// Output staging buffers (4 output rows each).  One suffices: the bulk store of a
// band has long finished reading smem by the time the next band (3 triples
// later) is emitted, and the saved space buys one more ring stage.
constexpr int kOutBufs = 1;
// Bytes of TMA loads to keep in flight per SM.  Measured on B200 (profiles/r01_stage_sweep*.jsonl): HD
// int32 throughput peaks at 5 row-triples (115 KB) per SM with the band-unrolled consumer (it was 6 with
// the slower first consumer); deeper rings are SLOWER (HBM efficiency drops), shallower starve HBM.
constexpr int kInflightBytesPerSM = 5 * 23552;

__device__ __forceinline__ int32_t task_T(int32_t S) {
    // Fig. 5: tmp/6 - tmp%6 == 7*(tmp/6) - tmp for C truncating division.
    return 7 * (S / 6) - S;
}

// Same for 0 <= S < 98304 (sums of six 8-bit samples are <= 1530): S/6 == (S * 43691) >> 18 exactly
// there without 32-bit overflow (43691 = (2^18 + 2) / 6; checked exhaustively in tests/test_abi.py).
__device__ __forceinline__ int32_t task_T_nonneg(int32_t S) {
    const int32_t q = int32_t((uint32_t(S) * 43691u) >> 18);
    return 7 * q - S;
}

// Same for |S| < 49152 of either sign (V-stage sums of 8-bit-sample frames lie in [-30, 1530]): the
// arithmetic shift floors S/6 - S/(3*2^18) (= floor(S/6) for S >= 0, = ceil(S/6) - 1 for S < 0, including
// multiples of 6), so adding the sign bit gives C's truncating S/6 without a multiply-high (IMAD.HI
// measured slower than IMAD + SHF in this issue-bound kernel; checked exhaustively in tests/test_abi.py).
__device__ __forceinline__ int32_t task_T_small(int32_t S) {
    const int32_t q = ((S * 43691) >> 18) + int32_t(uint32_t(S) >> 31);
    return 7 * q - S;
}

// Packed 24-bit pixels (AOL_RGB8): bytes c, c+3, c+6, c+9 of the 12-byte window (a, b, c) -- channel kCh of
// 4 consecutive pixels -- by two byte permutes.
template <int kCh>
__device__ __forceinline__ uint32_t rgb_channel_word(uint32_t a, uint32_t b, uint32_t c) {
    constexpr uint32_t o0 = kCh, o1 = kCh + 3, o2 = kCh + 6, o3 = kCh + 9;
    constexpr uint32_t s1 = (o0 < 8 ? o0 : 0) | (o1 < 8 ? o1 : 0) << 4 | (o2 < 8 ? o2 : 0) << 8 | (o3 < 8 ? o3 : 0) << 12;
    constexpr uint32_t s2 = (o0 < 8 ? 0u : o0 - 4) | (o1 < 8 ? 1u : o1 - 4) << 4 | (o2 < 8 ? 2u : o2 - 4) << 8 |
                            (o3 < 8 ? 3u : o3 - 4) << 12;
    return __byte_perm(__byte_perm(a, b, s1), c, s2);
}

struct FusedArgs {
    void* Z;                    // output, Tout elements (int32, or int16 for 8-bit samples)
    uint64_t* cs;
    const void* X;              // uint8 path: source of the 1-D bulk copies
    int64_t nunits;
    int32_t H, W, Ho, Wo;
    int32_t channels;
    int32_t reps;               // W/8  repetitions of the H tiler per row
    int32_t segs;               // int32 path: lines per row (W/32 of 128 B, or W/8 of 32 B with SWIZZLE_32B)
    int32_t triples_per_plane;  // H/3
    int32_t nbands;             // H/9
    int32_t bands_per_unit;
    int32_t units_per_plane;
    int32_t stages;
    uint32_t stage_bytes;   // bytes of one row triple (12W int32, 3W uint8)
    uint32_t stage_stride;  // stage_bytes rounded up (1024 for the swizzle atom, 128 for uint8)
    uint32_t out_bytes;     // 4 output rows: 4 * Wo * sizeof(Tout)
    int32_t n_consumer;     // consumer threads, multiple of 32
    int32_t u8_tensor;      // uint8 path: 1 = 3-D TMA tensor loads (W % 128 == 0), 0 = 1-D bulk copies
    int32_t rows_per_stage; // int32 path: 3 (a stage holds a row triple) or 1 (one row per stage: finer ring
                            // granularity for wide frames); always 3 for uint8
    int32_t row_pitch;      // uint8 paths: bytes per input row (W planar, 3W packed 24-bit pixels)
};

// Byte offset of 16-byte chunk `chunk` (0..7) of 128-byte line `line` under SWIZZLE_128B
// (chunk index XOR line index mod 8; stage buffers are 1024-byte aligned).
__device__ __forceinline__ uint32_t swz(uint32_t line, uint32_t chunk) {
    return (line << 7) | (((chunk ^ line) & 7u) << 4);
}

// k-th work unit of this CTA: round-robin, so concurrently running CTAs stream adjacent units (a contiguous
// block of units per CTA measured no faster, profiles/r01_blocked_units_ab.jsonl).  >= nunits when done.
__device__ __forceinline__ int64_t unit_of(const FusedArgs&, int64_t k) {
    return int64_t(blockIdx.x) + k * gridDim.x;
}

// Per-thread constants of the H stage (which repetition, where its bytes live).
struct RepGeom {
    uint32_t off0, off1;  // int32: swizzled offsets of the two chunks within a row's lines (kSwz = 0: byte
                          // offsets of the first / second chunk LOADED); uint8: 8r
    uint32_t offn;        // neighbour repetition's first chunk / word
    uint32_t seg, segn;   // int32: 128-byte segment of the repetition / neighbour
    bool fix;             // read the neighbour from smem instead of the shuffle
    bool swap;            // int32, kSwz = 0: the thread loads its upper chunk first (bank rotation)
};

// H stage of one input row: the three 6-tap window sums of each of the thread's kR repetitions, T() applied:
// y[3j + k] = T(window k of repetition j).
template <typename Tin, int kR, int kSwz>
__device__ __forceinline__ void h_row(uint32_t row_base, uint32_t rr, const RepGeom& g, uint32_t segs, uint32_t W,
                                      int32_t (&y)[3 * kR]) {
    if constexpr (std::is_same<Tin, int32_t>::value) {
        static_assert(kR == 1, "int32 path: one repetition per thread");
        const uint32_t line = rr * segs + g.seg;
        int4 q0, q1;
        if constexpr (kSwz == 0 || kSwz == 1) {
            // linear rows (1-D bulk copies): a thread's 32 bytes sit at 32r, so a quarter-warp's first loads
            // would hit each 16-byte bank group twice; lanes with bit 2 set load their upper chunk first,
            // which spreads every quarter-warp's 8 chunks over all 8 bank groups (conflict-free LDS.128)
            const uint32_t rowa = row_base + rr * (4u * W);
            const int4 A = ptx::lds128(rowa + g.off0);
            const int4 B = ptx::lds128(rowa + g.off1);
            q0 = g.swap ? B : A;
            q1 = g.swap ? A : B;
        } else {
            q0 = ptx::lds128(row_base + swz(line, g.off0));
            q1 = ptx::lds128(row_base + swz(line, g.off1));
        }
        const int32_t e = q0.x + q0.y;
        const int32_t d = e + q0.z;                 // cols 8r..8r+2: the left neighbour's overlap
        const int32_t q = q0.z + q0.w;
        const int32_t p = q1.x + q1.y;
        const int32_t f = q1.z + q1.w;
        const int32_t qp = q + p;
        int32_t dn = __shfl_down_sync(0xffffffffu, d, 1);
        int4 qn = q0;   // lane 31 / wrapping repetition: neighbour chunk from smem (predicated, no branch)
        if constexpr (kSwz == 0 || kSwz == 1)
            ptx::lds128_if(qn, row_base + rr * (4u * W) + g.offn, g.fix);
        else
            ptx::lds128_if(qn, row_base + swz(rr * segs + g.segn, g.offn), g.fix);
        dn = g.fix ? qn.x + qn.y + qn.z : dn;
        y[0] = task_T(e + qp);            // window cols 0..5
        y[1] = task_T(qp + f);            // window cols 2..7
        y[2] = task_T(q1.y + f + dn);     // window cols 5..10
    } else if constexpr (kSwz == 3) {
        // packed 24-bit pixels (kR = 3 channels of ONE repetition): the repetition's 8 pixels are 24 bytes at
        // 24r, the next repetition's first 3 pixels 9 of the 12 bytes at 24(r+1) (0 for the row-wrapping one);
        // each channel's samples are gathered into words by byte permutes, then summed like planar samples
        static_assert(kR == 3, "packed pixels: 3 channels per thread");
        const uint32_t rowa = row_base + rr * (3u * W);
        const uint2 v0 = ptx::lds64(rowa + g.off0), v1 = ptx::lds64(rowa + g.off0 + 8u),
                    v2 = ptx::lds64(rowa + g.off0 + 16u);
        const uint2 n01 = ptx::lds64(rowa + g.offn);
        const uint32_t n2 = ptx::lds32(rowa + g.offn + 8u);
        uint32_t lo[3], hi[3], nw[3];
        lo[0] = rgb_channel_word<0>(v0.x, v0.y, v1.x);
        lo[1] = rgb_channel_word<1>(v0.x, v0.y, v1.x);
        lo[2] = rgb_channel_word<2>(v0.x, v0.y, v1.x);
        hi[0] = rgb_channel_word<0>(v1.y, v2.x, v2.y);
        hi[1] = rgb_channel_word<1>(v1.y, v2.x, v2.y);
        hi[2] = rgb_channel_word<2>(v1.y, v2.x, v2.y);
        nw[0] = rgb_channel_word<0>(n01.x, n01.y, n2);
        nw[1] = rgb_channel_word<1>(n01.x, n01.y, n2);
        nw[2] = rgb_channel_word<2>(n01.x, n01.y, n2);
#pragma unroll
        for (int j = 0; j < 3; ++j) {
            const int32_t S0 = int32_t(__dp4a(lo[j], 0x01010101u, __dp4a(hi[j], 0x00000101u, 0u)));
            const int32_t S1 = int32_t(__dp4a(lo[j], 0x01010000u, __dp4a(hi[j], 0x01010101u, 0u)));
            const int32_t S2 = int32_t(__dp4a(hi[j], 0x01010100u, __dp4a(nw[j], 0x00010101u, 0u)));
            y[3 * j + 0] = task_T_nonneg(S0);
            y[3 * j + 1] = task_T_nonneg(S1);
            y[3 * j + 2] = task_T_nonneg(S2);
        }
    } else {
        // uint8 samples: the kR repetitions' 8*kR bytes in 2*kR words, then the next repetition's first word
        // (columns 8(r+kR)..; word 0 for the row-wrapping repetition); dp4a(x, m, c) = c + sum of the bytes
        // of x selected by the 0/1 bytes of m (byte k = bits 8k..8k+7 = column 8r+k).
        const uint32_t rowa = row_base + rr * W;
        uint32_t x[2 * kR + 1];
        if constexpr (kR == 1) {
            const uint2 v = ptx::lds64(rowa + g.off0);
            x[0] = v.x;
            x[1] = v.y;
        } else {
            static_assert(kR == 2, "uint8 path: 1 or 2 repetitions per thread");
            const int4 v = ptx::lds128(rowa + g.off0);
            x[0] = uint32_t(v.x);
            x[1] = uint32_t(v.y);
            x[2] = uint32_t(v.z);
            x[3] = uint32_t(v.w);
        }
#ifndef AOL_U8_NBR_SHFL
        // the next repetition's first word by one LDS.32 per lane: at the 8kR-byte lane stride a 2-way (kR = 1) /
        // 4-way (kR = 2) bank conflict, but the kernel is issue-bound, not LSU-bound: a shuffle plus a predicated
        // LDS for lane 31 removes the conflicts and costs 16 M more instructions, 2 % slower
        // (profiles/r02_u8_nbr_ab.jsonl; A/B build flag AOL_U8_NBR_SHFL)
        x[2 * kR] = ptx::lds32(rowa + g.offn);
#else
        {
            uint32_t nw = __shfl_down_sync(0xffffffffu, x[0], 1);
            uint32_t nl = 0;
            ptx::lds32_if(nl, rowa + g.offn, g.fix);
            x[2 * kR] = g.fix ? nl : nw;
        }
#endif
#pragma unroll
        for (int j = 0; j < kR; ++j) {
            const uint32_t lo = x[2 * j], hi = x[2 * j + 1], nw = x[2 * j + 2];
            const int32_t S0 = int32_t(__dp4a(lo, 0x01010101u, __dp4a(hi, 0x00000101u, 0u)));  // cols 0..5
            const int32_t S1 = int32_t(__dp4a(lo, 0x01010000u, __dp4a(hi, 0x01010101u, 0u)));  // cols 2..7
            const int32_t S2 = int32_t(__dp4a(hi, 0x01010100u, __dp4a(nw, 0x00010101u, 0u)));  // cols 5..10
            y[3 * j + 0] = task_T_nonneg(S0);   // 8-bit samples: 0 <= S <= 1530
            y[3 * j + 1] = task_T_nonneg(S1);
            y[3 * j + 2] = task_T_nonneg(S2);
        }
    }
}

// kR = repetitions of the H tiler per consumer thread: 1 for int32 (two LDS.128 already cover one repetition's
// 8 columns); 1 or 2 for uint8 input, whose 16 bytes for two repetitions come in one LDS.128 and whose per-stage
// bookkeeping (mbarrier wait/arrive, addressing) two repetitions then share (the host picks, fused.cu).
// kSwz = the int32 smem layout: 128 (TMA tensor loads under SWIZZLE_128B, W % 32 == 0) or 0 (1-D bulk copies,
// linear rows, any W % 8 == 0; the default when W % 32 != 0) or 1 (column strips for frames wider than one CTA's
// 992 consumer threads, W % 32 == 0: a unit is (plane, strip of a.segs repetitions, run of bands); a stage is
// one row of the strip, 1-D bulk copies of the strip's 32 bytes per repetition plus 16 bytes of the next
// repetition -- the row-wrapping strip's from column 0 -- into linear rows; each band's 4 output rows leave as
// 4 row-segment bulk stores); 3 = packed 24-bit pixels; 0 for planar uint8.
// (SWIZZLE_32B tensor lines for W % 32 != 0 measured no faster than linear rows and were removed,
// profiles/r01_i32_layout_ab.jsonl.)  Tout = output element: int32, or int16 for 8-bit samples ([-5, 255]).
template <typename Tin, typename Tout, int kR, int kSwz, bool kChecksum, int kMaxThreads, int kMinBlocks>
__global__ void __launch_bounds__(kMaxThreads, kMinBlocks)
    fused_tma_kernel(const __grid_constant__ CUtensorMap tmap, const FusedArgs a) {
    constexpr bool kI32 = std::is_same<Tin, int32_t>::value;
    constexpr bool kIL = !kI32 && kSwz == 3;   // packed 24-bit pixels: a unit covers the 3 planes of a frame
    constexpr bool kStrip = kI32 && kSwz == 1; // column strips (a.segs repetitions each, one row per stage)
    // 8-bit samples with int16 outputs: outputs stored directly from registers instead of through the smem
    // staging buffer and a bulk store, whose two CTA barriers per band the issue-bound consumer waited on (HD
    // uint8 0.416 -> 0.401 ms, packed pixels 0.516 -> 0.479, CIF 0.290 -> 0.284).  int32 outputs keep the bulk
    // store: direct 8-byte stores cost DRAM efficiency there (uint8 HD 0.481 -> 0.555 ms, packed 0.503 -> 0.511;
    // profiles/r02_direct_store_ab.jsonl)
    constexpr bool kDirectStore = !kI32 && sizeof(Tout) == 2;
    // Packed pixels, and planar 8-bit samples with two repetitions per thread in the multi-CTA int16-output
    // instantiations (HD: 4 CTAs/SM of 160 threads; 4K: 2 of 288), stream the unit's halo triple LAST instead of
    // first: its values (rows 9 and 9..11 of the last band) are then consumed at once instead of held in
    // registers through the unit -- the 3-channel consumer spilled at 2 CTAs/SM, and the planar one fits 96
    // registers without spills only this way (HD uint8 -> int16 0.403 -> 0.395 ms at 4 CTAs/SM, 4K 0.362 ->
    // 0.343 at 2; halo-last at 3 CTAs/SM, or for int32 outputs and CIF: no gain or up to 3 % slower;
    // profiles/r02_u8_cps4_ab.jsonl, profiles/r02_u8_4k_cps2_ab.jsonl).  Halo-first makes the halo read coincide
    // with the neighbouring unit's read of the same rows (an L2 hit) -- what the HBM-bound paths need.
    constexpr bool kHaloLast = kIL || (kDirectStore && kR == 2 && kMinBlocks * kMaxThreads >= 576);
    constexpr int kC = 3 * kR;                 // Y / Z columns per consumer thread (kIL: 3 channels x 3)
    constexpr int kRP = kIL ? 1 : kR;          // H-tiler repetitions per consumer thread
    extern __shared__ uint8_t smem_raw[];
    uint8_t* smem = reinterpret_cast<uint8_t*>((reinterpret_cast<uintptr_t>(smem_raw) + 1023) & ~uintptr_t(1023));
    uint8_t* stage_base = smem;
    uint8_t* outbuf = smem + size_t(a.stages) * a.stage_stride;
    uint64_t* full = reinterpret_cast<uint64_t*>(smem + size_t(a.stages) * a.stage_stride + kOutBufs * a.out_bytes);
    uint64_t* empty = full + a.stages;
    unsigned long long* red = reinterpret_cast<unsigned long long*>(empty + a.stages);   // [32] checksum partials

    // Let a programmatic dependent of this launch (the next call's checksum-zeroing kernel, which waits for
    // this grid's completion before touching anything) become resident now instead of after the drain.
    ptx::griddep_launch_dependents();
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
            if ((kI32 && kSwz != 0) || a.u8_tensor) ptx::prefetch_tensormap(&tmap);
            int s = 0;
            uint32_t ph = 0;
            for (int64_t k = 0, u = unit_of(a, 0); u < a.nunits; u = unit_of(a, ++k)) {
                const int64_t plane = u / a.units_per_plane;
                int32_t run = int32_t(u - plane * a.units_per_plane), rs0 = 0, rs1 = a.reps;
                if constexpr (kStrip) {   // unit = (plane, strip, run of bands), runs innermost
                    const int32_t nstrips = (a.reps + a.segs - 1) / a.segs;
                    const int32_t runs = a.units_per_plane / nstrips;
                    const int32_t strip = run / runs;
                    run -= strip * runs;
                    rs0 = strip * a.segs;
                    rs1 = min(rs0 + a.segs, a.reps);
                }
                const int32_t b0 = run * a.bands_per_unit;
                const int32_t b1 = min(b0 + a.bands_per_unit, a.nbands);
                const int32_t ntrip = 3 * (b1 - b0) + 1;
                const int64_t row0 = plane * a.H;
                // halo triple: rows 9*b1 .. 9*b1+2 (mod H -- the V tiler's toroidal wrap for the last band)
                const int32_t halo = (3 * b1 == a.triples_per_plane) ? 0 : 3 * b1;
                // (packed pixels load the halo LAST: see kHaloLast)
                for (int32_t t = 0; t < ntrip; ++t) {
                    const int32_t trip = kHaloLast ? (t == ntrip - 1 ? halo : 3 * b0 + t)
                                                   : (t == 0 ? halo : 3 * b0 + t - 1);
                    if constexpr (kI32) {
                        if (a.rows_per_stage == 1) {   // one row per stage, three stages per triple
                            for (int32_t q = 0; q < 3; ++q) {
                                ptx::mbar_wait_sleep(&empty[s], ph ^ 1u);
                                uint8_t* dst = stage_base + size_t(s) * a.stage_stride;
                                const int64_t row = row0 + 3 * trip + q;
                                if constexpr (kStrip) {
                                    // the strip's repetitions, then the next repetition's first 16 bytes (its
                                    // first 3 columns are the last pattern overlap; column 0 for the last strip)
                                    const uint32_t main = 32u * uint32_t(rs1 - rs0);
                                    const uint8_t* xr = static_cast<const uint8_t*>(a.X) + size_t(row) * 4u * a.W;
                                    ptx::mbar_arrive_expect_tx(&full[s], main + 16u);
                                    ptx::bulk_load(dst, xr + 32u * uint32_t(rs0), main, &full[s]);
                                    ptx::bulk_load(dst + main, xr + (rs1 == a.reps ? 0u : 32u * uint32_t(rs1)), 16u,
                                                   &full[s]);
                                    if (++s == a.stages) {
                                        s = 0;
                                        ph ^= 1u;
                                    }
                                    continue;
                                }
                                ptx::mbar_arrive_expect_tx(&full[s], a.stage_bytes);
                                if constexpr (kSwz == 0)
                                    ptx::bulk_load(dst, static_cast<const uint8_t*>(a.X) + size_t(row) * 4u * a.W,
                                                   a.stage_bytes, &full[s]);
                                else
                                    ptx::tma_load_3d(dst, &tmap, &full[s], 0, 0, int32_t(row));
                                if (++s == a.stages) {
                                    s = 0;
                                    ph ^= 1u;
                                }
                            }
                            continue;
                        }
                    }
                    ptx::mbar_wait_sleep(&empty[s], ph ^ 1u);   // suspended, not spinning, while the ring is full
                    ptx::mbar_arrive_expect_tx(&full[s], a.stage_bytes);
                    uint8_t* dst = stage_base + size_t(s) * a.stage_stride;
                    if constexpr (kI32 && kSwz == 0) {
                        // linear layout: the triple is 12W contiguous bytes (16-byte multiple for W % 4 == 0)
                        const uint8_t* src = static_cast<const uint8_t*>(a.X) + size_t(row0 + 3 * trip) * 4u * a.W;
                        ptx::bulk_load(dst, src, a.stage_bytes, &full[s]);
                    } else if constexpr (kI32) {
                        ptx::tma_load_3d(dst, &tmap, &full[s], 0, 0, int32_t(row0 + 3 * trip));
                    } else if (a.u8_tensor) {
                        // {128 B, W/128, rows} tensor, no swizzle: same linear smem layout as the bulk copy
                        ptx::tma_load_3d(dst, &tmap, &full[s], 0, 0, int32_t(row0 + 3 * trip));
                    } else {
                        const uint8_t* src = static_cast<const uint8_t*>(a.X) + size_t(row0 + 3 * trip) * a.row_pitch;
                        ptx::bulk_load(dst, src, a.stage_bytes, &full[s]);
                    }
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
    bool active = kRP * tid < a.reps;
    int r = active ? kRP * tid : a.reps - kRP;   // first repetition owned (clamped for idle lanes)
    const int rn = (r + kRP == a.reps) ? 0 : r + kRP;  // next thread's repetition (toroidal, Fig. 11 '% 1920')
    RepGeom g;
    g.fix = (lane == 31) || (r + 1 == a.reps);
    g.swap = false;
    if constexpr (kI32 && kSwz == 0) {
        g.seg = g.segn = 0;
        g.swap = ((lane >> 2) & 1) != 0;   // r = tid, so r mod 8 = lane mod 8
        g.off0 = 32u * uint32_t(r) + (g.swap ? 16u : 0u);
        g.off1 = 32u * uint32_t(r) + (g.swap ? 0u : 16u);
        g.offn = 32u * uint32_t(rn);
    } else if constexpr (kI32) {
        g.seg = uint32_t(r) >> 2;
        g.segn = uint32_t(rn) >> 2;
        g.off0 = (uint32_t(r) & 3u) << 1;   // chunk indices within the 128-byte line
        g.off1 = g.off0 + 1;
        g.offn = (uint32_t(rn) & 3u) << 1;
    } else if constexpr (kIL) {
        g.seg = g.segn = 0;
        g.off0 = 24u * uint32_t(r);
        g.off1 = g.off0 + 8;
        g.offn = 24u * uint32_t(rn);
        g.fix = false;
    } else {
        g.seg = g.segn = 0;
        g.off0 = 8u * uint32_t(r);
        g.off1 = g.off0 + 4;
        g.offn = 8u * uint32_t(rn);
        g.fix = (lane == 31) || (r + kRP == a.reps);   // neighbour word not in lane+1 (see h_row)
    }
    const uint32_t segs = uint32_t(a.segs);
    const uint32_t Wu = uint32_t(a.W);
    const int Wo = a.Wo;
    int ow = Wo, rl = r;   // output staging: row pitch (elements) and the thread's repetition within it
    const uint32_t stage_s32 = ptx::smem_u32(stage_base);

    int s = 0;
    uint32_t ph = 0;
    uint32_t emit_idx = 0;

    for (int64_t k = 0, u = unit_of(a, 0); u < a.nunits; u = unit_of(a, ++k)) {
        const int64_t plane = u / a.units_per_plane;
        int32_t run = int32_t(u - plane * a.units_per_plane), rs0 = 0;
        if constexpr (kStrip) {   // this unit's strip: repetitions rs0 .. rs0 + nr - 1, rows of 32 nr + 16 bytes
            const int32_t nstrips = (a.reps + a.segs - 1) / a.segs;
            const int32_t runs = a.units_per_plane / nstrips;
            const int32_t strip = run / runs;
            run -= strip * runs;
            rs0 = strip * a.segs;
            const int32_t nr = min(a.segs, a.reps - rs0);
            active = tid < nr;
            rl = active ? tid : nr - 1;
            r = rs0 + rl;
            ow = 3 * nr;
            g.seg = g.segn = 0;
            g.swap = ((lane >> 2) & 1) != 0;   // as kSwz = 0 (rs0 is a multiple of 32)
            g.off0 = 32u * uint32_t(rl) + (g.swap ? 16u : 0u);
            g.off1 = 32u * uint32_t(rl) + (g.swap ? 0u : 16u);
            g.offn = 32u * uint32_t(rl + 1);   // the last thread: the 16 bytes after the strip
            g.fix = (lane == 31) || (rl + 1 == nr);
        }
        const int32_t b0 = run * a.bands_per_unit;
        const int32_t b1 = min(b0 + a.bands_per_unit, a.nbands);
        const int32_t chan = int32_t(plane % a.channels);
        uint64_t csacc = 0;

        int32_t A0[kC], A1[kC], A2[kC], A3[kC];   // running V window sums of the current band
        int32_t Hr9[kC], Hr911[kC];               // halo: Y row 9 and rows 9..11 of the unit's last band
#pragma unroll
        for (int m = 0; m < kC; ++m) A0[m] = A1[m] = A2[m] = A3[m] = Hr9[m] = Hr911[m] = 0;

        // Band `band` is complete once rows 9..11 of its pattern are known: z = T(window sums).
        auto emit = [&](int32_t band, const int32_t* add9, const int32_t* add911) {
            int32_t z[4][kC];
#pragma unroll
            for (int m = 0; m < kC; ++m) {
                if constexpr (kI32) {
                    z[0][m] = task_T(A0[m]);
                    z[1][m] = task_T(A1[m]);
                    z[2][m] = task_T(A2[m] + add9[m]);
                    z[3][m] = task_T(A3[m] + add911[m]);
                } else {   // 8-bit samples: V sums in [-30, 1530]
                    z[0][m] = task_T_small(A0[m]);
                    z[1][m] = task_T_small(A1[m]);
                    z[2][m] = task_T_small(A2[m] + add9[m]);
                    z[3][m] = task_T_small(A3[m] + add911[m]);
                }
            }
            if constexpr (kDirectStore) {
                // each thread stores its outputs straight to Z from registers (per plane and row: its 3 kR columns
                // at column 3r, coalesced across the warp in the widest aligned words) -- no staging, no barriers
                if (active) {
                    constexpr int kPl = kIL ? 3 : 1;       // planes per unit
                    constexpr int kCols = kC / kPl;        // columns per plane and row: 3 kR (or 3)
#pragma unroll
                    for (int j = 0; j < kPl; ++j) {
                        Tout* gz = static_cast<Tout*>(a.Z) +
                                   (size_t(kPl * plane + j) * a.Ho + size_t(4 * band)) * size_t(Wo) + 3 * r;
#pragma unroll
                        for (int k = 0; k < 4; ++k) {
                            Tout* row = gz + size_t(k) * Wo;
                            const int32_t* v = &z[k][kCols * j];
                            if constexpr (sizeof(Tout) == 2 && kCols % 2 == 0) {   // 12 r bytes: 4-byte words
#pragma unroll
                                for (int m = 0; m < kCols; m += 2)
                                    reinterpret_cast<uint32_t*>(row)[m / 2] =
                                        __byte_perm(uint32_t(v[m]), uint32_t(v[m + 1]), 0x5410u);
                            } else if constexpr (sizeof(Tout) == 4 && kCols % 2 == 0) {   // 24 tid bytes: 8-byte words
#pragma unroll
                                for (int m = 0; m < kCols; m += 2)
                                    reinterpret_cast<int2*>(row)[m / 2] = make_int2(v[m], v[m + 1]);
                            } else {
#pragma unroll
                                for (int m = 0; m < kCols; ++m) row[m] = Tout(v[m]);
                            }
                        }
                    }
                }
            } else {
            if (tid == 0) ptx::bulk_wait_read<kOutBufs - 1>();   // the out buffer we reuse is free again
            ptx::named_bar_sync(1, NC);
            const uint32_t ob = ptx::smem_u32(outbuf) + (emit_idx % kOutBufs) * a.out_bytes;
            if constexpr (kIL) {
              if (active) {
                // packed pixels: channel j's 4 output rows are region j of the staging buffer (one plane each)
#pragma unroll
                for (int j = 0; j < 3; ++j)
#pragma unroll
                    for (int k = 0; k < 4; ++k) {
                        const uint32_t e0 = uint32_t((4 * j + k) * Wo + 3 * r);
#pragma unroll
                        for (int m = 0; m < 3; ++m) {
                            if constexpr (sizeof(Tout) == 4)
                                ptx::sts32(ob + 4u * (e0 + m), z[k][3 * j + m]);
                            else
                                ptx::sts16(ob + 2u * (e0 + m), z[k][3 * j + m]);
                        }
                    }
              }
            } else if (active) {
#pragma unroll
                for (int k = 0; k < 4; ++k) {
                    const uint32_t e0 = uint32_t(k * ow + 3 * rl);   // element index of the thread's first column
                    if constexpr (sizeof(Tout) == 4 && kR == 1) {
#pragma unroll
                        for (int m = 0; m < 3; ++m) ptx::sts32(ob + 4u * (e0 + m), z[k][m]);
                    } else if constexpr (sizeof(Tout) == 4) {   // 8-byte aligned pairs: Wo = 6 (W/16) and 3r even
#pragma unroll
                        for (int m = 0; m < kC; m += 2) ptx::sts64(ob + 4u * (e0 + m), z[k][m], z[k][m + 1]);
                    } else if constexpr (kR == 1) {             // int16
#pragma unroll
                        for (int m = 0; m < 3; ++m) ptx::sts16(ob + 2u * (e0 + m), z[k][m]);
                    } else {   // int16 pairs packed into 32-bit stores (e0 even)
#pragma unroll
                        for (int m = 0; m < kC; m += 2)
                            ptx::sts32(ob + 2u * (e0 + m),   // low halves of both values: one PRMT
                                       int32_t(__byte_perm(uint32_t(z[k][m]), uint32_t(z[k][m + 1]), 0x5410u)));
                    }
                }
            }
            ptx::fence_proxy_async_smem();
            ptx::named_bar_sync(1, NC);
            if (kIL && tid == 0) {   // one 4-row store per plane of the frame (kIL: compile-time)
                const uint32_t pb = a.out_bytes / 3u;
#pragma unroll
                for (int j = 0; j < 3; ++j) {
                    Tout* gz = static_cast<Tout*>(a.Z) + (size_t(3 * plane + j) * a.Ho + size_t(4 * band)) * size_t(Wo);
                    ptx::bulk_store(gz, outbuf + (emit_idx % kOutBufs) * a.out_bytes + j * pb, pb);
                }
                ptx::bulk_commit();
            } else if (kStrip && tid == 0) {   // 4 row segments of the strip
                Tout* gz = static_cast<Tout*>(a.Z) + (size_t(plane) * a.Ho + size_t(4 * band)) * size_t(Wo) + 3 * rs0;
                const uint8_t* src = outbuf + (emit_idx % kOutBufs) * a.out_bytes;
#pragma unroll
                for (int k = 0; k < 4; ++k)
                    ptx::bulk_store(gz + size_t(k) * Wo, src + k * ow * int(sizeof(Tout)), uint32_t(ow * sizeof(Tout)));
                ptx::bulk_commit();
            } else if (tid == 0) {
                Tout* gz = static_cast<Tout*>(a.Z) + (size_t(plane) * a.Ho + size_t(4 * band)) * size_t(Wo);
                const uint8_t* src = outbuf + (emit_idx % kOutBufs) * a.out_bytes;
                ptx::bulk_store(gz, src, a.out_bytes);   // 4 rows
                ptx::bulk_commit();
            }
            }   // !kDirectStore
            ++emit_idx;
            if constexpr (kChecksum && kIL) {
              if (active) {
#pragma unroll
                for (int j = 0; j < 3; ++j) {
                    const uint32_t w0 = 1u + (uint32_t(j) * uint32_t(a.Ho) + uint32_t(4 * band)) * uint32_t(Wo) +
                                        uint32_t(3 * r);
#pragma unroll
                    for (int k = 0; k < 4; ++k)
#pragma unroll
                        for (int m = 0; m < 3; ++m)
                            csacc += uint64_t(uint32_t(z[k][3 * j + m])) * uint64_t(w0 + uint32_t(k * Wo + m));
                }
              }
            } else if (kChecksum && active) {
                // weight = 1 + frame-local flat index < 2^32 (the planner guarantees C*Ho*Wo < 2^32), so each
                // term is one 32x32->64 multiply-add (IMAD.WIDE.U32 with a 64-bit addend)
                const uint32_t w0 = 1u + (uint32_t(chan) * uint32_t(a.Ho) + uint32_t(4 * band)) * uint32_t(Wo) +
                                    uint32_t(3 * r);
#pragma unroll
                for (int k = 0; k < 4; ++k)
#pragma unroll
                    for (int m = 0; m < kC; ++m)
                        csacc += uint64_t(uint32_t(z[k][m])) * uint64_t(w0 + uint32_t(k * Wo + m));
            }
        };

        // Wait for the next ring stage, run the H stage on its 3 rows (y[row][col]), release the stage.
        auto triple = [&](int32_t (&y)[3][kC]) {
            if constexpr (kI32) {
                if (a.rows_per_stage == 1) {   // three one-row stages
#pragma unroll
                    for (int rr = 0; rr < 3; ++rr) {
                        ptx::mbar_wait_sleep(&full[s], ph);
                        h_row<Tin, kR, kSwz>(stage_s32 + uint32_t(s) * a.stage_stride, 0u, g, segs, Wu, y[rr]);
                        __syncwarp();
                        if (lane == 0) ptx::mbar_arrive(&empty[s]);
                        if (++s == a.stages) {
                            s = 0;
                            ph ^= 1u;
                        }
                    }
                    return;
                }
            }
            ptx::mbar_wait_sleep(&full[s], ph);
            const uint32_t sb = stage_s32 + uint32_t(s) * a.stage_stride;   // 32-bit shared address
#pragma unroll
            for (int rr = 0; rr < 3; ++rr) {
#ifdef AOL_PROBE_STREAM_ONLY
                // measurement build only (tools/stream_probe.sh): skip the smem reads and H arithmetic to
                // expose the pure TMA streaming rate of this access pattern.  Never in libaol.so.
#pragma unroll
                for (int m = 0; m < kC; ++m) y[rr][m] = int32_t(sb) + rr;
#else
                h_row<Tin, kR, kSwz>(sb, uint32_t(rr), g, segs, Wu, y[rr]);
#endif
            }
            __syncwarp();
            if (lane == 0) ptx::mbar_arrive(&empty[s]);
            if (++s == a.stages) {
                s = 0;
                ph ^= 1u;
            }
        };

        if (!kHaloLast) {   // the halo triple comes first: keep what the unit's last band needs (rows 9 and 9..11)
            int32_t y[3][kC];
            triple(y);
#pragma unroll
            for (int m = 0; m < kC; ++m) {
                Hr9[m] = y[0][m];
                Hr911[m] = y[0][m] + y[1][m] + y[2][m];
            }
        }
        // ---- one band per iteration; V stage = running sums of the 12-row pattern (windows at rows 0,2,4,6)
        for (int32_t band = b0; band < b1; ++band) {
            int32_t y[3][kC];
            triple(y);   // rows 0..2
            if (band > b0) {
                // rows 0..2 of this band are rows 9..11 of the previous one: emit it
                int32_t r9[kC], r911[kC];
#pragma unroll
                for (int m = 0; m < kC; ++m) {
                    r9[m] = y[0][m];
                    r911[m] = y[0][m] + y[1][m] + y[2][m];
                }
                emit(band - 1, r9, r911);
            }
#pragma unroll
            for (int m = 0; m < kC; ++m) {
                A0[m] = y[0][m] + y[1][m] + y[2][m];   // rows 0..2 of window 0..5
                A1[m] = y[2][m];                        // row 2 of window 2..7
            }
            triple(y);   // rows 3..5
#pragma unroll
            for (int m = 0; m < kC; ++m) {
                const int32_t s3 = y[0][m] + y[1][m] + y[2][m];
                A0[m] += s3;
                A1[m] += s3;
                A2[m] = y[1][m] + y[2][m];                        // rows 4,5 of window 4..9
            }
            triple(y);   // rows 6..8
#pragma unroll
            for (int m = 0; m < kC; ++m) {
                const int32_t s2 = y[0][m] + y[1][m];
                A1[m] += s2;
                A2[m] += s2 + y[2][m];
                A3[m] = s2 + y[2][m];                             // rows 6..8 of window 6..11
            }
        }
        if (kHaloLast) {   // the halo triple now: it completes the unit's last band
            int32_t y[3][kC];
            triple(y);
#pragma unroll
            for (int m = 0; m < kC; ++m) {
                Hr9[m] = y[0][m];
                Hr911[m] = y[0][m] + y[1][m] + y[2][m];
            }
        }
        emit(b1 - 1, Hr9, Hr911);   // the unit's last band, completed by the halo rows

        if (kChecksum) {
            // warp -> CTA reduction, then ONE atomic per unit (many units of one frame hit the same address)
#pragma unroll
            for (int off = 16; off > 0; off >>= 1) csacc += __shfl_xor_sync(0xffffffffu, csacc, off);
            if (lane == 0) red[tid >> 5] = csacc;
            ptx::named_bar_sync(2, NC);
            if (tid == 0) {
                unsigned long long sum = 0;
                for (int w = 0; w < NC / 32; ++w) sum += red[w];
                // the checksums were zeroed by the preceding zero_checksums_kernel, which this launch may
                // overlap (programmatic dependent launch): wait for it before the first atomic (no-op when
                // the kernel was launched without the PDL attribute, and after the first wait)
                ptx::griddep_wait();
                atomicAdd(reinterpret_cast<unsigned long long*>(a.cs + plane / a.channels), sum);
            }
            ptx::named_bar_sync(2, NC);   // red[] is reused by the next unit
        }
    }
    if (tid == 0) ptx::bulk_wait<0>();
}

// -------------------------------------------------------------------------
// Generic fused kernel: any W % 8 == 0, H % 9 == 0, int32 or uint8 input.
// One thread per (plane, band, output column): recomputes the 12 Y values it
// needs straight from global memory (L1/L2 absorb the overlap).  Correct for
// every shape; used when the TMA kernel's geometry constraints do not hold.
template <typename Tin, typename Tout, bool kChecksum>
__global__ void __launch_bounds__(256)
    fused_generic_kernel(const Tin* __restrict__ X, Tout* __restrict__ Z, uint64_t* __restrict__ cs,
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
            Tout* Zp = Z + size_t(plane) * Ho * Wo;
            const int32_t chan = int32_t(plane % channels);
#pragma unroll
            for (int kk = 0; kk < 4; ++kk) {
                int32_t S = 0;
#pragma unroll
                for (int t = 0; t < 6; ++t) S += yv[2 * kk + t];
                const int32_t z = task_T(S);
                const int32_t yo = 4 * b + kk;
                Zp[size_t(yo) * Wo + xo] = Tout(z);
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

using KernelFn = void (*)(const CUtensorMap, const FusedArgs);

// A resolved fused-kernel launch (kernel 1): tensor map, arguments, the kernels without / with the checksum
// epilogue (k[0] / k[1], smem attributes set), launch shape.  Built by prepare_fused (fused.cu), enqueued by
// enqueue_fused (zero_checksums_kernel + the fused kernel as its programmatic dependent).  Plans (plan.cu) keep
// one and re-enqueue it.  (A one-launch plan variant -- per-unit checksum partials with self-resetting counters,
// extra FusedArgs fields -- measured slower on device and perturbed the register allocation of the packed-pixel
// and int16-output instantiations by 2-9 %, profiles/r02_plan_epilogue_ab.jsonl; removed.)
struct FusedLaunch {
    CUtensorMap map;
    FusedArgs args;
    KernelFn k[2];
    int grid, block, smem, flags;
    int64_t frames;
};

// Explicit instantiations live in fused_k_*.cu (compiled in parallel); these pick one.
KernelFn tma_kernel_i32(bool checksum, int layout, int block, int cps);   // layout = kSwz (128, 0 or 1)
KernelFn tma_kernel_u8(bool checksum, bool out16, int reps_per_thread, int block, int cps);
KernelFn tma_kernel_rgb8(bool checksum, bool out16, int block, int cps);   // packed 24-bit pixels

}  // namespace fused

aol_status_t prepare_fused(const FusedPlan& plan, const void* d_in, aol_dtype_t in_dtype, void* d_out,
                           int64_t frames, int64_t channels, int64_t H, int64_t W, fused::FusedLaunch* L);
aol_status_t enqueue_fused(const fused::FusedLaunch& L, uint64_t* d_cs, cudaStream_t s);

namespace fused {

template <typename Tin, typename Tout, int kR, int kSwz, bool kChecksum>
KernelFn pick_tma_kernel(int block, int cps) {
    if constexpr (kR == 3) {   // packed 24-bit pixels: 3 channels per thread
        if (block <= 288 && cps >= 2) return fused_tma_kernel<Tin, Tout, kR, kSwz, kChecksum, 288, 2>;
        if (block <= 512) return fused_tma_kernel<Tin, Tout, kR, kSwz, kChecksum, 512, 1>;
        return fused_tma_kernel<Tin, Tout, kR, kSwz, kChecksum, 1024, 1>;
    } else if constexpr (kR == 2) {
        // two repetitions per thread take ~126 registers: bounds that never force spills below 1024 threads
        // int16 outputs at 4 CTAs/SM (HD) / 2 CTAs/SM (4K): 96 registers, no spills with the halo triple streamed
        // last (see kHaloLast)
        if constexpr (std::is_same<Tout, int16_t>::value) {
            if (block <= 160 && cps >= 4) return fused_tma_kernel<Tin, Tout, kR, kSwz, kChecksum, 160, 4>;
            if (block > 256 && block <= 288 && cps >= 2) return fused_tma_kernel<Tin, Tout, kR, kSwz, kChecksum, 288, 2>;
        }
        if (block <= 160 && cps >= 3) return fused_tma_kernel<Tin, Tout, kR, kSwz, kChecksum, 160, 3>;
        if (block <= 256 && cps >= 2) return fused_tma_kernel<Tin, Tout, kR, kSwz, kChecksum, 256, 2>;
        if (block <= 512) return fused_tma_kernel<Tin, Tout, kR, kSwz, kChecksum, 512, 1>;
        return fused_tma_kernel<Tin, Tout, kR, kSwz, kChecksum, 1024, 1>;
    } else {
        if (block <= 128 && cps >= 3) return fused_tma_kernel<Tin, Tout, kR, kSwz, kChecksum, 128, 4>;
        if (block <= 320 && cps >= 3) return fused_tma_kernel<Tin, Tout, kR, kSwz, kChecksum, 320, 3>;
        if (block <= 320 && cps >= 2) return fused_tma_kernel<Tin, Tout, kR, kSwz, kChecksum, 320, 2>;
        if (block <= 512) return fused_tma_kernel<Tin, Tout, kR, kSwz, kChecksum, 512, 1>;
        return fused_tma_kernel<Tin, Tout, kR, kSwz, kChecksum, 1024, 1>;
    }
}

}  // namespace fused
}  // namespace aol
