// fused.cu -- K-5 host side: launch planning (residency, ring depth, work units) and launch.
// The kernels are in fused_kernel.cuh (see its header comment for the design).
#include <cuda.h>
#include <cuda_runtime.h>

#include <algorithm>
#include <cstdint>
#include <cstdlib>
#include <cstring>

#include "common.h"
#include "fused_kernel.cuh"

namespace aol {

using namespace fused;

namespace {

// Zeroes the per-frame checksums ahead of a fused launch.  It is itself launched as a programmatic dependent
// of whatever precedes it in the stream (the previous fused kernel triggers its dependents at its start), so
// its one CTA is already resident when that kernel drains; griddepcontrol.wait then holds it until the
// preceding grid has completed and its writes are visible (the previous call may still be adding into the
// same checksums, or producing X).  Only after that wait does it let the fused launch start
// (griddepcontrol.launch_dependents): the fused kernel's prologue, TMA ring fill and whole first work unit
// overlap the zeroing, and only its first checksum atomic waits for it (ptx::griddep_wait).
__global__ void __launch_bounds__(256) zero_checksums_kernel(uint64_t* __restrict__ cs, int64_t n) {
    ptx::griddep_wait();
    ptx::griddep_launch_dependents();
    for (int64_t i = threadIdx.x; i < n; i += blockDim.x) cs[i] = 0;
}

// ------------------------------------------------------------ TMA descriptor
using EncodeTiledFn = CUresult (*)(CUtensorMap*, CUtensorMapDataType, cuuint32_t, void*, const cuuint64_t*,
                                   const cuuint64_t*, const cuuint32_t*, const cuuint32_t*, CUtensorMapInterleave,
                                   CUtensorMapSwizzle, CUtensorMapL2promotion, CUtensorMapFloatOOBfill);

aol_status_t get_encode_fn(EncodeTiledFn* fn) {
    // The driver entry point is immutable for the process: resolve it once (thread-safe static init).
    static void* cached = [] {
        void* p = nullptr;
        cudaDriverEntryPointQueryResult q;
        if (cudaGetDriverEntryPoint("cuTensorMapEncodeTiled", &p, cudaEnableDefault, &q) != cudaSuccess ||
            q != cudaDriverEntryPointSuccess)
            p = nullptr;
        return p;
    }();
    if (!cached) {
        set_error("cuTensorMapEncodeTiled unavailable from the CUDA driver");
        return AOL_E_CUDA;
    }
    *fn = reinterpret_cast<EncodeTiledFn>(cached);
    return AOL_OK;
}

// Column strips (int32, W % 32 == 0): repetitions per strip, a multiple of 32 (0: no strips).  Frames wider than
// one CTA's 992 consumer threads (W > 7936) run as strips of <= 480 repetitions (8K DCI: 352 + 352 + 320); the
// strips of a row are balanced.  AOL_FLAG_I32_STRIPS forces ~64-repetition strips (tests: several strips at small widths).
int i32_strip_reps(aol_dtype_t dt, int64_t W, int flags) {
    if (dt != AOL_I32 || W % 32 != 0) return 0;
    const int64_t reps = W / 8;
    static const int per_env = [] {   // AOL_STRIP_REPS=n: strips of <= n repetitions (A/B measurements only)
        const char* e = std::getenv("AOL_STRIP_REPS");
        return e ? std::max(32, std::min(kMaxConsumers, std::atoi(e))) : 0;
    }();
    int64_t per = 0;
    if (flags & AOL_FLAG_I32_STRIPS)
        per = 64;
    else if (reps > kMaxConsumers)
        per = per_env > 0 ? per_env : 480;   // <= 512 threads per CTA: the 64-register 1024-thread build spills
    else
        return 0;
    const int64_t n = (reps + per - 1) / per;
    return int(((reps + n - 1) / n + 31) / 32 * 32);
}

// Shared-memory layout of an int32 row triple (the kernel's kSwz): 128 = TMA tensor loads of 128-byte lines
// under SWIZZLE_128B (W % 32 == 0); 0 = one 1-D bulk copy of the contiguous triple into linear rows (W % 32 != 0,
// or forced by AOL_FLAG_I32_LINEAR); 1 = column strips (i32_strip_reps), one row per stage.  -1 for uint8 input.
int i32_layout(aol_dtype_t dt, int64_t W, int flags) {
    if (dt != AOL_I32) return -1;
    if (i32_strip_reps(dt, W, flags) > 0) return 1;
    if (flags & AOL_FLAG_I32_LINEAR) return 0;
    return W % 32 == 0 ? 128 : 0;
}

bool tma_shape_ok(aol_dtype_t dt, int64_t planes, int64_t channels, int64_t H, int64_t W, int flags) {
    if (H < 9 || (W / 8 > kMaxConsumers && i32_layout(dt, W, flags) != 1)) return false;
    // checksum weights (1 + frame-local output index) are computed in 32 bits
    if (channels * (4 * (H / 9)) * (3 * (W / 8)) >= (int64_t(1) << 32) - 1) return false;
    // int32 tensor layout: {32, W/32, 3}-element boxes under SWIZZLE_128B (a box dimension holds at most 256
    // elements; tensor row coordinates are int32); linear rows: 1-D bulk copies of 12W bytes (16-byte multiple
    // since W % 8 == 0)
    if (dt == AOL_I32) {
        if (i32_layout(dt, W, flags) <= 1) return true;   // 1-D bulk copies
        return W / 32 <= 256 && planes * H < (int64_t(1) << 31);
    }
    if (dt == AOL_U8) return W % 16 == 0;   // 1-D bulk copies: 16-byte granularity
    if (dt == AOL_RGB8) return W % 16 == 0;  // packed pixels: 9W-byte triples, 24-byte repetitions
    return false;
}

KernelFn pick(aol_dtype_t dt, int out_es, bool checksum, int kr, int64_t W, int flags, int block, int cps) {
    if (dt == AOL_RGB8) return tma_kernel_rgb8(checksum, out_es == 2, block, cps);
    return dt == AOL_U8 ? tma_kernel_u8(checksum, out_es == 2, kr, block, cps)
                        : tma_kernel_i32(checksum, i32_layout(dt, W, flags), block, cps);
}

// Rows per ring stage: a row triple, or (int32) one row when a triple would be coarser than a third of the
// bytes the ring keeps in flight (4K: 46 KB triples vs 115 KB per SM), unless forced by a flag.
int rows_per_stage(aol_dtype_t dt, int64_t W, int flags) {
    if (dt != AOL_I32) return 3;
    if (i32_layout(dt, W, flags) == 1) return 1;   // column strips: one row (of the strip) per stage
    if (flags & AOL_FLAG_ROW_STAGES) return 1;
    if (flags & AOL_FLAG_TRIPLE_STAGES) return 3;
    return 12 * W > kInflightBytesPerSM / 3 ? 1 : 3;
}

// Shared-memory geometry of the TMA ring: one stage = one row triple (or one row, rows_per_stage).
struct RingGeom {
    uint32_t stage_bytes;   // rows_per_stage rows of the input
    uint32_t stage_stride;  // rounded up: 1024 B (SWIZZLE_128B atom) for int32, 128 B for uint8
    uint32_t out_bytes;     // one band of output: 4 rows of Wo output elements
};

RingGeom ring_geom(aol_dtype_t dt, int out_es, int64_t W, int flags) {
    // swizzled layouts need 1024-byte aligned stages (the swizzle atom); bulk copies 16 bytes (128 kept)
    // bytes per input row: W int32 / W uint8 / 3W packed 24-bit pixels
    const uint32_t es = dt == AOL_I32 ? 4u : (dt == AOL_RGB8 ? 3u : 1u), align = i32_layout(dt, W, flags) > 0 ? 1024u : 128u;
    RingGeom g;
    g.stage_bytes = uint32_t(rows_per_stage(dt, W, flags) * W) * es;
    g.stage_stride = (g.stage_bytes + align - 1) & ~(align - 1);
    g.out_bytes = uint32_t(4 * out_es * (3 * (W / 8))) * (dt == AOL_RGB8 ? 3u : 1u);   // packed: 3 planes
    if (dt != AOL_I32 && out_es == 2) g.out_bytes = 0;   // int16 outputs leave from registers (no staging)
    if (const int sr = i32_strip_reps(dt, W, flags)) {   // a strip row + the next repetition's first 16 bytes
        g.stage_bytes = uint32_t(32 * sr + 16);
        g.stage_stride = (g.stage_bytes + align - 1) & ~(align - 1);
        g.out_bytes = uint32_t(4 * out_es * 3 * sr);
    }
    return g;
}

// ring + output staging + full/empty mbarriers + checksum partials + 1 KB alignment slack
int smem_bytes(const RingGeom& g, int stages) {
    return stages * int(g.stage_stride) + kOutBufs * int(g.out_bytes) + 2 * stages * 8 + 256 + 1024;
}

// L2 sector promotion of the TMA loads: none (the rows are streamed once; 256-byte promotion measured 0.2-0.4 %
// slower on HD / 4K int32 and HD uint8, profiles/r01_l2promo_ab.jsonl).  AOL_TMA_L2_PROMO=1/2/3 selects
// 64 / 128 / 256 B (A/B measurements only).
CUtensorMapL2promotion l2_promotion() {
    static const CUtensorMapL2promotion v = [] {
        const char* e = std::getenv("AOL_TMA_L2_PROMO");
        if (e && e[0] == '1') return CU_TENSOR_MAP_L2_PROMOTION_L2_64B;
        if (e && e[0] == '2') return CU_TENSOR_MAP_L2_PROMOTION_L2_128B;
        if (e && e[0] == '3') return CU_TENSOR_MAP_L2_PROMOTION_L2_256B;
        return CU_TENSOR_MAP_L2_PROMOTION_NONE;
    }();
    return v;
}

// TMA descriptor for row triples of a [rows][W] array viewed as {inner, W/inner, rows}: int32 with a
// 128 B swizzle (inner = 32 elements), uint8 unswizzled (inner = 128 elements).
aol_status_t encode_row_map(CUtensorMap* map, aol_dtype_t dt, const void* base, int64_t rows, int64_t W, int flags) {
    EncodeTiledFn encode;
    aol_status_t st = get_encode_fn(&encode);
    if (st != AOL_OK) return st;
    const bool i32 = dt == AOL_I32;
    const cuuint64_t inner = i32 ? 32 : 128, es = i32 ? 4 : 1;
    const cuuint64_t gdim[3] = {inner, cuuint64_t(W) / inner, cuuint64_t(rows)};
    const cuuint64_t gstride[2] = {inner * es, cuuint64_t(W) * es};
    const cuuint32_t box[3] = {cuuint32_t(inner), cuuint32_t(W / int64_t(inner)), cuuint32_t(rows_per_stage(dt, W, flags))};
    const cuuint32_t estr[3] = {1, 1, 1};
    CUresult cr = encode(map, i32 ? CU_TENSOR_MAP_DATA_TYPE_INT32 : CU_TENSOR_MAP_DATA_TYPE_UINT8, 3,
                         const_cast<void*>(base), gdim, gstride, box, estr, CU_TENSOR_MAP_INTERLEAVE_NONE,
                         i32 ? CU_TENSOR_MAP_SWIZZLE_128B : CU_TENSOR_MAP_SWIZZLE_NONE,
                         l2_promotion(), CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
    if (cr != CUDA_SUCCESS) {
        set_error("cuTensorMapEncodeTiled failed (CUresult %d)", int(cr));
        return AOL_E_CUDA;
    }
    return AOL_OK;
}

// The generic fused kernel (kernel 2): pre-flight, then zero the checksums and launch.
template <typename Tin, typename Tout>
aol_status_t launch_generic(const FusedPlan& plan, const void* d_in, void* d_out, uint64_t* d_cs, int64_t frames,
                            int64_t planes, int64_t H, int64_t W, int32_t Ho, int32_t Wo, int64_t channels,
                            cudaStream_t s) {
    auto k = d_cs ? fused_generic_kernel<Tin, Tout, true> : fused_generic_kernel<Tin, Tout, false>;
    aol_status_t st = launch_preflight(reinterpret_cast<const void*>(k), plan.block, 0, "fused_generic_kernel");
    if (st != AOL_OK) return st;   // nothing enqueued yet
    if (d_cs) AOL_CUDA_TRY(cudaMemsetAsync(d_cs, 0, size_t(frames) * sizeof(uint64_t), s));
    k<<<plan.grid, plan.block, 0, s>>>(static_cast<const Tin*>(d_in), static_cast<Tout*>(d_out), d_cs, planes,
                                       int32_t(H), int32_t(W), Ho, Wo, int32_t(channels));
    AOL_LAUNCH_CHECK("fused_generic_kernel");
    return AOL_OK;
}

}  // namespace

aol_status_t plan_fused(aol_dtype_t in_dtype, aol_dtype_t out_dtype, const void* d_in, const void* d_out,
                        int64_t frames, int64_t channels, int64_t H, int64_t W, const aol_launch_opts_t* opts,
                        FusedPlan* plan, bool checksum) {
    DeviceInfo dev;
    aol_status_t st = device_info(&dev);
    if (st != AOL_OK) return st;
    const aol_launch_opts_t o = opts ? *opts : aol_launch_opts_t{0, 0, 0, 0, 0};
    const bool rgb = in_dtype == AOL_RGB8;              // packed 24-bit pixels: a unit covers a frame's 3 planes
    const bool u8like = in_dtype == AOL_U8 || rgb;     // 8-bit samples: issue-bound consumer
    const int64_t planes = rgb ? frames : frames * channels;
    const int64_t Wo = 3 * (W / 8);
    *plan = FusedPlan{};
    plan->num_sms = dev.num_sms;
    plan->out_es = out_dtype == AOL_I16 ? 2 : 4;

    bool tma_ok = tma_shape_ok(in_dtype, planes, channels, H, W, o.flags) && (d_in == nullptr || aligned16(d_in)) &&
                  (d_out == nullptr || aligned16(d_out));
    const int out_es = out_dtype == AOL_I16 ? 2 : 4;
    const RingGeom geom = ring_geom(in_dtype, out_es, W, o.flags);
    // repetitions per consumer thread: 2 for uint8 frames at least 1024 wide (HD: 0.498 vs 0.520 ms; 4K: equal),
    // 1 for narrower ones (CIF: 0.361 vs 0.315 ms -- one half-idle warp per CTA) and for int32
    // (profiles/r01_u8_r2_ab.jsonl)
    const int kr = rgb ? 3 : (in_dtype == AOL_U8 && W >= 1024 && !(o.flags & AOL_FLAG_U8_ONE_REP)) ? 2 : 1;
    const int strip = i32_strip_reps(in_dtype, W, o.flags);   // column strips: consumers = repetitions per strip
    const int64_t nstrips = strip > 0 ? (W / 8 + strip - 1) / strip : 1;
    const int nc = strip > 0 ? strip : int(((W / 8 / (rgb ? 1 : kr)) + 31) / 32 * 32);   // packed: one repetition (3 channels) per thread
    const int block = nc + 32;
    int stages = 0, cps = 1;
    if (tma_ok) {
        // CTAs per SM: enough consumer warps to hide the per-row dependency chains (narrow frames
        // such as CIF have only 2 consumer warps per CTA), unless the caller fixed it, but no more
        // concurrent row streams than that: DRAM efficiency falls as streams are added.  int32
        // (HBM-bound): 8 consumer warps per SM.  uint8 (issue-bound): 16 warps of one repetition each,
        // or 8 warps of two (HD: 2 CTAs/SM, 0.499 ms vs 0.567 at 3 and 0.738 at 1;
        // profiles/r01_u8_r2_ab.jsonl) -- 16 with int16 outputs, whose halved write traffic leaves DRAM room
        // for more row streams per SM (HD: 0.431 ms at 3 CTAs/SM vs 0.503 at 2, profiles/r01_u8_i16.jsonl; 0.397
        // at 4 with the 96-register instantiation, profiles/r02_u8_cps4_ab.jsonl).
        const int cwarps = nc / 32;
        // packed 24-bit pixels (3 channels per thread, ~100 registers): 16 warps (HD: 2 CTAs/SM 0.513 ms vs 0.608
        // at 1; profiles/r01_rgb_sweep.jsonl)
        const int want_warps = rgb ? 16 : (in_dtype == AOL_U8 && (kr == 1 || out_es == 2)) ? 16 : 8;
        cps = o.ctas_per_sm > 0 ? o.ctas_per_sm
                                : std::max(1, std::min(8, (want_warps + cwarps - 1) / cwarps));
        for (;; --cps) {
            const int budget = std::min(dev.smem_optin, dev.smem_per_sm / cps - 1024);
            const int fixed = smem_bytes(geom, 0) + 2 * kMaxStages * 8;   // everything but the ring itself
            stages = std::min((budget - fixed) / int(geom.stage_stride), kMaxStages);
            if (o.stages > 0) {
                stages = std::min(stages, o.stages);
            } else {
                // nearest whole number of stages to the in-flight target; one-row stages round down (4K: 7 rows =
                // 1.065 ms, 8 = 1.070, 9 = 1.13-1.16: HBM efficiency falls off a cliff above ~120 KB per SM)
                // (8-bit samples, issue-bound: rounded up -- packed pixels with int16 outputs 0.479 ms at 3
                // stages, 0.464 at 4; planar uint8 4K 0.434 -> 0.417; except packed pixels with int32 outputs,
                // whose 4th stage costs the 2nd CTA's room: 0.503 -> 0.530; profiles/r02_stage_round_ab.jsonl)
                const bool up = u8like && !(rgb && out_es == 4);
                const int half = up ? int(geom.stage_stride) - 1
                                    : rows_per_stage(in_dtype, W, o.flags) == 1 ? 0 : int(geom.stage_stride) / 2;
                const int target = (kInflightBytesPerSM / cps + half) / int(geom.stage_stride);
                stages = std::min(stages, std::max(2, target));
                // planar 8-bit samples with int32 outputs and no checksum epilogue: the lighter consumer runs
                // ahead of the memory side and a ring of half that depth keeps DRAM efficiency (HD 0.567 -> 0.488
                // ms at 6 stages instead of 11; with the epilogue 11 stays best, 0.478;
                // profiles/r02_nocs_stage_sweep.jsonl)
                if (!checksum && in_dtype == AOL_U8 && out_es == 4) stages = std::min(stages, std::max(2, (target + 1) / 2));
            }
            int occ = 0;
            const int smem = smem_bytes(geom, stages);
            if (stages >= 2 && cps > 1)
                occ = kernel_occupancy(reinterpret_cast<const void*>(pick(in_dtype, out_es, true, kr, W, o.flags, block, cps)),
                                       block, smem);
            if (cps == 1) occ = 1;   // one CTA always fits once its shared memory does
            if ((stages >= 2 && occ >= cps) || cps == 1 || o.ctas_per_sm > 0) {
                if (stages < 2) tma_ok = false;
                break;
            }
        }
    }
    if (o.kernel == 1 && !tma_ok) {
        set_error("TMA fused kernel requested but unsupported for this shape/dtype/alignment "
                  "(W <= 7936, or int32 with W %% 32 == 0 (column strips), and a 2-stage ring within shared memory; "
                  "uint8: W %% 16 == 0; 16-byte aligned buffers)");
        return AOL_E_SHAPE;
    }
    if (o.kernel == 2) tma_ok = false;
    if (rgb && !tma_ok) {
        // a CTA holds two 9W-byte ring stages plus the 3-plane 4-row output staging (18W bytes for int32, 9W for
        // int16 outputs) within the 227 KB opt-in: W <= 6400 (int32 outputs) / 7936 (int16 outputs)
        set_error("packed 24-bit pixels (AOL_RGB8) need the TMA fused kernel: W %% 16 == 0, W <= %d with %s outputs "
                  "(two ring stages and the output staging in shared memory), 16-byte aligned buffers",
                  out_es == 4 ? 6400 : 7936, out_es == 4 ? "int32" : "int16");
        return AOL_E_SHAPE;
    }

    if (tma_ok) {
        const int nbands = int(H / 9);
        const int64_t max_ctas = int64_t(dev.num_sms) * cps;
        int nb = o.bands_per_unit;
        if (nb <= 0) {
            // Cost of a candidate: (units the busiest CTA runs) x (row triples per unit + a fixed per-unit cost in
            // triple-equivalents).  int32 (HBM-bound): no fixed cost, and the SMALLEST unit within 2 % of the
            // cheapest wins (a shorter last unit = a shorter tail; HD 1.240 ms at 10-12 bands vs 1.248 at 15, 4K
            // 1.083 at 12 vs 1.089 at 24).  uint8 (issue-bound): the per-unit epilogue (checksum reduction,
            // barriers) costs ~2 triples of a 1920-wide frame, inversely proportional to the row width, and the
            // cheapest (largest on ties) wins (HD 0.479 ms at 20 bands vs 0.497 at 12, CIF 0.289 at 32 vs 0.310
            // at 8; profiles/r01_nb_sweep.jsonl).
            // (int16 outputs run 3 CTAs/SM: the epilogue weighs ~1.5x more; HD 0.421 ms at 20 vs 0.425 at 15)
            const double ovh = u8like ? (out_es == 2 ? 5760.0 : 3840.0) / double(W) : 0.0;
            constexpr int kMaxNb = 120;
            const int max_nb = std::min(nbands, kMaxNb);
            double cost[kMaxNb + 1] = {};
            double best = 1e300;
            for (int cand = 1; cand <= max_nb; ++cand) {
                const int64_t units = planes * nstrips * ((nbands + cand - 1) / cand);
                const int64_t waves = (units + max_ctas - 1) / max_ctas;
                cost[cand] = double(waves) * (3.0 * cand + 1.0 + ovh);
                best = std::min(best, cost[cand]);
            }
            for (int cand = 1; cand <= max_nb; ++cand) {
                if (u8like) {
                    if (cost[cand] <= best) nb = cand;   // largest of the cheapest
                } else if (cost[cand] <= 1.02 * best) {
                    nb = cand;                                   // smallest within 2 %
                    break;
                }
            }
        }
        nb = std::max(1, std::min(nb, nbands));
        plan->kernel = 1;
        plan->bands_per_unit = nb;
        plan->units_per_plane = int(nstrips * ((nbands + nb - 1) / nb));
        plan->units = planes * plan->units_per_plane;
        plan->grid = int(std::min<int64_t>(plan->units, max_ctas));
        plan->block = block;
        plan->stages = stages;
        // The grid is persistent (cps CTAs per SM, units assigned round-robin): pad the shared memory so
        // that no SM can take a (cps+1)-th CTA, which would leave another SM short and stretch the tail.
        const int exclusive = dev.smem_per_sm / (cps + 1) - 1024 + 128;
        plan->smem = std::max(smem_bytes(geom, stages), std::min(exclusive, dev.smem_optin));
        plan->ctas_per_sm = cps;
        plan->reps_per_thread = kr;
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

aol_status_t prepare_fused(const FusedPlan& plan, const void* d_in, aol_dtype_t in_dtype, void* d_out,
                           int64_t frames, int64_t channels, int64_t H, int64_t W, FusedLaunch* L) {
    const bool rgb = in_dtype == AOL_RGB8;
    const int64_t planes = rgb ? frames : frames * channels;   // packed pixels: work units per frame
    std::memset(&L->map, 0, sizeof L->map);
    const bool u8_tensor = in_dtype == AOL_U8 && W % 128 == 0 && W / 128 <= 256 && planes * H < (int64_t(1) << 31);
    const int layout = i32_layout(in_dtype, W, plan.flags);
    if (layout == 128 || u8_tensor) {
        aol_status_t st = encode_row_map(&L->map, in_dtype, d_in, planes * H, W, plan.flags);
        if (st != AOL_OK) return st;
    }
    FusedArgs& a = L->args;
    std::memset(&a, 0, sizeof a);
    a.u8_tensor = u8_tensor ? 1 : 0;
    a.rows_per_stage = rows_per_stage(in_dtype, W, plan.flags);
    a.Z = d_out;
    a.X = d_in;
    // units from THIS call's frame count (a plan may be reused for a shorter batch, e.g. the last chunk of
    // the host-streamed path): never more units, or CTAs, than the batch has
    a.nunits = planes * plan.units_per_plane;
    L->grid = int(std::min<int64_t>(plan.grid, a.nunits));
    L->block = plan.block;
    L->smem = plan.smem;
    L->frames = frames;
    L->flags = plan.flags;
    a.H = int32_t(H);
    a.W = int32_t(W);
    a.Ho = int32_t(4 * (H / 9));
    a.Wo = int32_t(3 * (W / 8));
    a.channels = rgb ? 1 : int32_t(channels);   // packed: the unit index is the frame index
    a.row_pitch = int32_t(rgb ? 3 * W : W);
    a.reps = int32_t(W / 8);
    a.segs = int32_t(W / 32);   // int32 swizzled 128-byte lines per row (unused for linear rows)
    if (layout == 1) a.segs = i32_strip_reps(in_dtype, W, plan.flags);   // column strips: repetitions per strip
    a.triples_per_plane = int32_t(H / 3);
    a.nbands = int32_t(H / 9);
    a.bands_per_unit = plan.bands_per_unit;
    a.units_per_plane = plan.units_per_plane;
    a.stages = plan.stages;
    const RingGeom geom = ring_geom(in_dtype, plan.out_es, W, plan.flags);
    a.stage_bytes = geom.stage_bytes;
    a.stage_stride = geom.stage_stride;
    a.out_bytes = geom.out_bytes;
    a.n_consumer = plan.block - 32;
    for (int c = 0; c < 2; ++c) {
        L->k[c] = pick(in_dtype, plan.out_es, c == 1, plan.reps_per_thread, W, plan.flags, plan.block,
                       plan.ctas_per_sm);
        aol_status_t st = kernel_smem(reinterpret_cast<const void*>(L->k[c]), plan.smem);
        if (st != AOL_OK) return st;
    }
    return AOL_OK;
}

aol_status_t enqueue_fused(const FusedLaunch& L, uint64_t* d_cs, cudaStream_t s) {
    FusedArgs a = L.args;
    a.cs = d_cs;
    KernelFn k = L.k[d_cs ? 1 : 0];
    // With checksums: zero them in a one-CTA kernel and launch the fused kernel as its programmatic
    // dependent, so the zeroing (and the launch gap after it) overlaps the fused kernel's start instead of
    // preceding it (single-frame latency).  Only the zero kernel can be the primary: it
    // is an ordinary launch, so everything earlier in the stream (e.g. the producer of X) has completed.
    // PDL invariant: the fused kernel issues its TMA loads and bulk stores without griddepcontrol.wait, so it
    // may only be a programmatic dependent of zero_checksums_kernel (which touches nothing but cs and waits
    // for its own predecessor); pdl therefore requires d_cs, and the zero kernel is launched right before it.
    const bool zero = d_cs != nullptr;
    const bool pdl = zero && !(L.flags & AOL_FLAG_NO_PDL);
    if (zero) {
        cudaLaunchConfig_t zc;
        std::memset(&zc, 0, sizeof zc);
        zc.gridDim = dim3(1);
        zc.blockDim = dim3(256);
        zc.stream = s;
        cudaLaunchAttribute za[1];
        za[0].id = cudaLaunchAttributeProgrammaticStreamSerialization;
        za[0].val.programmaticStreamSerializationAllowed = 1;
        zc.attrs = za;
        zc.numAttrs = pdl ? 1 : 0;
        cudaError_t ze = cudaLaunchKernelEx(&zc, zero_checksums_kernel, d_cs, int64_t(L.frames));
        if (ze != cudaSuccess) {
            set_error("launch of zero_checksums_kernel failed: %s", cudaGetErrorString(ze));
            return AOL_E_CUDA;
        }
    }
    cudaLaunchConfig_t cfg;
    std::memset(&cfg, 0, sizeof cfg);
    cfg.gridDim = dim3(unsigned(L.grid));
    cfg.blockDim = dim3(unsigned(L.block));
    cfg.dynamicSmemBytes = size_t(L.smem);
    cfg.stream = s;
    cudaLaunchAttribute attr[1];
    attr[0].id = cudaLaunchAttributeProgrammaticStreamSerialization;
    attr[0].val.programmaticStreamSerializationAllowed = 1;
    cfg.attrs = attr;
    cfg.numAttrs = pdl ? 1 : 0;
    cudaError_t le = cudaLaunchKernelEx(&cfg, k, L.map, a);
    note_launch("fused_tma_kernel");
    if (le != cudaSuccess) {
        set_error("launch of fused_tma_kernel failed: %s", cudaGetErrorString(le));
        return AOL_E_CUDA;
    }
    return AOL_OK;
}

aol_status_t launch_fused(const FusedPlan& plan, const void* d_in, aol_dtype_t in_dtype, void* d_out,
                          int64_t frames, int64_t channels, int64_t H, int64_t W, uint64_t* d_cs, cudaStream_t s) {
    if (plan.kernel == 2) {
        const bool rgb = in_dtype == AOL_RGB8;
        const int64_t planes = rgb ? frames : frames * channels;
        const int32_t Ho = int32_t(4 * (H / 9)), Wo = int32_t(3 * (W / 8));
        if (in_dtype == AOL_U8 && plan.out_es == 2)
            return launch_generic<uint8_t, int16_t>(plan, d_in, d_out, d_cs, frames, planes, H, W, Ho, Wo, channels, s);
        if (in_dtype == AOL_U8)
            return launch_generic<uint8_t, int32_t>(plan, d_in, d_out, d_cs, frames, planes, H, W, Ho, Wo, channels, s);
        return launch_generic<int32_t, int32_t>(plan, d_in, d_out, d_cs, frames, planes, H, W, Ho, Wo, channels, s);
    }
    FusedLaunch L;
    aol_status_t st = prepare_fused(plan, d_in, in_dtype, d_out, frames, channels, H, W, &L);
    if (st != AOL_OK) return st;
    // Everything that can fail before the kernels run has been resolved (plan, tensor map, smem attributes);
    // the pre-flight checks the configuration is runnable.  Nothing has been enqueued yet.
    st = launch_preflight(reinterpret_cast<const void*>(L.k[d_cs ? 1 : 0]), L.block, L.smem, "fused_tma_kernel");
    if (st != AOL_OK) return st;
    return enqueue_fused(L, d_cs, s);
}

}  // namespace aol
