/*
 * aol.h -- C ABI of the B200 (sm_100a) ArrayOL downscaler library (libaol.so).
 *
 * What it computes: the data-parallel hot path of Guo et al., "Harnessing the
 * Power of GPUs without Losing Abstractions in SaC and ArrayOL" (HIPS 2011),
 * /root/reference/PAPER.md ("P:Lnnn" = line nnn).  The paper's running
 * example is a two-stage HD->SD video downscaler (Fig. 2; task
 * graph Fig. 3) whose stages are ArrayOL repetitions connected by
 * tilers (Section IV):
 *
 *   pattern element  e(r, i) = (o + P.r + F.i) mod s_array
 *   horizontal filter: pattern {11} every 8 columns -> 3 outputs   (Fig. 10)
 *   vertical filter:   pattern {12} every 9 rows    -> 4 outputs   (reading Z1)
 *   task: tile[k] = tmp/6 - tmp%6, tmp = 6-tap window sum          (Fig. 5)
 *
 * Conventions for every entry point:
 *  - Device pointers ("d_") are owned by the caller (e.g. PyTorch); the library
 *    allocates no device memory.  Its only global state is a thread-local
 *    error string and mutex-guarded memos of immutable per-process facts
 *    (device attributes, kernel attributes it set, occupancy), so it is
 *    re-entrant and thread-safe.
 *  - Device calls are stream-ordered on the given stream and return after
 *    launch (asynchronous).  Kernel faults surface at the caller's next sync.
 *  - Errors are returned synchronously as aol_status_t for invalid arguments,
 *    shapes, dtypes, alignment, and launch failures; aol_last_error() then
 *    holds a message.  A device call that returns an error has enqueued
 *    nothing: arguments, the launch plan, the TMA descriptor, kernel
 *    attributes and the launch configuration are all checked before the first
 *    enqueue (tested with aol_debug_fail_next_launches, aol_tuning.h).  The one
 *    exception is a CUDA launch that fails after that pre-flight (a broken CUDA
 *    context): then an earlier kernel of the same call (the checksum zeroing) may
 *    already be enqueued.  aol_downscale_frame_host is a pipeline of many
 *    enqueues: see its comment.
 *  - Integer arithmetic is exact: results are bit-identical to the CPU oracle.
 *  - Arrays are dense row-major; a batch of frames is planar
 *    [frames][channels][H][W] (reading Z8: one plane per colour channel,
 *    P:L671-675).
 */
#ifndef AOL_H
#define AOL_H

#include <stddef.h>
#include <stdint.h>

/* The one CUDA type in these signatures, declared as cuda_runtime_api.h declares it (an identical
 * typedef may be repeated in C11 and C++), so this header needs no CUDA include path. */
typedef struct CUstream_st* cudaStream_t;

#ifdef __cplusplus
extern "C" {
#endif

#define AOL_VERSION 100 /* 1.0.0 */

#if defined(__GNUC__)
#define AOL_API __attribute__((visibility("default")))
#else
#define AOL_API
#endif
#define AOL_MAX_RANK 8

typedef enum {
    AOL_OK = 0,
    AOL_E_INVALID = -1,   /* null pointer, rank or extent out of range, bad enum        */
    AOL_E_SHAPE = -2,     /* W % 8 != 0, H % 9 != 0, or a shape the call cannot pave     */
    AOL_E_DTYPE = -3,     /* element type not supported by this entry point              */
    AOL_E_ALIGN = -4,     /* pointer not 16-byte aligned (TMA / vector access)          */
    AOL_E_WORKSPACE = -5, /* workspace missing or too small                              */
    AOL_E_RANGE = -6,     /* index arithmetic would overflow int64                       */
    AOL_E_CUDA = -7       /* CUDA runtime / driver error (message in aol_last_error())   */
} aol_status_t;

typedef enum {
    AOL_U8 = 1, AOL_I16 = 2, AOL_I32 = 3, AOL_I64 = 4, /* typed elements            */
    AOL_RAW8 = 5, AOL_RAW16 = 6, AOL_RAW32 = 7, AOL_RAW64 = 8, /* raw bytes, same sizes */
    AOL_RGB8 = 9 /* fused downscaler input only: packed 24-bit pixels, frames [N][H][W][3] of 8-bit samples
                    (P:L260's 24-bit RGB as OpenCV delivers it); channels must be 3 */
} aol_dtype_t;

typedef enum {
    AOL_SCATTER_FAST = 0,      /* caller asserts the output tiler is injective (ArrayOL single
                                  assignment); one pass                             */
    AOL_SCATTER_SEQUENTIAL = 1 /* Fig. 6 semantics: the LAST (r, i) in row-major
                                  loop order wins on collisions; needs a workspace              */
} aol_scatter_mode_t;

/* ArrayOL tiler record (Fig. 10; Section IV).
 * Shapes are extents > 0.  Matrices are row-major [array_dim][column]:
 * paving[a][j] multiplies repetition index r_j, fitting[a][k] multiplies
 * pattern index i_k (reading Z6: the paper prints matrices by columns; Fig. 11
 * P:L720-725 pins the orientation).  origin and all matrix entries may be
 * negative; the modulo is Euclidean, giving [0, s) (reading Z4).
 * rep_rank / pattern_rank may be 0 (a single repetition / a scalar pattern). */
typedef struct {
    int32_t array_rank, rep_rank, pattern_rank; /* 1..8, 0..8, 0..8 */
    int64_t array_shape[AOL_MAX_RANK];
    int64_t rep_shape[AOL_MAX_RANK];
    int64_t pattern_shape[AOL_MAX_RANK];
    int64_t origin[AOL_MAX_RANK];
    int64_t paving[AOL_MAX_RANK][AOL_MAX_RANK];
    int64_t fitting[AOL_MAX_RANK][AOL_MAX_RANK];
} aol_tiler_t;

typedef enum {
    AOL_PRESET_H_IN = 0,  /* Fig. 10 input tiler:  array {H,W}, pattern {11}, F=(0,1)^T, P=diag(1,8), rep {H,W/8} */
    AOL_PRESET_H_OUT = 1, /* Fig. 10 output tiler: array {H,3W/8}, pattern {3}, F=(0,1)^T, P=diag(1,3), rep {H,W/8} */
    AOL_PRESET_V_IN = 2,  /* reading Z1: array {H,W}, pattern {12}, F=(1,0)^T, P=diag(9,1), rep {H/9,W}            */
    AOL_PRESET_V_OUT = 3  /* reading Z1: array {4H/9,W}, pattern {4}, F=(1,0)^T, P=diag(4,1), rep {H/9,W}           */
} aol_preset_t;

/* Optional launch tuning for aol_downscale_frame_ex (all zero = automatic). */
typedef struct {
    int32_t ctas_per_sm;    /* resident CTAs per SM for the fused kernel (1..8), 0 = auto       */
    int32_t stages;         /* TMA ring depth in 3-row stages, 0 = as many as fit              */
    int32_t bands_per_unit; /* 9-row bands per work unit, 0 = auto (balance waves vs halo)     */
    int32_t kernel;         /* 0 = auto, 1 = TMA fused kernel (error if shape unsupported),
                               2 = generic fused kernel (any W%8==0, H%9==0)                   */
    int32_t flags;          /* 0 in production; A/B experiment bits of aol_tuning.h (results are
                               identical whatever the bits)                                    */
} aol_launch_opts_t;

/* The launch configuration aol_downscale_frame_ex would use (for reports/tests). */
typedef struct {
    int32_t kernel;          /* 1 = TMA fused, 2 = generic fused                      */
    int32_t grid, block;     /* CTAs, threads per CTA                                 */
    int32_t smem_bytes;      /* dynamic shared memory per CTA                         */
    int32_t stages;          /* TMA ring depth (kernel 1)                              */
    int32_t bands_per_unit;  /* kernel 1                                               */
    int64_t units;           /* work units (kernel 1)                                  */
    int32_t ctas_per_sm;     /* kernel 1                                               */
    int32_t num_sms;
} aol_plan_t;

/* ------------------------------------------------------------------ misc */

/* Library version (AOL_VERSION). Never fails. */
AOL_API int aol_version(void);

/* Thread-local message describing the last error on this thread ("" if none).
 * The pointer stays valid until the next aol_* call on the same thread. */
AOL_API const char* aol_last_error(void);

/* ------------------------------------------------------- tiler descriptors */

/* Fill *out with the paper's tiler `which` for one plane.  H_IN/H_OUT take the
 * input plane H x W (W % 8 == 0); V_IN/V_OUT take the intermediate plane
 * H x W (H % 9 == 0).  Host only.  AOL_E_INVALID / AOL_E_SHAPE on bad input. */
AOL_API aol_status_t aol_tiler_preset(aol_preset_t which, int64_t H, int64_t W, aol_tiler_t* out);

/* Check ranks, extents, and that every index computation fits in int64.
 * Host only.  Returns AOL_OK, AOL_E_INVALID or AOL_E_RANGE. */
AOL_API aol_status_t aol_tiler_validate(const aol_tiler_t* t);

/* *injective = 1 if no two (r, i) pairs address the same array element
 * (brute force over the repetition x pattern space; a test helper meant for
 * small descriptors).  Host only. */
AOL_API aol_status_t aol_tiler_is_injective(const aol_tiler_t* t, int* injective);

/* --------------------------------------------------- generic gather/scatter */

/* Input tiler (Fig. 4; Section IV):
 *   d_tiles[r][i] = d_array[(o + P.r + F.i) mod s]
 * d_array: device, array_shape row-major, element type el (size 1/2/4/8 B).
 * d_tiles: device, [rep_shape..., pattern_shape...] row-major, same element type.
 * Both must be aligned to the element size.  Async on s. */
AOL_API aol_status_t aol_tiler_gather(const aol_tiler_t* t, aol_dtype_t el, const void* d_array, void* d_tiles,
                              cudaStream_t s);

/* Bytes of device workspace aol_tiler_scatter needs in SEQUENTIAL mode
 * (8 bytes per array element; 0 for a NULL/invalid tiler). */
AOL_API size_t aol_tiler_scatter_workspace_bytes(const aol_tiler_t* t);

/* Output tiler (Fig. 6; modarray): d_array[(o+P.r+F.i) mod s] = d_tiles[r][i],
 * in place -- elements no (r, i) addresses keep their value.
 * FAST: caller asserts injectivity (ArrayOL single assignment); collisions are
 * then unspecified.  SEQUENTIAL: Fig. 6's loop order, the last writer wins;
 * d_workspace must hold aol_tiler_scatter_workspace_bytes(t) bytes (it is
 * overwritten).  Async on s. */
AOL_API aol_status_t aol_tiler_scatter(const aol_tiler_t* t, aol_dtype_t el, const void* d_tiles, void* d_array,
                               aol_scatter_mode_t mode, void* d_workspace, size_t ws_bytes, cudaStream_t s);

/* ------------------------------------------------------------- the filters */

/* Horizontal filter alone (the SaC/GASPARD2 "HorizontalFilter", Fig. 10 tilers
 * + Fig. 5 task): d_in int32 [planes][H][W] -> d_out int32 [planes][H][3W/8].
 * W % 8 == 0 else AOL_E_SHAPE.  Pointers 4-byte aligned (a 16-byte aligned input takes the
 * 128-bit vector path).  Async on s. */
AOL_API aol_status_t aol_downscale_h(const int32_t* d_in, int32_t* d_out, int64_t planes, int64_t H, int64_t W,
                             cudaStream_t s);

/* Vertical filter alone (reading Z1/Z2): d_in int32 [planes][H][W] ->
 * d_out int32 [planes][4H/9][W].  H % 9 == 0 else AOL_E_SHAPE.  Async on s. */
AOL_API aol_status_t aol_downscale_v(const int32_t* d_in, int32_t* d_out, int64_t planes, int64_t H, int64_t W,
                             cudaStream_t s);

/* The fused downscaler (hf -> vf of Fig. 3 in one kernel, the intermediate
 * never touches HBM -- the hand-written analogue of SaC's WITH-loop folding,
 * P:L528-546): d_in [frames][channels][H][W] -> d_out int32
 * [frames][channels][4H/9][3W/8], H filter first (Fig. 2).
 * in_dtype: AOL_I32 (values must lie in (-2^27, 2^27), reading Z12), AOL_U8
 * (8-bit samples) or AOL_RGB8 (packed pixels: d_in [frames][H][W][3] bytes, channels == 3,
 * W % 16 == 0, W <= 6400 with int32 outputs / 7936 with int16 outputs; the output is still planar).  d_frame_checksums: nullable device u64 [frames],
 * 8-byte aligned, overwritten with
 * sum (u64)(u32)Z[n][c][y][x] * (1 + (c*Ho + y)*Wo + x)  mod 2^64.
 * frames == 0 is a no-op.  d_in/d_out 16-byte aligned.  Async on s. */
AOL_API aol_status_t aol_downscale_frame(const void* d_in, aol_dtype_t in_dtype, int32_t* d_out, int64_t frames,
                                 int64_t channels, int64_t H, int64_t W, uint64_t* d_frame_checksums,
                                 cudaStream_t s);

/* Same, with explicit launch options (NULL = automatic). */
AOL_API aol_status_t aol_downscale_frame_ex(const void* d_in, aol_dtype_t in_dtype, int32_t* d_out, int64_t frames,
                                    int64_t channels, int64_t H, int64_t W, uint64_t* d_frame_checksums,
                                    const aol_launch_opts_t* opts, cudaStream_t s);

/* Report the launch aol_downscale_frame_ex would make on the current device. */
AOL_API aol_status_t aol_downscale_frame_plan(aol_dtype_t in_dtype, int64_t frames, int64_t channels, int64_t H,
                                      int64_t W, const aol_launch_opts_t* opts, aol_plan_t* out);

/* The fused downscaler with the output element type chosen (NEXT row f1): out_dtype AOL_I32 (as
 * aol_downscale_frame_ex) or AOL_I16 -- only with in_dtype AOL_U8, whose outputs lie in [-5, 255]
 * (P:L260, 8-bit samples): d_out int16 [frames][channels][4H/9][3W/8], 2 bytes per output instead of 4.
 * The checksums are those of the same integer outputs (identical for both output types).  AOL_E_DTYPE
 * for other combinations; otherwise as aol_downscale_frame_ex. */
AOL_API aol_status_t aol_downscale_frame_out(const void* d_in, aol_dtype_t in_dtype, void* d_out,
                                             aol_dtype_t out_dtype, int64_t frames, int64_t channels, int64_t H,
                                             int64_t W, uint64_t* d_frame_checksums, const aol_launch_opts_t* opts,
                                             cudaStream_t s);

/* Report the launch aol_downscale_frame_out would make on the current device. */
AOL_API aol_status_t aol_downscale_frame_plan_out(aol_dtype_t in_dtype, aol_dtype_t out_dtype, int64_t frames,
                                                  int64_t channels, int64_t H, int64_t W,
                                                  const aol_launch_opts_t* opts, aol_plan_t* out);

/* ------------------------------------------------ persistent launch plans */

/* A fused-downscale launch resolved once for fixed device buffers and shape (the d1 single-frame case,
 * where per-call host planning outweighs the kernel: the launch-overhead argument of P:L776-779).
 * aol_frame_plan_create checks the arguments exactly as aol_downscale_frame_out, plans the launch, encodes
 * the TMA descriptor of d_in, sets kernel attributes and records the launches as a CUDA graph (on a private
 * stream), once.  Host only; frames > 0; the plan allocates no buffers of its own. */
typedef struct aol_frame_plan* aol_frame_plan_t;
AOL_API aol_status_t aol_frame_plan_create(const void* d_in, aol_dtype_t in_dtype, void* d_out, aol_dtype_t out_dtype,
                                           int64_t frames, int64_t channels, int64_t H, int64_t W,
                                           const aol_launch_opts_t* opts, aol_frame_plan_t* plan);

/* Enqueue the planned downscale on s (the device current at creation): d_in -> d_out as
 * aol_downscale_frame_out, with d_frame_checksums (nullable, 8-byte aligned, [frames], overwritten).
 * ONE cudaGraphLaunch of the recorded launches (checksum zeroing + the fused kernel as its programmatic
 * dependent); the first call with a new checksum pointer records that graph first; into a stream that is
 * being captured the two launches are enqueued directly.  Not thread-safe for one plan.  Argument errors are those of a NULL plan or a misaligned checksum pointer. */
AOL_API aol_status_t aol_frame_plan_launch(aol_frame_plan_t plan, uint64_t* d_frame_checksums, cudaStream_t s);

/* The launch configuration the plan uses. */
AOL_API aol_status_t aol_frame_plan_info(aol_frame_plan_t plan, aol_plan_t* out);

/* Free the plan and its recorded graphs (launches already enqueued are unaffected).  NULL is a no-op. */
AOL_API aol_status_t aol_frame_plan_destroy(aol_frame_plan_t plan);

/* Per-frame checksum of an existing output batch (for the unfused paths):
 * d_out int32 [frames][channels][Ho][Wo] -> d_checksums u64 [frames] (overwritten). */
AOL_API aol_status_t aol_frame_checksum(const int32_t* d_out, int64_t frames, int64_t channels, int64_t Ho, int64_t Wo,
                                uint64_t* d_checksums, cudaStream_t s);

/* ------------------------------------------------- host-streamed end to end */

/* Device workspace aol_downscale_frame_host needs for chunks of chunk_frames frames. */
AOL_API size_t aol_downscale_frame_host_workspace_bytes(aol_dtype_t in_dtype, int64_t chunk_frames, int64_t channels,
                                                int64_t H, int64_t W);

/* The downscaler fed from and drained to HOST memory (the paper's runtime loop:
 * H2D, filters, D2H per frame, Table I), pipelined in chunks of
 * chunk_frames frames over three caller streams: s_h2d copies chunk k+1 in while
 * s_compute downscales chunk k and s_d2h copies chunk k-1 out.
 * h_in / h_out / h_frame_checksums: host buffers (pinned memory gives overlap;
 * pageable memory works but serialises).  d_workspace: device, at least
 * aol_downscale_frame_host_workspace_bytes(...) bytes.  BLOCKING: returns when
 * h_out (and h_frame_checksums, nullable) are complete. */
/* On an error in the middle of the pipeline, the chunks enqueued before it still complete (the call
 * synchronises the three streams before returning); h_out then holds those chunks' results, the rest
 * is unspecified. */
AOL_API aol_status_t aol_downscale_frame_host(const void* h_in, aol_dtype_t in_dtype, int32_t* h_out, int64_t frames,
                                      int64_t channels, int64_t H, int64_t W, uint64_t* h_frame_checksums,
                                      int64_t chunk_frames, void* d_workspace, size_t ws_bytes,
                                      cudaStream_t s_h2d, cudaStream_t s_compute, cudaStream_t s_d2h);

/* ------------------------------------ generic fused repetition (NEXT row f3) */

#define AOL_MAX_FILTER_PATTERN 64 /* input pattern elements */
#define AOL_MAX_WINDOWS 16        /* output pattern elements */

/* One ArrayOL repetition, fully described at run time: an input tiler, a
 * windowed-sum task and an output tiler -- the SaC "generic" downscaler of
 * Fig. 4 (input_tiler) + Fig. 5 (task) + Fig. 6 (generic_output_tiler),
 * P:L384-471, generalised to any window layout:
 *   for every repetition r (in.rep_shape == out.rep_shape):
 *     p      = the in.pattern elements gathered at r (flattened row-major)
 *     tile[k] = S/divisor - S%divisor,  S = sum_{t<window_len} p[window_start[k] + t]   (C int)
 *     out[(o' + P'.r + F'.k) mod s'] = tile[k]          (k < n_windows = out pattern elements)
 * The paper's filters are presets (aol_filter_preset).  Gather, task and
 * scatter run in ONE kernel (no intermediate arrays: WLF for arbitrary
 * tilers).  Array extents must be < 2^31; the output tiler must be injective
 * (ArrayOL single assignment) or results at colliding cells are unspecified. */
typedef struct {
    aol_tiler_t in;
    aol_tiler_t out;
    int32_t n_windows;  /* 1..AOL_MAX_WINDOWS, = out pattern element count          */
    int32_t window_len; /* >= 1; window_start[k] + window_len <= in pattern elements */
    int32_t divisor;    /* != 0                                                       */
    int32_t window_start[AOL_MAX_WINDOWS];
} aol_filter_t;

typedef enum {
    AOL_FILTER_H = 0, /* horizontal filter of Fig. 10 + Fig. 5 on [planes][H][W]   -> [planes][H][3W/8]  */
    AOL_FILTER_V = 1  /* vertical filter (reading Z1/Z2) on [planes][H][W]         -> [planes][4H/9][W]  */
} aol_filter_kind_t;

/* The paper's filters as 3-D repetitions over a stack of planes (the plane index is one more
 * repetition dimension with paving 1 -- time/channels as array dimensions). */
AOL_API aol_status_t aol_filter_preset(aol_filter_kind_t which, int64_t planes, int64_t H, int64_t W,
                                       aol_filter_t* out);

/* Check a filter description (ranks, shapes, windows, divisor, int32 ranges).  Host only. */
AOL_API aol_status_t aol_filter_validate(const aol_filter_t* f);

/* Apply a filter: d_in int32 shaped f->in.array_shape, d_out int32 shaped f->out.array_shape
 * (cells no repetition writes keep their value).  4-byte aligned.  Async on s.
 * A row filter or a column filter (pattern along the last / second-to-last dimension, diagonal paving,
 * dense output -- the paper's H and V with any parameters) runs a kernel specialised for its
 * parameters at run time: compiled with NVRTC on the first call for that filter and array shape
 * (a fraction of a second, host side), cached for the process.  Without NVRTC, and for every other
 * filter, a statically compiled generic kernel runs.  Results are identical either way. */
AOL_API aol_status_t aol_filter_apply(const aol_filter_t* f, const int32_t* d_in, int32_t* d_out, cudaStream_t s);

/* Two repetitions chained -- f2 consumes f1's output array -- in ONE kernel: d_out = f2(f1(d_in)), the
 * intermediate array never stored (WITH-loop folding across repetitions, for run-time
 * descriptors; the paper's generic filters ran as separate kernels with host-side tilers).
 * Fused when f1's output tiler is a bijection onto its array whose window digits are the low digits of
 * each dimension (the paper's H and V output tilers are), f2's output tiler does not wrap, ranks <= 4 and
 * patterns <= 16 elements; otherwise the two filters run as two launches through d_workspace (>= the
 * intermediate array's bytes; NULL -> AOL_E_WORKSPACE naming the reason).  f1.out.array_shape must equal
 * f2.in.array_shape.  d_in / d_out int32 shaped f1.in / f2.out arrays, 4-byte aligned.  Async on s.
 * A row filter followed by a column filter (the paper's H -> V shape, any parameters) runs a kernel
 * specialised at run time as for aol_filter_apply (first call per filter pair and shape compiles). */
AOL_API aol_status_t aol_filter_chain_apply(const aol_filter_t* f1, const aol_filter_t* f2, const int32_t* d_in,
                                            int32_t* d_out, void* d_workspace, size_t ws_bytes, cudaStream_t s);

/* ------------------------------------------- synthetic input (test support) */

/* Fill d_out [nframes][channels][H][W] with the counter-based synthetic frames
 * of synth/ (the seeded generator shared with the oracle side; it stands in
 * for the paper's OpenCV FrameGenerator):
 *   u = splitmix64(seed*0x9E3779B97F4A7C15 + (((frame0+n)*channels + c)*H + y)*W + x)
 *   kind 0 uniform u>>56 | 1 dark u>>61 | 2 signed (u>>37) - 2^26 | 3 ramp x | 4 constant value
 * out_dtype AOL_I32 or AOL_U8 (kinds whose values fit).  Async on s. */
AOL_API aol_status_t aol_synth_frames(uint64_t seed, int64_t frame0, int64_t nframes, int64_t channels, int64_t H,
                              int64_t W, int32_t kind, int32_t value, aol_dtype_t out_dtype, void* d_out,
                              cudaStream_t s);

#ifdef __cplusplus
}
#endif
#endif /* AOL_H */
