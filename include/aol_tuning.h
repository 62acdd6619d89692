/*
 * aol_tuning.h -- A/B experiment switches of libaol.so (not part of the stable API).
 *
 * Bits for aol_launch_opts_t.flags (include/aol.h).  Each selects an alternative
 * launch or shared-memory layout of the fused downscaler that was measured against the
 * default on B200 (profiles/); results are bit-identical whatever the bits.  Production
 * callers pass 0.  Round-1 dead ends (L2 evict_first hints, blocked unit order, forced
 * 1-D uint8 copies, SWIZZLE_32B int32 lines) were measured no faster and removed.
 */
#ifndef AOL_TUNING_H
#define AOL_TUNING_H

#include "aol.h"

#define AOL_FLAG_U8_ONE_REP 32      /* uint8 input: one H repetition per consumer thread even for W >= 1024
                                       (default there: two; profiles/r01_u8_r2_ab.jsonl)                   */
#define AOL_FLAG_NO_PDL 64          /* launch the fused kernel after the checksum zeroing completes (default:
                                       programmatic dependent launch, overlapped; profiles/r01_pdl_ab.jsonl) */
#define AOL_FLAG_I32_LINEAR 128     /* int32 input: 1-D bulk copies into linear smem rows even when W % 32 == 0
                                       (default there: TMA tensor loads, SWIZZLE_128B)                       */
#define AOL_FLAG_ROW_STAGES 512     /* int32 input: one row per TMA ring stage (default when a row triple
                                       exceeds a third of the ring's bytes: W > 3271)                        */
#define AOL_FLAG_TRIPLE_STAGES 1024 /* int32 input: one row triple per ring stage for any W                  */
#define AOL_FLAG_I32_STRIPS 2048    /* int32 input, W % 32 == 0: column strips of ~64 repetitions (default:
                                       strips of <= 512 only when W / 8 exceeds one CTA's 992 consumers, i.e.
                                       W > 7936; lets the tests exercise several strips at small widths)     */

#ifdef __cplusplus
extern "C" {
#endif

/* Test hook: the next n fused-downscaler launches on this thread fail in their pre-flight check (after
 * planning and tensor-map encoding, immediately before the first enqueue) with AOL_E_CUDA.  Lets a test
 * check that a failing call enqueues nothing -- the caller's output and checksum buffers stay untouched. */
AOL_API void aol_debug_fail_next_launches(int n);

/* Name of the last kernel an aol_* call launched on this thread (e.g. "tiler_box_kernel",
 * "fused_tma_kernel"); "" before any launch.  Lets tests and reports check which kernel path a
 * descriptor or shape takes. */
AOL_API const char* aol_debug_last_kernel(void);

/* Test hook: aol_filter_chain_apply's separable chains run the kernel specialised at run time by NVRTC (on,
 * the default unless AOL_CHAIN_JIT=0) or the statically compiled generic one (off).  Same results. */
AOL_API void aol_debug_set_chain_jit(int on);

/* Test hook, no GPU needed: compile (with NVRTC, without loading) the run-time specialised separable chain kernel
 * aol_filter_chain_apply would build for f1 -> f2.  Returns 1 (compiled; log = "register-resident" or "ring", the
 * kernel body chosen), 0 (not a separable chain; log = why), -1 (NVRTC not available), -2 (compilation failed;
 * log = the NVRTC log).  log may be NULL. */
AOL_API int aol_debug_sep_jit_compile(const aol_filter_t* f1, const aol_filter_t* f2, char* log, size_t cap);

#ifdef __cplusplus
}
#endif
#endif /* AOL_TUNING_H */
