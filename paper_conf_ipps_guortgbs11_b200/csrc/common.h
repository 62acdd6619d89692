// common.h -- host-side internals shared by the library's translation units.
#pragma once
#include <cstdint>
#include <cstdio>
#include <string>

#include <cuda_runtime.h>

#include "../../include/aol.h"
#include "../../include/aol_tuning.h"

namespace aol {

// Thread-local last-error message (besides the memos in api.cu, the library's only mutable state).
void set_error(const char* fmt, ...) __attribute__((format(printf, 1, 2)));
void clear_error();
const char* last_error_cstr();

inline aol_status_t fail(aol_status_t st, const char* what) {
    set_error("%s", what);
    return st;
}

// Check a CUDA runtime call; on failure record the message and return AOL_E_CUDA.
#define AOL_CUDA_TRY(call)                                                                            \
    do {                                                                                              \
        cudaError_t err__ = (call);                                                                   \
        if (err__ != cudaSuccess) {                                                                   \
            ::aol::set_error("%s failed: %s (%s:%d)", #call, cudaGetErrorString(err__), __FILE__,     \
                             __LINE__);                                                               \
            return AOL_E_CUDA;                                                                        \
        }                                                                                             \
    } while (0)

// Name of the last kernel this thread launched (aol_debug_last_kernel, a test / report hook).
void note_launch(const char* what);

// After a launch: report launch-configuration errors synchronously.
#define AOL_LAUNCH_CHECK(what)                                                                        \
    do {                                                                                              \
        ::aol::note_launch(what);                                                                     \
        cudaError_t err__ = cudaGetLastError();                                                       \
        if (err__ != cudaSuccess) {                                                                   \
            ::aol::set_error("launch of %s failed: %s", what, cudaGetErrorString(err__));             \
            return AOL_E_CUDA;                                                                        \
        }                                                                                             \
    } while (0)

inline bool aligned16(const void* p) { return (reinterpret_cast<uintptr_t>(p) & 15u) == 0; }

struct DeviceInfo {
    int device;
    int num_sms;
    int smem_optin;   // max dynamic smem per block (opt-in)
    int smem_per_sm;  // shared memory per multiprocessor
};
aol_status_t device_info(DeviceInfo* out);               // memoised per device
aol_status_t kernel_smem(const void* fn, int smem_bytes);   // cudaFuncSetAttribute(MaxDynamicSmem), memoised
int kernel_occupancy(const void* fn, int block, int smem);  // resident CTAs per SM, memoised (0 on error)
// Pre-flight of a launch about to be enqueued: the configuration must be runnable (occupancy >= 1 CTA/SM),
// and the test hook aol_debug_fail_next_launches() may force a failure here.  Called before the FIRST
// enqueue of an entry point, so a failing call leaves the caller's buffers untouched.
aol_status_t launch_preflight(const void* fn, int block, int smem, const char* what);
aol_status_t debug_injected_failure(const char* what);   // the test hook alone (AOL_OK unless armed)

// ---- launchers implemented in the .cu files (all validate nothing; callers do)
struct FusedPlan {
    int kernel;  // 1 = TMA fused, 2 = generic fused
    int grid, block, smem, stages, bands_per_unit, ctas_per_sm, num_sms, units_per_plane, flags;
    int reps_per_thread;  // kernel 1: H-tiler repetitions per consumer thread (1, or 2 for wide uint8 frames)
    int out_es;           // output element bytes: 4 (int32) or 2 (int16, uint8 input only)
    int64_t units;
};

// Argument checks of the fused entry points (shapes, dtypes, alignment incl. the checksum pointer, options).
aol_status_t validate_frame_call(const void* d_in, aol_dtype_t in_dtype, const void* d_out, aol_dtype_t out_dtype,
                                 int64_t frames, int64_t channels, int64_t H, int64_t W, const uint64_t* d_cs,
                                 const aol_launch_opts_t* opts);
struct FusedPlan;
void fill_plan_info(const FusedPlan& p, aol_plan_t* out);

aol_status_t plan_fused(aol_dtype_t in_dtype, aol_dtype_t out_dtype, const void* d_in, const void* d_out,
                        int64_t frames, int64_t channels, int64_t H, int64_t W, const aol_launch_opts_t* opts,
                        FusedPlan* plan, bool checksum = true);
aol_status_t launch_fused(const FusedPlan& plan, const void* d_in, aol_dtype_t in_dtype, void* d_out,
                          int64_t frames, int64_t channels, int64_t H, int64_t W, uint64_t* d_cs, cudaStream_t s);

// chain_sep.cu: aol_filter_chain_apply's separable case (a row filter then a column filter).  false: not that
// case (nothing done); true: handled, *st = the outcome.
bool launch_sep_chain(const aol_filter_t* f1, const aol_filter_t* f2, const int32_t* d_in, int32_t* d_out,
                      cudaStream_t s, aol_status_t* st);
// aol_filter_apply for a single row filter or column filter: the separable chain kernel with an identity partner
// filter, specialised at run time (false when NVRTC is absent or the filter is not of that shape).
bool launch_sep_single(const aol_filter_t* f, const int32_t* d_in, int32_t* d_out, cudaStream_t s, aol_status_t* st);

aol_status_t launch_downscale_h(const int32_t* d_in, int32_t* d_out, int64_t planes, int64_t H, int64_t W,
                                cudaStream_t s);
aol_status_t launch_downscale_v(const int32_t* d_in, int32_t* d_out, int64_t planes, int64_t H, int64_t W,
                                cudaStream_t s);
aol_status_t launch_checksum(const int32_t* d_out, int64_t frames, int64_t per_frame, uint64_t* d_cs,
                             cudaStream_t s);

// Generic tiler: device-ready descriptor (coefficients reduced mod the array extents).
struct TilerDev {
    int32_t ra, nd;             // array rank, combined (rep ++ pattern) rank
    int32_t linear;             // 1: no coordinate can wrap -> offset is affine in the tile index
    int32_t fast32;             // 1: total < 2^31 -> 32-bit magic-number division
    int32_t small32;            // 1: linear, total and array offsets < 2^31 -> all-32-bit linear kernel
    uint32_t nowrap_mask;       // bit a: array dim a never wraps
    int64_t ext[2 * AOL_MAX_RANK];
    int64_t coef[AOL_MAX_RANK][2 * AOL_MAX_RANK];
    int64_t org[AOL_MAX_RANK];
    int64_t ashape[AOL_MAX_RANK];
    int64_t astride[AOL_MAX_RANK];
    int64_t lin[2 * AOL_MAX_RANK];  // element offset per unit of combined index d (linear tilers)
    int64_t base;                   // element offset of the origin
    uint32_t fd_mul[2 * AOL_MAX_RANK], fd_shift[2 * AOL_MAX_RANK];
    // Linear tilers are walked in an order that makes the ARRAY side contiguous (dims sorted by
    // array stride, smallest innermost); p_* describe the permuted dims: extent, array stride,
    // tile stride (row-major over the natural [rep..., pattern...] order) and magic divisors.
    int64_t p_ext[2 * AOL_MAX_RANK], p_lin[2 * AOL_MAX_RANK], p_gst[2 * AOL_MAX_RANK];
    uint32_t p_fd_mul[2 * AOL_MAX_RANK], p_fd_shift[2 * AOL_MAX_RANK];
    int64_t total;              // rep elements * pattern elements
    int64_t array_elems;
    int32_t proven_injective;   // 1: the host proved no two (r, i) address the same element (see api.cu);
                                // SEQUENTIAL scatters then take the one-pass FAST kernels
};
// Bytes per array element of the SEQUENTIAL scatter's claim workspace: 0 when proven injective, 4 when every
// claim (flat tile index + 1) fits 32 bits, else 8.
int claim_bytes(const TilerDev& td);
aol_status_t make_tiler_dev(const aol_tiler_t* t, TilerDev* out);
aol_status_t launch_gather(const TilerDev& td, int elsize, const void* d_array, void* d_tiles, cudaStream_t s);
aol_status_t launch_scatter(const TilerDev& td, int elsize, const void* d_tiles, void* d_array, int sequential,
                            void* d_ws, cudaStream_t s);

aol_status_t launch_synth(uint64_t seed, int64_t frame0, int64_t nframes, int64_t channels, int64_t H, int64_t W,
                          int32_t kind, int32_t value, int out_u8, void* d_out, cudaStream_t s);

int elsize_of(aol_dtype_t el);

}  // namespace aol
