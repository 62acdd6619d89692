// api.cu -- the C ABI (include/aol.h): argument validation, tiler descriptors,
// dispatch to the kernels, and the host-streamed end-to-end driver.
#include <cuda_runtime.h>

#include <algorithm>
#include <cstdarg>
#include <cstdint>
#include <cstring>
#include <mutex>
#include <string>
#include <unordered_map>
#include <vector>

#include "common.h"

namespace aol {

namespace {
thread_local std::string g_err;
}

void set_error(const char* fmt, ...) {
    char buf[512];
    va_list ap;
    va_start(ap, fmt);
    vsnprintf(buf, sizeof buf, fmt, ap);
    va_end(ap);
    g_err = buf;
}

void clear_error() { g_err.clear(); }

const char* last_error_cstr() { return g_err.c_str(); }

// Immutable per-process facts (device attributes, kernel attributes the library has set, occupancy
// of a kernel configuration) are memoised: they never change for a process, and querying them on
// every call made the host side of a launch several microseconds longer than a one-frame kernel.
namespace {
std::mutex g_cache_mu;
std::unordered_map<int, DeviceInfo> g_dev_cache;
std::unordered_map<std::string, int> g_kernel_cache;   // "dev:fn:smem" -> applied, "dev:fn:block:smem" -> occ

std::string key_of(int dev, const void* fn, int a, int b) {
    char buf[96];
    snprintf(buf, sizeof buf, "%d:%p:%d:%d", dev, fn, a, b);
    return buf;
}
}  // namespace

aol_status_t device_info(DeviceInfo* out) {
    int dev = 0;
    AOL_CUDA_TRY(cudaGetDevice(&dev));
    {
        std::lock_guard<std::mutex> lk(g_cache_mu);
        auto it = g_dev_cache.find(dev);
        if (it != g_dev_cache.end()) {
            *out = it->second;
            return AOL_OK;
        }
    }
    DeviceInfo d;
    d.device = dev;
    AOL_CUDA_TRY(cudaDeviceGetAttribute(&d.num_sms, cudaDevAttrMultiProcessorCount, dev));
    AOL_CUDA_TRY(cudaDeviceGetAttribute(&d.smem_optin, cudaDevAttrMaxSharedMemoryPerBlockOptin, dev));
    AOL_CUDA_TRY(cudaDeviceGetAttribute(&d.smem_per_sm, cudaDevAttrMaxSharedMemoryPerMultiprocessor, dev));
    std::lock_guard<std::mutex> lk(g_cache_mu);
    g_dev_cache[dev] = d;
    *out = d;
    return AOL_OK;
}

aol_status_t kernel_smem(const void* fn, int smem) {
    // the attribute is an upper bound: only ever raise it, and remember the largest value applied
    int dev = 0;
    AOL_CUDA_TRY(cudaGetDevice(&dev));
    const std::string k = key_of(dev, fn, -1, -1);
    std::lock_guard<std::mutex> lk(g_cache_mu);
    auto it = g_kernel_cache.find(k);
    if (it != g_kernel_cache.end() && it->second >= smem) return AOL_OK;
    AOL_CUDA_TRY(cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, smem));
    g_kernel_cache[k] = smem;
    return AOL_OK;
}

int kernel_occupancy(const void* fn, int block, int smem) {
    int dev = 0;
    if (cudaGetDevice(&dev) != cudaSuccess) return 0;
    const std::string k = key_of(dev, fn, block, smem);
    {
        std::lock_guard<std::mutex> lk(g_cache_mu);
        auto it = g_kernel_cache.find(k);
        if (it != g_kernel_cache.end()) return it->second;
    }
    int occ = 0;
    if (kernel_smem(fn, smem) != AOL_OK ||
        cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, fn, block, smem) != cudaSuccess) {
        (void)cudaGetLastError();
        return 0;
    }
    std::lock_guard<std::mutex> lk(g_cache_mu);
    g_kernel_cache[k] = occ;
    return occ;
}

namespace {
thread_local int g_fail_launches = 0;   // aol_debug_fail_next_launches (test hook)
thread_local const char* g_last_kernel = "";
}

void note_launch(const char* what) { g_last_kernel = what; }

aol_status_t debug_injected_failure(const char* what) {
    if (g_fail_launches > 0) {
        --g_fail_launches;
        set_error("launch of %s failed: injected failure (aol_debug_fail_next_launches)", what);
        return AOL_E_CUDA;
    }
    return AOL_OK;
}

aol_status_t launch_preflight(const void* fn, int block, int smem, const char* what) {
    aol_status_t st = debug_injected_failure(what);
    if (st != AOL_OK) return st;
    if (kernel_occupancy(fn, block, smem) < 1) {
        set_error("launch of %s is not runnable: %d threads with %d bytes of dynamic shared memory", what, block,
                  smem);
        return AOL_E_CUDA;
    }
    return AOL_OK;
}

int elsize_of(aol_dtype_t el) {
    switch (el) {
        case AOL_U8: case AOL_RAW8: return 1;
        case AOL_I16: case AOL_RAW16: return 2;
        case AOL_I32: case AOL_RAW32: return 4;
        case AOL_I64: case AOL_RAW64: return 8;
    }
    return 0;
}

namespace {

using i128 = __int128;
constexpr i128 kI64Max = i128(INT64_MAX);

int64_t emod(int64_t a, int64_t m) {
    int64_t r = a % m;
    return r < 0 ? r + m : r;
}

aol_status_t validate_tiler(const aol_tiler_t* t) {
    if (!t) return fail(AOL_E_INVALID, "tiler is NULL");
    if (t->array_rank < 1 || t->array_rank > AOL_MAX_RANK) return fail(AOL_E_INVALID, "array_rank must be 1..8");
    if (t->rep_rank < 0 || t->rep_rank > AOL_MAX_RANK) return fail(AOL_E_INVALID, "rep_rank must be 0..8");
    if (t->pattern_rank < 0 || t->pattern_rank > AOL_MAX_RANK)
        return fail(AOL_E_INVALID, "pattern_rank must be 0..8");
    i128 arr = 1, total = 1;
    for (int a = 0; a < t->array_rank; ++a) {
        if (t->array_shape[a] <= 0) return fail(AOL_E_INVALID, "array extents must be > 0");
        arr *= t->array_shape[a];
        if (arr > kI64Max / 8) return fail(AOL_E_RANGE, "array too large");
    }
    for (int j = 0; j < t->rep_rank; ++j) {
        if (t->rep_shape[j] <= 0) return fail(AOL_E_INVALID, "repetition extents must be > 0");
        total *= t->rep_shape[j];
        if (total > kI64Max / 8) return fail(AOL_E_RANGE, "repetition x pattern space too large");
    }
    for (int k = 0; k < t->pattern_rank; ++k) {
        if (t->pattern_shape[k] <= 0) return fail(AOL_E_INVALID, "pattern extents must be > 0");
        total *= t->pattern_shape[k];
        if (total > kI64Max / 8) return fail(AOL_E_RANGE, "repetition x pattern space too large");
    }
    // after reducing coefficients mod s_a, every coordinate sum is < s_a * (1 + sum of extents)
    for (int a = 0; a < t->array_rank; ++a) {
        i128 bound = t->array_shape[a];
        for (int j = 0; j < t->rep_rank; ++j) bound += i128(t->array_shape[a]) * t->rep_shape[j];
        for (int k = 0; k < t->pattern_rank; ++k) bound += i128(t->array_shape[a]) * t->pattern_shape[k];
        if (bound > kI64Max) return fail(AOL_E_RANGE, "tiler index arithmetic would overflow int64");
    }
    return AOL_OK;
}

// A sufficient condition for injectivity of (r, i) -> (o + P.r + F.i) mod s, checked on the host in
// O(rank^2): every combined (repetition or pattern) dim d with extent > 1 moves exactly ONE array dim a(d),
// with signed coefficient c_d (the representative of c mod s_a nearest 0); per array dim, the coefficients
// of its dims, sorted by |c|, dominate (|c_d| > sum over smaller ones of |c_e| (ext_e - 1): mixed-radix
// digits, so distinct index vectors give distinct raw coordinates), and the raw coordinates span at most
// s_a values (so the modulo keeps them distinct).  The paper's output tilers, blockings and their wrapping
// variants qualify; anything it cannot prove takes the two-pass claim path.
bool prove_injective(const TilerDev& td) {
    int owner[2 * AOL_MAX_RANK];
    int64_t sc[2 * AOL_MAX_RANK];
    for (int d = 0; d < td.nd; ++d) {
        owner[d] = -1;
        if (td.ext[d] == 1) continue;
        for (int a = 0; a < td.ra; ++a) {
            int64_t c = td.coef[a][d];
            if (c == 0) continue;
            if (owner[d] >= 0) return false;   // moves two array dims: not provable here
            if (2 * c > td.ashape[a]) c -= td.ashape[a];
            owner[d] = a;
            sc[d] = c < 0 ? -c : c;
        }
        if (owner[d] < 0) return false;         // broadcast dim: two indices hit the same element
    }
    for (int a = 0; a < td.ra; ++a) {
        int ds[2 * AOL_MAX_RANK], n = 0;
        for (int d = 0; d < td.nd; ++d)
            if (td.ext[d] > 1 && owner[d] == a) ds[n++] = d;
        std::sort(ds, ds + n, [&](int x, int y) { return sc[x] < sc[y]; });
        __int128 acc = 0;   // largest |raw offset| the smaller digits reach
        for (int k = 0; k < n; ++k) {
            if (__int128(sc[ds[k]]) <= acc) return false;
            acc += __int128(sc[ds[k]]) * (td.ext[ds[k]] - 1);
        }
        if (acc + 1 > td.ashape[a]) return false;
    }
    return true;
}

}  // namespace

int claim_bytes(const TilerDev& td) {
    if (td.proven_injective) return 0;
    return td.total < (int64_t(1) << 32) - 1 ? 4 : 8;
}

aol_status_t make_tiler_dev(const aol_tiler_t* t, TilerDev* td) {
    aol_status_t st = validate_tiler(t);
    if (st != AOL_OK) return st;
    std::memset(td, 0, sizeof *td);
    td->ra = t->array_rank;
    td->nd = t->rep_rank + t->pattern_rank;
    int64_t total = 1;
    for (int j = 0; j < t->rep_rank; ++j) {
        td->ext[j] = t->rep_shape[j];
        total *= t->rep_shape[j];
    }
    for (int k = 0; k < t->pattern_rank; ++k) {
        td->ext[t->rep_rank + k] = t->pattern_shape[k];
        total *= t->pattern_shape[k];
    }
    td->total = total;
    int64_t stride = 1;
    for (int a = t->array_rank - 1; a >= 0; --a) {
        const int64_t s = t->array_shape[a];
        td->ashape[a] = s;
        td->astride[a] = stride;
        stride *= s;
        td->org[a] = emod(t->origin[a], s);
        for (int j = 0; j < t->rep_rank; ++j) td->coef[a][j] = emod(t->paving[a][j], s);
        for (int k = 0; k < t->pattern_rank; ++k) td->coef[a][t->rep_rank + k] = emod(t->fitting[a][k], s);
    }
    td->array_elems = stride;
    // classify: which array dims can wrap, affine offsets, fast 32-bit division
    td->linear = 1;
    td->nowrap_mask = 0;
    td->base = 0;
    for (int a = 0; a < td->ra; ++a) {
        __int128 mx = td->org[a];
        for (int d = 0; d < td->nd; ++d) mx += __int128(td->coef[a][d]) * (td->ext[d] - 1);
        if (mx < td->ashape[a]) td->nowrap_mask |= 1u << a;
        else td->linear = 0;
        td->base += td->org[a] * td->astride[a];
    }
    for (int d = 0; d < td->nd; ++d) {
        int64_t l = 0;
        for (int a = 0; a < td->ra; ++a) l += td->coef[a][d] * td->astride[a];
        td->lin[d] = td->linear ? l : 0;
    }
    td->fast32 = total < (int64_t(1) << 31) ? 1 : 0;
    for (int d = 0; d < td->nd; ++d) {
        // n / ext == (umulhi(n, mul) + n) >> shift for n, ext < 2^31
        uint32_t shift = 0;
        while (shift < 32 && (uint64_t(1) << shift) < uint64_t(td->ext[d])) ++shift;
        const uint64_t magic = ((uint64_t(1) << 32) * ((uint64_t(1) << shift) - uint64_t(td->ext[d]))) /
                                   uint64_t(td->ext[d]) + 1;
        td->fd_mul[d] = td->fast32 ? uint32_t(magic) : 0u;
        td->fd_shift[d] = shift;
    }
    // Walk order for linear tilers: array-side strides ascending (innermost = smallest), dims that
    // do not move on the array side (stride 0, broadcast) outermost; the natural last dim stays
    // innermost when it is unit-stride on the array side so 16-byte vectors remain possible.
    int order[2 * AOL_MAX_RANK];
    for (int d = 0; d < td->nd; ++d) order[d] = d;
    if (td->linear) {
        auto key = [&](int d) { return td->lin[d] == 0 ? INT64_MAX : td->lin[d]; };
        // stable insertion sort, descending key = outermost first
        for (int i = 1; i < td->nd; ++i)
            for (int j = i; j > 0 && key(order[j - 1]) < key(order[j]); --j) std::swap(order[j - 1], order[j]);
        const int last = td->nd - 1;
        if (td->nd > 0 && td->lin[last] == 1) {
            int pos = 0;
            while (order[pos] != last) ++pos;
            for (; pos < last; ++pos) order[pos] = order[pos + 1];
            order[last] = last;
        }
    }
    td->small32 = td->linear && td->fast32 && td->array_elems < (int64_t(1) << 31) ? 1 : 0;
    int64_t gst[2 * AOL_MAX_RANK];
    int64_t g = 1;
    for (int d = td->nd - 1; d >= 0; --d) {
        gst[d] = g;
        g *= td->ext[d];
    }
    for (int i = 0; i < td->nd; ++i) {
        const int d = order[i];
        td->p_ext[i] = td->ext[d];
        td->p_lin[i] = td->lin[d];
        td->p_gst[i] = gst[d];
        td->p_fd_mul[i] = td->fd_mul[d];
        td->p_fd_shift[i] = td->fd_shift[d];
    }
    td->proven_injective = prove_injective(*td) ? 1 : 0;
    return AOL_OK;
}

}  // namespace aol

using namespace aol;

namespace {

aol_status_t check_frame_args(const void* d_in, aol_dtype_t in_dtype, const void* d_out, int64_t frames,
                              int64_t channels, int64_t H, int64_t W, aol_dtype_t out_dtype = AOL_I32,
                              const uint64_t* d_cs = nullptr) {
    if (frames < 0 || channels <= 0 || H <= 0 || W <= 0)
        return fail(AOL_E_INVALID, "frames must be >= 0 and channels, H, W > 0");
    if (in_dtype != AOL_I32 && in_dtype != AOL_U8 && in_dtype != AOL_RGB8)
        return fail(AOL_E_DTYPE, "in_dtype must be AOL_I32, AOL_U8 or AOL_RGB8");
    if (out_dtype != AOL_I32 && out_dtype != AOL_I16) return fail(AOL_E_DTYPE, "out_dtype must be AOL_I32 or AOL_I16");
    if (out_dtype == AOL_I16 && in_dtype == AOL_I32)
        return fail(AOL_E_DTYPE, "AOL_I16 output needs 8-bit input (8-bit samples give outputs in [-5, 255])");
    if (in_dtype == AOL_RGB8 && channels != 3) return fail(AOL_E_SHAPE, "AOL_RGB8 (packed pixels) needs channels == 3");
    if (in_dtype == AOL_RGB8 && W % 16) return fail(AOL_E_SHAPE, "AOL_RGB8 needs W % 16 == 0");
    if (W % 8) return fail(AOL_E_SHAPE, "W must be a multiple of 8 (H tiler paving step, Fig. 10)");
    if (H % 9) return fail(AOL_E_SHAPE, "H must be a multiple of 9 (V tiler paving step, reading Z1)");
    const __int128 in_elems = __int128(frames) * channels * H * W;
    if (in_elems > (__int128(1) << 60)) return fail(AOL_E_RANGE, "batch too large");
    if (frames > 0 && (!d_in || !d_out)) return fail(AOL_E_INVALID, "null buffer");
    if (frames > 0 && (!aligned16(d_in) || !aligned16(d_out)))
        return fail(AOL_E_ALIGN, "d_in and d_out must be 16-byte aligned");
    if (reinterpret_cast<uintptr_t>(d_cs) % 8) return fail(AOL_E_ALIGN, "d_frame_checksums must be 8-byte aligned");
    return AOL_OK;
}

constexpr int32_t kKnownFlags = AOL_FLAG_U8_ONE_REP | AOL_FLAG_NO_PDL | AOL_FLAG_I32_LINEAR | AOL_FLAG_ROW_STAGES |
                                AOL_FLAG_TRIPLE_STAGES | AOL_FLAG_I32_STRIPS;

aol_status_t check_opts(const aol_launch_opts_t* opts) {
    if (opts && (opts->ctas_per_sm < 0 || opts->ctas_per_sm > 8 || opts->stages < 0 || opts->bands_per_unit < 0 ||
                 opts->kernel < 0 || opts->kernel > 2))
        return fail(AOL_E_INVALID, "launch options out of range");
    if (opts && (opts->flags & ~kKnownFlags))
        return fail(AOL_E_INVALID, "unknown launch-option flag bits (see include/aol_tuning.h)");
    return AOL_OK;
}

}  // namespace

aol_status_t aol::validate_frame_call(const void* d_in, aol_dtype_t in_dtype, const void* d_out,
                                      aol_dtype_t out_dtype, int64_t frames, int64_t channels, int64_t H, int64_t W,
                                      const uint64_t* d_cs, const aol_launch_opts_t* opts) {
    aol_status_t st = check_frame_args(d_in, in_dtype, d_out, frames, channels, H, W, out_dtype, d_cs);
    if (st != AOL_OK) return st;
    return check_opts(opts);
}

void aol::fill_plan_info(const FusedPlan& p, aol_plan_t* out) {
    out->kernel = p.kernel;
    out->grid = p.grid;
    out->block = p.block;
    out->smem_bytes = p.smem;
    out->stages = p.stages;
    out->bands_per_unit = p.bands_per_unit;
    out->units = p.units;
    out->ctas_per_sm = p.ctas_per_sm;
    out->num_sms = p.num_sms;
}

namespace {

aol_status_t frame_ex(const void* d_in, aol_dtype_t in_dtype, void* d_out, aol_dtype_t out_dtype, int64_t frames,
                      int64_t channels, int64_t H, int64_t W, uint64_t* d_cs, const aol_launch_opts_t* opts,
                      cudaStream_t s) {
    aol_status_t st = validate_frame_call(d_in, in_dtype, d_out, out_dtype, frames, channels, H, W, d_cs, opts);
    if (st != AOL_OK) return st;
    if (frames == 0) return AOL_OK;
    FusedPlan plan;
    st = plan_fused(in_dtype, out_dtype, d_in, d_out, frames, channels, H, W, opts, &plan, d_cs != nullptr);
    if (st != AOL_OK) return st;
    return launch_fused(plan, d_in, in_dtype, d_out, frames, channels, H, W, d_cs, s);
}

}  // namespace

extern "C" {

int aol_version(void) { return AOL_VERSION; }

void aol_debug_fail_next_launches(int n) { g_fail_launches = n > 0 ? n : 0; }

const char* aol_debug_last_kernel(void) { return g_last_kernel; }

const char* aol_last_error(void) { return aol::last_error_cstr(); }

aol_status_t aol_tiler_preset(aol_preset_t which, int64_t H, int64_t W, aol_tiler_t* out) {
    if (!out) return fail(AOL_E_INVALID, "out is NULL");
    if (H <= 0 || W <= 0) return fail(AOL_E_INVALID, "H and W must be > 0");
    aol_tiler_t t;
    std::memset(&t, 0, sizeof t);
    t.array_rank = 2;
    t.rep_rank = 2;
    t.pattern_rank = 1;
    switch (which) {
        case AOL_PRESET_H_IN:  // Fig. 10
            if (W % 8) return fail(AOL_E_SHAPE, "W % 8 != 0");
            t.array_shape[0] = H; t.array_shape[1] = W;
            t.pattern_shape[0] = 11;
            t.fitting[1][0] = 1;
            t.paving[0][0] = 1; t.paving[1][1] = 8;
            t.rep_shape[0] = H; t.rep_shape[1] = W / 8;
            break;
        case AOL_PRESET_H_OUT:  // Fig. 10
            if (W % 8) return fail(AOL_E_SHAPE, "W % 8 != 0");
            t.array_shape[0] = H; t.array_shape[1] = 3 * (W / 8);
            t.pattern_shape[0] = 3;
            t.fitting[1][0] = 1;
            t.paving[0][0] = 1; t.paving[1][1] = 3;
            t.rep_shape[0] = H; t.rep_shape[1] = W / 8;
            break;
        case AOL_PRESET_V_IN:  // reading Z1
            if (H % 9) return fail(AOL_E_SHAPE, "H % 9 != 0");
            t.array_shape[0] = H; t.array_shape[1] = W;
            t.pattern_shape[0] = 12;
            t.fitting[0][0] = 1;
            t.paving[0][0] = 9; t.paving[1][1] = 1;
            t.rep_shape[0] = H / 9; t.rep_shape[1] = W;
            break;
        case AOL_PRESET_V_OUT:  // reading Z1
            if (H % 9) return fail(AOL_E_SHAPE, "H % 9 != 0");
            t.array_shape[0] = 4 * (H / 9); t.array_shape[1] = W;
            t.pattern_shape[0] = 4;
            t.fitting[0][0] = 1;
            t.paving[0][0] = 4; t.paving[1][1] = 1;
            t.rep_shape[0] = H / 9; t.rep_shape[1] = W;
            break;
        default:
            return fail(AOL_E_INVALID, "unknown preset");
    }
    *out = t;
    return AOL_OK;
}

aol_status_t aol_tiler_validate(const aol_tiler_t* t) {
    TilerDev td;
    return make_tiler_dev(t, &td);
}

aol_status_t aol_tiler_is_injective(const aol_tiler_t* t, int* injective) {
    if (!injective) return fail(AOL_E_INVALID, "injective is NULL");
    TilerDev td;
    aol_status_t st = make_tiler_dev(t, &td);
    if (st != AOL_OK) return st;
    if (td.proven_injective) {   // the host proof (prove_injective) is sound: no enumeration needed
        *injective = 1;
        return AOL_OK;
    }
    if (td.array_elems > (int64_t(1) << 32) || td.total > (int64_t(1) << 32))
        return fail(AOL_E_RANGE, "brute-force injectivity check limited to 2^32 elements");
    std::vector<uint64_t> seen;   // one bit per array element (<= 512 MiB)
    try {
        seen.assign(size_t((td.array_elems + 63) / 64), 0);
    } catch (...) {
        return fail(AOL_E_RANGE, "not enough host memory for the injectivity bitmap");
    }
    int64_t idx[2 * AOL_MAX_RANK] = {0};
    *injective = 1;
    for (int64_t g = 0; g < td.total; ++g) {
        int64_t off = 0;
        for (int a = 0; a < td.ra; ++a) {
            __int128 v = td.org[a];
            for (int d = 0; d < td.nd; ++d) v += __int128(td.coef[a][d]) * idx[d];
            off += int64_t(v % td.ashape[a]) * td.astride[a];
        }
        const uint64_t bit = uint64_t(1) << (off & 63);
        if (seen[size_t(off >> 6)] & bit) {
            *injective = 0;
            return AOL_OK;
        }
        seen[size_t(off >> 6)] |= bit;
        for (int d = td.nd - 1; d >= 0; --d) {
            if (++idx[d] < td.ext[d]) break;
            idx[d] = 0;
        }
    }
    return AOL_OK;
}

aol_status_t aol_tiler_gather(const aol_tiler_t* t, aol_dtype_t el, const void* d_array, void* d_tiles,
                              cudaStream_t s) {
    TilerDev td;
    aol_status_t st = make_tiler_dev(t, &td);
    if (st != AOL_OK) return st;
    const int es = elsize_of(el);
    if (!es) return fail(AOL_E_DTYPE, "unknown element type");
    if (!d_array || !d_tiles) return fail(AOL_E_INVALID, "null buffer");
    if ((reinterpret_cast<uintptr_t>(d_array) | reinterpret_cast<uintptr_t>(d_tiles)) % es)
        return fail(AOL_E_ALIGN, "buffers must be aligned to the element size");
    return launch_gather(td, es, d_array, d_tiles, s);
}

size_t aol_tiler_scatter_workspace_bytes(const aol_tiler_t* t) {
    TilerDev td;
    if (make_tiler_dev(t, &td) != AOL_OK) return 0;
    return size_t(td.array_elems) * size_t(claim_bytes(td));
}

aol_status_t aol_tiler_scatter(const aol_tiler_t* t, aol_dtype_t el, const void* d_tiles, void* d_array,
                               aol_scatter_mode_t mode, void* d_workspace, size_t ws_bytes, cudaStream_t s) {
    TilerDev td;
    aol_status_t st = make_tiler_dev(t, &td);
    if (st != AOL_OK) return st;
    const int es = elsize_of(el);
    if (!es) return fail(AOL_E_DTYPE, "unknown element type");
    if (!d_array || !d_tiles) return fail(AOL_E_INVALID, "null buffer");
    if ((reinterpret_cast<uintptr_t>(d_array) | reinterpret_cast<uintptr_t>(d_tiles)) % es)
        return fail(AOL_E_ALIGN, "buffers must be aligned to the element size");
    if (mode != AOL_SCATTER_FAST && mode != AOL_SCATTER_SEQUENTIAL) return fail(AOL_E_INVALID, "bad scatter mode");
    if (mode == AOL_SCATTER_SEQUENTIAL && claim_bytes(td) > 0) {
        if (!d_workspace || ws_bytes < size_t(td.array_elems) * size_t(claim_bytes(td)))
            return fail(AOL_E_WORKSPACE, "SEQUENTIAL scatter needs aol_tiler_scatter_workspace_bytes() of workspace");
        if (reinterpret_cast<uintptr_t>(d_workspace) % 8) return fail(AOL_E_ALIGN, "workspace must be 8-byte aligned");
    }
    return launch_scatter(td, es, d_tiles, d_array, mode == AOL_SCATTER_SEQUENTIAL, d_workspace, s);
}

aol_status_t aol_downscale_h(const int32_t* d_in, int32_t* d_out, int64_t planes, int64_t H, int64_t W,
                             cudaStream_t s) {
    if (planes < 0 || H <= 0 || W <= 0) return fail(AOL_E_INVALID, "planes >= 0, H > 0, W > 0 required");
    if (W % 8) return fail(AOL_E_SHAPE, "W must be a multiple of 8 (Fig. 10 paving step)");
    if (planes == 0) return AOL_OK;
    if (!d_in || !d_out) return fail(AOL_E_INVALID, "null buffer");
    if (reinterpret_cast<uintptr_t>(d_out) % 4 || reinterpret_cast<uintptr_t>(d_in) % 4)
        return fail(AOL_E_ALIGN, "buffers must be 4-byte aligned");
    return launch_downscale_h(d_in, d_out, planes, H, W, s);
}

aol_status_t aol_downscale_v(const int32_t* d_in, int32_t* d_out, int64_t planes, int64_t H, int64_t W,
                             cudaStream_t s) {
    if (planes < 0 || H <= 0 || W <= 0) return fail(AOL_E_INVALID, "planes >= 0, H > 0, W > 0 required");
    if (H % 9) return fail(AOL_E_SHAPE, "H must be a multiple of 9 (V paving step, reading Z1)");
    if (planes == 0) return AOL_OK;
    if (!d_in || !d_out) return fail(AOL_E_INVALID, "null buffer");
    if (reinterpret_cast<uintptr_t>(d_out) % 4 || reinterpret_cast<uintptr_t>(d_in) % 4)
        return fail(AOL_E_ALIGN, "buffers must be 4-byte aligned");
    return launch_downscale_v(d_in, d_out, planes, H, W, s);
}

aol_status_t aol_downscale_frame(const void* d_in, aol_dtype_t in_dtype, int32_t* d_out, int64_t frames,
                                 int64_t channels, int64_t H, int64_t W, uint64_t* d_frame_checksums,
                                 cudaStream_t s) {
    return frame_ex(d_in, in_dtype, d_out, AOL_I32, frames, channels, H, W, d_frame_checksums, nullptr, s);
}

aol_status_t aol_downscale_frame_ex(const void* d_in, aol_dtype_t in_dtype, int32_t* d_out, int64_t frames,
                                    int64_t channels, int64_t H, int64_t W, uint64_t* d_frame_checksums,
                                    const aol_launch_opts_t* opts, cudaStream_t s) {
    return frame_ex(d_in, in_dtype, d_out, AOL_I32, frames, channels, H, W, d_frame_checksums, opts, s);
}

aol_status_t aol_downscale_frame_out(const void* d_in, aol_dtype_t in_dtype, void* d_out, aol_dtype_t out_dtype,
                                     int64_t frames, int64_t channels, int64_t H, int64_t W,
                                     uint64_t* d_frame_checksums, const aol_launch_opts_t* opts, cudaStream_t s) {
    return frame_ex(d_in, in_dtype, d_out, out_dtype, frames, channels, H, W, d_frame_checksums, opts, s);
}

aol_status_t aol_downscale_frame_plan_out(aol_dtype_t in_dtype, aol_dtype_t out_dtype, int64_t frames,
                                          int64_t channels, int64_t H, int64_t W, const aol_launch_opts_t* opts,
                                          aol_plan_t* out) {
    if (!out) return fail(AOL_E_INVALID, "out is NULL");
    aol_status_t st = check_frame_args(nullptr, in_dtype, nullptr, 0, channels, H, W, out_dtype);
    if (st != AOL_OK) return st;
    st = check_opts(opts);
    if (st != AOL_OK) return st;
    if (frames <= 0) return fail(AOL_E_INVALID, "frames must be > 0 to plan");
    FusedPlan p;
    st = plan_fused(in_dtype, out_dtype, nullptr, nullptr, frames, channels, H, W, opts, &p);
    if (st != AOL_OK) return st;
    fill_plan_info(p, out);
    return AOL_OK;
}

aol_status_t aol_downscale_frame_plan(aol_dtype_t in_dtype, int64_t frames, int64_t channels, int64_t H,
                                      int64_t W, const aol_launch_opts_t* opts, aol_plan_t* out) {
    return aol_downscale_frame_plan_out(in_dtype, AOL_I32, frames, channels, H, W, opts, out);
}

aol_status_t aol_frame_checksum(const int32_t* d_out, int64_t frames, int64_t channels, int64_t Ho, int64_t Wo,
                                uint64_t* d_checksums, cudaStream_t s) {
    if (frames < 0 || channels <= 0 || Ho <= 0 || Wo <= 0) return fail(AOL_E_INVALID, "bad extents");
    if (frames == 0) return AOL_OK;
    if (!d_out || !d_checksums) return fail(AOL_E_INVALID, "null buffer");
    if (reinterpret_cast<uintptr_t>(d_checksums) % 8 || reinterpret_cast<uintptr_t>(d_out) % 4)
        return fail(AOL_E_ALIGN, "d_checksums must be 8-byte and d_out 4-byte aligned");
    return launch_checksum(d_out, frames, channels * Ho * Wo, d_checksums, s);
}

size_t aol_downscale_frame_host_workspace_bytes(aol_dtype_t in_dtype, int64_t chunk_frames, int64_t channels,
                                                int64_t H, int64_t W) {
    const int es = (in_dtype == AOL_U8 || in_dtype == AOL_RGB8) ? 1 : (in_dtype == AOL_I32 ? 4 : 0);
    if (!es || chunk_frames <= 0 || channels <= 0 || H <= 0 || W <= 0 || W % 8 || H % 9) return 0;
    const size_t in_b = (size_t(chunk_frames) * channels * H * W * es + 255) & ~size_t(255);
    const size_t out_b = (size_t(chunk_frames) * channels * (4 * (H / 9)) * (3 * (W / 8)) * 4 + 255) & ~size_t(255);
    const size_t cs_b = (size_t(chunk_frames) * 8 + 255) & ~size_t(255);
    return 2 * (in_b + out_b + cs_b);
}

aol_status_t aol_downscale_frame_host(const void* h_in, aol_dtype_t in_dtype, int32_t* h_out, int64_t frames,
                                      int64_t channels, int64_t H, int64_t W, uint64_t* h_frame_checksums,
                                      int64_t chunk_frames, void* d_workspace, size_t ws_bytes, cudaStream_t s_h2d,
                                      cudaStream_t s_compute, cudaStream_t s_d2h) {
    aol_status_t st = check_frame_args(nullptr, in_dtype, nullptr, 0, channels, H, W);
    if (st != AOL_OK) return st;
    if (frames == 0) return AOL_OK;
    if (!h_in || !h_out) return fail(AOL_E_INVALID, "null host buffer");
    if (chunk_frames <= 0) return fail(AOL_E_INVALID, "chunk_frames must be > 0");
    chunk_frames = std::min(chunk_frames, frames);
    const size_t need = aol_downscale_frame_host_workspace_bytes(in_dtype, chunk_frames, channels, H, W);
    if (!d_workspace || ws_bytes < need) return fail(AOL_E_WORKSPACE, "device workspace too small");
    if (!aligned16(d_workspace)) return fail(AOL_E_ALIGN, "workspace must be 16-byte aligned");

    const int es = (in_dtype == AOL_U8 || in_dtype == AOL_RGB8) ? 1 : 4;
    const int64_t Ho = 4 * (H / 9), Wo = 3 * (W / 8);
    const size_t in_frame = size_t(channels) * H * W * es, out_frame = size_t(channels) * Ho * Wo * 4;
    const size_t in_b = (size_t(chunk_frames) * in_frame + 255) & ~size_t(255);
    const size_t out_b = (size_t(chunk_frames) * out_frame + 255) & ~size_t(255);
    const size_t cs_b = (size_t(chunk_frames) * 8 + 255) & ~size_t(255);
    uint8_t* ws = static_cast<uint8_t*>(d_workspace);
    uint8_t* d_in[2] = {ws, ws + in_b};
    int32_t* d_out[2] = {reinterpret_cast<int32_t*>(ws + 2 * in_b), reinterpret_cast<int32_t*>(ws + 2 * in_b + out_b)};
    uint64_t* d_cs[2] = {reinterpret_cast<uint64_t*>(ws + 2 * in_b + 2 * out_b),
                         reinterpret_cast<uint64_t*>(ws + 2 * in_b + 2 * out_b + cs_b)};

    FusedPlan plan;
    st = plan_fused(in_dtype, AOL_I32, d_in[0], d_out[0], chunk_frames, channels, H, W, nullptr, &plan);
    if (st != AOL_OK) return st;

    cudaEvent_t ev_in[2] = {}, ev_comp[2] = {}, ev_out[2] = {};
    auto destroy_events = [&] {
        for (int b = 0; b < 2; ++b)
            for (cudaEvent_t ev : {ev_in[b], ev_comp[b], ev_out[b]})
                if (ev) cudaEventDestroy(ev);
    };
    for (int b = 0; b < 2; ++b) {
        cudaError_t ce = cudaEventCreateWithFlags(&ev_in[b], cudaEventDisableTiming);
        if (ce == cudaSuccess) ce = cudaEventCreateWithFlags(&ev_comp[b], cudaEventDisableTiming);
        if (ce == cudaSuccess) ce = cudaEventCreateWithFlags(&ev_out[b], cudaEventDisableTiming);
        if (ce != cudaSuccess) {
            destroy_events();
            set_error("cudaEventCreate failed: %s", cudaGetErrorString(ce));
            return AOL_E_CUDA;
        }
    }
    aol_status_t result = AOL_OK;
    const uint8_t* hin = static_cast<const uint8_t*>(h_in);
    uint8_t* hout = reinterpret_cast<uint8_t*>(h_out);
    int k = 0;
    for (int64_t f0 = 0; f0 < frames; f0 += chunk_frames, ++k) {
        const int b = k & 1;
        const int64_t nf = std::min(chunk_frames, frames - f0);
        cudaError_t e = cudaSuccess;
        // input buffer b is free once the compute of chunk k-2 finished
        if (e == cudaSuccess) e = cudaStreamWaitEvent(s_h2d, ev_comp[b], 0);
        if (e == cudaSuccess)
            e = cudaMemcpyAsync(d_in[b], hin + size_t(f0) * in_frame, size_t(nf) * in_frame, cudaMemcpyHostToDevice,
                                s_h2d);
        if (e == cudaSuccess) e = cudaEventRecord(ev_in[b], s_h2d);
        if (e == cudaSuccess) e = cudaStreamWaitEvent(s_compute, ev_in[b], 0);
        // output buffer b is free once the D2H of chunk k-2 finished
        if (e == cudaSuccess) e = cudaStreamWaitEvent(s_compute, ev_out[b], 0);
        if (e != cudaSuccess) {
            set_error("host stream enqueue failed: %s", cudaGetErrorString(e));
            result = AOL_E_CUDA;
            break;
        }
        result = launch_fused(plan, d_in[b], in_dtype, d_out[b], nf, channels, H, W,
                              h_frame_checksums ? d_cs[b] : nullptr, s_compute);
        if (result != AOL_OK) break;
        e = cudaEventRecord(ev_comp[b], s_compute);
        if (e == cudaSuccess) e = cudaStreamWaitEvent(s_d2h, ev_comp[b], 0);
        if (e == cudaSuccess)
            e = cudaMemcpyAsync(hout + size_t(f0) * out_frame, d_out[b], size_t(nf) * out_frame,
                                cudaMemcpyDeviceToHost, s_d2h);
        if (e == cudaSuccess && h_frame_checksums)
            e = cudaMemcpyAsync(h_frame_checksums + f0, d_cs[b], size_t(nf) * 8, cudaMemcpyDeviceToHost, s_d2h);
        if (e == cudaSuccess) e = cudaEventRecord(ev_out[b], s_d2h);
        if (e != cudaSuccess) {
            set_error("host stream enqueue failed: %s", cudaGetErrorString(e));
            result = AOL_E_CUDA;
            break;
        }
    }
    cudaError_t e1 = cudaStreamSynchronize(s_d2h);
    cudaError_t e2 = cudaStreamSynchronize(s_compute);
    cudaError_t e3 = cudaStreamSynchronize(s_h2d);
    destroy_events();
    if (result == AOL_OK) {
        for (cudaError_t e : {e1, e2, e3})
            if (e != cudaSuccess) {
                set_error("host-streamed downscale failed: %s", cudaGetErrorString(e));
                return AOL_E_CUDA;
            }
    }
    return result;
}

aol_status_t aol_synth_frames(uint64_t seed, int64_t frame0, int64_t nframes, int64_t channels, int64_t H,
                              int64_t W, int32_t kind, int32_t value, aol_dtype_t out_dtype, void* d_out,
                              cudaStream_t s) {
    if (frame0 < 0 || nframes < 0 || channels <= 0 || H <= 0 || W <= 0) return fail(AOL_E_INVALID, "bad extents");
    if (kind < 0 || kind > 4) return fail(AOL_E_INVALID, "kind must be 0..4");
    if (out_dtype != AOL_I32 && out_dtype != AOL_U8) return fail(AOL_E_DTYPE, "out_dtype must be AOL_I32 or AOL_U8");
    if (out_dtype == AOL_U8 && (kind == 2 || (kind == 3 && W > 256) || (kind == 4 && (value < 0 || value > 255))))
        return fail(AOL_E_DTYPE, "values of this kind do not fit in uint8");
    if (nframes == 0) return AOL_OK;
    if (!d_out) return fail(AOL_E_INVALID, "null buffer");
    return launch_synth(seed, frame0, nframes, channels, H, W, kind, value, out_dtype == AOL_U8, d_out, s);
}

}  // extern "C"
