// tiler.cu -- K-1 generic ArrayOL tiler gather and K-2 scatter (any rank <= 8,
// element size 1/2/4/8 bytes, Euclidean modulo).
//
//   gather : tiles[r][i]  = array[(o + P.r + F.i) mod s]     (Section IV, Fig. 4)
//   scatter: array[(o + P.r + F.i) mod s] = tiles[r][i]      (Fig. 6, modarray P:L479)
//
// The host reduces o, P and F modulo the array extents (every partial sum is
// then non-negative) and classifies each array dimension: if no (r, i) can
// push its coordinate past the extent, the `mod` is the identity there.  When
// that holds for every dimension the tiler is an affine map of the flat tile
// index -- offset = base + sum_d lin[d] * idx[d] -- and the LINEAR kernels
// apply: one fast 32-bit division chain per thread and, when the innermost
// pattern dimension walks contiguous memory, 16-byte vector accesses on both
// sides.  Linear tilers are walked in array-stride order (the host sorts the
// combined dims so consecutive threads touch consecutive ARRAY addresses, the
// side whose locality is not guaranteed); the tile side is then written in
// contiguous runs of the innermost dim.  Otherwise the GENERAL kernels walk the
// natural tile order (tile accesses coalesced) and evaluate the modulo per
// wrapping dimension.
#include <cuda_runtime.h>

#include <cstdint>

#include "common.h"

namespace aol {

// per-element-size launchers (tiler_es{1,2,4,8}.cu); mode 0 gather, 1 FAST scatter, 2/3 SEQUENTIAL passes with
// 8-byte claims, 4/5 the same with 4-byte claims
aol_status_t tiler_launch_es1(int mode, const TilerDev& td, int vec, const void* src, void* dst,
                              unsigned long long* ws, int num_sms, cudaStream_t s);
aol_status_t tiler_launch_es2(int mode, const TilerDev& td, int vec, const void* src, void* dst,
                              unsigned long long* ws, int num_sms, cudaStream_t s);
aol_status_t tiler_launch_es4(int mode, const TilerDev& td, int vec, const void* src, void* dst,
                              unsigned long long* ws, int num_sms, cudaStream_t s);
aol_status_t tiler_launch_es8(int mode, const TilerDev& td, int vec, const void* src, void* dst,
                              unsigned long long* ws, int num_sms, cudaStream_t s);

namespace {

template <int MODE>
aol_status_t launch_mode(const TilerDev& td, int elsize, int vec, const void* src, void* dst,
                         unsigned long long* ws, int num_sms, cudaStream_t s) {
    switch (elsize) {
        case 1: return tiler_launch_es1(MODE, td, vec, src, dst, ws, num_sms, s);
        case 2: return tiler_launch_es2(MODE, td, vec, src, dst, ws, num_sms, s);
        case 4: return tiler_launch_es4(MODE, td, vec, src, dst, ws, num_sms, s);
        case 8: return tiler_launch_es8(MODE, td, vec, src, dst, ws, num_sms, s);
    }
    return fail(AOL_E_DTYPE, "element size must be 1, 2, 4 or 8 bytes");
}

// Largest usable vector (elements; 16, 8, 4 or 2 bytes): the permuted innermost dim is the natural last dim,
// unit-stride on both sides; every other stride, the origin and the pointers keep V-element alignment.
int vector_width(const TilerDev& td, int elsize, const void* p_array, const void* p_tiles) {
    if (!td.linear || td.nd == 0) return 1;
    const int last = td.nd - 1;
    if (td.p_lin[last] != 1 || td.p_gst[last] != 1) return 1;
    const uintptr_t ptrs = reinterpret_cast<uintptr_t>(p_array) | reinterpret_cast<uintptr_t>(p_tiles);
    for (int vb = 16; vb > elsize; vb /= 2) {
        const int v = vb / elsize;
        bool ok = td.p_ext[last] % v == 0 && td.base % v == 0 && ptrs % vb == 0;
        for (int d = 0; d < last && ok; ++d) ok = td.p_lin[d] % v == 0 && td.p_gst[d] % v == 0;
        if (ok) return v;
    }
    return 1;
}

}  // namespace

aol_status_t launch_gather(const TilerDev& td, int elsize, const void* d_array, void* d_tiles, cudaStream_t s) {
    if (td.total == 0) return AOL_OK;
    DeviceInfo dev;
    aol_status_t st = device_info(&dev);
    if (st != AOL_OK) return st;
    return launch_mode<0>(td, elsize, vector_width(td, elsize, d_array, d_tiles), d_array, d_tiles, nullptr,
                          dev.num_sms, s);
}

aol_status_t launch_scatter(const TilerDev& td, int elsize, const void* d_tiles, void* d_array, int sequential,
                            void* d_ws, cudaStream_t s) {
    if (td.total == 0) return AOL_OK;
    DeviceInfo dev;
    aol_status_t st = device_info(&dev);
    if (st != AOL_OK) return st;
    auto* ws = static_cast<unsigned long long*>(d_ws);
    // a SEQUENTIAL scatter whose tiler the host proved injective has no collisions: Fig. 6's loop order cannot
    // change the result, so it takes the one-pass FAST kernels (no workspace)
    const int cb = claim_bytes(td);
    if (!sequential || cb == 0)
        return launch_mode<1>(td, elsize, vector_width(td, elsize, d_array, d_tiles), d_tiles, d_array, nullptr,
                              dev.num_sms, s);
    // two passes: claim (the largest flat tile index + 1 per target: the last writer in Fig. 6 order), then
    // write where this element holds the claim; 4-byte claims when every claim fits 32 bits
    AOL_CUDA_TRY(cudaMemsetAsync(d_ws, 0, size_t(td.array_elems) * size_t(cb), s));
    st = cb == 4 ? launch_mode<4>(td, elsize, 1, d_tiles, d_array, ws, dev.num_sms, s)
                 : launch_mode<2>(td, elsize, 1, d_tiles, d_array, ws, dev.num_sms, s);
    if (st != AOL_OK) return st;
    return cb == 4 ? launch_mode<5>(td, elsize, 1, d_tiles, d_array, ws, dev.num_sms, s)
                   : launch_mode<3>(td, elsize, 1, d_tiles, d_array, ws, dev.num_sms, s);
}

}  // namespace aol
