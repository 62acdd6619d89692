// tiler_kernels.cuh -- the generic tiler kernels and their per-element-size launchers, compiled once per
// element size (tiler_es{1,2,4,8}.cu, in parallel); tiler.cu holds the host entry points.
// K-1 generic ArrayOL tiler gather and K-2 scatter (any rank <= 8,
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
#pragma once
#include <cuda_runtime.h>

#include <algorithm>
#include <cstdint>
#include <cstdlib>
#include <cstring>
#include <vector>

#include "common.h"
#include "ptx.cuh"

namespace aol {

namespace {

template <int ES>
struct Elem;
template <>
struct Elem<1> {
    using T = uint8_t;
};
template <>
struct Elem<2> {
    using T = uint16_t;
};
template <>
struct Elem<4> {
    using T = uint32_t;
};
template <>
struct Elem<8> {
    using T = unsigned long long;
};

template <int BYTES>
struct Vec;
template <>
struct Vec<1> {
    using T = uint8_t;
};
template <>
struct Vec<2> {
    using T = uint16_t;
};
template <>
struct Vec<4> {
    using T = uint32_t;
};
template <>
struct Vec<8> {
    using T = uint2;
};
template <>
struct Vec<16> {
    using T = uint4;
};

constexpr int kND = 2 * AOL_MAX_RANK;

// Decompose flat index g over extents ext (last dim fastest).
template <bool kFast32>
__device__ __forceinline__ void decompose(int nd, const int64_t* ext, const uint32_t* fmul, const uint32_t* fshift,
                                          int64_t g, int64_t (&idx)[kND]) {
#pragma unroll
    for (int d = kND - 1; d >= 0; --d) {
        if (d < nd) {
            if (kFast32) {
                const uint32_t n = uint32_t(g);
                const uint32_t q = (__umulhi(n, fmul[d]) + n) >> fshift[d];
                idx[d] = int64_t(n - q * uint32_t(ext[d]));
                g = q;
            } else {
                const int64_t q = g / ext[d];
                idx[d] = g - q * ext[d];
                g = q;
            }
        } else {
            idx[d] = 0;
        }
    }
}

__device__ __forceinline__ int64_t general_offset(const TilerDev& td, const int64_t (&idx)[kND]) {
    int64_t off = 0;
#pragma unroll
    for (int a = 0; a < AOL_MAX_RANK; ++a) {
        if (a < td.ra) {
            int64_t v = td.org[a];
#pragma unroll
            for (int d = 0; d < kND; ++d)
                if (d < td.nd) v += td.coef[a][d] * idx[d];
            if (!((td.nowrap_mask >> a) & 1)) v %= td.ashape[a];   // all terms >= 0: % == Euclidean mod
            off += v * td.astride[a];
        }
    }
    return off;
}

// mode 0: gather; 1: FAST scatter; 2: SEQUENTIAL claim (max flat index + 1 per target);
// 3: SEQUENTIAL write (store iff this element holds the claim); 4 / 5: the same with 4-byte claims.
template <int MODE>
__device__ __forceinline__ void seq_pass(void* ws, int64_t off, int64_t g, bool& write) {
    if constexpr (MODE == 2) {
        atomicMax(static_cast<unsigned long long*>(ws) + off, (unsigned long long)g + 1ull);
    } else if constexpr (MODE == 4) {
        atomicMax(static_cast<unsigned int*>(ws) + off, unsigned(g) + 1u);
    } else if constexpr (MODE == 3) {
        write = static_cast<const unsigned long long*>(ws)[off] == (unsigned long long)g + 1ull;
    } else if constexpr (MODE == 5) {
        write = static_cast<const unsigned int*>(ws)[off] == unsigned(g) + 1u;
    }
}
template <int ES, int V, bool kFast32, bool kLinear, int MODE>
__global__ void __launch_bounds__(256) tiler_kernel(const TilerDev td, const void* __restrict__ src,
                                                    void* __restrict__ dst, unsigned long long* __restrict__ ws) {
    using T = typename Elem<ES>::T;
    using VT = typename Vec<ES * V>::T;
    const int64_t nvec = td.total / V;
    const int64_t stride = int64_t(gridDim.x) * blockDim.x;
    // kU independent elements per thread per iteration: all loads issued before the stores, so each
    // thread keeps kU requests in flight (Little's law at ~43 GB/s per SM needs tens of KB per SM).
    constexpr int kU = (MODE <= 1) ? 4 : 1;
    // a warp owns kU*32 consecutive vectors per iteration (lane + 32u): locality is kept on both sides
    const int64_t warp_first = (int64_t(blockIdx.x) * blockDim.x + (threadIdx.x & ~31u)) * kU + (threadIdx.x & 31u);
    for (int64_t v0 = warp_first; v0 < nvec; v0 += kU * stride) {
        int64_t off[kU], g[kU];   // array-side and tile-side element offsets
#pragma unroll
        for (int u = 0; u < kU; ++u) {
            const int64_t v = v0 + 32 * u;
            if (kLinear) {
                // permuted walk (array side contiguous): both offsets are affine in the permuted index;
                // a runtime-rank loop that folds each digit straight into the two offsets (no index array)
                int64_t o = td.base, gg = 0;
                if (kFast32) {
                    uint32_t n = v < nvec ? uint32_t(v * V) : 0u;
#pragma unroll 1
                    for (int d = td.nd - 1; d >= 0; --d) {
                        const uint32_t q = (__umulhi(n, td.p_fd_mul[d]) + n) >> td.p_fd_shift[d];
                        const uint32_t i = n - q * uint32_t(td.p_ext[d]);
                        n = q;
                        o += td.p_lin[d] * int64_t(i);
                        gg += td.p_gst[d] * int64_t(i);
                    }
                } else {
                    int64_t n = v < nvec ? v * V : 0;
#pragma unroll 1
                    for (int d = td.nd - 1; d >= 0; --d) {
                        const int64_t q = n / td.p_ext[d];
                        const int64_t i = n - q * td.p_ext[d];
                        n = q;
                        o += td.p_lin[d] * i;
                        gg += td.p_gst[d] * i;
                    }
                }
                off[u] = o;
                g[u] = gg;
            } else {
                int64_t idx[kND];
                g[u] = v < nvec ? v * V : 0;
                decompose<kFast32>(td.nd, td.ext, td.fd_mul, td.fd_shift, g[u], idx);
                off[u] = general_offset(td, idx);
            }
        }
        if (MODE == 0) {
            // tiles[g .. g+V) = array[off .. off+V)   (V > 1 only when contiguous and aligned)
            VT val[kU];
#pragma unroll
            for (int u = 0; u < kU; ++u)
                if (v0 + 32 * u < nvec) val[u] = reinterpret_cast<const VT*>(static_cast<const T*>(src) + off[u])[0];
#pragma unroll
            for (int u = 0; u < kU; ++u)
                if (v0 + 32 * u < nvec) reinterpret_cast<VT*>(static_cast<T*>(dst) + g[u])[0] = val[u];
        } else if (MODE == 1) {
            VT val[kU];
#pragma unroll
            for (int u = 0; u < kU; ++u)
                if (v0 + 32 * u < nvec) val[u] = reinterpret_cast<const VT*>(static_cast<const T*>(src) + g[u])[0];
#pragma unroll
            for (int u = 0; u < kU; ++u)
                if (v0 + 32 * u < nvec) reinterpret_cast<VT*>(static_cast<T*>(dst) + off[u])[0] = val[u];
        } else if (v0 < nvec) {   // SEQUENTIAL passes (V == 1, kU == 1)
            bool write = false;
            seq_pass<MODE>(ws, off[0], g[0], write);
            if (write) static_cast<T*>(dst)[off[0]] = static_cast<const T*>(src)[g[0]];
        }
    }
}

// Linear tilers whose array and tile offsets fit in 31 bits (the common case): the permuted walk with
// all-32-bit digit arithmetic, the per-dimension constants loaded once per thread into registers and the digit
// loop fully unrolled for NDU dims (the tiler's, padded with unit extents on the outside): the walk's instruction
// count is what bounds these kernels (round 2: a loop over constants staged in shared memory issued ~1.9x the
// instructions; d3 affine gather 0.0878 ms there).
template <int ES, int V, int MODE, int NDU>
__global__ void __launch_bounds__(256) tiler_linear32_kernel(const TilerDev td, const void* __restrict__ src,
                                                             void* __restrict__ dst) {
    using T = typename Elem<ES>::T;
    using VT = typename Vec<ES * V>::T;
    int32_t L[NDU], AL[NDU], GS[NDU];
    uint32_t M[NDU], S[NDU];
#pragma unroll
    for (int d = 0; d < NDU; ++d) {
        const int e = d - (NDU - td.nd);
        L[d] = e >= 0 ? int32_t(td.p_ext[e]) : 1;
        M[d] = e >= 0 ? uint32_t(td.p_fd_mul[e]) : 0u;
        S[d] = e >= 0 ? uint32_t(td.p_fd_shift[e]) : 0u;
        AL[d] = e >= 0 ? int32_t(td.p_lin[e]) : 0;
        GS[d] = e >= 0 ? int32_t(td.p_gst[e]) : 0;
    }
    const int32_t nvec = int32_t(td.total / V);
    const int32_t stride = int32_t(gridDim.x * blockDim.x);
    const int32_t base = int32_t(td.base);
    // 2 vectors per thread per iteration with a 4x larger grid than the general kernels (tools/tiler_probe2.py,
    // profiles/r01_tiler_variants.jsonl: d3 gather 5.01 -> 5.22 TB/s; kU = 1, 4, 8 and grids x8..x512 are slower)
    constexpr int kU = 2;
    const int32_t warp_first = int32_t((blockIdx.x * blockDim.x + (threadIdx.x & ~31u)) * kU + (threadIdx.x & 31u));
    for (int32_t v0 = warp_first; v0 < nvec; v0 += kU * stride) {
        int32_t off[kU], g[kU];
#pragma unroll
        for (int u = 0; u < kU; ++u) {
            const int32_t v = v0 + 32 * u;
            uint32_t n = v < nvec ? uint32_t(v) * V : 0u;
            int32_t o = base, gg = 0;
#pragma unroll
            for (int d = NDU - 1; d >= 1; --d) {
                const uint32_t q = (__umulhi(n, M[d]) + n) >> S[d];
                const int32_t i = int32_t(n - q * uint32_t(L[d]));
                n = q;
                o += AL[d] * i;
                gg += GS[d] * i;
            }
            o += AL[0] * int32_t(n);   // the outermost digit is what is left (n < L[0] for every valid vector)
            gg += GS[0] * int32_t(n);
            off[u] = o;
            g[u] = gg;
        }
        VT val[kU];
        if (MODE == 0) {
#pragma unroll
            for (int u = 0; u < kU; ++u)
                if (v0 + 32 * u < nvec) val[u] = reinterpret_cast<const VT*>(static_cast<const T*>(src) + off[u])[0];
#pragma unroll
            for (int u = 0; u < kU; ++u)
                if (v0 + 32 * u < nvec) reinterpret_cast<VT*>(static_cast<T*>(dst) + g[u])[0] = val[u];
        } else {
#pragma unroll
            for (int u = 0; u < kU; ++u)
                if (v0 + 32 * u < nvec) val[u] = reinterpret_cast<const VT*>(static_cast<const T*>(src) + g[u])[0];
#pragma unroll
            for (int u = 0; u < kU; ++u)
                if (v0 + 32 * u < nvec) reinterpret_cast<VT*>(static_cast<T*>(dst) + off[u])[0] = val[u];
        }
    }
}

// ------------------------------------------------------------ wrapping tilers, 32-bit
// Tilers whose pattern can leave the array (the paper's H/V input tilers wrap at the last repetition, Fig. 10
// P:L681-687) with at most two wrapping array dims and all offsets < 2^31.  The flat offset is computed as if
// nothing wrapped (one IMAD per combined dim, like the linear kernels) together with the raw coordinate of each
// wrapping dim; the toroidal wrap is then one magic-number division per wrapping dim:
//   (v mod s) * stride = v * stride - floor(v / s) * (s * stride).
// Walked in tile order (tile side coalesced), all-32-bit, constants staged in shared memory.
struct Wrap32Dev {
    int32_t nd, nw;                                    // combined dims, wrapping array dims (0..2)
    int32_t ext[2 * AOL_MAX_RANK], lin[2 * AOL_MAX_RANK];
    uint32_t mul[2 * AOL_MAX_RANK], shift[2 * AOL_MAX_RANK];
    int32_t wc[2][2 * AOL_MAX_RANK];                   // coefficient of combined dim d in wrapping dim k
    int32_t worg[2], wext[2], wstep[2];                // origin, extent, extent * array stride
    uint32_t wmul[2], wshift[2];
    int32_t base, total;
};

template <int ES, int MODE>
__global__ void __launch_bounds__(256) tiler_wrap32_kernel(const Wrap32Dev wd, const void* __restrict__ src,
                                                           void* __restrict__ dst, unsigned long long* __restrict__ ws) {
    using T = typename Elem<ES>::T;
    __shared__ int4 pk[kND];   // {extent, magic multiplier, shift, flat-offset coefficient}
    __shared__ int2 pw[kND];   // coefficients in the two wrapping dims
    if (threadIdx.x < wd.nd) {
        const int d = threadIdx.x;
        pk[d] = make_int4(wd.ext[d], int32_t(wd.mul[d]), int32_t(wd.shift[d]), wd.lin[d]);
        pw[d] = make_int2(wd.wc[0][d], wd.wc[1][d]);
    }
    __syncthreads();
    const int32_t n_el = wd.total;
    const int32_t stride = int32_t(gridDim.x * blockDim.x);
    constexpr int kU = (MODE <= 1) ? 2 : 1;
    const int32_t warp_first = int32_t((blockIdx.x * blockDim.x + (threadIdx.x & ~31u)) * kU + (threadIdx.x & 31u));
    for (int32_t v0 = warp_first; v0 < n_el; v0 += kU * stride) {
        int32_t off[kU], g[kU];
#pragma unroll
        for (int u = 0; u < kU; ++u) {
            g[u] = v0 + 32 * u;
            uint32_t n = g[u] < n_el ? uint32_t(g[u]) : 0u;
            int32_t o = wd.base, w0 = wd.worg[0], w1 = wd.worg[1];
#pragma unroll 1
            for (int d = wd.nd - 1; d >= 0; --d) {
                const int4 p = pk[d];
                const int2 c = pw[d];
                const uint32_t q = (__umulhi(n, uint32_t(p.y)) + n) >> p.z;
                const int32_t i = int32_t(n - q * uint32_t(p.x));
                n = q;
                o += p.w * i;
                w0 += c.x * i;
                w1 += c.y * i;
            }
            if (wd.nw > 0) o -= int32_t((__umulhi(uint32_t(w0), wd.wmul[0]) + uint32_t(w0)) >> wd.wshift[0]) * wd.wstep[0];
            if (wd.nw > 1) o -= int32_t((__umulhi(uint32_t(w1), wd.wmul[1]) + uint32_t(w1)) >> wd.wshift[1]) * wd.wstep[1];
            off[u] = o;
        }
        if (MODE == 0) {   // gather: tiles[g] = array[off]
            T val[kU];
#pragma unroll
            for (int u = 0; u < kU; ++u)
                if (g[u] < n_el) val[u] = static_cast<const T*>(src)[off[u]];
#pragma unroll
            for (int u = 0; u < kU; ++u)
                if (g[u] < n_el) static_cast<T*>(dst)[g[u]] = val[u];
        } else if (MODE == 1) {   // FAST scatter: array[off] = tiles[g]
            T val[kU];
#pragma unroll
            for (int u = 0; u < kU; ++u)
                if (g[u] < n_el) val[u] = static_cast<const T*>(src)[g[u]];
#pragma unroll
            for (int u = 0; u < kU; ++u)
                if (g[u] < n_el) static_cast<T*>(dst)[off[u]] = val[u];
        } else if (g[0] < n_el) {   // SEQUENTIAL claim / write: the last (r, i) in row-major order wins
            bool write = false;
            seq_pass<MODE>(ws, off[0], g[0], write);
            if (write) static_cast<T*>(dst)[off[0]] = static_cast<const T*>(src)[g[0]];
        }
    }
}

// Fill *wd for a non-linear tiler if it qualifies (<= 2 wrapping dims, every unwrapped offset < 2^31).
bool make_wrap32(const TilerDev& td, Wrap32Dev* wd) {
    if (td.linear || !td.fast32 || td.array_elems >= (int64_t(1) << 31)) return false;
    std::memset(wd, 0, sizeof *wd);
    int wa[2], nw = 0;
    for (int a = 0; a < td.ra; ++a)
        if (!((td.nowrap_mask >> a) & 1)) {
            if (nw == 2) return false;
            wa[nw++] = a;
        }
    // the largest unwrapped flat offset: sum over array dims of (max raw coordinate) * stride
    __int128 bound = 0;
    for (int a = 0; a < td.ra; ++a) {
        __int128 mx = td.org[a];
        for (int d = 0; d < td.nd; ++d) mx += __int128(td.coef[a][d]) * (td.ext[d] - 1);
        bound += mx * td.astride[a];
    }
    if (bound >= (__int128(1) << 31)) return false;
    wd->nd = td.nd;
    wd->nw = nw;
    wd->total = int32_t(td.total);
    int64_t base = 0;
    for (int a = 0; a < td.ra; ++a) base += td.org[a] * td.astride[a];
    wd->base = int32_t(base);
    for (int d = 0; d < td.nd; ++d) {
        int64_t l = 0;
        for (int a = 0; a < td.ra; ++a) l += td.coef[a][d] * td.astride[a];
        wd->ext[d] = int32_t(td.ext[d]);
        wd->lin[d] = int32_t(l);
        wd->mul[d] = td.fd_mul[d];
        wd->shift[d] = td.fd_shift[d];
        for (int k = 0; k < nw; ++k) wd->wc[k][d] = int32_t(td.coef[wa[k]][d]);
    }
    for (int k = 0; k < nw; ++k) {
        const int a = wa[k];
        const int64_t sa = td.ashape[a];
        wd->worg[k] = int32_t(td.org[a]);
        wd->wext[k] = int32_t(sa);
        wd->wstep[k] = int32_t(sa * td.astride[a]);
        uint32_t sh = 0;   // floor(v / s) == (umulhi(v, mul) + v) >> sh for v, s < 2^31
        while (sh < 32 && (uint64_t(1) << sh) < uint64_t(sa)) ++sh;
        wd->wmul[k] = uint32_t(((uint64_t(1) << 32) * ((uint64_t(1) << sh) - uint64_t(sa))) / uint64_t(sa) + 1);
        wd->wshift[k] = sh;
    }
    return true;
}

// Gather / FAST scatter of the same tilers in blocks: the tile index space (natural order, tile side
// contiguous) splits into INNER dims (the innermost ones, the outermost of them possibly in chunks) whose
// product fills a block of <= kWTab elements, and OUTER dims enumerating the blocks.  Every block shares the
// inner parts of the unwrapped flat offset and of the wrapping coordinates, so each CTA tabulates them once in
// shared memory; an element then costs one LDS.128, three adds and the wrap fix-up instead of a digit-by-digit
// decomposition (the per-element kernel above is issue/latency-bound on exactly that).
constexpr int kWTab = 2048;   // 32 KB of int4 per CTA: 1024 entries 2.84 / 4096 2.61 / 2048 3.29 TB/s (wrapping d3)

struct WrapTabDev {
    int32_t n_in, n_out, nw;
    int32_t in_ext[2 * AOL_MAX_RANK], in_lin[2 * AOL_MAX_RANK], in_w0[2 * AOL_MAX_RANK], in_w1[2 * AOL_MAX_RANK];
    uint32_t in_mul[2 * AOL_MAX_RANK], in_shift[2 * AOL_MAX_RANK];
    int32_t out_ext[2 * AOL_MAX_RANK + 1], out_lin[2 * AOL_MAX_RANK + 1], out_w0[2 * AOL_MAX_RANK + 1],
        out_w1[2 * AOL_MAX_RANK + 1], out_g[2 * AOL_MAX_RANK + 1];
    uint32_t out_mul[2 * AOL_MAX_RANK + 1], out_shift[2 * AOL_MAX_RANK + 1];
    int32_t chunk_ext, chunk_len, inner, inner_tail, nblocks;
    int32_t base, worg0, worg1, wext0, wext1, wstep0, wstep1;
    uint32_t wmul0, wshift0, wmul1, wshift1;
};

template <int ES, int MODE>
__global__ void __launch_bounds__(256) tiler_wraptab_kernel(const WrapTabDev wt, const void* __restrict__ src,
                                                            void* __restrict__ dst) {
    using T = typename Elem<ES>::T;
    constexpr int kPer = kWTab / 256;
    __shared__ int4 tab[kWTab];   // {flat offset, wrapping coordinate 0, wrapping coordinate 1} of the inner index
    for (int e = threadIdx.x; e < wt.inner; e += 256) {
        uint32_t n = uint32_t(e);
        int32_t o = 0, w0 = 0, w1 = 0;
        for (int d = wt.n_in - 1; d >= 0; --d) {
            const uint32_t q = (__umulhi(n, wt.in_mul[d]) + n) >> wt.in_shift[d];
            const int32_t i = int32_t(n - q * uint32_t(wt.in_ext[d]));
            n = q;
            o += wt.in_lin[d] * i;
            w0 += wt.in_w0[d] * i;
            w1 += wt.in_w1[d] * i;
        }
        tab[e] = make_int4(o, w0, w1, 0);
    }
    __syncthreads();
    for (int32_t blk = blockIdx.x; blk < wt.nblocks; blk += gridDim.x) {
        uint32_t n = uint32_t(blk);
        int32_t bo = wt.base, b0 = wt.worg0, b1 = wt.worg1, bg = 0, count = wt.inner;
        for (int d = wt.n_out - 1; d >= 0; --d) {
            const uint32_t q = (__umulhi(n, wt.out_mul[d]) + n) >> wt.out_shift[d];
            const int32_t i = int32_t(n - q * uint32_t(wt.out_ext[d]));
            n = q;
            bo += wt.out_lin[d] * i;
            b0 += wt.out_w0[d] * i;
            b1 += wt.out_w1[d] * i;
            bg += wt.out_g[d] * i;
            if (d == wt.n_out - 1)   // the chunk index: a partial last chunk holds fewer elements
                count = min(wt.chunk_len, wt.chunk_ext - i * wt.chunk_len) * wt.inner_tail;
        }
        int32_t off[kPer];
        T val[kPer];
#pragma unroll
        for (int k = 0; k < kPer; ++k) {
            const int e = threadIdx.x + 256 * k;
            const int4 t = tab[e < count ? e : 0];
            int32_t o = bo + t.x;
            const uint32_t w0 = uint32_t(b0 + t.y), w1 = uint32_t(b1 + t.z);
            if (wt.nw > 0) o -= int32_t((__umulhi(w0, wt.wmul0) + w0) >> wt.wshift0) * wt.wstep0;
            if (wt.nw > 1) o -= int32_t((__umulhi(w1, wt.wmul1) + w1) >> wt.wshift1) * wt.wstep1;
            off[k] = o;
        }
#pragma unroll
        for (int k = 0; k < kPer; ++k) {
            const int e = threadIdx.x + 256 * k;
            if (e < count) val[k] = MODE == 0 ? static_cast<const T*>(src)[off[k]] : static_cast<const T*>(src)[bg + e];
        }
#pragma unroll
        for (int k = 0; k < kPer; ++k) {
            const int e = threadIdx.x + 256 * k;
            if (e < count) {
                if (MODE == 0)
                    static_cast<T*>(dst)[bg + e] = val[k];
                else
                    static_cast<T*>(dst)[off[k]] = val[k];
            }
        }
    }
}

void magic32(int64_t ext, uint32_t* mul, uint32_t* shift) {
    // n / ext == (umulhi(n, mul) + n) >> shift for n, ext < 2^31
    uint32_t sh = 0;
    while (sh < 32 && (uint64_t(1) << sh) < uint64_t(ext)) ++sh;
    *mul = uint32_t(((uint64_t(1) << 32) * ((uint64_t(1) << sh) - uint64_t(ext))) / uint64_t(ext) + 1);
    *shift = sh;
}

// Blocked form of a Wrap32Dev (natural tile order; tile strides from the extents).
WrapTabDev make_wraptab(const Wrap32Dev& wd) {
    WrapTabDev wt;
    std::memset(&wt, 0, sizeof wt);
    const int nd = wd.nd;
    int64_t gst[2 * AOL_MAX_RANK];
    int64_t g = 1;
    for (int d = nd - 1; d >= 0; --d) {
        gst[d] = g;
        g *= wd.ext[d];
    }
    int k = nd - 1;
    int64_t prod = 1;
    while (k >= 0 && prod * wd.ext[k] <= kWTab) prod *= wd.ext[k--];
    const int64_t c = k >= 0 ? std::max<int64_t>(1, kWTab / prod) : 1;
    auto put_in = [&](int d, int64_t ext) {
        wt.in_ext[wt.n_in] = int32_t(ext);
        wt.in_lin[wt.n_in] = wd.lin[d];
        wt.in_w0[wt.n_in] = wd.wc[0][d];
        wt.in_w1[wt.n_in] = wd.wc[1][d];
        magic32(ext, &wt.in_mul[wt.n_in], &wt.in_shift[wt.n_in]);
        ++wt.n_in;
    };
    if (k >= 0) put_in(k, c);
    for (int d = k + 1; d < nd; ++d) put_in(d, wd.ext[d]);
    wt.inner = int32_t(prod * c);
    wt.inner_tail = int32_t(prod);
    wt.chunk_len = int32_t(c);
    int64_t nblocks = 1;
    auto put_out = [&](int64_t ext, int64_t lin, int64_t w0, int64_t w1, int64_t gs) {
        wt.out_ext[wt.n_out] = int32_t(ext);
        wt.out_lin[wt.n_out] = int32_t(lin);
        wt.out_w0[wt.n_out] = int32_t(w0);
        wt.out_w1[wt.n_out] = int32_t(w1);
        wt.out_g[wt.n_out] = int32_t(gs);
        magic32(ext, &wt.out_mul[wt.n_out], &wt.out_shift[wt.n_out]);
        ++wt.n_out;
        nblocks *= ext;
    };
    for (int d = 0; d < k; ++d) put_out(wd.ext[d], wd.lin[d], wd.wc[0][d], wd.wc[1][d], gst[d]);
    const int64_t cext = k >= 0 ? wd.ext[k] : 1;
    if (k >= 0)
        put_out((cext + c - 1) / c, int64_t(wd.lin[k]) * c, int64_t(wd.wc[0][k]) * c, int64_t(wd.wc[1][k]) * c,
                gst[k] * c);
    else
        put_out(1, 0, 0, 0, 0);
    wt.chunk_ext = int32_t(cext);
    wt.nblocks = int32_t(nblocks);
    wt.base = wd.base;
    wt.nw = wd.nw;
    wt.worg0 = wd.worg[0];
    wt.worg1 = wd.worg[1];
    wt.wext0 = wd.wext[0];
    wt.wext1 = wd.wext[1];
    wt.wstep0 = wd.wstep[0];
    wt.wstep1 = wd.wstep[1];
    wt.wmul0 = wd.wmul[0];
    wt.wshift0 = wd.wshift[0];
    wt.wmul1 = wd.wmul[1];
    wt.wshift1 = wd.wshift[1];
    return wt;
}

// ------------------------------------------------------------ footprint-staged (box) tilers
// Gathers / FAST scatters of tilers that wrap (the paper's H/V input tilers, Fig. 10; d3's wrapping
// blockings) staged through shared memory.  The tile index space (natural order) splits into OUTER dims and
// INNER dims (the innermost ones, the outermost of them possibly in chunks); for a fixed outer index the inner
// block is CONTIGUOUS on the tile side and its array-side footprint lies in a BOX of raw coordinates
//   [base_a, base_a + E_a)   per array dim a,   E_a = 1 + sum over inner dims |c_ad| (len_d - 1),
// which wraps toroidally only when the box is loaded or stored (element (b_a) <-> array ((base_a + b_a) mod s_a)).
// A CTA per block: (gather) load the box with coalesced row reads, the modulo applied once per row and per
// row wrap point, into smem; then write the tile block with 16-byte vector stores, each element's smem offset
// an affine function of its inner index (no modulo).  FAST scatter runs the same in reverse (tile block read
// with vector loads, box written out row by row) when the inner block covers its box exactly (injective
// tilers, ArrayOL single assignment).  Replaces the per-element offset arithmetic of the kernels above with
// ~10 instructions per element and keeps both global sides streaming.
constexpr int kBoxMaxInner = 4;           // inner dims (incl. the chunked one)
constexpr int kBoxBytes = 36 * 1024;      // smem per box buffer (gather: two, + the offset table: 2 CTAs per SM; 16 KB boxes measured slower: barrier-bound)
constexpr int kBoxTab = 8192;             // entries of the per-CTA inner offset table (32 KB)

// Array dims are stored REVERSED in the box descriptors (r = 0 is the innermost, contiguous array dim: the box
// row), so that every per-dim array is indexed by compile-time constants after unrolling (registers, no local
// memory).
struct BoxDev {
    int32_t ra;                                            // array rank
    int32_t ashape[AOL_MAX_RANK], astride[AOL_MAX_RANK];   // reversed
    int32_t org[AOL_MAX_RANK];                             // origin (reduced mod s), reversed
    // outer dims (enumerating blocks; the last one is the chunk index of the chunked inner dim)
    int32_t n_out;
    int32_t out_ext[2 * AOL_MAX_RANK + 1], out_g[2 * AOL_MAX_RANK + 1];
    uint32_t out_mul[2 * AOL_MAX_RANK + 1], out_shift[2 * AOL_MAX_RANK + 1];
    int32_t out_c[2 * AOL_MAX_RANK + 1][AOL_MAX_RANK];      // raw-coordinate step per outer dim (reversed)
    // inner dims, outermost first: inner dim 0 is the chunked dim (length chunk_len, last chunk shorter)
    int32_t n_in;
    int32_t in_len[kBoxMaxInner];                          // full lengths (dim 0: chunk_len)
    int32_t in_c[kBoxMaxInner][AOL_MAX_RANK];              // signed raw-coordinate step per inner dim (reversed)
    int32_t chunk_ext, chunk_len;                          // extent of the chunked dim, chunk length
    int32_t tail_prod;                                     // product of inner lengths after dim 0
    uint32_t tail_mul, tail_shift;                         // magic division by tail_prod
    uint32_t in_mul[kBoxMaxInner], in_shift[kBoxMaxInner]; // magic division by in_len (dims >= 1)
    int32_t nblocks;
    int32_t pitch_pad;                                     // extra elements per smem box row
    int32_t vec16;                                         // 1: rows load as 16-byte async copies (below)
    int32_t vs;                                            // 1: a 16-byte output vector's elements are 16 contiguous
                                                           // smem bytes at one phase: 16-byte shared reads
};

__device__ __forceinline__ uint32_t magic_div(uint32_t n, uint32_t mul, uint32_t shift) {
    return (__umulhi(n, mul) + n) >> shift;
}

// Per-block geometry: box extents / base coordinates (reversed dims) and the smem strides of the inner dims.
struct BoxBlock {
    int32_t g0, count;                 // tile-side start, elements in the block
    int32_t len0;                      // this block's length of inner dim 0
    int32_t E[AOL_MAX_RANK];           // box extents (E[0]: the row length)
    int32_t base[AOL_MAX_RANK];        // box origin, reduced into [0, s)
    int32_t step[kBoxMaxInner];        // smem offset per unit of inner dim d
    int32_t off0;                      // smem offset of inner index 0
    int32_t rows, pitch;
    int32_t phase;                     // vec16: box element x of a row sits at smem x + phase (same 16-byte phase as
                                       // its global address)
};

__device__ __forceinline__ void box_block(const BoxDev& bd, int32_t blk, BoxBlock& b) {
    uint32_t n = uint32_t(blk);
    int64_t raw[AOL_MAX_RANK];   // raw coordinates of the outer index (64-bit: sums of coef x index)
#pragma unroll
    for (int r = 0; r < AOL_MAX_RANK; ++r) raw[r] = r < bd.ra ? bd.org[r] : 0;
    b.g0 = 0;
    int32_t ck = 0;
    for (int d = bd.n_out - 1; d >= 0; --d) {
        const uint32_t q = magic_div(n, bd.out_mul[d], bd.out_shift[d]);
        const int32_t i = int32_t(n - q * uint32_t(bd.out_ext[d]));
        n = q;
        if (d == bd.n_out - 1) ck = i;
        b.g0 += bd.out_g[d] * i;
#pragma unroll
        for (int r = 0; r < AOL_MAX_RANK; ++r)
            if (r < bd.ra) raw[r] += int64_t(bd.out_c[d][r]) * i;
    }
    b.len0 = min(bd.chunk_len, bd.chunk_ext - ck * bd.chunk_len);
    b.count = b.len0 * bd.tail_prod;
    // box extents, the corner's raw offset (negative steps reach below the outer index's raw point) and smem
    // strides (r = 0: stride 1 along a row of pitch E[0] + pad; r > 0: products)
    int32_t st = 1;
    b.rows = 1;
    b.off0 = 0;
    int32_t bstride[AOL_MAX_RANK];
#pragma unroll
    for (int r = 0; r < AOL_MAX_RANK; ++r) {
        b.E[r] = 1;
        b.base[r] = 0;
        bstride[r] = 0;
        if (r >= bd.ra) continue;
        int32_t lo = 0, hi = 0;
#pragma unroll
        for (int d = 0; d < kBoxMaxInner; ++d) {
            if (d >= bd.n_in) continue;
            const int32_t c = bd.in_c[d][r], l = (d == 0 ? b.len0 : bd.in_len[d]) - 1;
            if (c < 0) lo += c * l; else hi += c * l;
        }
        b.E[r] = hi - lo + 1;
        const int32_t v = int32_t((raw[r] + lo) % bd.ashape[r]);
        b.base[r] = v < 0 ? v + bd.ashape[r] : v;
        bstride[r] = st;
        if (r == 0) {
            if (bd.vec16) {
                // 16-byte async row copies: box element x sits at smem x + phase, the 16-byte phase of its global
                // address (every row start has phase 0 and the row extent is a multiple of 16 bytes: host-checked);
                // the pitch keeps row starts 16-byte aligned and is padded off multiples of 128 bytes
                const int32_t V = bd.vec16;
                b.phase = b.base[0] % V;
                b.pitch = (b.E[0] + 2 * V - 2) / V * V;
                if (bd.vs) {
                    // 16-byte reads: rows 8 words (mod 32) apart, so a quarter-warp reading chunks of 4 consecutive
                    // rows x 2 adjacent chunks hits 8 different bank groups (the d3 blocking's access shape)
                    const int32_t wpe = 16 / V / 4 > 0 ? 16 / V / 4 : 1;   // 4-byte words per element (ES >= 4)
                    while ((b.pitch * wpe) % 32 != 8) b.pitch += V;
                } else if ((b.pitch * (16 / V)) % 128 == 0) {
                    b.pitch += V;
                }
            } else {
                b.phase = 0;
                b.pitch = b.E[0] + bd.pitch_pad;
            }
            st = b.pitch;
        } else {
            st *= b.E[r];
            b.rows *= b.E[r];
        }
        b.off0 += -lo * bstride[r];   // smem offset of inner index 0
    }
    b.off0 += b.phase;
#pragma unroll
    for (int d = 0; d < kBoxMaxInner; ++d) {
        int32_t o = 0;
#pragma unroll
        for (int r = 0; r < AOL_MAX_RANK; ++r)
            if (r < bd.ra && d < bd.n_in) o += bd.in_c[d][r] * bstride[r];
        b.step[d] = o;
    }
}

// Global element offset of box row `row` (box dims r >= 1; r = 1 varies fastest).
__device__ __forceinline__ int32_t box_row_offset(const BoxDev& bd, const BoxBlock& b, int32_t row) {
    int32_t off = 0;
#pragma unroll
    for (int r = 1; r < AOL_MAX_RANK; ++r) {
        if (r >= bd.ra) continue;
        const int32_t q = row / b.E[r];
        int32_t v = b.base[r] + (row - q * b.E[r]);
        row = q;
        while (v >= bd.ashape[r]) v -= bd.ashape[r];
        off += v * bd.astride[r];
    }
    return off;
}

// Smem offsets of the TAIL of the inner block (inner dims >= 1, tail_prod elements, row-major) relative to the
// offset of its inner-dim-0 index: tab[t] = sum_{d >= 1} step[d] idx_d(t).  Built per CTA whenever the box
// layout changes (only between a full and the ragged last chunk), so an element's box offset is then
// off0 + step[0] i0 + tab[t]: one magic division per 16-byte vector and two shared loads per element.
__device__ __forceinline__ void box_build_table(const BoxDev& bd, const BoxBlock& b, int16_t* tab) {
    for (int32_t t = threadIdx.x; t < bd.tail_prod; t += blockDim.x) {
        uint32_t rem = uint32_t(t);
        int32_t off = 0;
#pragma unroll
        for (int d = kBoxMaxInner - 1; d >= 1; --d) {
            if (d >= bd.n_in) continue;
            const uint32_t q = magic_div(rem, bd.in_mul[d], bd.in_shift[d]);
            off += b.step[d] * int32_t(rem - q * uint32_t(bd.in_len[d]));
            rem = q;
        }
        tab[t] = int16_t(off);   // |off| < box elements <= 32767
    }
}

// Issue the loads of a block's box into smem buffer `buf`: a warp per box row, lanes along the row (coalesced),
// wrapped at the row's end.  4- and 8-byte elements: asynchronous copies (cp.async, committed as one group by
// the caller: the whole box in flight at once); 1- and 2-byte elements: plain loads and stores.
template <int ES>
__device__ __forceinline__ void box_issue_load(const BoxDev& bd, const BoxBlock& b, const void* src, uint8_t* buf) {
    using T = typename Elem<ES>::T;
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    const int sl = bd.ashape[0];
    const int32_t El = b.E[0], c0 = b.base[0];
    const T* A = static_cast<const T*>(src);
    for (int32_t row = warp; row < b.rows; row += 8) {
        const int32_t roff = box_row_offset(bd, b, row);
        if constexpr (ES >= 4) {
            const uint32_t srow = ptx::smem_u32(buf) + uint32_t(row * b.pitch + b.phase) * ES;
            if (bd.vec16) {
                // the row as contiguous global segments (the wrap restarts at column 0), each copied as an unaligned
                // head, 16-byte chunks and a tail; smem and global share the 16-byte phase
                constexpr int32_t V = 16 / ES;
                int32_t x = 0, gc = c0;
                while (x < El) {
                    const int32_t len = min(El - x, sl - gc);
                    const int32_t head = min(len, (V - gc % V) % V);
                    const int32_t nch = (len - head) / V;
                    const int32_t tail = len - head - nch * V;
                    const uint32_t sseg = srow + uint32_t(x) * ES;
                    const T* gseg = A + roff + gc;
                    if (lane < head) ptx::cp_async<ES>(sseg + uint32_t(lane) * ES, gseg + lane);
                    for (int32_t c = lane; c < nch; c += 32)
                        ptx::cp_async<16>(sseg + uint32_t(head + c * V) * ES, gseg + head + c * V);
                    if (lane < tail)
                        ptx::cp_async<ES>(sseg + uint32_t(head + nch * V + lane) * ES, gseg + head + nch * V + lane);
                    x += len;
                    gc = 0;
                }
            } else {
                for (int32_t x = lane; x < El; x += 32) {
                    int32_t gc = c0 + x;
                    while (gc >= sl) gc -= sl;
                    ptx::cp_async<ES>(srow + uint32_t(x) * ES, A + roff + gc);
                }
            }
        } else {
            T* srow = reinterpret_cast<T*>(buf) + row * b.pitch;
            constexpr int kU = 8;
            for (int32_t x0 = lane; x0 < El; x0 += 32 * kU) {
                T v[kU];
#pragma unroll
                for (int u = 0; u < kU; ++u) {
                    const int32_t x = x0 + 32 * u;
                    int32_t gc = c0 + x;
                    while (gc >= sl) gc -= sl;
                    if (x < El) v[u] = A[roff + gc];
                }
#pragma unroll
                for (int u = 0; u < kU; ++u)
                    if (x0 + 32 * u < El) srow[x0 + 32 * u] = v[u];
            }
        }
    }
}

// The VW table entries of a 16-byte output vector (t is a multiple of VW): one 16-byte (or two / four) shared
// load(s) instead of VW scalar ones (those hit the same bank group from every quarter-warp).
template <int VW>
__device__ __forceinline__ void box_tab_vec(const int16_t* tab, int32_t t, int32_t (&o)[VW]) {
    // VW int16 entries at t (a multiple of VW): one shared load of 2 VW bytes (two 16-byte loads for VW = 16)
    if constexpr (VW >= 8) {
#pragma unroll
        for (int q = 0; q < VW / 8; ++q) {
            const int4 v = *reinterpret_cast<const int4*>(tab + t + 8 * q);
            const uint32_t w[4] = {uint32_t(v.x), uint32_t(v.y), uint32_t(v.z), uint32_t(v.w)};
#pragma unroll
            for (int i = 0; i < 4; ++i) {
                o[8 * q + 2 * i] = int32_t(int16_t(w[i] & 0xffffu));
                o[8 * q + 2 * i + 1] = int32_t(w[i]) >> 16;
            }
        }
    } else if constexpr (VW == 4) {
        const int2 v = *reinterpret_cast<const int2*>(tab + t);
        o[0] = int32_t(int16_t(uint32_t(v.x) & 0xffffu));
        o[1] = v.x >> 16;
        o[2] = int32_t(int16_t(uint32_t(v.y) & 0xffffu));
        o[3] = v.y >> 16;
    } else if constexpr (VW == 2) {
        const int32_t v = *reinterpret_cast<const int32_t*>(tab + t);
        o[0] = int32_t(int16_t(uint32_t(v) & 0xffffu));
        o[1] = v >> 16;
    } else {
        o[0] = tab[t];
    }
}

// smem: [tail_prod] int16 offset table, then one box buffer (FAST scatter; gather with nbuf = 1) or two (gather,
// nbuf = 2: the next block's box loads asynchronously while the current one is written out), 16-byte aligned.  A block's geometry is
// computed once, by thread 0, into shared memory (every thread computing it cost ~20 instructions per element).
template <int ES, int VW, int MODE>
__global__ void __launch_bounds__(256) tiler_box_kernel(const __grid_constant__ BoxDev bd, const void* __restrict__ src,
                                                        void* __restrict__ dst, int32_t buf_bytes, int32_t nbuf) {
    using T = typename Elem<ES>::T;
    using VT = typename Vec<ES * VW>::T;
    extern __shared__ __align__(16) uint8_t box_raw[];
    __shared__ BoxBlock geo[2];
    int16_t* tab = reinterpret_cast<int16_t*>(box_raw);
    uint8_t* bufs = box_raw + ((size_t(bd.tail_prod) * 2 + 15) & ~size_t(15));
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    const int sl = bd.ashape[0];
    int32_t tab_len0 = -1;   // len0 the table was built for
    if (MODE == 0) {
        // nbuf = 2: software pipeline over this CTA's blocks, box k+1 loads while box k is emitted; nbuf = 1: one
        // buffer (less smem, more CTAs per SM: the overlap comes from the other CTAs)
        int32_t blk = blockIdx.x;
        if (threadIdx.x == 0 && blk < bd.nblocks) box_block(bd, blk, geo[0]);
        __syncthreads();
        if (nbuf == 2 && blk < bd.nblocks) box_issue_load<ES>(bd, geo[0], src, bufs);
        ptx::cp_async_commit();
        for (int32_t k = 0; blk < bd.nblocks; ++k, blk += gridDim.x) {
            const int32_t nxt = blk + gridDim.x;
            const int slot = nbuf == 2 ? (k & 1) : 0;
            const BoxBlock& b = geo[slot];
            if (nbuf == 2) {
                BoxBlock& gn = geo[(k + 1) & 1];
                if (threadIdx.x == 0 && nxt < bd.nblocks) box_block(bd, nxt, gn);
                __syncthreads();
                if (nxt < bd.nblocks) box_issue_load<ES>(bd, gn, src, bufs + ((k + 1) & 1) * buf_bytes);
                ptx::cp_async_commit();
            } else {
                box_issue_load<ES>(bd, b, src, bufs);
                ptx::cp_async_commit();
            }
            if (b.len0 != tab_len0) {   // uniform across the CTA; the previous block's reads of tab have finished
                box_build_table(bd, b, tab);
                tab_len0 = b.len0;
            }
            if (nbuf == 2)
                ptx::cp_async_wait<1>();   // this block's box has landed (the next one may still be in flight)
            else
                ptx::cp_async_wait<0>();
            __syncthreads();
            const T* box = reinterpret_cast<const T*>(bufs + slot * buf_bytes);
            T* Tg = static_cast<T*>(dst) + b.g0;
            const int32_t count = b.count, off0 = b.off0, step0 = b.step[0];
            // four independent vectors per thread per iteration: their table and data loads overlap (one vector
            // at a time left the loop waiting on shared-memory latency)
            constexpr int kU = 4;
            for (int32_t v0 = threadIdx.x; v0 * VW < count; v0 += 256 * kU) {
                int32_t o[kU], to[kU][VW];
#pragma unroll
                for (int u = 0; u < kU; ++u) {
                    const int32_t v = min(v0 + 256 * u, count / VW - 1);
                    const uint32_t e = uint32_t(v * VW);
                    const uint32_t i0 = magic_div(e, bd.tail_mul, bd.tail_shift);
                    const int32_t t = int32_t(e - i0 * uint32_t(bd.tail_prod));
                    o[u] = off0 + step0 * int32_t(i0);
                    box_tab_vec<VW>(tab, t, to[u]);
                }
                union { VT vec; T e[VW]; } pk[kU];
                if constexpr (ES >= 4 && VW * ES == 16) {
                    if (bd.vs) {
                        // the vector's elements are contiguous in smem at a block-uniform phase: one 16-byte read
                        // (phase 0) or two and a selection
                        const int32_t ph = b.phase;
#pragma unroll
                        for (int u = 0; u < kU; ++u) {
                            const int32_t a0 = o[u] + to[u][0] - ph;   // 16-byte aligned
                            const uint4 c0 = *reinterpret_cast<const uint4*>(box + a0);
                            if (ph == 0) {
                                pk[u].vec = *reinterpret_cast<const VT*>(&c0);
                            } else {
                                const uint4 c1 = *reinterpret_cast<const uint4*>(box + a0 + VW);
                                const uint32_t w[8] = {c0.x, c0.y, c0.z, c0.w, c1.x, c1.y, c1.z, c1.w};
                                const int sh = ph * (ES / 4);   // in 4-byte words
                                uint32_t r[4];
#pragma unroll
                                for (int q = 0; q < 4; ++q)
                                    r[q] = sh == 1 ? w[q + 1] : sh == 2 ? w[q + 2] : w[q + 3];
                                pk[u].vec = *reinterpret_cast<const VT*>(r);
                            }
                        }
                    } else {
#pragma unroll
                        for (int u = 0; u < kU; ++u)
#pragma unroll
                            for (int j = 0; j < VW; ++j) pk[u].e[j] = box[o[u] + to[u][j]];
                    }
                } else {
#pragma unroll
                    for (int u = 0; u < kU; ++u)
#pragma unroll
                        for (int j = 0; j < VW; ++j) pk[u].e[j] = box[o[u] + to[u][j]];
                }
#pragma unroll
                for (int u = 0; u < kU; ++u)
                    if ((v0 + 256 * u) * VW < count) reinterpret_cast<VT*>(Tg)[v0 + 256 * u] = pk[u].vec;
            }
            __syncthreads();   // this buffer, its geometry slot and tab may be overwritten from here on
            if (nbuf == 1 && threadIdx.x == 0 && nxt < bd.nblocks) box_block(bd, nxt, geo[0]);
            if (nbuf == 1) __syncthreads();
        }
        ptx::cp_async_wait<0>();
    } else {
        T* box = reinterpret_cast<T*>(bufs);
        for (int32_t blk = blockIdx.x; blk < bd.nblocks; blk += gridDim.x) {
            if (threadIdx.x == 0) box_block(bd, blk, geo[0]);
            __syncthreads();
            const BoxBlock& b = geo[0];
            const int32_t El = b.E[0], c0 = b.base[0];
            if (b.len0 != tab_len0) {
                box_build_table(bd, b, tab);
                tab_len0 = b.len0;
                __syncthreads();
            }
            // ---- FAST scatter: the tile block into the box (it covers the box exactly), then the box out;
            // four 16-byte tile loads in flight per thread
            const T* Tg = static_cast<const T*>(src) + b.g0;
            const int32_t count = b.count, off0 = b.off0, step0 = b.step[0];
            constexpr int kU = 4;
            for (int32_t v0 = threadIdx.x; v0 * VW < count; v0 += 256 * kU) {
                union { VT vec; T e[VW]; } pk[kU];
#pragma unroll
                for (int u = 0; u < kU; ++u)
                    if ((v0 + 256 * u) * VW < count) pk[u].vec = reinterpret_cast<const VT*>(Tg)[v0 + 256 * u];
                int32_t o[kU], to[kU][VW];
#pragma unroll
                for (int u = 0; u < kU; ++u) {
                    const int32_t v = min(v0 + 256 * u, count / VW - 1);
                    const uint32_t e = uint32_t(v * VW);
                    const uint32_t i0 = magic_div(e, bd.tail_mul, bd.tail_shift);
                    const int32_t t = int32_t(e - i0 * uint32_t(bd.tail_prod));
                    o[u] = off0 + step0 * int32_t(i0);
                    box_tab_vec<VW>(tab, t, to[u]);
                }
#pragma unroll
                for (int u = 0; u < kU; ++u)
                    if ((v0 + 256 * u) * VW < count)
#pragma unroll
                        for (int j = 0; j < VW; ++j) box[o[u] + to[u][j]] = pk[u].e[j];
            }
            __syncthreads();
            T* A = static_cast<T*>(dst);
            for (int32_t row = warp; row < b.rows; row += 8) {
                const int32_t roff = box_row_offset(bd, b, row);
                const T* srow = box + row * b.pitch + b.phase;
                for (int32_t x = lane; x < El; x += 32) {
                    int32_t gc = c0 + x;
                    while (gc >= sl) gc -= sl;
                    A[roff + gc] = srow[x];
                }
            }
            __syncthreads();   // the box and geo[0] are rewritten by the next block
        }
    }
}

// Plan the box form of a tiler (fast32, every offset < 2^31); false if it does not qualify: the inner block
// must be dense in its box (gather: box <= 1.5 x inner elements; scatter: exactly equal), box rows >= 32
// elements long, <= kBoxMaxInner inner dims, box within kBoxBytes.
bool make_box(const TilerDev& td, int es, int mode, BoxDev* bd, int* smem_bytes, int* buf_bytes) {
    if (!td.fast32 || td.array_elems >= (int64_t(1) << 31) || td.nd == 0) return false;
    std::memset(bd, 0, sizeof *bd);
    const int nd = td.nd, ra = td.ra;
    int64_t sc[2 * AOL_MAX_RANK][AOL_MAX_RANK];   // signed raw steps (representative nearest 0)
    for (int d = 0; d < nd; ++d)
        for (int a = 0; a < ra; ++a) {
            int64_t c = td.coef[a][d];
            if (2 * c > td.ashape[a]) c -= td.ashape[a];
            sc[d][a] = c;
        }
    auto box_of = [&](int k, int64_t lenk, int64_t* E) {   // inner = (chunk of dim k of length lenk), k+1..nd-1
        int64_t vol = 1;
        for (int a = 0; a < ra; ++a) {
            int64_t span = 0;
            for (int d = k; d < nd; ++d) {
                const int64_t l = (d == k ? lenk : td.ext[d]) - 1;
                span += (sc[d][a] < 0 ? -sc[d][a] : sc[d][a]) * l;
            }
            E[a] = span + 1;
            vol *= E[a];
            if (vol > (int64_t(1) << 40)) vol = int64_t(1) << 40;
        }
        return vol;
    };
    const int64_t budget = std::min<int64_t>(kBoxBytes / es, 32767 - 4 * 32);   // int16 table offsets
    // grow the inner block from the innermost dim outwards while the box fits; the first dim that does not fit
    // entirely is chunked
    int k = nd - 1;
    int64_t E[AOL_MAX_RANK], lenk = td.ext[k];
    for (;;) {
        const int64_t pitch_extra = 4;
        int64_t vol = box_of(k, td.ext[k], E);
        if (vol + pitch_extra * (vol / std::max<int64_t>(1, E[ra - 1])) <= budget) {   // all of dim k fits
            lenk = td.ext[k];
            if (k == 0 || nd - (k - 1) > kBoxMaxInner) break;
            int64_t tail = 1;   // the table would cover dims k..nd-1 once dim k-1 is the chunked one
            for (int d = k; d < nd; ++d) tail *= td.ext[d];
            if (tail > kBoxTab) break;
            int64_t E2[AOL_MAX_RANK];
            const int64_t v2 = box_of(k - 1, 1, E2);   // would one slice of dim k-1 still fit?
            if (v2 + pitch_extra * (v2 / std::max<int64_t>(1, E2[ra - 1])) > budget) break;
            --k;
            continue;
        }
        // chunk dim k: the largest length that fits
        int64_t lo = 1, hi = td.ext[k];
        while (lo < hi) {
            const int64_t mid = (lo + hi + 1) / 2;
            const int64_t v = box_of(k, mid, E);
            if (v + pitch_extra * (v / std::max<int64_t>(1, E[ra - 1])) <= budget) lo = mid; else hi = mid - 1;
        }
        lenk = lo;
        const int64_t v = box_of(k, lenk, E);
        if (v + pitch_extra * (v / std::max<int64_t>(1, E[ra - 1])) > budget) return false;
        break;
    }
    if (nd - k > kBoxMaxInner) return false;
    const int64_t vol = box_of(k, lenk, E);
    int64_t inner = lenk;
    for (int d = k + 1; d < nd; ++d) inner *= td.ext[d];
    if (inner / lenk > kBoxTab) return false;
    if (mode == 0 ? (2 * vol > 3 * inner) : (vol != inner)) return false;
    if (E[ra - 1] < 32) return false;
    if (E[ra - 1] > 2 * td.ashape[ra - 1]) return false;   // the row wrap takes at most two subtractions
    bd->ra = ra;
    for (int a = 0; a < ra; ++a) {   // reversed: r = ra - 1 - a
        bd->ashape[ra - 1 - a] = int32_t(td.ashape[a]);
        bd->astride[ra - 1 - a] = int32_t(td.astride[a]);
        bd->org[ra - 1 - a] = int32_t(td.org[a]);
    }
    int64_t gst[2 * AOL_MAX_RANK];
    int64_t g = 1;
    for (int d = nd - 1; d >= 0; --d) {
        gst[d] = g;
        g *= td.ext[d];
    }
    int no = 0;
    for (int d = 0; d < k; ++d, ++no) {
        bd->out_ext[no] = int32_t(td.ext[d]);
        bd->out_g[no] = int32_t(gst[d]);
        magic32(td.ext[d], &bd->out_mul[no], &bd->out_shift[no]);
        for (int a = 0; a < ra; ++a) bd->out_c[no][ra - 1 - a] = int32_t(td.coef[a][d]);
    }
    const int64_t nch = (td.ext[k] + lenk - 1) / lenk;   // chunks of dim k (the last outer dim, possibly 1)
    bd->out_ext[no] = int32_t(nch);
    bd->out_g[no] = int32_t(gst[k] * lenk);
    magic32(nch, &bd->out_mul[no], &bd->out_shift[no]);
    for (int a = 0; a < ra; ++a) bd->out_c[no][ra - 1 - a] = int32_t((int64_t(td.coef[a][k]) * lenk) % td.ashape[a]);
    ++no;
    bd->n_out = no;
    int64_t nblocks = nch;
    for (int d = 0; d < k; ++d) nblocks *= td.ext[d];
    if (nblocks >= (int64_t(1) << 31)) return false;
    bd->nblocks = int32_t(nblocks);
    bd->n_in = nd - k;
    bd->chunk_ext = int32_t(td.ext[k]);
    bd->chunk_len = int32_t(lenk);
    for (int j = 0; j < bd->n_in; ++j) {
        const int d = k + j;
        bd->in_len[j] = int32_t(j == 0 ? lenk : td.ext[d]);
        for (int a = 0; a < ra; ++a) bd->in_c[j][ra - 1 - a] = int32_t(sc[d][a]);
        if (j >= 1) magic32(td.ext[d], &bd->in_mul[j], &bd->in_shift[j]);
    }
    bd->tail_prod = int32_t(inner / lenk);
    magic32(bd->tail_prod, &bd->tail_mul, &bd->tail_shift);
    bd->pitch_pad = (E[ra - 1] % 32 == 0) ? 1 : 0;   // rows of 32-multiple length: odd pitch, fewer bank conflicts
    // 16-byte async row copies: 4- or 8-byte elements, every row start 16-byte aligned (row strides and the
    // row length multiples of 16 bytes) so that a box row shares its global addresses' 16-byte phase
    if (es >= 4) {
        const int V = 16 / es;
        bool ok = td.ashape[ra - 1] % V == 0;
        for (int a = 0; a < ra - 1; ++a) ok = ok && td.astride[a] % V == 0;
        bd->vec16 = ok ? V : 0;
        // 16-byte shared reads of an output vector: the innermost inner dim walks the row (+1 per element) and
        // its length is a multiple of V, every other inner dim steps the row by multiples of V (its steps along
        // other array dims are multiples of the pitch, itself a multiple of V)
        const int j_last = nd - 1;
        bool vs = ok && (mode == 0) && td.ext[j_last] % V == 0 && (nd - k) >= 1;
        for (int a = 0; a < ra && vs; ++a) {
            const int64_t c = sc[j_last][a];
            vs = (a == ra - 1) ? c == 1 : c == 0;
        }
        for (int d = k; d < j_last && vs; ++d) vs = sc[d][ra - 1] % V == 0;
        bd->vs = vs ? 1 : 0;
    }
    const int64_t rows = vol / E[ra - 1];
    const int64_t pitch_max = bd->vec16 ? E[ra - 1] + 3 * bd->vec16 + (bd->vs ? 32 : 0) : E[ra - 1] + bd->pitch_pad;
    const int64_t buf = (rows * pitch_max * es + 15) / 16 * 16;
    *buf_bytes = int(buf);
    *smem_bytes = int(((inner / lenk) * 2 + 15) / 16 * 16 + (mode == 0 ? 2 : 1) * buf);   // (2 buffers: see caller)
    return true;
}

// AOL_TILER_BOX=0 disables the staged box kernels (A/B measurements only).
bool tiler_box_enabled() {
    static const bool v = [] {
        const char* e = std::getenv("AOL_TILER_BOX");
        return !(e && e[0] == '0');
    }();
    return v;
}

// ------------------------------------------------------------ affine pieces of wrapping tilers
// A wrapping tiler is affine on each region of its index space where no coordinate crosses the array edge.  When
// every wrapping array dim is driven by at most two combined dims (an outer one and an inner one, used by no other
// wrapping dim) and wraps at most once, those regions are a few boxes of the index space: for the outer index
// values whose whole inner range stays inside (or wraps), one box; for the few boundary values, a split of the
// inner range.  Each box is a LINEAR tiler on a sub-range (its own array base, the wrap folded in as -s_a *
// stride_a), so the pieces run through the affine kernel's permuted walk with 16-byte vectors -- the d3 blocking
// shifted to wrap in both image dims is 1 big piece + 8 slivers.  Pieces are cut into chunks of 1024 vectors, one
// per CTA, which stages its piece's constants in shared memory (like the affine kernel's large grid).
constexpr int kMaxPieces = 32;   // (a blocking wrapping in 3 dims: 3 x 3 x 2 = 18)
constexpr int kPieceChunk = 1024;   // vectors per chunk (= per CTA: 2 iterations of 256 threads x 2 vectors)

struct PiecesDev {
    int32_t nd, npieces, nchunks;
    int32_t p_lin[2 * AOL_MAX_RANK], p_gst[2 * AOL_MAX_RANK];    // permuted strides (the parent's)
    int32_t len[kMaxPieces][2 * AOL_MAX_RANK];                   // permuted extents of each piece
    uint32_t mul[kMaxPieces][2 * AOL_MAX_RANK], shift[kMaxPieces][2 * AOL_MAX_RANK];
    int32_t abase[kMaxPieces], tbase[kMaxPieces];
    int32_t nvec[kMaxPieces];                                    // vectors in the piece
    int32_t phase[kMaxPieces];                                   // array-side misalignment (elements)
    int32_t vec[kMaxPieces];                                     // 1: walked with vectors, 0: element by element
    int32_t chunk0[kMaxPieces + 1];                              // first chunk of each piece (prefix)
};

// 16 bytes starting `b` bytes (0..15) into the 32 bytes (lo, hi): the misaligned array-side read of a vector
// whose aligned neighbours were loaded instead (funnel shifts; b is uniform across the CTA, so the word offset is a
// uniform branch rather than a select chain per word).
__device__ __forceinline__ uint4 shift16(const uint4& lo, const uint4& hi, uint32_t b) {
    const uint32_t sh = (b & 3u) * 8u;
    switch (b >> 2) {
        case 0:
            return make_uint4(__funnelshift_r(lo.x, lo.y, sh), __funnelshift_r(lo.y, lo.z, sh),
                              __funnelshift_r(lo.z, lo.w, sh), __funnelshift_r(lo.w, hi.x, sh));
        case 1:
            return make_uint4(__funnelshift_r(lo.y, lo.z, sh), __funnelshift_r(lo.z, lo.w, sh),
                              __funnelshift_r(lo.w, hi.x, sh), __funnelshift_r(hi.x, hi.y, sh));
        case 2:
            return make_uint4(__funnelshift_r(lo.z, lo.w, sh), __funnelshift_r(lo.w, hi.x, sh),
                              __funnelshift_r(hi.x, hi.y, sh), __funnelshift_r(hi.y, hi.z, sh));
        default:
            return make_uint4(__funnelshift_r(lo.w, hi.x, sh), __funnelshift_r(hi.x, hi.y, sh),
                              __funnelshift_r(hi.y, hi.z, sh), __funnelshift_r(hi.z, hi.w, sh));
    }
}

// The walk of one chunk of a piece with W-element accesses (W = the vector width, or 1 for a piece that cannot
// be vectorised), the digit constants in registers.
template <int ES, int W, int MODE, int NDU>
__device__ __forceinline__ void pieces_walk(const int32_t (&L)[NDU], const uint32_t (&M)[NDU], const uint32_t (&S)[NDU],
                                            const int32_t (&AL)[NDU], const int32_t (&GS)[NDU], int32_t v_begin,
                                            int32_t v_end, int32_t ab, int32_t tb, int32_t ph,
                                            const void* __restrict__ src, void* __restrict__ dst) {
    constexpr int V = W;
    using T = typename Elem<ES>::T;
    using VT = typename Vec<ES * V>::T;
    const uint32_t lane = threadIdx.x & 31u;
    constexpr int kU = 2;
    for (int32_t v0 = v_begin + int32_t((threadIdx.x & ~31u) * kU + lane); v0 < v_end + int32_t(lane);
         v0 += 256 * kU) {   // (whole warps iterate together: the realignment below shuffles)
        int32_t off[kU], g[kU];
#pragma unroll
        for (int u = 0; u < kU; ++u) {
            const int32_t v = v0 + 32 * u;
            uint32_t n = v < v_end ? uint32_t(v) * V : 0u;
            int32_t o = ab, gg = tb;
#pragma unroll
            for (int d = NDU - 1; d >= 1; --d) {
                const uint32_t q = (__umulhi(n, M[d]) + n) >> S[d];
                const int32_t i = int32_t(n - q * uint32_t(L[d]));
                n = q;
                o += AL[d] * i;
                gg += GS[d] * i;
            }
            o += AL[0] * int32_t(n);   // the outermost digit is what is left (n < L[0] for every valid vector)
            gg += GS[0] * int32_t(n);
            off[u] = o;
            g[u] = gg;
        }
        VT val[kU];
        if constexpr (MODE == 0 && V * ES == 16) {
            if (ph != 0) {
                // array side misaligned by ph elements: each lane loads the aligned 16 bytes holding its vector's
                // head; the tail comes from the next lane's load when that lane's vector follows on in the array
                // (runs of tiles along a row), else from a second load of its own, issued together with the first
                // (known from the decoded offsets alone).  Lanes past the end load the piece's first vector (in
                // bounds) so that the whole warp takes part in the shuffles.
                bool own[kU];
#pragma unroll
                for (int u = 0; u < kU; ++u) {
                    const int32_t noff = __shfl_down_sync(0xffffffffu, off[u], 1);
                    own[u] = v0 + 32 * u < v_end && (lane == 31 || noff != off[u] + V);
                }
                uint4 lo[kU], hi[kU];
#pragma unroll
                for (int u = 0; u < kU; ++u) {
                    const uint4* a = reinterpret_cast<const uint4*>(static_cast<const T*>(src) + off[u] - ph);
                    lo[u] = a[0];
                    if (own[u]) hi[u] = a[1];
                }
#pragma unroll
                for (int u = 0; u < kU; ++u) {
                    uint4 h;
                    h.x = __shfl_down_sync(0xffffffffu, lo[u].x, 1);
                    h.y = __shfl_down_sync(0xffffffffu, lo[u].y, 1);
                    h.z = __shfl_down_sync(0xffffffffu, lo[u].z, 1);
                    h.w = __shfl_down_sync(0xffffffffu, lo[u].w, 1);
                    if (!own[u]) hi[u] = h;
                    const uint4 r = shift16(lo[u], hi[u], uint32_t(ph * ES));
                    val[u] = *reinterpret_cast<const VT*>(&r);
                }
            } else {
#pragma unroll
                for (int u = 0; u < kU; ++u)
                    if (v0 + 32 * u < v_end) val[u] = reinterpret_cast<const VT*>(static_cast<const T*>(src) + off[u])[0];
            }
        } else {
#pragma unroll
            for (int u = 0; u < kU; ++u)
                if (v0 + 32 * u < v_end)
                    val[u] = reinterpret_cast<const VT*>(static_cast<const T*>(src) + (MODE == 0 ? off[u] : g[u]))[0];
        }
        if constexpr (MODE == 1 && V * ES == 16) {
            if (ph != 0) {
                // array side misaligned by ph elements: lane L stores the aligned 16 bytes that start inside its
                // vector (its last ph elements + the next lane's first V - ph) when the next lane's vector follows
                // on in the array; a vector without such a neighbour stores its tail, one without an array-side
                // predecessor its head, element by element.  Every element is stored exactly once.
#pragma unroll
                for (int u = 0; u < kU; ++u) {
                    const bool valid = v0 + 32 * u < v_end;
                    const uint4 lo = *reinterpret_cast<const uint4*>(&val[u]);
                    uint4 hi;
                    hi.x = __shfl_down_sync(0xffffffffu, lo.x, 1);
                    hi.y = __shfl_down_sync(0xffffffffu, lo.y, 1);
                    hi.z = __shfl_down_sync(0xffffffffu, lo.z, 1);
                    hi.w = __shfl_down_sync(0xffffffffu, lo.w, 1);
                    const int32_t noff = __shfl_down_sync(0xffffffffu, off[u], 1);
                    const int32_t poff = __shfl_up_sync(0xffffffffu, off[u], 1);
                    const bool nvalid = __shfl_down_sync(0xffffffffu, int(valid), 1) != 0;
                    if (!valid) continue;
                    const bool next = lane != 31 && nvalid && noff == off[u] + V;
                    const bool prev = lane != 0 && poff + V == off[u];
                    T* a = static_cast<T*>(dst) + off[u];
                    if (next) {
                        *reinterpret_cast<uint4*>(a - ph + V) = shift16(lo, hi, uint32_t((V - ph) * ES));
                    } else {
                        T e[V];
                        memcpy(e, &val[u], sizeof e);
#pragma unroll
                        for (int k = 1; k < V; ++k)
                            if (k >= V - ph) a[k] = e[k];
                    }
                    if (!prev) {
                        T e[V];
                        memcpy(e, &val[u], sizeof e);
#pragma unroll
                        for (int k = 0; k < V - 1; ++k)
                            if (k < V - ph) a[k] = e[k];
                    }
                }
                continue;
            }
        }
#pragma unroll
        for (int u = 0; u < kU; ++u)
            if (v0 + 32 * u < v_end)
                reinterpret_cast<VT*>(static_cast<T*>(dst) + (MODE == 0 ? g[u] : off[u]))[0] = val[u];
    }
}

template <int ES, int V, int MODE, int NDU>
__global__ void __launch_bounds__(256) tiler_pieces_kernel(const __grid_constant__ PiecesDev pd,
                                                           const void* __restrict__ src, void* __restrict__ dst) {
    const int32_t c = int32_t(blockIdx.x);   // one chunk per CTA (a persistent chunk loop measured slower)
    int pc = 0;
    while (pc + 1 < pd.npieces && pd.chunk0[pc + 1] <= c) ++pc;
    // the piece's walk constants in registers, padded to NDU dims with unit extents on the outside: the digit
    // loop is then fully unrolled without loads (the walk's instruction count bounds this kernel)
    int32_t L[NDU], AL[NDU], GS[NDU];
    uint32_t M[NDU], S[NDU];
#pragma unroll
    for (int d = 0; d < NDU; ++d) {
        const int e = d - (NDU - pd.nd);
        L[d] = e >= 0 ? pd.len[pc][e] : 1;
        M[d] = e >= 0 ? pd.mul[pc][e] : 0u;
        S[d] = e >= 0 ? pd.shift[pc][e] : 0u;
        AL[d] = e >= 0 ? pd.p_lin[e] : 0;
        GS[d] = e >= 0 ? pd.p_gst[e] : 0;
    }
    const int32_t v_begin = (c - pd.chunk0[pc]) * kPieceChunk;
    const int32_t v_end = min(pd.nvec[pc], v_begin + kPieceChunk);
    // vector pieces and the scalar slivers in one launch (a second launch for the slivers cost ~8 us)
    if (V > 1 && pd.vec[pc])
        pieces_walk<ES, V, MODE, NDU>(L, M, S, AL, GS, v_begin, v_end, pd.abase[pc], pd.tbase[pc], pd.phase[pc],
                                      src, dst);
    else
        pieces_walk<ES, 1, MODE, NDU>(L, M, S, AL, GS, v_begin, v_end, pd.abase[pc], pd.tbase[pc], 0, src, dst);
}

// One piece under construction: a sub-range per combined dim, a wrap flag per array dim.
struct PieceBox {
    int64_t start[2 * AOL_MAX_RANK], len[2 * AOL_MAX_RANK];
    uint32_t wrapped;   // bit a: array dim a wrapped once inside this piece
};

// Split the parent tiler into affine pieces; false if it does not have the structure above (or needs more than
// kMaxPieces pieces, or would not fit 31-bit offsets).  Each piece is marked for V-element vectors or not;
// *vec_elems counts the elements of the vector pieces.
bool make_pieces(const TilerDev& td, int es, int mode, const void* arr, const void* tiles, int V, PiecesDev* P,
                 int64_t* vec_elems) {
    if (td.linear || !td.fast32 || td.array_elems >= (int64_t(1) << 31) || td.total >= (int64_t(1) << 31)) return false;
    const int nd = td.nd, ra = td.ra;
    std::vector<PieceBox> boxes(1);
    for (int d = 0; d < nd; ++d) {
        boxes[0].start[d] = 0;
        boxes[0].len[d] = td.ext[d];
    }
    boxes[0].wrapped = 0;
    int used_by[2 * AOL_MAX_RANK];
    for (int d = 0; d < nd; ++d) used_by[d] = -1;
    for (int a = 0; a < ra; ++a) {
        if ((td.nowrap_mask >> a) & 1) continue;
        int ds[2], n = 0;
        int64_t maxraw = td.org[a];
        for (int d = 0; d < nd; ++d) {
            if (td.coef[a][d] == 0 || td.ext[d] == 1) continue;
            if (n == 2 || used_by[d] >= 0) return false;
            used_by[d] = a;
            ds[n++] = d;
            maxraw += td.coef[a][d] * (td.ext[d] - 1);
        }
        if (n == 0 || maxraw >= 2 * td.ashape[a]) return false;   // at most one wrap
        if (n == 2 && td.coef[a][ds[0]] < td.coef[a][ds[1]]) std::swap(ds[0], ds[1]);   // ds[0] outer
        const int64_t T = td.ashape[a] - td.org[a];   // wrap iff sum of coef * idx >= T
        std::vector<PieceBox> next;
        for (const PieceBox& b : boxes) {
            auto push = [&](int64_t s0, int64_t l0, int64_t s1, int64_t l1, bool w) {
                if (l0 <= 0 || (n == 2 && l1 <= 0)) return;
                PieceBox q = b;
                q.start[ds[0]] = s0;
                q.len[ds[0]] = l0;
                if (n == 2) {
                    q.start[ds[1]] = s1;
                    q.len[ds[1]] = l1;
                }
                if (w) q.wrapped |= 1u << a;
                next.push_back(q);
            };
            const int64_t Co = td.coef[a][ds[0]], So = b.start[ds[0]], Lo = b.len[ds[0]];
            if (n == 1) {
                const int64_t istar = std::min(std::max<int64_t>((T + Co - 1) / Co, So), So + Lo);   // first wrapping index
                push(So, istar - So, 0, 0, false);
                push(istar, So + Lo - istar, 0, 0, true);
                continue;
            }
            const int64_t Cn = td.coef[a][ds[1]], Sn = b.start[ds[1]], Ln = b.len[ds[1]];
            // threshold on the inner index for outer value io: inner >= t(io) wraps, t non-increasing in io
            auto t_of = [&](int64_t io) {
                const int64_t r = T - Co * io;
                const int64_t t = r <= 0 ? 0 : (r + Cn - 1) / Cn;
                return std::min(std::max(t, Sn), Sn + Ln);
            };
            int64_t io = So;
            while (io < So + Lo) {
                const int64_t t = t_of(io);
                int64_t j = io + 1;   // extend while the same inner split applies
                while (j < So + Lo && t_of(j) == t) ++j;
                push(io, j - io, Sn, t - Sn, false);
                push(io, j - io, t, Sn + Ln - t, true);
                io = j;
            }
        }
        boxes.swap(next);
        if (boxes.size() > size_t(2 * kMaxPieces)) return false;
    }
    // build the piece table
    int64_t lin[2 * AOL_MAX_RANK], gst[2 * AOL_MAX_RANK];
    {
        int64_t g = 1;
        for (int d = nd - 1; d >= 0; --d) {
            gst[d] = g;
            g *= td.ext[d];
        }
        for (int d = 0; d < nd; ++d) {
            lin[d] = 0;
            for (int a = 0; a < ra; ++a) lin[d] += td.coef[a][d] * td.astride[a];
        }
    }
    // walk order: array strides ascending (innermost = smallest), broadcast dims outermost -- as make_tiler_dev
    int order[2 * AOL_MAX_RANK];
    for (int d = 0; d < nd; ++d) order[d] = d;
    auto key = [&](int d) { return lin[d] == 0 ? INT64_MAX : lin[d]; };
    for (int i = 1; i < nd; ++i)
        for (int j = i; j > 0 && key(order[j - 1]) < key(order[j]); --j) std::swap(order[j - 1], order[j]);
    if (nd > 0 && lin[nd - 1] == 1) {
        int pos = 0;
        while (order[pos] != nd - 1) ++pos;
        for (; pos < nd - 1; ++pos) order[pos] = order[pos + 1];
        order[nd - 1] = nd - 1;
    }
    std::memset(P, 0, sizeof *P);
    *vec_elems = 0;
    P->nd = nd;
    for (int i = 0; i < nd; ++i) {
        P->p_lin[i] = int32_t(lin[order[i]]);
        P->p_gst[i] = int32_t(gst[order[i]]);
    }
    const uintptr_t ptrs = reinterpret_cast<uintptr_t>(arr) | reinterpret_cast<uintptr_t>(tiles);
    for (const PieceBox& b : boxes) {
        int64_t count = 1, ab = 0, tb = 0;
        for (int d = 0; d < nd; ++d) {
            count *= b.len[d];
            ab += lin[d] * b.start[d];
            tb += gst[d] * b.start[d];
        }
        if (count == 0) continue;
        for (int a = 0; a < ra; ++a) ab += (td.org[a] - (((b.wrapped >> a) & 1) ? td.ashape[a] : 0)) * td.astride[a];
        // vectors: the innermost walked dim unit-stride on both sides, extents / bases / strides multiples of V
        // (a piece may start misaligned on the array side: every vector of the piece then shares the phase
        // ab mod V; gathers read, and scatters write, the aligned 16 bytes around each vector, exchanging the
        // overlap with the neighbouring lanes; a gather's second aligned load stays inside the allocation because
        // the array's rows are a multiple of V elements long)
        const int last = order[nd - 1];
        bool vec = V > 1 && lin[last] == 1 && gst[last] == 1 && b.len[last] % V == 0 && tb % V == 0 &&
                   ptrs % uintptr_t(V * es) == 0 && (ab % V == 0 || mode == 1 || td.ashape[ra - 1] % V == 0);
        for (int i = 0; i < nd - 1 && vec; ++i) vec = lin[order[i]] % V == 0 && gst[order[i]] % V == 0;
        if (P->npieces == kMaxPieces) return false;
        const int k = P->npieces++;
        for (int i = 0; i < nd; ++i) {
            P->len[k][i] = int32_t(b.len[order[i]]);
            magic32(b.len[order[i]], &P->mul[k][i], &P->shift[k][i]);
        }
        P->abase[k] = int32_t(ab);
        P->tbase[k] = int32_t(tb);
        P->nvec[k] = int32_t(count / (vec ? V : 1));
        P->phase[k] = vec ? int32_t(ab % V) : 0;
        P->vec[k] = vec ? 1 : 0;
        if (vec) *vec_elems += count;
    }
    P->chunk0[0] = 0;
    for (int k = 0; k < P->npieces; ++k) P->chunk0[k + 1] = P->chunk0[k] + (P->nvec[k] + kPieceChunk - 1) / kPieceChunk;
    P->nchunks = P->chunk0[P->npieces];
    return P->npieces > 0;
}

// The digit loop unrolled for the smallest of 4 / 5 / 6 / 8 / 16 dims that holds the tiler's (5: a blocking of
// a stack of planes, as in d3).
template <int ES, int V, int MODE>
void launch_pieces(const PiecesDev& p, const void* src, void* dst, cudaStream_t s) {
    if (p.nd <= 4)
        tiler_pieces_kernel<ES, V, MODE, 4><<<p.nchunks, 256, 0, s>>>(p, src, dst);
    else if (p.nd == 5)
        tiler_pieces_kernel<ES, V, MODE, 5><<<p.nchunks, 256, 0, s>>>(p, src, dst);
    else if (p.nd <= 6)
        tiler_pieces_kernel<ES, V, MODE, 6><<<p.nchunks, 256, 0, s>>>(p, src, dst);
    else if (p.nd <= 8)
        tiler_pieces_kernel<ES, V, MODE, 8><<<p.nchunks, 256, 0, s>>>(p, src, dst);
    else
        tiler_pieces_kernel<ES, V, MODE, kND><<<p.nchunks, 256, 0, s>>>(p, src, dst);
}

// AOL_TILER_PIECES=0 disables the affine-piece path (A/B measurements only).
bool tiler_pieces_enabled() {
    static const bool v = [] {
        const char* e = std::getenv("AOL_TILER_PIECES");
        return !(e && e[0] == '0');
    }();
    return v;
}

// AOL_TILER_WRAPTAB=0 runs wrapping gathers / FAST scatters element by element (A/B measurements only).
bool tiler_wraptab_enabled() {
    static const bool v = [] {
        const char* e = std::getenv("AOL_TILER_WRAPTAB");
        return !(e && e[0] == '0');
    }();
    return v;
}

// AOL_TILER_WRAP32=0 keeps wrapping tilers on the 64-bit general kernel (A/B measurements only).
bool tiler_wrap32_enabled() {
    static const bool v = [] {
        const char* e = std::getenv("AOL_TILER_WRAP32");
        return !(e && e[0] == '0');
    }();
    return v;
}

// ------------------------------------------------ deinterleave / interleave (linear tilers)
// Linear tilers whose two innermost array-order dims are C (<= 8) interleaved channels of unit array stride
// inside runs of X >= 64 positions that are contiguous on the TILE side, e.g. [N][H][W][3] video frames ->
// [N][3][H][W] planes (SURVEY 8(f) f2's split, as a tiler gather) or back (the FAST scatter).  Element-wise
// either the array side (stride-C reads) or the tile side (stride-S writes) is strided; here each CTA stages a
// chunk of X positions x C channels in shared memory so both global sides are read / written contiguously.
struct DeintDev {
    int32_t n_out;                               // outer dims (array-order dims 0 .. nd-3)
    int32_t out_ext[2 * AOL_MAX_RANK], out_lin[2 * AOL_MAX_RANK], out_gst[2 * AOL_MAX_RANK];
    uint32_t out_mul[2 * AOL_MAX_RANK], out_shift[2 * AOL_MAX_RANK];
    int32_t C, X, S;                             // channels, positions per run, tile stride of a channel
    int32_t chunk, nchunks, nitems, base;        // positions per smem chunk, chunks per run, runs x chunks
    uint32_t chunk_mul, chunk_shift;             // magic division by nchunks
};

constexpr int kDeintBytes = 16384;   // smem staging per CTA

template <int ES, int MODE>
__global__ void __launch_bounds__(256) tiler_deint_kernel(const DeintDev dd, const void* __restrict__ src,
                                                          void* __restrict__ dst) {
    using T = typename Elem<ES>::T;
    constexpr int kV = 16 / ES;   // elements per 16-byte vector
    __shared__ __align__(16) T buf[kDeintBytes / ES];
    const int C = dd.C;
    for (int32_t item = blockIdx.x; item < dd.nitems; item += gridDim.x) {
        uint32_t n = uint32_t(item);
        const uint32_t run = (__umulhi(n, dd.chunk_mul) + n) >> dd.chunk_shift;
        const int32_t ck = int32_t(n - run * uint32_t(dd.nchunks));
        n = run;
        int32_t a0 = dd.base, t0 = 0;
        for (int d = dd.n_out - 1; d >= 0; --d) {
            const uint32_t q = (__umulhi(n, dd.out_mul[d]) + n) >> dd.out_shift[d];
            const int32_t i = int32_t(n - q * uint32_t(dd.out_ext[d]));
            n = q;
            a0 += dd.out_lin[d] * i;
            t0 += dd.out_gst[d] * i;
        }
        const int32_t x0 = ck * dd.chunk;
        const int32_t nx = min(dd.chunk, dd.X - x0);
        const int32_t ne = nx * C;
        a0 += x0 * C;   // array: positions x0 .. x0+nx, all channels, contiguous
        t0 += x0;       // tile: channel c run at t0 + c*S
        // 16-byte vectors on a global side when its run starts 16-byte aligned and spans whole vectors
        // (HD [N][H][W][3] bytes: always); element by element otherwise
        const T* gsrc = static_cast<const T*>(src);
        T* gdst = static_cast<T*>(dst);
        const bool va = ((reinterpret_cast<uintptr_t>(MODE == 0 ? gsrc + a0 : gdst + a0)) & 15) == 0 && ne % kV == 0;
        bool vt = nx % kV == 0 && (dd.S % kV) == 0;
        vt = vt && ((reinterpret_cast<uintptr_t>(MODE == 0 ? gdst + t0 : gsrc + t0)) & 15) == 0;
        if (MODE == 0) {
            if (va) {
                const uint4* A = reinterpret_cast<const uint4*>(gsrc + a0);
                for (int32_t e = threadIdx.x; e < ne / kV; e += 256) reinterpret_cast<uint4*>(buf)[e] = A[e];
            } else {
                for (int32_t e = threadIdx.x; e < ne; e += 256) buf[e] = gsrc[a0 + e];
            }
            __syncthreads();
            for (int c = 0; c < C; ++c) {
                T* Tl = gdst + t0 + c * dd.S;
                if (vt) {
                    for (int32_t v = threadIdx.x; v < nx / kV; v += 256) {
                        union { uint4 u; T e[kV]; } pk;
#pragma unroll
                        for (int j = 0; j < kV; ++j) pk.e[j] = buf[(v * kV + j) * C + c];
                        reinterpret_cast<uint4*>(Tl)[v] = pk.u;
                    }
                } else {
                    for (int32_t x = threadIdx.x; x < nx; x += 256) Tl[x] = buf[x * C + c];
                }
            }
        } else {
            for (int c = 0; c < C; ++c) {
                const T* Tl = gsrc + t0 + c * dd.S;
                if (vt) {
                    for (int32_t v = threadIdx.x; v < nx / kV; v += 256) {
                        union { uint4 u; T e[kV]; } pk;
                        pk.u = reinterpret_cast<const uint4*>(Tl)[v];
#pragma unroll
                        for (int j = 0; j < kV; ++j) buf[(v * kV + j) * C + c] = pk.e[j];
                    }
                } else {
                    for (int32_t x = threadIdx.x; x < nx; x += 256) buf[x * C + c] = Tl[x];
                }
            }
            __syncthreads();
            if (va) {
                uint4* A = reinterpret_cast<uint4*>(gdst + a0);
                for (int32_t e = threadIdx.x; e < ne / kV; e += 256) A[e] = reinterpret_cast<const uint4*>(buf)[e];
            } else {
                for (int32_t e = threadIdx.x; e < ne; e += 256) gdst[a0 + e] = buf[e];
            }
        }
        __syncthreads();   // buf is reused by the next item
    }
}

// The common video case of the above -- 3 interleaved 8-bit channels (24-bit RGB/BGR pixels), every
// run 16-byte aligned on both sides -- needs no shared memory: a thread moves 16 pixels, three 16-byte loads of
// packed pixels <-> one 16-byte vector per channel plane, the byte transpose done in registers with two PRMTs
// per output word.  Lanes take consecutive 16-pixel groups, so both global sides stay coalesced.
template <int kC>
__device__ __forceinline__ uint32_t rgb_deint_word(uint32_t a, uint32_t b, uint32_t c) {
    // bytes kC, kC+3, kC+6, kC+9 of the 12-byte window (a, b, c)
    constexpr uint32_t o0 = kC, o1 = kC + 3, o2 = kC + 6, o3 = kC + 9;
    constexpr uint32_t s1 = (o0 < 8 ? o0 : 0) | (o1 < 8 ? o1 : 0) << 4 | (o2 < 8 ? o2 : 0) << 8 | (o3 < 8 ? o3 : 0) << 12;
    constexpr uint32_t s2 = (o0 < 8 ? 0u : o0 - 4) | (o1 < 8 ? 1u : o1 - 4) << 4 | (o2 < 8 ? 2u : o2 - 4) << 8 |
                            (o3 < 8 ? 3u : o3 - 4) << 12;
    return __byte_perm(__byte_perm(a, b, s1), c, s2);
}

// packed bytes 4k .. 4k+3 of a 12-byte group (4 pixels) from the three channel words p0, p1, p2
template <int kK>
__device__ __forceinline__ uint32_t rgb_int_word(uint32_t p0, uint32_t p1, uint32_t p2) {
    // packed byte j = pixel (4kK + j) / 3, channel (4kK + j) % 3; first merge channels 0 and 1, then 2
    constexpr int b0 = 4 * kK, b1 = b0 + 1, b2 = b0 + 2, b3 = b0 + 3;
    constexpr uint32_t s1 = ((b0 % 3 == 2) ? 0u : uint32_t((b0 % 3) * 4 + b0 / 3)) |
                            ((b1 % 3 == 2) ? 0u : uint32_t((b1 % 3) * 4 + b1 / 3)) << 4 |
                            ((b2 % 3 == 2) ? 0u : uint32_t((b2 % 3) * 4 + b2 / 3)) << 8 |
                            ((b3 % 3 == 2) ? 0u : uint32_t((b3 % 3) * 4 + b3 / 3)) << 12;
    constexpr uint32_t s2 = ((b0 % 3 == 2) ? uint32_t(4 + b0 / 3) : 0u) | ((b1 % 3 == 2) ? uint32_t(4 + b1 / 3) : 1u) << 4 |
                            ((b2 % 3 == 2) ? uint32_t(4 + b2 / 3) : 2u) << 8 | ((b3 % 3 == 2) ? uint32_t(4 + b3 / 3) : 3u) << 12;
    return __byte_perm(__byte_perm(p0, p1, s1), p2, s2);
}

template <int MODE>
__global__ void __launch_bounds__(256) tiler_rgb8_kernel(const DeintDev dd, const void* __restrict__ src,
                                                         void* __restrict__ dst) {
    const int32_t groups = dd.X / 16;   // 16-pixel groups per run
    const int32_t total = dd.nitems;    // runs x groups
    for (int32_t g = int32_t(blockIdx.x * blockDim.x + threadIdx.x); g < total; g += int32_t(gridDim.x * blockDim.x)) {
        uint32_t n = uint32_t(g);
        const uint32_t run = (__umulhi(n, dd.chunk_mul) + n) >> dd.chunk_shift;   // chunk_* = division by groups
        const int32_t grp = int32_t(n - run * uint32_t(groups));
        n = run;
        int32_t a0 = dd.base, t0 = 0;
        for (int d = dd.n_out - 1; d >= 0; --d) {
            const uint32_t q = (__umulhi(n, dd.out_mul[d]) + n) >> dd.out_shift[d];
            const int32_t i = int32_t(n - q * uint32_t(dd.out_ext[d]));
            n = q;
            a0 += dd.out_lin[d] * i;
            t0 += dd.out_gst[d] * i;
        }
        a0 += 48 * grp;
        t0 += 16 * grp;
        if (MODE == 0) {
            const uint4* A = reinterpret_cast<const uint4*>(static_cast<const uint8_t*>(src) + a0);
            const uint4 u0 = A[0], u1 = A[1], u2 = A[2];
            const uint32_t w[12] = {u0.x, u0.y, u0.z, u0.w, u1.x, u1.y, u1.z, u1.w, u2.x, u2.y, u2.z, u2.w};
            uint8_t* T = static_cast<uint8_t*>(dst) + t0;
            *reinterpret_cast<uint4*>(T) =
                make_uint4(rgb_deint_word<0>(w[0], w[1], w[2]), rgb_deint_word<0>(w[3], w[4], w[5]),
                           rgb_deint_word<0>(w[6], w[7], w[8]), rgb_deint_word<0>(w[9], w[10], w[11]));
            *reinterpret_cast<uint4*>(T + dd.S) =
                make_uint4(rgb_deint_word<1>(w[0], w[1], w[2]), rgb_deint_word<1>(w[3], w[4], w[5]),
                           rgb_deint_word<1>(w[6], w[7], w[8]), rgb_deint_word<1>(w[9], w[10], w[11]));
            *reinterpret_cast<uint4*>(T + 2 * dd.S) =
                make_uint4(rgb_deint_word<2>(w[0], w[1], w[2]), rgb_deint_word<2>(w[3], w[4], w[5]),
                           rgb_deint_word<2>(w[6], w[7], w[8]), rgb_deint_word<2>(w[9], w[10], w[11]));
        } else {
            const uint8_t* T = static_cast<const uint8_t*>(src) + t0;
            const uint4 c0 = *reinterpret_cast<const uint4*>(T), c1 = *reinterpret_cast<const uint4*>(T + dd.S),
                        c2 = *reinterpret_cast<const uint4*>(T + 2 * dd.S);
            const uint32_t p0[4] = {c0.x, c0.y, c0.z, c0.w}, p1[4] = {c1.x, c1.y, c1.z, c1.w},
                           p2[4] = {c2.x, c2.y, c2.z, c2.w};
            uint32_t o[12];
#pragma unroll
            for (int q = 0; q < 4; ++q) {   // pixels 4q .. 4q+3 -> packed words 3q .. 3q+2
                o[3 * q + 0] = rgb_int_word<0>(p0[q], p1[q], p2[q]);
                o[3 * q + 1] = rgb_int_word<1>(p0[q], p1[q], p2[q]);
                o[3 * q + 2] = rgb_int_word<2>(p0[q], p1[q], p2[q]);
            }
            uint4* A = reinterpret_cast<uint4*>(static_cast<uint8_t*>(dst) + a0);
            A[0] = make_uint4(o[0], o[1], o[2], o[3]);
            A[1] = make_uint4(o[4], o[5], o[6], o[7]);
            A[2] = make_uint4(o[8], o[9], o[10], o[11]);
        }
    }
}

// AOL_TILER_DEINT=0 disables the staged (de)interleave kernel (A/B measurements only).
bool tiler_deint_enabled() {
    static const bool v = [] {
        const char* e = std::getenv("AOL_TILER_DEINT");
        return !(e && e[0] == '0');
    }();
    return v;
}

bool make_deint(const TilerDev& td, int es, DeintDev* dd) {
    const int nd = td.nd;
    if (!td.linear || !td.small32 || nd < 2) return false;
    const int l = nd - 1, p = nd - 2;
    if (td.p_lin[l] != 1 || td.p_ext[l] < 2 || td.p_ext[l] > 8) return false;
    if (td.p_lin[p] != td.p_ext[l] || td.p_gst[p] != 1 || td.p_ext[p] < 64) return false;
    if (td.p_gst[l] < td.p_ext[p]) return false;   // channel runs on the tile side must not interleave
    std::memset(dd, 0, sizeof *dd);
    dd->C = int32_t(td.p_ext[l]);
    dd->X = int32_t(td.p_ext[p]);
    dd->S = int32_t(td.p_gst[l]);
    dd->chunk = std::max(32, (kDeintBytes / (dd->C * es)) & ~31);
    dd->nchunks = (dd->X + dd->chunk - 1) / dd->chunk;
    int64_t runs = 1;
    for (int d = 0; d < p; ++d) {
        dd->out_ext[d] = int32_t(td.p_ext[d]);
        dd->out_lin[d] = int32_t(td.p_lin[d]);
        dd->out_gst[d] = int32_t(td.p_gst[d]);
        magic32(td.p_ext[d], &dd->out_mul[d], &dd->out_shift[d]);
        runs *= td.p_ext[d];
    }
    dd->n_out = p;
    magic32(dd->nchunks, &dd->chunk_mul, &dd->chunk_shift);
    if (runs * dd->nchunks >= (int64_t(1) << 31)) return false;
    dd->nitems = int32_t(runs * dd->nchunks);
    dd->base = int32_t(td.base);
    return true;
}

int grid_for(int64_t n, int num_sms) {
    return int(std::max<int64_t>(1, std::min<int64_t>((n + 255) / 256, int64_t(num_sms) * 32)));
}

template <int ES, int V, int MODE>
aol_status_t launch_v(const TilerDev& td, const void* src, void* dst, unsigned long long* ws, int grid,
                      cudaStream_t s) {
    const bool fast = td.fast32 != 0, lin = td.linear != 0;
    if (MODE <= 1 && lin && td.small32) {
        DeviceInfo dev;
        aol_status_t st = device_info(&dev);
        if (st != AOL_OK) return st;
        DeintDev dd;
        if (V == 1 && tiler_deint_enabled() && make_deint(td, ES, &dd)) {
            if constexpr (ES == 1) {
                // 24-bit pixels with every run 16-byte aligned on both sides: the register transpose
                const uintptr_t pa = reinterpret_cast<uintptr_t>(MODE == 0 ? src : dst);
                const uintptr_t pt = reinterpret_cast<uintptr_t>(MODE == 0 ? dst : src);
                bool ok = dd.C == 3 && dd.X % 16 == 0 && dd.S % 16 == 0 && dd.base % 16 == 0 && (pa | pt) % 16 == 0;
                for (int d = 0; d < dd.n_out && ok; ++d) ok = dd.out_lin[d] % 16 == 0 && dd.out_gst[d] % 16 == 0;
                const int64_t total = int64_t(dd.nitems / dd.nchunks) * (dd.X / 16);
                if (ok && total < (int64_t(1) << 31)) {
                    DeintDev rd = dd;
                    rd.nitems = int32_t(total);
                    magic32(dd.X / 16, &rd.chunk_mul, &rd.chunk_shift);
                    const int gr = int(std::max<int64_t>(1, std::min<int64_t>((total + 255) / 256, int64_t(dev.num_sms) * 16)));
                    tiler_rgb8_kernel<MODE><<<gr, 256, 0, s>>>(rd, src, dst);
                    AOL_LAUNCH_CHECK("tiler_rgb8_kernel");
                    return AOL_OK;
                }
            }
            const int gd = int(std::max<int64_t>(1, std::min<int64_t>(dd.nitems, int64_t(dev.num_sms) * 8)));
            tiler_deint_kernel<ES, MODE><<<gd, 256, 0, s>>>(dd, src, dst);
            AOL_LAUNCH_CHECK("tiler_deint_kernel");
            return AOL_OK;
        }
        const int g32 = int(std::max<int64_t>(1, std::min<int64_t>((td.total / V + 255) / 256, int64_t(dev.num_sms) * 128)));
        if (td.nd <= 3)
            tiler_linear32_kernel<ES, V, MODE, 3><<<g32, 256, 0, s>>>(td, src, dst);
        else if (td.nd <= 5)
            tiler_linear32_kernel<ES, V, MODE, 5><<<g32, 256, 0, s>>>(td, src, dst);
        else if (td.nd <= 8)
            tiler_linear32_kernel<ES, V, MODE, 8><<<g32, 256, 0, s>>>(td, src, dst);
        else
            tiler_linear32_kernel<ES, V, MODE, kND><<<g32, 256, 0, s>>>(td, src, dst);
        AOL_LAUNCH_CHECK("tiler_linear32_kernel");
        return AOL_OK;
    }
    if constexpr (V == 1) {
        if (MODE <= 1 && !lin && tiler_pieces_enabled()) {
            constexpr int VV = 16 / ES;
            PiecesDev pd;
            int64_t nv = 0;
            // only when (nearly) all elements run as 16-byte vectors: scalar pieces lose to the box kernel
            const bool use = VV > 1 && make_pieces(td, ES, MODE, MODE == 0 ? src : dst, MODE == 0 ? dst : src, VV,
                                                   &pd, &nv) && 10 * nv >= 9 * td.total;
            if (use) {
                if constexpr (VV > 1) launch_pieces<ES, VV, MODE>(pd, src, dst, s);
                AOL_LAUNCH_CHECK("tiler_pieces_kernel");
                return AOL_OK;
            }
        }
        BoxDev bd;
        int box_smem = 0, box_buf = 0;
        if (MODE <= 1 && !lin && tiler_box_enabled() && make_box(td, ES, MODE, &bd, &box_smem, &box_buf)) {
          if constexpr (MODE <= 1) {
            DeviceInfo dev;
            aol_status_t st = device_info(&dev);
            if (st != AOL_OK) return st;
            // 16-byte vectors on the tile side when every block starts and ends on a 16-byte boundary
            constexpr int VW = 16 / ES;
            const void* tp = MODE == 0 ? dst : src;
            const void* ap = MODE == 0 ? src : dst;   // the array side: 16-byte row copies need an aligned base
            if (reinterpret_cast<uintptr_t>(ap) % 16) bd.vec16 = bd.vs = 0;
            bool vec = reinterpret_cast<uintptr_t>(tp) % 16 == 0 && (int64_t(bd.tail_prod) * ES) % 16 == 0;
            for (int d = 0; d < bd.n_out && vec; ++d) vec = (int64_t(bd.out_g[d]) * ES) % 16 == 0;
            auto kern = vec ? tiler_box_kernel<ES, VW, MODE> : tiler_box_kernel<ES, 1, MODE>;
            // gathers: one box buffer per CTA whenever that buys more CTAs per SM (the overlap then comes from the
            // other CTAs: H_IN 0.278 -> 0.220 ms, wrapping d3 0.145 -> 0.142, profiles/r02_box_nbuf_ab.jsonl), else
            // double-buffered (AOL_TILER_BOX_NBUF forces 1 or 2 for A/B measurements)
            int nbuf = MODE == 0 ? 2 : 1;
            if (MODE == 0) {
                const int one = box_smem - box_buf;
                const int cps2 = kernel_occupancy(reinterpret_cast<const void*>(kern), 256, box_smem);
                const int cps1 = kernel_occupancy(reinterpret_cast<const void*>(kern), 256, one);
                if (cps1 > cps2) nbuf = 1;
                const char* e = std::getenv("AOL_TILER_BOX_NBUF");
                if (e && (e[0] == '1' || e[0] == '2')) nbuf = e[0] - '0';
                if (nbuf == 1) box_smem = one;
            }
            st = kernel_smem(reinterpret_cast<const void*>(kern), box_smem);
            if (st != AOL_OK) return st;
            const int per_sm = std::max(1, kernel_occupancy(reinterpret_cast<const void*>(kern), 256, box_smem));
            const int gb = int(std::max<int64_t>(1, std::min<int64_t>(bd.nblocks, int64_t(dev.num_sms) * per_sm)));
            kern<<<gb, 256, box_smem, s>>>(bd, src, dst, box_buf, nbuf);
            AOL_LAUNCH_CHECK("tiler_box_kernel");
            return AOL_OK;
          }
        }
        Wrap32Dev wd;
        if (!lin && tiler_wrap32_enabled() && make_wrap32(td, &wd)) {
            DeviceInfo dev;
            aol_status_t st = device_info(&dev);
            if (st != AOL_OK) return st;
            if (MODE <= 1 && tiler_wraptab_enabled()) {
                const WrapTabDev wt = make_wraptab(wd);
                const int gt = int(std::max<int64_t>(1, std::min<int64_t>(wt.nblocks, int64_t(dev.num_sms) * 8)));
                tiler_wraptab_kernel<ES, MODE><<<gt, 256, 0, s>>>(wt, src, dst);
                AOL_LAUNCH_CHECK("tiler_wraptab_kernel");
                return AOL_OK;
            }
            const int gw = int(std::max<int64_t>(1, std::min<int64_t>((td.total + 255) / 256, int64_t(dev.num_sms) * 128)));
            tiler_wrap32_kernel<ES, MODE><<<gw, 256, 0, s>>>(wd, src, dst, ws);
            AOL_LAUNCH_CHECK("tiler_wrap32_kernel");
            return AOL_OK;
        }
    }
    if (fast && lin)
        tiler_kernel<ES, V, true, true, MODE><<<grid, 256, 0, s>>>(td, src, dst, ws);
    else if (fast)
        tiler_kernel<ES, V, true, false, MODE><<<grid, 256, 0, s>>>(td, src, dst, ws);
    else if (lin)
        tiler_kernel<ES, V, false, true, MODE><<<grid, 256, 0, s>>>(td, src, dst, ws);
    else
        tiler_kernel<ES, V, false, false, MODE><<<grid, 256, 0, s>>>(td, src, dst, ws);
    AOL_LAUNCH_CHECK("tiler_kernel");
    return AOL_OK;
}

template <int ES, int MODE>
aol_status_t launch_es(const TilerDev& td, int vec, const void* src, void* dst, unsigned long long* ws,
                       int num_sms, cudaStream_t s) {
    const int grid = grid_for(td.total / vec, num_sms);
    // vector width in elements (16, 8, 4 or 2 bytes) when the host proved contiguity + alignment, else 1
    if (vec > 1) {
        const int vb = ES * vec;
        if constexpr (ES == 1) {
            if (vb == 16) return launch_v<1, 16, MODE>(td, src, dst, ws, grid, s);
            if (vb == 8) return launch_v<1, 8, MODE>(td, src, dst, ws, grid, s);
            if (vb == 4) return launch_v<1, 4, MODE>(td, src, dst, ws, grid, s);
            if (vb == 2) return launch_v<1, 2, MODE>(td, src, dst, ws, grid, s);
        }
        if constexpr (ES == 2) {
            if (vb == 16) return launch_v<2, 8, MODE>(td, src, dst, ws, grid, s);
            if (vb == 8) return launch_v<2, 4, MODE>(td, src, dst, ws, grid, s);
            if (vb == 4) return launch_v<2, 2, MODE>(td, src, dst, ws, grid, s);
        }
        if constexpr (ES == 4) {
            if (vb == 16) return launch_v<4, 4, MODE>(td, src, dst, ws, grid, s);
            if (vb == 8) return launch_v<4, 2, MODE>(td, src, dst, ws, grid, s);
        }
        if constexpr (ES == 8) {
            if (vb == 16) return launch_v<8, 2, MODE>(td, src, dst, ws, grid, s);
        }
    }
    return launch_v<ES, 1, MODE>(td, src, dst, ws, grid_for(td.total, num_sms), s);
}

}  // namespace
}  // namespace aol
