// filter.cu -- NEXT row f3: one ArrayOL repetition (input tiler -> windowed-sum task -> output
// tiler) described at RUN TIME and executed by one fused kernel.  This is the "generic"
// formulation of the paper's SaC downscaler (Fig. 4 input_tiler, Fig. 5 task, Fig. 6
// generic_output_tiler), whose GPU version lost 4.5x (H) / 3x (V) to the
// non-generic one because the generic output tiler ran on the host.  Here all
// three steps stay on the device in a single kernel, so the comparison with the specialised
// K-5 measures what generality costs on B200 (tools/bench_configs.py, config f3).
//
// Per repetition r (one thread): base coordinates of both tilers are o' + P'.r reduced mod
// the extents once; the pattern-element and output-element offsets F'.i are host-precomputed
// tables already reduced mod the extents.  A repetition whose whole pattern stays inside the
// array (every repetition of a non-wrapping tiler; all but the last repetition of a row for the
// paper's H tiler) takes the fast path: element = base + lin[p], one add per element.  The
// others apply the toroidal wrap per dimension (add, conditional subtract, FMA).
#include <cuda_runtime.h>

#include <algorithm>
#include <cstdint>
#include <cstdlib>
#include <cstring>
#include <type_traits>

#include "common.h"

namespace aol {

namespace {

struct FilterDev {
    int32_t ra_in, ra_out, rr, n_in, n_win, len, divisor, fast32;
    int64_t nrep;
    int32_t rep_ext[AOL_MAX_RANK];
    uint32_t fd_mul[AOL_MAX_RANK], fd_shift[AOL_MAX_RANK];
    int32_t s_in[AOL_MAX_RANK], s_out[AOL_MAX_RANK];
    int64_t st_in[AOL_MAX_RANK], st_out[AOL_MAX_RANK];
    int32_t o_in[AOL_MAX_RANK], o_out[AOL_MAX_RANK];
    int32_t P_in[AOL_MAX_RANK][AOL_MAX_RANK], P_out[AOL_MAX_RANK][AOL_MAX_RANK];
    int32_t start[AOL_MAX_WINDOWS];
    int32_t f_in[AOL_MAX_FILTER_PATTERN][AOL_MAX_RANK];  // F'.i(p) mod s, per input pattern element
    int32_t f_out[AOL_MAX_WINDOWS][AOL_MAX_RANK];        // F'.i(k) mod s, per output element
    // fast path: a repetition whose reference point + the largest pattern coordinate stays inside every
    // extent needs no modulo, and its elements sit at base + lin[p] (row-major element offsets)
    int32_t fmax_in[AOL_MAX_RANK], fmax_out[AOL_MAX_RANK];
    int64_t lin_in[AOL_MAX_FILTER_PATTERN], lin_out[AOL_MAX_WINDOWS];
    // magic numbers: x mod s_in/s_out (x < 2^31) and |S| / |divisor| (|S| <= 2^31) as (umulhi(x, mul) + x) >> sh
    uint32_t mi_mul[AOL_MAX_RANK], mi_sh[AOL_MAX_RANK], mo_mul[AOL_MAX_RANK], mo_sh[AOL_MAX_RANK];
    uint32_t dv_mul, dv_sh;
    // (32 * P[a][last rep dim]) mod s: reference-point step between a lane's consecutive repetitions
    int32_t st32_in[AOL_MAX_RANK], st32_out[AOL_MAX_RANK];
};

// floor(x / d) for 0 <= x <= 2^31 and the host-computed (mul, sh) of d (1 <= d < 2^31)
__device__ __forceinline__ uint32_t udiv_magic(uint32_t x, uint32_t mul, uint32_t sh) {
    return (__umulhi(x, mul) + x) >> sh;
}

// D bounds every rank involved (array ranks of both tilers, repetition rank): loops unroll to D.
template <int D, bool kFast32>
__global__ void __launch_bounds__(256) filter_kernel(const FilterDev fd, const int32_t* __restrict__ in,
                                                     int32_t* __restrict__ out) {
    for (int64_t r = int64_t(blockIdx.x) * blockDim.x + threadIdx.x; r < fd.nrep;
         r += int64_t(gridDim.x) * blockDim.x) {
        // repetition multi-index (last dim fastest)
        int64_t ridx[D];
        int64_t g = r;
#pragma unroll
        for (int j = D - 1; j >= 0; --j) {
            if (j < fd.rr) {
                if (kFast32) {
                    const uint32_t n = uint32_t(g);
                    const uint32_t q = (__umulhi(n, fd.fd_mul[j]) + n) >> fd.fd_shift[j];
                    ridx[j] = int64_t(n - q * uint32_t(fd.rep_ext[j]));
                    g = q;
                } else {
                    const int64_t q = g / fd.rep_ext[j];
                    ridx[j] = g - q * fd.rep_ext[j];
                    g = q;
                }
            } else {
                ridx[j] = 0;
            }
        }
        // reference points o' + P'.r  (mod s), Section IV
        int32_t bin[D], bout[D];
#pragma unroll
        for (int a = 0; a < D; ++a) {
            int64_t vi = fd.o_in[a], vo = fd.o_out[a];
#pragma unroll
            for (int j = 0; j < D; ++j) {
                if (j < fd.rr) {
                    vi += int64_t(fd.P_in[a][j]) * ridx[j];
                    vo += int64_t(fd.P_out[a][j]) * ridx[j];
                }
            }
            bin[a] = a < fd.ra_in ? int32_t(vi % fd.s_in[a]) : 0;
            bout[a] = a < fd.ra_out ? int32_t(vo % fd.s_out[a]) : 0;
        }
        bool in_ok = true, out_ok = true;
        int64_t base_in = 0, base_out = 0;
#pragma unroll
        for (int a = 0; a < D; ++a) {
            if (a < fd.ra_in) {
                in_ok &= bin[a] + fd.fmax_in[a] < fd.s_in[a];
                base_in += int64_t(bin[a]) * fd.st_in[a];
            }
            if (a < fd.ra_out) {
                out_ok &= bout[a] + fd.fmax_out[a] < fd.s_out[a];
                base_out += int64_t(bout[a]) * fd.st_out[a];
            }
        }
        const int32_t* inb = in + base_in;
        for (int k = 0; k < fd.n_win; ++k) {
            // task (Fig. 5): S over the window, tile = S/d - S%d
            int32_t S = 0;
            if (in_ok) {
                for (int t = 0; t < fd.len; ++t) S += __ldg(inb + fd.lin_in[fd.start[k] + t]);
            } else {
                for (int t = 0; t < fd.len; ++t) {
                    const int p = fd.start[k] + t;
                    int64_t off = 0;
#pragma unroll
                    for (int a = 0; a < D; ++a) {
                        if (a < fd.ra_in) {
                            int32_t c = bin[a] + fd.f_in[p][a];   // pattern element, toroidal
                            if (c >= fd.s_in[a]) c -= fd.s_in[a];
                            off += int64_t(c) * fd.st_in[a];
                        }
                    }
                    S += __ldg(in + off);
                }
            }
            const int32_t tile = S / fd.divisor - S % fd.divisor;
            int64_t off = base_out + fd.lin_out[k];
            if (!out_ok) {
                off = 0;
#pragma unroll
                for (int a = 0; a < D; ++a) {
                    if (a < fd.ra_out) {
                        int32_t c = bout[a] + fd.f_out[k][a];       // output tiler (Fig. 6), toroidal
                        if (c >= fd.s_out[a]) c -= fd.s_out[a];
                        off += int64_t(c) * fd.st_out[a];
                    }
                }
            }
            out[off] = tile;
        }
    }
}

// All-32-bit variant for arrays < 2^31 elements whose reference-point sums fit in 31 bits (the usual
// case): the pattern/output offset tables, read with a data-dependent index, are staged in shared
// memory once per CTA instead of being fetched from the constant bank per element.
template <int D>
__global__ void __launch_bounds__(256) filter32_kernel(const FilterDev fd, const int32_t* __restrict__ in,
                                                       int32_t* __restrict__ out) {
    __shared__ int32_t lin_in[AOL_MAX_FILTER_PATTERN], lin_out[AOL_MAX_WINDOWS], start[AOL_MAX_WINDOWS];
    if (threadIdx.x < AOL_MAX_FILTER_PATTERN) lin_in[threadIdx.x] = int32_t(fd.lin_in[threadIdx.x]);
    if (threadIdx.x < AOL_MAX_WINDOWS) {
        lin_out[threadIdx.x] = int32_t(fd.lin_out[threadIdx.x]);
        start[threadIdx.x] = fd.start[threadIdx.x];
    }
    __syncthreads();
    const int32_t nrep = int32_t(fd.nrep);
    for (int32_t r = int32_t(blockIdx.x * blockDim.x + threadIdx.x); r < nrep; r += int32_t(gridDim.x * blockDim.x)) {
        int32_t vi[D], vo[D];
#pragma unroll
        for (int a = 0; a < D; ++a) {
            vi[a] = fd.o_in[a];
            vo[a] = fd.o_out[a];
        }
        uint32_t n = uint32_t(r);
#pragma unroll
        for (int j = D - 1; j >= 0; --j) {
            if (j < fd.rr) {
                const uint32_t q = (__umulhi(n, fd.fd_mul[j]) + n) >> fd.fd_shift[j];
                const int32_t i = int32_t(n - q * uint32_t(fd.rep_ext[j]));
                n = q;
#pragma unroll
                for (int a = 0; a < D; ++a) {   // reference points o' + P'.r (Section IV)
                    vi[a] += fd.P_in[a][j] * i;
                    vo[a] += fd.P_out[a][j] * i;
                }
            }
        }
        bool in_ok = true, out_ok = true;
        int32_t base_in = 0, base_out = 0;
#pragma unroll
        for (int a = 0; a < D; ++a) {
            if (a < fd.ra_in) {
                vi[a] %= fd.s_in[a];
                in_ok &= vi[a] + fd.fmax_in[a] < fd.s_in[a];
                base_in += vi[a] * int32_t(fd.st_in[a]);
            }
            if (a < fd.ra_out) {
                vo[a] %= fd.s_out[a];
                out_ok &= vo[a] + fd.fmax_out[a] < fd.s_out[a];
                base_out += vo[a] * int32_t(fd.st_out[a]);
            }
        }
        for (int k = 0; k < fd.n_win; ++k) {
            int32_t S = 0;                                      // task (Fig. 5): tile = S/d - S%d
            const int p0 = start[k];
            if (in_ok) {
                for (int t = 0; t < fd.len; ++t) S += __ldg(in + base_in + lin_in[p0 + t]);
            } else {
                for (int t = 0; t < fd.len; ++t) {
                    int32_t off = 0;
#pragma unroll
                    for (int a = 0; a < D; ++a) {
                        if (a < fd.ra_in) {
                            int32_t c = vi[a] + fd.f_in[p0 + t][a];   // toroidal pattern element
                            if (c >= fd.s_in[a]) c -= fd.s_in[a];
                            off += c * int32_t(fd.st_in[a]);
                        }
                    }
                    S += __ldg(in + off);
                }
            }
            const int32_t tile = S / fd.divisor - S % fd.divisor;
            int32_t off = base_out + lin_out[k];
            if (!out_ok) {
                off = 0;
#pragma unroll
                for (int a = 0; a < D; ++a) {
                    if (a < fd.ra_out) {
                        int32_t c = vo[a] + fd.f_out[k][a];
                        if (c >= fd.s_out[a]) c -= fd.s_out[a];
                        off += c * int32_t(fd.st_out[a]);
                    }
                }
            }
            out[off] = tile;
        }
    }
}

// Register-pattern variant for input patterns of at most 16 elements (the paper's filters: 11 and 12):
// each pattern element is loaded ONCE per repetition into registers -- four at a time with 128-bit loads
// when the pattern is a contiguous run of the array (lin_in[p] == p, e.g. the H filter's 11 columns) and
// the repetition's run is 16-byte aligned -- and every window sum is then formed from registers by a
// predicated walk over the NP elements (no dynamic register indexing).  The generic kernel above instead
// issues window_len loads per window (18 for H, 24 for V), most of them L1 hits of a scattered warp access.
template <int D, int NP>
__global__ void __launch_bounds__(256) filter32_reg_kernel(const FilterDev fd, const int32_t* __restrict__ in,
                                                           int32_t* __restrict__ out, int32_t in_elems,
                                                           int32_t contig) {
    __shared__ int32_t lin_out[AOL_MAX_WINDOWS], start[AOL_MAX_WINDOWS];
    // per-thread prefix sums of the pattern, [p][thread] (conflict-free: a warp reads one row at a time)
    __shared__ int32_t pre[(NP + 1) * 256];
    if (threadIdx.x < AOL_MAX_WINDOWS) {
        lin_out[threadIdx.x] = int32_t(fd.lin_out[threadIdx.x]);
        start[threadIdx.x] = fd.start[threadIdx.x];
    }
    __syncthreads();
    int32_t* my = pre + threadIdx.x;
    const int32_t nrep = int32_t(fd.nrep);
    // Each warp takes chunks of 32 * kT consecutive repetitions; lane l handles l, l + 32, ...  (coalesced
    // across the warp).  Only a lane's first repetition of a chunk, and one whose innermost repetition index
    // carries into the next dimension, decomposes its index (magic-number divisions + mod); the others step
    // the reference points o' + P'.r by 32 columns of P' with one conditional subtract per dimension.
    constexpr int kT = 8;
    const int32_t lane = int32_t(threadIdx.x & 31u);
    const int32_t nchunks = (nrep + 32 * kT - 1) / (32 * kT);
    const int32_t nwarps = int32_t((gridDim.x * blockDim.x) >> 5);
    const int32_t ext_last = fd.rr > 0 ? fd.rep_ext[fd.rr - 1] : 1;
    for (int32_t chunk = int32_t((blockIdx.x * blockDim.x + threadIdx.x) >> 5); chunk < nchunks; chunk += nwarps) {
    int32_t vi[D], vo[D], ilast = 0;
    bool have = false;
    for (int32_t t = 0, r = chunk * 32 * kT + lane; t < kT && r < nrep; ++t, r += 32) {
        if (have && ilast + 32 < ext_last) {
            ilast += 32;
#pragma unroll
            for (int a = 0; a < D; ++a) {
                if (a < fd.ra_in) {
                    vi[a] += fd.st32_in[a];
                    if (vi[a] >= fd.s_in[a]) vi[a] -= fd.s_in[a];
                }
                if (a < fd.ra_out) {
                    vo[a] += fd.st32_out[a];
                    if (vo[a] >= fd.s_out[a]) vo[a] -= fd.s_out[a];
                }
            }
        } else {
            have = true;
#pragma unroll
            for (int a = 0; a < D; ++a) {
                vi[a] = fd.o_in[a];
                vo[a] = fd.o_out[a];
            }
            uint32_t n = uint32_t(r);
#pragma unroll
            for (int j = D - 1; j >= 0; --j) {
                if (j < fd.rr) {
                    const uint32_t q = (__umulhi(n, fd.fd_mul[j]) + n) >> fd.fd_shift[j];
                    const int32_t i = int32_t(n - q * uint32_t(fd.rep_ext[j]));
                    n = q;
                    if (j == fd.rr - 1) ilast = i;
#pragma unroll
                    for (int a = 0; a < D; ++a) {   // reference points o' + P'.r (Section IV)
                        vi[a] += fd.P_in[a][j] * i;
                        vo[a] += fd.P_out[a][j] * i;
                    }
                }
            }
#pragma unroll
            for (int a = 0; a < D; ++a) {   // mod s (all terms >= 0 and < 2^31): magic-number division
                if (a < fd.ra_in) vi[a] -= int32_t(udiv_magic(uint32_t(vi[a]), fd.mi_mul[a], fd.mi_sh[a])) * fd.s_in[a];
                if (a < fd.ra_out)
                    vo[a] -= int32_t(udiv_magic(uint32_t(vo[a]), fd.mo_mul[a], fd.mo_sh[a])) * fd.s_out[a];
            }
        }
        bool in_ok = true, out_ok = true;
        int32_t base_in = 0, base_out = 0;
#pragma unroll
        for (int a = 0; a < D; ++a) {
            if (a < fd.ra_in) {
                in_ok &= vi[a] + fd.fmax_in[a] < fd.s_in[a];
                base_in += vi[a] * int32_t(fd.st_in[a]);
            }
            if (a < fd.ra_out) {
                out_ok &= vo[a] + fd.fmax_out[a] < fd.s_out[a];
                base_out += vo[a] * int32_t(fd.st_out[a]);
            }
        }
        // gather (Fig. 4): the repetition's pattern, each element once
        int32_t x[NP];
        if (contig && in_ok && (base_in & 3) == 0 && base_in + NP <= in_elems) {
#pragma unroll
            for (int v = 0; v < NP / 4; ++v) {
                const int4 q = __ldg(reinterpret_cast<const int4*>(in + base_in) + v);
                x[4 * v] = q.x;
                x[4 * v + 1] = q.y;
                x[4 * v + 2] = q.z;
                x[4 * v + 3] = q.w;
            }
        } else {
#pragma unroll
            for (int p = 0; p < NP; ++p) {
                x[p] = 0;
                if (p < fd.n_in) {
                    int32_t off;
                    if (in_ok) {
                        off = base_in + int32_t(fd.lin_in[p]);
                    } else {
                        off = 0;
#pragma unroll
                        for (int a = 0; a < D; ++a) {
                            if (a < fd.ra_in) {
                                int32_t c = vi[a] + fd.f_in[p][a];   // toroidal pattern element
                                if (c >= fd.s_in[a]) c -= fd.s_in[a];
                                off += c * int32_t(fd.st_in[a]);
                            }
                        }
                    }
                    x[p] = __ldg(in + off);
                }
            }
        }
        // prefix sums: window k's sum = pre[start_k + len] - pre[start_k] (two LDS, whatever the window)
        {
            int32_t acc = 0;
            my[0] = 0;
#pragma unroll
            for (int p = 0; p < NP; ++p) {
                acc += x[p];
                my[(p + 1) * 256] = acc;
            }
        }
        for (int k = 0; k < fd.n_win; ++k) {
            // task (Fig. 5): S over window k = elements start_k .. start_k + len - 1, tile = S/d - S%d
            const int32_t s0 = start[k];
            const int32_t S = my[(s0 + fd.len) * 256] - my[s0 * 256];
            // tile = S/d - S%d (C semantics) = q (1 + d) - S with q = trunc(S/d) = sign(S) sign(d) floor(|S|/|d|)
            const uint32_t qa = udiv_magic(uint32_t(abs(S)), fd.dv_mul, fd.dv_sh);   // |INT_MIN| = 2^31 ok
            const int32_t q = ((S < 0) != (fd.divisor < 0)) ? -int32_t(qa) : int32_t(qa);
            const int32_t tile = q * (1 + fd.divisor) - S;
            int32_t off = base_out + lin_out[k];
            if (!out_ok) {
                off = 0;
#pragma unroll
                for (int a = 0; a < D; ++a) {
                    if (a < fd.ra_out) {
                        int32_t c = vo[a] + fd.f_out[k][a];   // output tiler (Fig. 6), toroidal
                        if (c >= fd.s_out[a]) c -= fd.s_out[a];
                        off += c * int32_t(fd.st_out[a]);
                    }
                }
            }
            out[off] = tile;
        }
    }
    }
}

// (mul, sh) with floor(x / d) == (umulhi(x, mul) + x) >> sh for every 0 <= x <= 2^31 (1 <= d <= 2^31):
// sh = ceil(log2 d), mul = floor(2^32 (2^sh - d) / d) + 1 (the round-up method; the 33-bit sum
// umulhi + x stays below 2^32 because x <= 2^31).  Checked exhaustively for small d in tests/test_abi.py.
void magic_u31(uint32_t d, uint32_t* mul, uint32_t* sh) {
    uint32_t s = 0;
    while (s < 32 && (uint64_t(1) << s) < uint64_t(d)) ++s;
    *sh = s;
    *mul = uint32_t(((uint64_t(1) << 32) * ((uint64_t(1) << s) - uint64_t(d))) / uint64_t(d) + 1);
}

// AOL_FILTER_LEGACY=1 selects the per-window-load kernels (A/B measurements only).
bool getenv_flag_filter_legacy() {
    static const bool v = [] {
        const char* e = std::getenv("AOL_FILTER_LEGACY");
        return e && e[0] == '1';
    }();
    return v;
}

int64_t emod(int64_t a, int64_t m) {
    const int64_t r = a % m;
    return r < 0 ? r + m : r;
}

int64_t elems(const int64_t* s, int n) {
    int64_t p = 1;
    for (int k = 0; k < n; ++k) p *= s[k];
    return p;
}

// pattern element p (flattened row-major) -> its multi-index
void unflatten(int64_t p, const int64_t* shape, int n, int64_t* idx) {
    for (int k = n - 1; k >= 0; --k) {
        idx[k] = p % shape[k];
        p /= shape[k];
    }
}

aol_status_t check_filter(const aol_filter_t* f) {
    if (!f) return fail(AOL_E_INVALID, "filter is NULL");
    aol_status_t st = aol_tiler_validate(&f->in);
    if (st != AOL_OK) return st;
    st = aol_tiler_validate(&f->out);
    if (st != AOL_OK) return st;
    if (f->in.rep_rank != f->out.rep_rank) return fail(AOL_E_SHAPE, "input and output repetition spaces differ");
    for (int j = 0; j < f->in.rep_rank; ++j)
        if (f->in.rep_shape[j] != f->out.rep_shape[j])
            return fail(AOL_E_SHAPE, "input and output repetition spaces differ");
    const int64_t n_in = elems(f->in.pattern_shape, f->in.pattern_rank);
    const int64_t n_out = elems(f->out.pattern_shape, f->out.pattern_rank);
    if (n_in > AOL_MAX_FILTER_PATTERN) return fail(AOL_E_RANGE, "input pattern larger than AOL_MAX_FILTER_PATTERN");
    if (f->n_windows < 1 || f->n_windows > AOL_MAX_WINDOWS || n_out != f->n_windows)
        return fail(AOL_E_SHAPE, "n_windows must equal the output pattern size (1..AOL_MAX_WINDOWS)");
    if (f->window_len < 1 || f->divisor == 0) return fail(AOL_E_INVALID, "window_len >= 1 and divisor != 0");
    for (int k = 0; k < f->n_windows; ++k)
        if (f->window_start[k] < 0 || int64_t(f->window_start[k]) + f->window_len > n_in)
            return fail(AOL_E_SHAPE, "window outside the input pattern");
    for (const aol_tiler_t* t : {&f->in, &f->out}) {
        for (int a = 0; a < t->array_rank; ++a)
            if (t->array_shape[a] >= (int64_t(1) << 31)) return fail(AOL_E_RANGE, "filter array extents must be < 2^31");
        if (elems(t->array_shape, t->array_rank) >= (int64_t(1) << 62)) return fail(AOL_E_RANGE, "array too large");
    }
    return AOL_OK;
}

void fill_side(const aol_tiler_t* t, int32_t* s, int64_t* st, int32_t* o, int32_t (*P)[AOL_MAX_RANK]) {
    int64_t stride = 1;
    for (int a = t->array_rank - 1; a >= 0; --a) {
        s[a] = int32_t(t->array_shape[a]);
        st[a] = stride;
        stride *= t->array_shape[a];
        o[a] = int32_t(emod(t->origin[a], t->array_shape[a]));
        for (int j = 0; j < t->rep_rank; ++j) P[a][j] = int32_t(emod(t->paving[a][j], t->array_shape[a]));
    }
}

void fill_offsets(const aol_tiler_t* t, int64_t n, int32_t (*f)[AOL_MAX_RANK]) {
    for (int64_t p = 0; p < n; ++p) {
        int64_t idx[AOL_MAX_RANK] = {0};
        unflatten(p, t->pattern_shape, t->pattern_rank, idx);
        for (int a = 0; a < t->array_rank; ++a) {
            __int128 v = 0;
            for (int k = 0; k < t->pattern_rank; ++k) v += __int128(emod(t->fitting[a][k], t->array_shape[a])) * idx[k];
            f[p][a] = int32_t(v % t->array_shape[a]);
        }
    }
}

}  // namespace

}  // namespace aol

using namespace aol;

extern "C" {

aol_status_t aol_filter_validate(const aol_filter_t* f) { return check_filter(f); }

aol_status_t aol_filter_preset(aol_filter_kind_t which, int64_t planes, int64_t H, int64_t W, aol_filter_t* out) {
    if (!out) return fail(AOL_E_INVALID, "out is NULL");
    if (planes <= 0 || H <= 0 || W <= 0) return fail(AOL_E_INVALID, "planes, H, W must be > 0");
    aol_filter_t f;
    std::memset(&f, 0, sizeof f);
    // the per-plane tilers of Fig. 10 (H) / reading Z1 (V), lifted to a stack of planes:
    // array {planes, ...}, repetition {planes, ...}, paving 1 on the plane dimension
    aol_tiler_t tin, tout;
    aol_status_t st;
    if (which == AOL_FILTER_H) {
        if ((st = aol_tiler_preset(AOL_PRESET_H_IN, H, W, &tin)) != AOL_OK) return st;
        if ((st = aol_tiler_preset(AOL_PRESET_H_OUT, H, W, &tout)) != AOL_OK) return st;
        f.n_windows = 3;
        const int32_t s[3] = {0, 2, 5};   // Fig. 5: tmp0 over [0..5], tmp1 over [2..7], tmp2 over [5..10]
        for (int k = 0; k < 3; ++k) f.window_start[k] = s[k];
    } else if (which == AOL_FILTER_V) {
        if ((st = aol_tiler_preset(AOL_PRESET_V_IN, H, W, &tin)) != AOL_OK) return st;
        if ((st = aol_tiler_preset(AOL_PRESET_V_OUT, H, W, &tout)) != AOL_OK) return st;
        f.n_windows = 4;
        const int32_t s[4] = {0, 2, 4, 6};   // reading Z1
        for (int k = 0; k < 4; ++k) f.window_start[k] = s[k];
    } else {
        return fail(AOL_E_INVALID, "unknown filter kind");
    }
    f.window_len = 6;
    f.divisor = 6;
    for (aol_tiler_t* t : {&tin, &tout}) {
        aol_tiler_t l;
        std::memset(&l, 0, sizeof l);
        l.array_rank = 3;
        l.rep_rank = 3;
        l.pattern_rank = t->pattern_rank;
        l.array_shape[0] = planes;
        l.rep_shape[0] = planes;
        l.paving[0][0] = 1;
        for (int a = 0; a < 2; ++a) {
            l.array_shape[a + 1] = t->array_shape[a];
            l.origin[a + 1] = t->origin[a];
            for (int j = 0; j < 2; ++j) l.paving[a + 1][j + 1] = t->paving[a][j];
            for (int k = 0; k < t->pattern_rank; ++k) l.fitting[a + 1][k] = t->fitting[a][k];
        }
        for (int j = 0; j < 2; ++j) l.rep_shape[j + 1] = t->rep_shape[j];
        for (int k = 0; k < t->pattern_rank; ++k) l.pattern_shape[k] = t->pattern_shape[k];
        *t = l;
    }
    f.in = tin;
    f.out = tout;
    *out = f;
    return AOL_OK;
}

aol_status_t aol_filter_apply(const aol_filter_t* f, const int32_t* d_in, int32_t* d_out, cudaStream_t s) {
    aol_status_t st = check_filter(f);
    if (st != AOL_OK) return st;
    if (!d_in || !d_out) return fail(AOL_E_INVALID, "null buffer");
    if ((reinterpret_cast<uintptr_t>(d_in) | reinterpret_cast<uintptr_t>(d_out)) % 4)
        return fail(AOL_E_ALIGN, "buffers must be 4-byte aligned");
    // a row filter or a column filter (the paper's H and V, any run-time parameters): the separable chain kernel
    // specialised at run time, with an identity partner
    if (launch_sep_single(f, d_in, d_out, s, &st)) return st;
    FilterDev fd;
    std::memset(&fd, 0, sizeof fd);
    fd.ra_in = f->in.array_rank;
    fd.ra_out = f->out.array_rank;
    fd.rr = f->in.rep_rank;
    fd.n_in = int32_t(elems(f->in.pattern_shape, f->in.pattern_rank));
    fd.n_win = f->n_windows;
    fd.len = f->window_len;
    fd.divisor = f->divisor;
    fd.nrep = elems(f->in.rep_shape, f->in.rep_rank);
    if (fd.nrep == 0) return AOL_OK;
    fd.fast32 = fd.nrep < (int64_t(1) << 31);
    for (int j = 0; j < fd.rr; ++j) {
        fd.rep_ext[j] = int32_t(std::min<int64_t>(f->in.rep_shape[j], INT32_MAX));
        if (f->in.rep_shape[j] >= (int64_t(1) << 31)) fd.fast32 = 0;
    }
    for (int j = 0; j < fd.rr; ++j) {
        uint32_t shift = 0;
        while (shift < 32 && (uint64_t(1) << shift) < uint64_t(fd.rep_ext[j])) ++shift;
        fd.fd_shift[j] = shift;
        fd.fd_mul[j] = uint32_t(((uint64_t(1) << 32) * ((uint64_t(1) << shift) - uint64_t(fd.rep_ext[j]))) /
                                    uint64_t(fd.rep_ext[j]) + 1);
    }
    fill_side(&f->in, fd.s_in, fd.st_in, fd.o_in, fd.P_in);
    fill_side(&f->out, fd.s_out, fd.st_out, fd.o_out, fd.P_out);
    for (int a = 0; a < AOL_MAX_RANK; ++a) {
        if (a < fd.ra_in) magic_u31(uint32_t(fd.s_in[a]), &fd.mi_mul[a], &fd.mi_sh[a]);
        if (a < fd.ra_out) magic_u31(uint32_t(fd.s_out[a]), &fd.mo_mul[a], &fd.mo_sh[a]);
    }
    magic_u31(uint32_t(f->divisor < 0 ? -int64_t(f->divisor) : int64_t(f->divisor)), &fd.dv_mul, &fd.dv_sh);
    for (int a = 0; a < AOL_MAX_RANK && fd.rr > 0; ++a) {
        if (a < fd.ra_in) fd.st32_in[a] = int32_t(emod(32 * int64_t(fd.P_in[a][fd.rr - 1]), fd.s_in[a]));
        if (a < fd.ra_out) fd.st32_out[a] = int32_t(emod(32 * int64_t(fd.P_out[a][fd.rr - 1]), fd.s_out[a]));
    }
    for (int k = 0; k < fd.n_win; ++k) fd.start[k] = f->window_start[k];
    fill_offsets(&f->in, fd.n_in, fd.f_in);
    fill_offsets(&f->out, fd.n_win, fd.f_out);
    for (int a = 0; a < AOL_MAX_RANK; ++a) {
        for (int p = 0; p < fd.n_in; ++p) fd.fmax_in[a] = std::max(fd.fmax_in[a], fd.f_in[p][a]);
        for (int k = 0; k < fd.n_win; ++k) fd.fmax_out[a] = std::max(fd.fmax_out[a], fd.f_out[k][a]);
    }
    for (int p = 0; p < fd.n_in; ++p)
        for (int a = 0; a < fd.ra_in; ++a) fd.lin_in[p] += int64_t(fd.f_in[p][a]) * fd.st_in[a];
    for (int k = 0; k < fd.n_win; ++k)
        for (int a = 0; a < fd.ra_out; ++a) fd.lin_out[k] += int64_t(fd.f_out[k][a]) * fd.st_out[a];

    DeviceInfo dev;
    st = device_info(&dev);
    if (st != AOL_OK) return st;
    const int grid = int(std::max<int64_t>(1, std::min<int64_t>((fd.nrep + 255) / 256, int64_t(dev.num_sms) * 16)));
    const int D = std::max(fd.rr, std::max(fd.ra_in, fd.ra_out));
    // all-32-bit path: arrays < 2^31 elements, repetitions < 2^31, reference-point sums < 2^31
    bool small = fd.fast32 && elems(f->in.array_shape, f->in.array_rank) < (int64_t(1) << 31) &&
                 elems(f->out.array_shape, f->out.array_rank) < (int64_t(1) << 31);
    for (const aol_tiler_t* t : {&f->in, &f->out})
        for (int a = 0; a < t->array_rank; ++a) {
            __int128 bound = t->array_shape[a];
            for (int j = 0; j < t->rep_rank; ++j) bound += __int128(t->array_shape[a]) * t->rep_shape[j];
            if (bound >= (__int128(1) << 31)) small = false;
        }
    if (small && fd.n_in <= 16 && !(getenv_flag_filter_legacy())) {
        // pattern contiguous in the array (element p at base + p): 128-bit loads; the padded tail of the last
        // vector is read only when it stays inside the input array (checked per repetition in the kernel)
        int32_t contig = (reinterpret_cast<uintptr_t>(d_in) % 16) == 0;
        for (int p = 0; p < fd.n_in; ++p) contig &= fd.lin_in[p] == p;
        const int32_t in_elems = int32_t(elems(f->in.array_shape, f->in.array_rank));
        const int np = (fd.n_in + 3) / 4 * 4;
        auto go = [&](auto kd) {
            constexpr int DD = decltype(kd)::value;
            switch (np) {
                case 4: filter32_reg_kernel<DD, 4><<<grid, 256, 0, s>>>(fd, d_in, d_out, in_elems, contig); break;
                case 8: filter32_reg_kernel<DD, 8><<<grid, 256, 0, s>>>(fd, d_in, d_out, in_elems, contig); break;
                case 12: filter32_reg_kernel<DD, 12><<<grid, 256, 0, s>>>(fd, d_in, d_out, in_elems, contig); break;
                default: filter32_reg_kernel<DD, 16><<<grid, 256, 0, s>>>(fd, d_in, d_out, in_elems, contig); break;
            }
        };
        if (D <= 2) go(std::integral_constant<int, 2>{});
        else if (D <= 3) go(std::integral_constant<int, 3>{});
        else if (D <= 4) go(std::integral_constant<int, 4>{});
        else go(std::integral_constant<int, 8>{});
        AOL_LAUNCH_CHECK("filter32_reg_kernel");
        return AOL_OK;
    }
    if (small) {
        if (D <= 2) filter32_kernel<2><<<grid, 256, 0, s>>>(fd, d_in, d_out);
        else if (D <= 3) filter32_kernel<3><<<grid, 256, 0, s>>>(fd, d_in, d_out);
        else if (D <= 4) filter32_kernel<4><<<grid, 256, 0, s>>>(fd, d_in, d_out);
        else filter32_kernel<8><<<grid, 256, 0, s>>>(fd, d_in, d_out);
        AOL_LAUNCH_CHECK("filter32_kernel");
        return AOL_OK;
    }
    auto launch = [&](auto kfast, auto kd) {
        filter_kernel<decltype(kd)::value, decltype(kfast)::value><<<grid, 256, 0, s>>>(fd, d_in, d_out);
    };
    using T = std::true_type;
    using F = std::false_type;
    if (D <= 2) fd.fast32 ? launch(T{}, std::integral_constant<int, 2>{}) : launch(F{}, std::integral_constant<int, 2>{});
    else if (D <= 3) fd.fast32 ? launch(T{}, std::integral_constant<int, 3>{}) : launch(F{}, std::integral_constant<int, 3>{});
    else if (D <= 4) fd.fast32 ? launch(T{}, std::integral_constant<int, 4>{}) : launch(F{}, std::integral_constant<int, 4>{});
    else fd.fast32 ? launch(T{}, std::integral_constant<int, 8>{}) : launch(F{}, std::integral_constant<int, 8>{});
    AOL_LAUNCH_CHECK("filter_kernel");
    return AOL_OK;
}

}  // extern "C"
