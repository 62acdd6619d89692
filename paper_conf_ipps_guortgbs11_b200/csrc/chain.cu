// chain.cu -- NEXT row f3, fused: two run-time ArrayOL repetitions chained, f2 consuming f1's output array,
// in ONE kernel -- WITH-loop folding across repetitions for descriptors known only at run time (the paper's
// fusion, SaC WLF P:L528-546, applied to its generic formulation, Fig. 4-6, whose separately
// launched generic filters it compares in Section VIII-A).  The intermediate array Y never
// touches HBM.
//
// Work unit = a block of f2's repetitions (its inner repetition dims, the outermost of them in chunks).  The
// block's pattern elements lie in a BOX of Y's raw coordinates (the footprint box of tiler_kernels.cuh).  A CTA
//  (1) fills the box in shared memory by running f1 over exactly the f1 repetitions whose outputs land in it:
//      f1's output tiler must be a bijection whose window digits are the low digits of each Y dim, so the
//      repetitions covering a range of Y indices form a contiguous range per Y dim; each repetition gathers
//      its pattern from X once (16-byte loads when it is a contiguous aligned run), forms its window sums from
//      a shared-memory prefix array, applies the task and stores the outputs that fall inside the box;
//  (2) runs f2 over the block's repetitions, their patterns read from the box, outputs stored to Z through
//      f2's output tiler (linear: no wrap).
// Anything outside these conditions runs as two aol_filter_apply launches through a caller workspace.
#include <cuda_runtime.h>

#include <algorithm>
#include <cstdint>
#include <cstdlib>
#include <cstring>

#include "common.h"

namespace aol {
namespace {

constexpr int kCR = 4;       // array / repetition rank limit of the fused chain
constexpr int kCP = 16;      // pattern elements per repetition
constexpr int kCW = 16;      // windows per repetition
constexpr int kCIn = 3;      // f2 inner repetition dims per block
constexpr int kCDig = 3;     // digits of f1's output tiler per Y dim
constexpr int kChainBox = 48 * 1024;   // smem bytes of the Y box

struct ChainDev {
    // ---------------- f1: X -> Y
    int32_t rx, rr1;
    int32_t sX[kCR], stX[kCR];
    uint32_t mX_mul[kCR], mX_sh[kCR];          // floor(v / sX) for the reference point's mod
    int32_t o1[kCR], P1[kCR][kCR];             // f1.in origin and paving, reduced mod sX  [a][j]
    int32_t n_in1, len1, nwin1, div1;
    uint32_t dv1_mul, dv1_sh;
    int32_t start1[kCW];
    int32_t f_in1[kCP][kCR], fmax_in1[kCR], lin_in1[kCP];
    int32_t contig1, x_elems;
    // f1's output tiler, per Y dim a: dense index v = (y - yo) mod sY = R K + kk; R's digits are f1 repetition
    // indices (ascending, signed), kk(window) is a host table
    int32_t ry;
    int32_t sY[kCR], K[kCR], nRfull[kCR];       // nRfull = sY / K
    int32_t yo[kCR];
    int32_t nrd[kCR], rd_ext[kCR][kCDig], rd_neg[kCR][kCDig], rd_dim[kCR][kCDig];
    uint32_t rd_mul[kCR][kCDig], rd_sh[kCR][kCDig];
    int32_t xs[kCR][kCDig][kCR];                 // X reference-point step of digit g of Y dim a, per X dim
    int32_t kk[kCW][kCR];                        // window k's dense low part on each Y dim
    int32_t kkmin[kCR], kkmax[kCR];              // their range per Y dim
    // ---------------- f2: Y -> Z, blocked
    int32_t rr2, n_in2, len2, nwin2, div2;
    uint32_t dv2_mul, dv2_sh;
    int32_t start2[kCW];
    int32_t o2[kCR], P2[kCR][kCR];               // f2.in origin / paving mod sY  [a][j]
    int32_t F2[kCP][kCR];                        // f2 pattern element p's signed raw offset on Y dim a
    int32_t n_out, out_dim[kCR + 1], out_ext[kCR + 1], out_step[kCR + 1];   // outer rep dims (+ chunk index)
    uint32_t out_mul[kCR + 1], out_sh[kCR + 1];
    int32_t n_inr, in_dim[kCIn], in_len[kCIn];   // inner rep dims (0: chunked), full lengths
    uint32_t in_mul[kCIn], in_sh[kCIn];
    int32_t chunk_ext, chunk_len, tail_prod;
    uint32_t tail_mul, tail_sh;
    int32_t nblocks;
    // f2's output tiler (linear): Z offset = zo + sum_j zP[j] r_j + zF[k]
    int32_t zo, zP[kCR], zF[kCW];
    // the same steps per outer / inner repetition dim of the blocking (outer: raw Y steps reduced mod sY, the
    // chunk dim's per chunk; inner: signed Y steps)
    int32_t out_y[kCR + 1][kCR], out_z[kCR + 1];
    int32_t in_y[kCIn][kCR], in_z[kCIn];
};

// Per-block quantities, computed once by thread 0 into shared memory.
struct ChainBlk {
    int32_t E[kCR], base[kCR], bst[kCR], lo[kCR];   // Y box: extents, corner (mod sY), smem strides, corner offset
    int32_t v0[kCR], R0[kCR], nR[kCR];               // f1 repetitions covering the box: R0 .. R0 + nR - 1 per Y dim
    uint32_t nR_mul[kCR], nR_sh[kCR];
    int32_t nrep1, len0, count, zb;
    int32_t bstep[kCIn];                             // box offset per unit of inner repetition dim d
    int32_t poff[kCP];                               // box offset of f2 pattern element p (relative)
    int32_t kkoff[kCW];                              // box offset of f1 window k relative to its repetition
    int32_t nrow1;                                   // f1: rows of repetitions (all Y dims but the last)
    uint32_t nl_mul, nl_sh;                          // magic division by nR[last] (f1 row length)
    int32_t llast;                                   // f2 row length (innermost inner repetition dim)
    uint32_t ll_mul, ll_sh;
};

__device__ __forceinline__ uint32_t mdiv(uint32_t n, uint32_t mul, uint32_t sh) { return (__umulhi(n, mul) + n) >> sh; }

// C task: S/d - S%d (truncating), with |S| / |d| by a magic number.
__device__ __forceinline__ int32_t task_c(int32_t S, int32_t d, uint32_t mul, uint32_t sh) {
    const uint32_t qa = mdiv(uint32_t(abs(S)), mul, sh);
    const int32_t q = ((S < 0) != (d < 0)) ? -int32_t(qa) : int32_t(qa);
    return q * (1 + d) - S;
}

__device__ __forceinline__ void magic_dev(uint32_t d, uint32_t& mul, uint32_t& sh) {
    uint32_t s = 0;
    while (s < 32 && (1ull << s) < d) ++s;
    sh = s;
    mul = uint32_t(((1ull << 32) * ((1ull << s) - uint64_t(d))) / d + 1);
}

__device__ void chain_block(const ChainDev& cd, int32_t blk, ChainBlk& g, int RY) {
    int64_t raw[kCR];
    for (int a = 0; a < kCR; ++a) raw[a] = cd.o2[a];
    int32_t zb = cd.zo;
    uint32_t n = uint32_t(blk);
    int32_t ck = 0;
    for (int d = cd.n_out - 1; d >= 0; --d) {
        const uint32_t q = mdiv(n, cd.out_mul[d], cd.out_sh[d]);
        const int32_t i = int32_t(n - q * uint32_t(cd.out_ext[d]));
        n = q;
        if (d == cd.n_out - 1) ck = i;
        for (int a = 0; a < RY; ++a) raw[a] += int64_t(cd.out_y[d][a]) * i;
        zb += cd.out_z[d] * i;
    }
    g.len0 = min(cd.chunk_len, cd.chunk_ext - ck * cd.chunk_len);
    g.count = g.len0 * cd.tail_prod;
    g.zb = zb;
    int32_t st = 1;
    g.nrep1 = 1;
    for (int a = RY - 1; a >= 0; --a) {
        int32_t l = 0, h = 0;
        for (int d = 0; d < cd.n_inr; ++d) {
            const int32_t c = cd.in_y[d][a], ln = (d == 0 ? g.len0 : cd.in_len[d]) - 1;
            if (c < 0) l += c * ln; else h += c * ln;
        }
        int32_t pl = 0, ph = 0;
        for (int p = 0; p < cd.n_in2; ++p) {
            pl = min(pl, cd.F2[p][a]);
            ph = max(ph, cd.F2[p][a]);
        }
        l += pl;
        h += ph;
        g.E[a] = h - l + 1;
        int32_t v = int32_t((raw[a] + l) % cd.sY[a]);
        g.base[a] = v < 0 ? v + cd.sY[a] : v;
        g.lo[a] = l;
        g.bst[a] = st;
        st *= (a == RY - 1) ? g.E[a] + ((g.E[a] & 31) == 0 ? 1 : 0) : g.E[a];
        // f1 repetitions covering the dense index range [v0, v0 + E) of this Y dim
        v = g.base[a] - cd.yo[a];
        if (v < 0) v += cd.sY[a];
        g.v0[a] = v;
        g.R0[a] = v / cd.K[a];
        g.nR[a] = (v + g.E[a] - 1) / cd.K[a] - g.R0[a] + 1;
        magic_dev(uint32_t(g.nR[a]), g.nR_mul[a], g.nR_sh[a]);
        g.nrep1 *= g.nR[a];
    }
    for (int d = 0; d < cd.n_inr; ++d) {
        int32_t o = 0;
        for (int a = 0; a < RY; ++a) o += cd.in_y[d][a] * g.bst[a];
        g.bstep[d] = o;
    }
    for (int p = 0; p < cd.n_in2; ++p) {
        int32_t o = 0;
        for (int a = 0; a < RY; ++a) o += (cd.F2[p][a] - g.lo[a]) * g.bst[a];
        g.poff[p] = o;
    }
    for (int k = 0; k < cd.nwin1; ++k) {
        int32_t o = 0;
        for (int a = 0; a < RY; ++a) o += cd.kk[k][a] * g.bst[a];
        g.kkoff[k] = o;
    }
    g.nrow1 = g.nrep1 / g.nR[RY - 1];
    g.nl_mul = g.nR_mul[RY - 1];
    g.nl_sh = g.nR_sh[RY - 1];
    g.llast = cd.n_inr == 1 ? g.len0 : cd.in_len[cd.n_inr - 1];
    magic_dev(uint32_t(g.llast), g.ll_mul, g.ll_sh);
}

// f1's repetition at X reference point ref: gather its pattern, window sums, task; store the outputs into the
// box at dbase + kkoff[k] -- all of them when all_in, else only those whose dense position d0 + kk lies inside
// the box on every Y dim.
template <int RX, int RY, int NP1>
__device__ __forceinline__ void chain_f1_rep(const ChainDev& cd, const ChainBlk& g, const int32_t* __restrict__ X,
                                             int32_t* box, int32_t* my, int32_t (&ref)[RX], int32_t dbase,
                                             bool all_in, const int32_t (&d0)[RY]) {
    bool in_ok = true;
    int32_t xb = 0;
#pragma unroll
    for (int ax = 0; ax < RX; ++ax) {
        ref[ax] -= int32_t(mdiv(uint32_t(ref[ax]), cd.mX_mul[ax], cd.mX_sh[ax])) * cd.sX[ax];
        in_ok &= ref[ax] + cd.fmax_in1[ax] < cd.sX[ax];
        xb += ref[ax] * cd.stX[ax];
    }
    int32_t x[NP1];
    if (cd.contig1 && in_ok && (xb & 3) == 0 && xb + NP1 <= cd.x_elems) {
#pragma unroll
        for (int v = 0; v < NP1 / 4; ++v) {
            const int4 q = __ldg(reinterpret_cast<const int4*>(X + xb) + v);
            x[4 * v] = q.x;
            x[4 * v + 1] = q.y;
            x[4 * v + 2] = q.z;
            x[4 * v + 3] = q.w;
        }
    } else {
#pragma unroll
        for (int p = 0; p < NP1; ++p) {
            x[p] = 0;
            if (p >= cd.n_in1) continue;
            int32_t off;
            if (in_ok) {
                off = xb + cd.lin_in1[p];
            } else {
                off = 0;
#pragma unroll
                for (int ax = 0; ax < RX; ++ax) {
                    int32_t c = ref[ax] + cd.f_in1[p][ax];   // toroidal pattern element
                    if (c >= cd.sX[ax]) c -= cd.sX[ax];
                    off += c * cd.stX[ax];
                }
            }
            x[p] = __ldg(X + off);
        }
    }
    {   // prefix sums (elements past the pattern are never read by a window)
        int32_t acc = 0;
        my[0] = 0;
#pragma unroll
        for (int p = 0; p < NP1; ++p) {
            acc += x[p];
            my[(p + 1) * 256] = acc;
        }
    }
    for (int k = 0; k < cd.nwin1; ++k) {
        if (!all_in) {
            bool inside = true;
#pragma unroll
            for (int a = 0; a < RY; ++a) {
                const int32_t dpos = d0[a] + cd.kk[k][a];
                inside &= dpos >= 0 && dpos < g.E[a];
            }
            if (!inside) continue;
        }
        const int32_t s0 = cd.start1[k];
        box[dbase + g.kkoff[k]] = task_c(my[(s0 + cd.len1) * 256] - my[s0 * 256], cd.div1, cd.dv1_mul, cd.dv1_sh);
    }
}

// The f1 reference-point contribution of Y dim a's dense repetition coordinate Rraw (digits of R mod nRfull;
// a box taller than the Y dim -- small arrays, long patterns -- wraps Rraw around more than once).
template <int RX>
__device__ __forceinline__ void chain_digits(const ChainDev& cd, int a, int32_t Rraw, int32_t (&ref)[RX]) {
    uint32_t R = uint32_t(Rraw);
    while (R >= uint32_t(cd.nRfull[a])) R -= uint32_t(cd.nRfull[a]);
#pragma unroll
    for (int gg = 0; gg < kCDig; ++gg) {
        if (gg >= cd.nrd[a]) continue;
        uint32_t q2 = 0;
        int32_t dig = int32_t(R);
        if (gg + 1 < cd.nrd[a]) {   // the last digit is the remaining quotient itself
            q2 = mdiv(R, cd.rd_mul[a][gg], cd.rd_sh[a][gg]);
            dig = int32_t(R - q2 * uint32_t(cd.rd_ext[a][gg]));
        }
        R = q2;
        const int32_t idx = cd.rd_neg[a][gg] ? cd.rd_ext[a][gg] - 1 - dig : dig;
#pragma unroll
        for (int ax = 0; ax < RX; ++ax) ref[ax] += cd.xs[a][gg][ax] * idx;
    }
}

template <int RX, int RY, int NP1>
__global__ void __launch_bounds__(256) chain_kernel(const __grid_constant__ ChainDev cd, const int32_t* __restrict__ X,
                                                    int32_t* __restrict__ Z) {
    extern __shared__ __align__(16) int32_t sm[];
    __shared__ ChainBlk g;
    int32_t* pre = sm;                          // [kCP + 1][256] per-thread prefix sums
    int32_t* box = pre + (kCP + 1) * 256;
    int32_t* my = pre + threadIdx.x;
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    for (int32_t blk = blockIdx.x; blk < cd.nblocks; blk += gridDim.x) {
        if (threadIdx.x == 0) chain_block(cd, blk, g, RY);
        __syncthreads();
        // ---- (1) fill the box with f1 over the covering repetitions, flattened as (row, i): a row fixes every Y
        // dim but the last, i runs along the last Y dim's range.  Each warp walks a contiguous range of the
        // flattened index (lanes consecutive: coalesced X patterns), so a thread's row changes rarely and the row
        // part (digits, reference point, box offset, inside test) is recomputed only then.
        const int32_t nlast = g.nR[RY - 1], n1 = g.nrep1;
        {
            const int32_t per_warp = (n1 + 8 * 32 - 1) / (8 * 32) * 32;
            const int32_t e_end = min(n1, (warp + 1) * per_warp);
            int32_t rref[RX], d0[RY], cur_row = -1, rbase = 0;
            bool rin = true;
#pragma unroll
            for (int a = 0; a < RY; ++a) d0[a] = 0;
#pragma unroll
            for (int ax = 0; ax < RX; ++ax) rref[ax] = 0;
            for (int32_t e = warp * per_warp + lane; e < e_end; e += 32) {
                const uint32_t row = mdiv(uint32_t(e), g.nl_mul, g.nl_sh);
                const int32_t i = e - int32_t(row) * nlast;
                if (int32_t(row) != cur_row) {
                    cur_row = int32_t(row);
#pragma unroll
                    for (int ax = 0; ax < RX; ++ax) rref[ax] = cd.o1[ax];
                    rbase = 0;
                    rin = true;
                    uint32_t mm = row;
#pragma unroll
                    for (int a = RY - 2; a >= 0; --a) {
                        const uint32_t q = mdiv(mm, g.nR_mul[a], g.nR_sh[a]);
                        const int32_t ia = int32_t(mm - q * uint32_t(g.nR[a]));
                        mm = q;
                        const int32_t Rr = g.R0[a] + ia;
                        chain_digits<RX>(cd, a, Rr, rref);
                        d0[a] = Rr * cd.K[a] - g.v0[a];
                        rbase += d0[a] * g.bst[a];
                        rin &= d0[a] + cd.kkmin[a] >= 0 && d0[a] + cd.kkmax[a] < g.E[a];
                    }
                }
                int32_t ref[RX];
#pragma unroll
                for (int ax = 0; ax < RX; ++ax) ref[ax] = rref[ax];
                const int32_t Rl = g.R0[RY - 1] + i;
                chain_digits<RX>(cd, RY - 1, Rl, ref);
                d0[RY - 1] = Rl * cd.K[RY - 1] - g.v0[RY - 1];
                const bool all_in = rin && d0[RY - 1] + cd.kkmin[RY - 1] >= 0 &&
                                    d0[RY - 1] + cd.kkmax[RY - 1] < g.E[RY - 1];
                chain_f1_rep<RX, RY, NP1>(cd, g, X, box, my, ref, rbase + d0[RY - 1] * g.bst[RY - 1], all_in, d0);
            }
        }
        __syncthreads();
        // ---- (2) f2 over the block's repetitions, flattened as (row, i) along the innermost inner dim, warp-
        // contiguous ranges as above; patterns from the box, outputs to Z
        {
            const int32_t nin = cd.n_inr, llast = g.llast, count = g.count;
            const int32_t bl = g.bstep[nin - 1], zl = cd.in_z[nin - 1];
            const int32_t per_warp = (count + 8 * 32 - 1) / (8 * 32) * 32;
            const int32_t e_end = min(count, (warp + 1) * per_warp);
            int32_t cur_row = -1, boff = 0, zoff = 0;
            for (int32_t e = warp * per_warp + lane; e < e_end; e += 32) {
                const uint32_t row = mdiv(uint32_t(e), g.ll_mul, g.ll_sh);
                const int32_t i = e - int32_t(row) * llast;
                if (int32_t(row) != cur_row) {
                    cur_row = int32_t(row);
                    uint32_t rem = row;
                    boff = 0;
                    zoff = g.zb;
#pragma unroll
                    for (int d = kCIn - 2; d >= 1; --d) {
                        if (d >= nin - 1) continue;
                        const uint32_t q = mdiv(rem, cd.in_mul[d], cd.in_sh[d]);
                        const int32_t id = int32_t(rem - q * uint32_t(cd.in_len[d]));
                        rem = q;
                        boff += g.bstep[d] * id;
                        zoff += cd.in_z[d] * id;
                    }
                    if (nin > 1) {
                        boff += g.bstep[0] * int32_t(rem);
                        zoff += cd.in_z[0] * int32_t(rem);
                    }
                }
                const int32_t bo = boff + bl * i, zo = zoff + zl * i;
                int32_t acc = 0;
                my[0] = 0;
#pragma unroll
                for (int p = 0; p < kCP; ++p) {
                    if (p >= cd.n_in2) continue;
                    acc += box[bo + g.poff[p]];
                    my[(p + 1) * 256] = acc;
                }
                for (int k = 0; k < cd.nwin2; ++k) {
                    const int32_t s0 = cd.start2[k];
                    Z[zo + cd.zF[k]] = task_c(my[(s0 + cd.len2) * 256] - my[s0 * 256], cd.div2, cd.dv2_mul, cd.dv2_sh);
                }
            }
        }
        __syncthreads();   // the box and g are rewritten by the next block
    }
}

using ChainFn = void (*)(const ChainDev, const int32_t*, int32_t*);

template <int RX>
ChainFn chain_kernel_ry(int ry, int np) {
    const int q = (np + 3) / 4 - 1;   // pattern padded to 4, 8, 12 or 16 elements
#define AOL_CHAIN_NP(RY) \
    (q == 0 ? chain_kernel<RX, RY, 4> : q == 1 ? chain_kernel<RX, RY, 8> : q == 2 ? chain_kernel<RX, RY, 12> \
                                                                             : chain_kernel<RX, RY, 16>)
    switch (ry) {
        case 1: return AOL_CHAIN_NP(1);
        case 2: return AOL_CHAIN_NP(2);
        case 3: return AOL_CHAIN_NP(3);
        default: return AOL_CHAIN_NP(4);
    }
#undef AOL_CHAIN_NP
}

ChainFn chain_kernel_for(int rx, int ry, int np) {
    switch (rx) {
        case 1: return chain_kernel_ry<1>(ry, np);
        case 2: return chain_kernel_ry<2>(ry, np);
        case 3: return chain_kernel_ry<3>(ry, np);
        default: return chain_kernel_ry<4>(ry, np);
    }
}

int64_t emod(int64_t a, int64_t m) {
    const int64_t r = a % m;
    return r < 0 ? r + m : r;
}

int64_t signed_rep(int64_t c, int64_t s) {
    c = emod(c, s);
    return 2 * c > s ? c - s : c;
}

void magic_host(uint32_t d, uint32_t* mul, uint32_t* sh) {
    uint32_t s = 0;
    while (s < 32 && (uint64_t(1) << s) < uint64_t(d)) ++s;
    *sh = s;
    *mul = uint32_t(((uint64_t(1) << 32) * ((uint64_t(1) << s) - uint64_t(d))) / uint64_t(d) + 1);
}

int64_t prod(const int64_t* s, int n) {
    int64_t p = 1;
    for (int k = 0; k < n; ++k) p *= s[k];
    return p;
}

// Host plan of the fused chain; false (with a reason) when the chain does not qualify.
bool plan_chain(const aol_filter_t* f1, const aol_filter_t* f2, ChainDev* cd, int* smem, const char** why) {
    std::memset(cd, 0, sizeof *cd);
    const aol_tiler_t& ti = f1->in;
    const aol_tiler_t& to = f1->out;
    const aol_tiler_t& t2 = f2->in;
    const aol_tiler_t& t3 = f2->out;
    *why = "";
    if (ti.array_rank > kCR || to.array_rank > kCR || t3.array_rank > kCR || ti.rep_rank > kCR ||
        t2.rep_rank > kCR) {
        *why = "ranks above 4";
        return false;
    }
    const int64_t n_in1 = prod(ti.pattern_shape, ti.pattern_rank), n_in2 = prod(t2.pattern_shape, t2.pattern_rank);
    if (n_in1 > kCP || n_in2 > kCP || f1->n_windows > kCW || f2->n_windows > kCW) {
        *why = "patterns above 16 elements";
        return false;
    }
    for (const aol_tiler_t* t : {&ti, &to, &t3})
        if (prod(t->array_shape, t->array_rank) >= (int64_t(1) << 31)) {
            *why = "arrays of 2^31 elements or more";
            return false;
        }
    // ---- f1 input side (as filter.cu)
    cd->rx = ti.array_rank;
    cd->rr1 = ti.rep_rank;
    int64_t stride = 1;
    for (int a = ti.array_rank - 1; a >= 0; --a) {
        cd->sX[a] = int32_t(ti.array_shape[a]);
        cd->stX[a] = int32_t(stride);
        stride *= ti.array_shape[a];
        cd->o1[a] = int32_t(emod(ti.origin[a], ti.array_shape[a]));
        for (int j = 0; j < ti.rep_rank; ++j) cd->P1[a][j] = int32_t(emod(ti.paving[a][j], ti.array_shape[a]));
        // o1 + sum P1 r1 must stay below 2^31 before the mod
        __int128 bound = cd->o1[a];
        for (int j = 0; j < ti.rep_rank; ++j) bound += __int128(cd->P1[a][j]) * (ti.rep_shape[j] - 1);
        if (bound >= (__int128(1) << 31)) {
            *why = "f1 reference points beyond 2^31";
            return false;
        }
        magic_host(uint32_t(cd->sX[a]), &cd->mX_mul[a], &cd->mX_sh[a]);
    }
    cd->x_elems = int32_t(stride);
    cd->n_in1 = int32_t(n_in1);
    cd->len1 = f1->window_len;
    cd->nwin1 = f1->n_windows;
    cd->div1 = f1->divisor;
    magic_host(uint32_t(f1->divisor < 0 ? -int64_t(f1->divisor) : f1->divisor), &cd->dv1_mul, &cd->dv1_sh);
    for (int k = 0; k < f1->n_windows; ++k) cd->start1[k] = f1->window_start[k];
    cd->contig1 = 1;
    for (int p = 0; p < n_in1; ++p) {
        int64_t idx[AOL_MAX_RANK] = {0}, q = p;
        for (int k = ti.pattern_rank - 1; k >= 0; --k) {
            idx[k] = q % ti.pattern_shape[k];
            q /= ti.pattern_shape[k];
        }
        int64_t lin = 0;
        for (int a = 0; a < ti.array_rank; ++a) {
            __int128 v = 0;
            for (int k = 0; k < ti.pattern_rank; ++k) v += __int128(emod(ti.fitting[a][k], ti.array_shape[a])) * idx[k];
            cd->f_in1[p][a] = int32_t(v % ti.array_shape[a]);
            cd->fmax_in1[a] = std::max(cd->fmax_in1[a], cd->f_in1[p][a]);
            lin += int64_t(cd->f_in1[p][a]) * cd->stX[a];
        }
        cd->lin_in1[p] = int32_t(lin);
        cd->contig1 &= lin == p;
    }
    // ---- f1 output side: Y = f1.out.array == f2.in.array; bijective, block-diagonal, window digits low
    if (to.array_rank != t2.array_rank) {
        *why = "f1's output array is not f2's input array";
        return false;
    }
    for (int a = 0; a < to.array_rank; ++a)
        if (to.array_shape[a] != t2.array_shape[a]) {
            *why = "f1's output array is not f2's input array";
            return false;
        }
    if (prod(to.rep_shape, to.rep_rank) * prod(to.pattern_shape, to.pattern_rank) != prod(to.array_shape, to.array_rank)) {
        *why = "f1's output tiler does not cover its array exactly";
        return false;
    }
    cd->ry = to.array_rank;
    // digits: combined dims of f1.out (rep dims j, then pattern dims), each owning one Y dim
    const int nd = to.rep_rank + to.pattern_rank;
    int owner[2 * AOL_MAX_RANK];
    int64_t sstep[2 * AOL_MAX_RANK], ext[2 * AOL_MAX_RANK];
    for (int d = 0; d < nd; ++d) {
        ext[d] = d < to.rep_rank ? to.rep_shape[d] : to.pattern_shape[d - to.rep_rank];
        owner[d] = -1;
        sstep[d] = 0;
        if (ext[d] == 1) continue;
        for (int a = 0; a < to.array_rank; ++a) {
            const int64_t c = signed_rep(d < to.rep_rank ? to.paving[a][d] : to.fitting[a][d - to.rep_rank],
                                         to.array_shape[a]);
            if (c == 0) continue;
            if (owner[d] >= 0) {
                *why = "f1's output tiler is not block-diagonal";
                return false;
            }
            owner[d] = a;
            sstep[d] = c;
        }
        if (owner[d] < 0) {
            *why = "f1's output tiler is not injective";
            return false;
        }
    }
    // window index k (row-major over f1.out's pattern) -> dense low part per Y dim
    const int64_t nwin = prod(to.pattern_shape, to.pattern_rank);
    if (nwin != f1->n_windows) {
        *why = "f1 windows";
        return false;
    }
    for (int a = 0; a < to.array_rank; ++a) {
        int ds[2 * AOL_MAX_RANK], n = 0;
        for (int d = 0; d < nd; ++d)
            if (ext[d] > 1 && owner[d] == a) ds[n++] = d;
        std::sort(ds, ds + n, [&](int x, int y) { return std::llabs(sstep[x]) < std::llabs(sstep[y]); });
        int64_t expect = 1, minraw = 0;
        bool pattern_part = true;
        int64_t K = 1;
        int nrd = 0;
        for (int q = 0; q < n; ++q) {
            const int d = ds[q];
            if (std::llabs(sstep[d]) != expect) {
                *why = "f1's output tiler is not a dense mixed radix";
                return false;
            }
            expect *= ext[d];
            if (sstep[d] < 0) minraw += sstep[d] * (ext[d] - 1);
            if (d >= to.rep_rank) {   // a window (pattern) digit
                if (!pattern_part) {
                    *why = "f1's window digits are not the low digits of their Y dim";
                    return false;
                }
                K *= ext[d];
            } else {
                pattern_part = false;
                if (nrd == kCDig) {
                    *why = "more than 3 repetition digits on one Y dim";
                    return false;
                }
                cd->rd_ext[a][nrd] = int32_t(ext[d]);
                cd->rd_neg[a][nrd] = sstep[d] < 0;
                cd->rd_dim[a][nrd] = d;
                magic_host(uint32_t(ext[d]), &cd->rd_mul[a][nrd], &cd->rd_sh[a][nrd]);
                for (int ax = 0; ax < ti.array_rank; ++ax) cd->xs[a][nrd][ax] = cd->P1[ax][d];
                ++nrd;
            }
        }
        if (expect != to.array_shape[a]) {
            *why = "f1's output tiler does not cover its array exactly";
            return false;
        }
        cd->nrd[a] = nrd;
        cd->sY[a] = int32_t(to.array_shape[a]);
        cd->K[a] = int32_t(K);
        cd->nRfull[a] = int32_t(to.array_shape[a] / K);
        cd->yo[a] = int32_t(emod(to.origin[a] + minraw, to.array_shape[a]));
    }
    for (int a = to.array_rank; a < kCR; ++a) cd->rd_dim[a][0] = -1;
    for (int a = 0; a < kCR; ++a)
        for (int g = cd->nrd[a]; g < kCDig; ++g) cd->rd_dim[a][g] = -1;
    for (int64_t k = 0; k < nwin; ++k) {   // dense low part of window k on each Y dim
        int64_t idx[AOL_MAX_RANK] = {0}, q = k;
        for (int p = to.pattern_rank - 1; p >= 0; --p) {
            idx[p] = q % to.pattern_shape[p];
            q /= to.pattern_shape[p];
        }
        for (int a = 0; a < to.array_rank; ++a) {
            int64_t v = 0;
            for (int p = 0; p < to.pattern_rank; ++p) {
                const int d = to.rep_rank + p;
                if (owner[d] != a) continue;
                const int64_t dig = sstep[d] < 0 ? ext[d] - 1 - idx[p] : idx[p];
                v += std::llabs(sstep[d]) * dig;
            }
            cd->kk[k][a] = int32_t(v);
        }
    }
    for (int a = 0; a < kCR; ++a) {
        cd->kkmin[a] = 1 << 30;
        cd->kkmax[a] = -(1 << 30);
        for (int64_t k = 0; k < nwin; ++k) {
            cd->kkmin[a] = std::min(cd->kkmin[a], cd->kk[k][a]);
            cd->kkmax[a] = std::max(cd->kkmax[a], cd->kk[k][a]);
        }
    }
    // ---- f2 input side: blocks of repetitions over a box of Y
    cd->rr2 = t2.rep_rank;
    cd->n_in2 = int32_t(n_in2);
    cd->len2 = f2->window_len;
    cd->nwin2 = f2->n_windows;
    cd->div2 = f2->divisor;
    magic_host(uint32_t(f2->divisor < 0 ? -int64_t(f2->divisor) : f2->divisor), &cd->dv2_mul, &cd->dv2_sh);
    for (int k = 0; k < f2->n_windows; ++k) cd->start2[k] = f2->window_start[k];
    for (int a = 0; a < t2.array_rank; ++a) {
        cd->o2[a] = int32_t(emod(t2.origin[a], t2.array_shape[a]));
        for (int j = 0; j < t2.rep_rank; ++j) cd->P2[a][j] = int32_t(emod(t2.paving[a][j], t2.array_shape[a]));
        __int128 bound = cd->o2[a];
        for (int j = 0; j < t2.rep_rank; ++j) bound += __int128(cd->P2[a][j]) * (t2.rep_shape[j] - 1);
        if (bound >= (__int128(1) << 31)) {
            *why = "f2 reference points beyond 2^31";
            return false;
        }
    }
    int64_t pspan[kCR] = {0};
    for (int p = 0; p < n_in2; ++p) {
        int64_t idx[AOL_MAX_RANK] = {0}, q = p;
        for (int k = t2.pattern_rank - 1; k >= 0; --k) {
            idx[k] = q % t2.pattern_shape[k];
            q /= t2.pattern_shape[k];
        }
        for (int a = 0; a < t2.array_rank; ++a) {
            int64_t v = 0;
            for (int k = 0; k < t2.pattern_rank; ++k) v += signed_rep(t2.fitting[a][k], t2.array_shape[a]) * idx[k];
            if (std::llabs(v) >= (int64_t(1) << 20)) {
                *why = "f2 pattern offsets too large";
                return false;
            }
            cd->F2[p][a] = int32_t(v);
        }
    }
    for (int a = 0; a < t2.array_rank; ++a) {
        int64_t lo = 0, hi = 0;
        for (int p = 0; p < n_in2; ++p) {
            lo = std::min<int64_t>(lo, cd->F2[p][a]);
            hi = std::max<int64_t>(hi, cd->F2[p][a]);
        }
        pspan[a] = hi - lo;
    }
    // grow the inner repetition block from the innermost rep dim while the box fits; chunk the first that does not
    const int64_t budget = kChainBox / 4;
    auto box_vol = [&](int k, int64_t lenk) {
        int64_t v = 1, last = 1;
        for (int a = 0; a < t2.array_rank; ++a) {
            int64_t span = pspan[a];
            for (int j = k; j < t2.rep_rank; ++j)
                span += std::llabs(signed_rep(t2.paving[a][j], t2.array_shape[a])) *
                        ((j == k ? lenk : t2.rep_shape[j]) - 1);
            v *= span + 1;
            last = span + 1;
            if (v > (int64_t(1) << 40)) return int64_t(1) << 40;
        }
        return v + v / last;   // + one pad element per row
    };
    int k = t2.rep_rank - 1;
    if (k < 0) {
        *why = "f2 has no repetition dims";
        return false;
    }
    int64_t lenk = 1;
    if (box_vol(k, 1) > budget) {
        *why = "one f2 repetition's pattern box exceeds shared memory";
        return false;
    }
    for (;;) {
        if (box_vol(k, t2.rep_shape[k]) <= budget) {
            lenk = t2.rep_shape[k];
            if (k == 0 || t2.rep_rank - (k - 1) > kCIn || box_vol(k - 1, 1) > budget) break;
            --k;
            continue;
        }
        int64_t lo = 1, hi = t2.rep_shape[k];
        while (lo < hi) {
            const int64_t mid = (lo + hi + 1) / 2;
            if (box_vol(k, mid) <= budget) lo = mid; else hi = mid - 1;
        }
        lenk = lo;
        break;
    }
    cd->n_inr = t2.rep_rank - k;
    int no = 0;
    int64_t nblocks = 1;
    for (int j = 0; j < k; ++j, ++no) {
        cd->out_dim[no] = j;
        cd->out_ext[no] = int32_t(t2.rep_shape[j]);
        magic_host(uint32_t(t2.rep_shape[j]), &cd->out_mul[no], &cd->out_sh[no]);
        nblocks *= t2.rep_shape[j];
    }
    const int64_t nch = (t2.rep_shape[k] + lenk - 1) / lenk;
    cd->out_dim[no] = k;
    cd->out_ext[no] = int32_t(nch);
    magic_host(uint32_t(nch), &cd->out_mul[no], &cd->out_sh[no]);
    ++no;
    nblocks *= nch;
    cd->n_out = no;
    cd->nblocks = int32_t(nblocks);
    cd->chunk_ext = int32_t(t2.rep_shape[k]);
    cd->chunk_len = int32_t(lenk);
    int64_t tail = 1;
    for (int d = 0; d < kCIn; ++d) cd->in_dim[d] = -1;
    for (int d = 0; d < cd->n_inr; ++d) {
        const int j = k + d;
        cd->in_dim[d] = j;
        cd->in_len[d] = int32_t(d == 0 ? lenk : t2.rep_shape[j]);
        if (d > 0) {
            magic_host(uint32_t(t2.rep_shape[j]), &cd->in_mul[d], &cd->in_sh[d]);
            tail *= t2.rep_shape[j];
        }
    }
    cd->tail_prod = int32_t(tail);
    magic_host(uint32_t(tail), &cd->tail_mul, &cd->tail_sh);
    // ---- f2 output side: linear (no wrap) Z offsets
    {
        int64_t zst[kCR], s = 1;
        for (int a = t3.array_rank - 1; a >= 0; --a) {
            zst[a] = s;
            s *= t3.array_shape[a];
        }
        int64_t zo = 0;
        for (int a = 0; a < t3.array_rank; ++a) {
            const int64_t o = emod(t3.origin[a], t3.array_shape[a]);
            __int128 mx = o;
            for (int j = 0; j < t3.rep_rank; ++j) mx += __int128(emod(t3.paving[a][j], t3.array_shape[a])) * (t3.rep_shape[j] - 1);
            for (int q = 0; q < t3.pattern_rank; ++q)
                mx += __int128(emod(t3.fitting[a][q], t3.array_shape[a])) * (t3.pattern_shape[q] - 1);
            if (mx >= t3.array_shape[a]) {
                *why = "f2's output tiler wraps";
                return false;
            }
            zo += o * zst[a];
        }
        cd->zo = int32_t(zo);
        for (int j = 0; j < t3.rep_rank; ++j) {
            int64_t l = 0;
            for (int a = 0; a < t3.array_rank; ++a) l += emod(t3.paving[a][j], t3.array_shape[a]) * zst[a];
            cd->zP[j] = int32_t(l);
        }
        for (int64_t w = 0; w < f2->n_windows; ++w) {
            int64_t idx[AOL_MAX_RANK] = {0}, q = w;
            for (int p = t3.pattern_rank - 1; p >= 0; --p) {
                idx[p] = q % t3.pattern_shape[p];
                q /= t3.pattern_shape[p];
            }
            int64_t l = 0;
            for (int a = 0; a < t3.array_rank; ++a)
                for (int p = 0; p < t3.pattern_rank; ++p) l += emod(t3.fitting[a][p], t3.array_shape[a]) * idx[p] * zst[a];
            cd->zF[w] = int32_t(l);
        }
    }
    // per blocking dim: Y raw steps (outer: reduced mod sY, the chunk dim per chunk; inner: signed) and Z steps
    for (int d = 0; d < cd->n_out; ++d) {
        const int j = cd->out_dim[d];
        const int64_t mult = d == cd->n_out - 1 ? lenk : 1;
        for (int a = 0; a < t2.array_rank; ++a) cd->out_y[d][a] = int32_t(emod(int64_t(cd->P2[a][j]) * mult, t2.array_shape[a]));
        cd->out_z[d] = int32_t(int64_t(cd->zP[j]) * mult);
    }
    for (int d = 0; d < cd->n_inr; ++d) {
        const int j = cd->in_dim[d];
        for (int a = 0; a < t2.array_rank; ++a) cd->in_y[d][a] = int32_t(signed_rep(cd->P2[a][j], t2.array_shape[a]));
        cd->in_z[d] = cd->zP[j];
    }
    const int64_t box = box_vol(k, lenk);
    *smem = int((kCP + 1) * 256 * 4 + box * 4);
    return true;
}

}  // namespace
}  // namespace aol

using namespace aol;

extern "C" {

aol_status_t aol_filter_chain_apply(const aol_filter_t* f1, const aol_filter_t* f2, const int32_t* d_in, int32_t* d_out,
                                    void* d_workspace, size_t ws_bytes, cudaStream_t s) {
    aol_status_t st = aol_filter_validate(f1);
    if (st != AOL_OK) return st;
    st = aol_filter_validate(f2);
    if (st != AOL_OK) return st;
    if (!d_in || !d_out) return fail(AOL_E_INVALID, "null buffer");
    if ((reinterpret_cast<uintptr_t>(d_in) | reinterpret_cast<uintptr_t>(d_out)) % 4)
        return fail(AOL_E_ALIGN, "buffers must be 4-byte aligned");
    if (f1->out.array_rank != f2->in.array_rank) return fail(AOL_E_SHAPE, "f1's output array is not f2's input array");
    for (int a = 0; a < f1->out.array_rank; ++a)
        if (f1->out.array_shape[a] != f2->in.array_shape[a])
            return fail(AOL_E_SHAPE, "f1's output array is not f2's input array");
    const bool unfused = std::getenv("AOL_CHAIN_UNFUSED") != nullptr;
    // a row filter followed by a column filter (the paper's H -> V shape, any parameters): chain_sep.cu
    if (!unfused && launch_sep_chain(f1, f2, d_in, d_out, s, &st)) return st;
    ChainDev cd;
    int smem = 0;
    const char* why = "";
    const bool fused = !unfused && plan_chain(f1, f2, &cd, &smem, &why);
    if (!fused) {
        // two launches through the caller's workspace (the intermediate array)
        const size_t need = size_t(prod(f1->out.array_shape, f1->out.array_rank)) * 4;
        if (!d_workspace || ws_bytes < need) {
            set_error("this chain cannot be fused (%s): it needs a workspace of %zu bytes for the intermediate array",
                      why, need);
            return AOL_E_WORKSPACE;
        }
        if (reinterpret_cast<uintptr_t>(d_workspace) % 4) return fail(AOL_E_ALIGN, "workspace must be 4-byte aligned");
        st = aol_filter_apply(f1, d_in, static_cast<int32_t*>(d_workspace), s);
        if (st != AOL_OK) return st;
        return aol_filter_apply(f2, static_cast<const int32_t*>(d_workspace), d_out, s);
    }
    if (cd.nblocks == 0) return AOL_OK;
    if (!aligned16(d_in)) cd.contig1 = 0;   // 16-byte pattern loads need an aligned base
    DeviceInfo dev;
    st = device_info(&dev);
    if (st != AOL_OK) return st;
    const ChainFn kern = chain_kernel_for(cd.rx, cd.ry, cd.n_in1);
    st = kernel_smem(reinterpret_cast<const void*>(kern), smem);
    if (st != AOL_OK) return st;
    const int per_sm = std::max(1, kernel_occupancy(reinterpret_cast<const void*>(kern), 256, smem));
    const int grid = int(std::max<int64_t>(1, std::min<int64_t>(cd.nblocks, int64_t(dev.num_sms) * per_sm)));
    st = launch_preflight(reinterpret_cast<const void*>(kern), 256, smem, "chain_kernel");
    if (st != AOL_OK) return st;
    kern<<<grid, 256, smem, s>>>(cd, d_in, d_out);
    AOL_LAUNCH_CHECK("chain_kernel");
    return AOL_OK;
}

}  // extern "C"
