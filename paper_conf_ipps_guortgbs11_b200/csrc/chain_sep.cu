// chain_sep.cu -- NEXT row f3, fused, separable case: two run-time repetitions chained where f1 is a ROW filter
// and f2 a COLUMN filter over a stack of planes -- the paper's H -> V downscaler written generically (Fig. 4-6
// P:L384-471, the H and V tilers Fig. 10 P:L681-694 / reading Z1), with every filter parameter known only at
// run time: pattern lengths, paving steps, origins (incl. toroidal wraps), window starts / length, divisors.
//
// The class (checked on the descriptors by plan_sep; anything else takes chain.cu's general fused kernel or the
// two-launch path):
//   arrays [lead..., rows, cols]; every tiler is the identity on the lead dims (the plane index);
//   f1.in : pattern of L1 along cols, paving diag(1.., 1, p1), origin (0.., o1r, o1c)   (X -> windows)
//   f1.out: Y[.., r, nw1*q + k] (a dense bijection onto Y, origin 0)
//   f2.in : pattern of L2 along rows, paving diag(1.., p2, 1), origin (0.., o2r, 0), p2 <= L2
//   f2.out: Z[.., nw2*b + k, x] (dense, origin 0)
// so Y[r][nw1 q + k] = T1(sum_t X[(r + o1r) mod HX][(o1c + p1 q + s1_k + t) mod WX]) and
//    Z[nw2 b + k][x] = T2(sum_t Y[(o2r + p2 b + s2_k + t) mod HY][x]).
//
// Kernel (WITH-loop folding across the two repetitions, Y never in HBM): a CTA owns (plane, run of nb bands of
// f2).  It walks the Y rows the run needs, (nb - 1) p2 + L2 of them: each X row is staged in shared memory by
// cp.async (16-byte chunks when the column origin and width allow; the row rotated by o1c and extended past its
// end by the pattern overhang, so the wrapping repetition reads contiguously), kNB - 1 rows ahead; f1 turns it
// into one Y row of a ring of the last L2 rows; whenever a band's last row lands, f2 reads the band's L2 rows
// from the ring and writes its nw2 Z rows (coalesced).  Window sums are dot products with 0/1 masks held in the
// kernel's constant bank (one IMAD per pattern element and window, no dynamic register indexing); the task is
// C's S/d - S%d with d by a magic number.
#include <cuda_runtime.h>

#include <algorithm>
#include <cstdint>
#include <cstdlib>
#include <cstring>

#include "common.h"
#include "ptx.cuh"

namespace aol {
namespace {

constexpr int kSepNP = 16;    // pattern elements (L1, L2 <= 16)
constexpr int kSepNW = 8;     // windows per repetition
constexpr int kSepNB = 4;     // X row buffers (kSepNB - 1 rows in flight per CTA)
constexpr int kSepThreads = 256;

struct SepDev {
    int32_t HX, WX, HY, WY, HZ;
    int32_t p1, L1, nw1, o1r, o1c, R1;
    int32_t p2, L2, nw2, o2r, R2;
    int32_t d1, d2;
    uint32_t d1_mul, d1_sh, d2_mul, d2_sh;
    int32_t nb, runs, nunits;
    int32_t J, xstride, vec;   // staged row length, buffer stride (elements), 16-byte staging
    int32_t m1[kSepNW][kSepNP], m2[kSepNW][kSepNP];   // window masks
};

__device__ __forceinline__ int32_t sep_task(int32_t S, int32_t d, uint32_t mul, uint32_t sh) {
    // C: S/d - S%d = q (1 + d) - S with q = S/d truncated; |S| / |d| by a magic number
    const uint32_t a = uint32_t(S < 0 ? -S : S);
    const uint32_t qa = (__umulhi(a, mul) + a) >> sh;
    const int32_t q = ((S < 0) != (d < 0)) ? -int32_t(qa) : int32_t(qa);
    return q * (1 + d) - S;
}

// Window k's sum of a pattern held in registers: a dot product with the k-th 0/1 mask (constant bank).
template <int NP, int K>
__device__ __forceinline__ int32_t sep_dot(const int32_t (&x)[NP], const int32_t (&m)[kSepNW][kSepNP]) {
    int32_t S = 0;
#pragma unroll
    for (int p = 0; p < NP; ++p) S += x[p] * m[K][p];
    return S;
}

// out(k, task(window k)) for the first nw windows: a jump into a fall-through chain (nw is uniform), so only
// nw windows' multiply-adds issue (an unrolled loop guarded by k < nw was if-converted: all 8 issued).
template <int NP, typename Out>
__device__ __forceinline__ void sep_windows(const int32_t (&x)[NP], const int32_t (&m)[kSepNW][kSepNP], int nw,
                                            int32_t d, uint32_t mul, uint32_t sh, Out out) {
    switch (nw) {
        default:
        case 8: out(7, sep_task(sep_dot<NP, 7>(x, m), d, mul, sh)); [[fallthrough]];
        case 7: out(6, sep_task(sep_dot<NP, 6>(x, m), d, mul, sh)); [[fallthrough]];
        case 6: out(5, sep_task(sep_dot<NP, 5>(x, m), d, mul, sh)); [[fallthrough]];
        case 5: out(4, sep_task(sep_dot<NP, 4>(x, m), d, mul, sh)); [[fallthrough]];
        case 4: out(3, sep_task(sep_dot<NP, 3>(x, m), d, mul, sh)); [[fallthrough]];
        case 3: out(2, sep_task(sep_dot<NP, 2>(x, m), d, mul, sh)); [[fallthrough]];
        case 2: out(1, sep_task(sep_dot<NP, 1>(x, m), d, mul, sh)); [[fallthrough]];
        case 1: out(0, sep_task(sep_dot<NP, 0>(x, m), d, mul, sh));
    }
}

template <int NP1, int NP2>
__global__ void __launch_bounds__(kSepThreads) sep_chain_kernel(const __grid_constant__ SepDev sd,
                                                                const int32_t* __restrict__ X,
                                                                int32_t* __restrict__ Z) {
    extern __shared__ __align__(16) int32_t sm[];
    int32_t* ring = sm;                                             // [L2][WY]
    int32_t* xb = sm + ((sd.L2 * sd.WY + 3) & ~3);                  // [kSepNB][xstride]
    const int tid = threadIdx.x;
    for (int32_t unit = blockIdx.x; unit < sd.nunits; unit += gridDim.x) {
        const int32_t plane = unit / sd.runs, run = unit - plane * sd.runs;
        const int32_t b0 = run * sd.nb, b1 = min(b0 + sd.nb, sd.R2);
        const int32_t nrows = (b1 - b0 - 1) * sd.p2 + sd.L2;
        const int32_t* Xp = X + int64_t(plane) * sd.HX * sd.WX;
        int32_t* Zp = Z + int64_t(plane) * sd.HZ * sd.WY;
        // X row of the next row to stage: Y row (o2r + p2 b0 + j) mod HY comes from X row (that + o1r) mod HX
        int32_t xrow_next = int32_t((int64_t(sd.o2r) + int64_t(sd.p2) * b0) % sd.HY) + sd.o1r;
        if (xrow_next >= sd.HX) xrow_next -= sd.HX;
        int32_t staged = 0;

        auto issue = [&]() {
            if (staged < nrows) {
                const int32_t* src = Xp + int64_t(xrow_next) * sd.WX;
                const uint32_t dst = ptx::smem_u32(xb + (staged % kSepNB) * sd.xstride);
                if (sd.vec) {   // o1c, WX multiples of 4: every 16-byte chunk lies on one side of the wrap
                    for (int32_t c = tid; 4 * c < sd.J; c += kSepThreads) {
                        int32_t col = sd.o1c + 4 * c;
                        while (col >= sd.WX) col -= sd.WX;
                        ptx::cp_async<16>(dst + 16u * uint32_t(c), src + col);
                    }
                } else {
                    for (int32_t e = tid; e < sd.J; e += kSepThreads) {
                        int32_t col = sd.o1c + e;
                        while (col >= sd.WX) col -= sd.WX;
                        ptx::cp_async<4>(dst + 4u * uint32_t(e), src + col);
                    }
                }
                ++staged;
                if (++xrow_next == sd.HX) xrow_next = 0;   // Y rows (and so X rows) advance by one, toroidally
            }
            ptx::cp_async_commit();   // (empty groups keep the count uniform)
        };
#pragma unroll
        for (int i = 0; i < kSepNB - 1; ++i) issue();
        int32_t yslot = 0;        // ring slot of row j (= j mod L2)
        int32_t phase = -(sd.L2 - 1);   // j - (L2 - 1) mod p2 once >= 0: 0 when row j completes a band
        int32_t band = b0;
        for (int32_t j = 0; j < nrows; ++j) {
            issue();
            ptx::cp_async_wait<kSepNB - 1>();
            __syncthreads();   // row j staged by every thread; the previous band's ring reads are done
            // ---- f1: one Y row from the staged X row
            {
                const int32_t* xr = xb + (j % kSepNB) * sd.xstride;
                int32_t* yr = ring + yslot * sd.WY;
                for (int32_t q = tid; q < sd.R1; q += kSepThreads) {
                    int32_t x[NP1];
                    const int32_t* xp = xr + sd.p1 * q;
                    if (sd.p1 % 4 == 0) {   // 16-byte aligned pattern: NP1/4 LDS.128 (scalar loads at a stride of
                                            // p1 words conflict p1/gcd-way on the banks)
#pragma unroll
                        for (int v = 0; v < NP1 / 4; ++v) {
                            const int4 w = reinterpret_cast<const int4*>(xp)[v];
                            x[4 * v] = w.x;
                            x[4 * v + 1] = w.y;
                            x[4 * v + 2] = w.z;
                            x[4 * v + 3] = w.w;
                        }
                    } else {
#pragma unroll
                        for (int p = 0; p < NP1; ++p) x[p] = xp[p];
                    }
                    int32_t* yq = yr + sd.nw1 * q;
                    sep_windows<NP1>(x, sd.m1, sd.nw1, sd.d1, sd.d1_mul, sd.d1_sh,
                                     [&](int k, int32_t v) { yq[k] = v; });
                }
            }
            __syncthreads();   // the Y row is complete
            // ---- f2: the band whose last pattern row this was
            if (phase == 0) {
                int32_t roff[NP2];
                int32_t slot = yslot + 1 == sd.L2 ? 0 : yslot + 1;   // oldest row of the ring = the band's row 0
#pragma unroll
                for (int i = 0; i < NP2; ++i) {
                    roff[i] = slot * sd.WY;
                    if (++slot == sd.L2) slot = 0;
                }
                int32_t* zb = Zp + int64_t(sd.nw2) * band * sd.WY;
                for (int32_t x = tid; x < sd.WY; x += kSepThreads) {
                    int32_t y[NP2];
#pragma unroll
                    for (int i = 0; i < NP2; ++i) y[i] = i < sd.L2 ? ring[roff[i] + x] : 0;
                    sep_windows<NP2>(y, sd.m2, sd.nw2, sd.d2, sd.d2_mul, sd.d2_sh,
                                     [&](int k, int32_t v) { zb[int64_t(k) * sd.WY + x] = v; });
                }
                ++band;
            }
            if (++yslot == sd.L2) yslot = 0;
            if (++phase == sd.p2) phase = 0;
        }
        ptx::cp_async_wait<0>();
        __syncthreads();   // the next unit restages the buffers and the ring
    }
}

using SepFn = void (*)(const SepDev, const int32_t*, int32_t*);

template <int NP1>
SepFn sep_kernel_np2(int np2) {
    switch ((np2 + 3) / 4) {
        case 1: return sep_chain_kernel<NP1, 4>;
        case 2: return sep_chain_kernel<NP1, 8>;
        case 3: return sep_chain_kernel<NP1, 12>;
        default: return sep_chain_kernel<NP1, 16>;
    }
}

SepFn sep_kernel_for(int np1, int np2) {
    switch ((np1 + 3) / 4) {
        case 1: return sep_kernel_np2<4>(np2);
        case 2: return sep_kernel_np2<8>(np2);
        case 3: return sep_kernel_np2<12>(np2);
        default: return sep_kernel_np2<16>(np2);
    }
}

void sep_magic(uint32_t d, uint32_t* mul, uint32_t* sh) {
    uint32_t s = 0;
    while (s < 32 && (uint64_t(1) << s) < uint64_t(d)) ++s;
    *sh = s;
    *mul = uint32_t(((uint64_t(1) << 32) * ((uint64_t(1) << s) - uint64_t(d))) / uint64_t(d) + 1);
}

int64_t emod64(int64_t a, int64_t m) {
    const int64_t r = a % m;
    return r < 0 ? r + m : r;
}

// Identity on the lead dims, diagonal paving / single-dim fitting elsewhere.  `pav` = the diagonal of the
// paving on (row, col), `fit_dim` = the dim the pattern runs along.
bool sep_tiler(const aol_tiler_t& t, int n, int64_t pav_row, int64_t pav_col, int fit_dim, bool origin_zero) {
    const int row = n - 2, col = n - 1;
    if (t.array_rank != n || t.rep_rank != n || t.pattern_rank != 1) return false;
    for (int a = 0; a < n; ++a) {
        for (int j = 0; j < n; ++j) {
            const int64_t want = a != j ? 0 : a == row ? pav_row : a == col ? pav_col : 1;
            if (t.paving[a][j] != want) return false;
        }
        if (t.fitting[a][0] != (a == fit_dim ? 1 : 0)) return false;
        if (a < row && (t.origin[a] != 0 || t.rep_shape[a] != t.array_shape[a])) return false;
        if (origin_zero && t.origin[a] != 0) return false;
    }
    return true;
}

// Recognise the separable chain and fill the kernel descriptor; false (why set) when it does not apply.
bool plan_sep(const aol_filter_t* f1, const aol_filter_t* f2, const DeviceInfo& dev, SepDev* sd, int* smem,
              const char** why) {
    const aol_tiler_t &a = f1->in, &b = f1->out, &c = f2->in, &d = f2->out;
    const int n = a.array_rank, row = n - 2, col = n - 1;
    *why = "not a row filter followed by a column filter";
    if (n < 2) return false;
    const int64_t p1 = a.paving[col][col], nw1 = f1->n_windows, p2 = c.paving[row][row], nw2 = f2->n_windows;
    if (p1 < 1 || p2 < 1 || nw1 > kSepNW || nw2 > kSepNW) return false;
    if (!sep_tiler(a, n, 1, p1, col, false) || !sep_tiler(b, n, 1, nw1, col, true) ||
        !sep_tiler(c, n, p2, 1, row, false) || !sep_tiler(d, n, nw2, 1, row, true))
        return false;
    if (c.origin[col] != 0) return false;
    const int64_t HX = a.array_shape[row], WX = a.array_shape[col], HY = b.array_shape[row], WY = b.array_shape[col];
    const int64_t L1 = a.pattern_shape[0], L2 = c.pattern_shape[0], R1 = a.rep_shape[col], R2 = c.rep_shape[row];
    for (int i = 0; i < row; ++i)
        if (b.array_shape[i] != a.array_shape[i] || c.array_shape[i] != a.array_shape[i] ||
            d.array_shape[i] != a.array_shape[i])
            return false;
    if (a.rep_shape[row] != HX || HY != HX || WY != nw1 * R1 || b.rep_shape[row] != HX || b.rep_shape[col] != R1)
        return false;
    if (b.pattern_shape[0] != nw1 || d.pattern_shape[0] != nw2 || c.array_shape[row] != HY ||
        c.array_shape[col] != WY || c.rep_shape[col] != WY || d.rep_shape[row] != R2 || d.rep_shape[col] != WY ||
        d.array_shape[row] != nw2 * R2 || d.array_shape[col] != WY)
        return false;
    if (L1 > kSepNP || L2 > kSepNP || p2 > L2) {
        *why = "patterns longer than 16 or a column paving step beyond the pattern";
        return false;
    }
    int64_t planes = 1;
    for (int i = 0; i < row; ++i) planes *= a.array_shape[i];
    if (planes * HX * WX >= (int64_t(1) << 31) || planes * d.array_shape[row] * WY >= (int64_t(1) << 31)) {
        *why = "arrays of 2^31 elements or more";
        return false;
    }
    std::memset(sd, 0, sizeof *sd);
    sd->HX = int32_t(HX);
    sd->WX = int32_t(WX);
    sd->HY = int32_t(HY);
    sd->WY = int32_t(WY);
    sd->HZ = int32_t(d.array_shape[row]);
    sd->p1 = int32_t(p1);
    sd->L1 = int32_t(L1);
    sd->nw1 = int32_t(nw1);
    sd->o1r = int32_t(emod64(a.origin[row], HX));
    sd->o1c = int32_t(emod64(a.origin[col], WX));
    sd->R1 = int32_t(R1);
    sd->p2 = int32_t(p2);
    sd->L2 = int32_t(L2);
    sd->nw2 = int32_t(nw2);
    sd->o2r = int32_t(emod64(c.origin[row], HY));
    sd->R2 = int32_t(R2);
    sd->d1 = f1->divisor;
    sd->d2 = f2->divisor;
    sep_magic(uint32_t(std::abs(int64_t(f1->divisor))), &sd->d1_mul, &sd->d1_sh);
    sep_magic(uint32_t(std::abs(int64_t(f2->divisor))), &sd->d2_mul, &sd->d2_sh);
    for (int k = 0; k < nw1; ++k)
        for (int p = 0; p < L1; ++p)
            sd->m1[k][p] = p >= f1->window_start[k] && p < f1->window_start[k] + f1->window_len;
    for (int k = 0; k < nw2; ++k)
        for (int p = 0; p < L2; ++p)
            sd->m2[k][p] = p >= f2->window_start[k] && p < f2->window_start[k] + f2->window_len;
    // staged row: p1 (R1 - 1) + L1 elements from column o1c on (mod WX), + kSepNP of slack the unrolled
    // pattern loads may touch (masked out)
    const int64_t J = p1 * (R1 - 1) + L1;
    sd->J = int32_t(J);
    sd->vec = sd->o1c % 4 == 0 && WX % 4 == 0;
    sd->xstride = int32_t((J + 3) / 4 * 4 + kSepNP);
    const int64_t bytes = 4 * (((L2 * WY + 3) & ~int64_t(3)) + int64_t(kSepNB) * sd->xstride);
    if (bytes > dev.smem_optin) {
        *why = "rows too wide for the shared-memory ring";
        return false;
    }
    *smem = int(bytes);
    // bands per unit: 8 (the run re-reads L2 - p2 rows of its neighbour: 4 % for the paper's V filter), fewer
    // when that leaves fewer than 4 units per SM
    int64_t nb = std::min<int64_t>(8, R2);
    while (nb > 1 && planes * ((R2 + nb - 1) / nb) < int64_t(dev.num_sms) * 4) --nb;
    sd->nb = int32_t(nb);
    sd->runs = int32_t((R2 + nb - 1) / nb);
    sd->nunits = int32_t(planes * sd->runs);
    return true;
}

}  // namespace

// AOL_CHAIN_SEP=0 disables the separable chain kernel (A/B measurements only).
bool launch_sep_chain(const aol_filter_t* f1, const aol_filter_t* f2, const int32_t* d_in, int32_t* d_out,
                      cudaStream_t s, aol_status_t* st) {
    static const bool enabled = [] {
        const char* e = std::getenv("AOL_CHAIN_SEP");
        return !(e && e[0] == '0');
    }();
    if (!enabled) return false;
    DeviceInfo dev;
    *st = device_info(&dev);
    if (*st != AOL_OK) return true;
    SepDev sd;
    int smem = 0;
    const char* why = "";
    if (!plan_sep(f1, f2, dev, &sd, &smem, &why)) return false;
    if (sd.vec && reinterpret_cast<uintptr_t>(d_in) % 16) sd.vec = 0;
    *st = AOL_OK;
    if (sd.nunits == 0) return true;
    const SepFn kern = sep_kernel_for(sd.L1, sd.L2);
    *st = kernel_smem(reinterpret_cast<const void*>(kern), smem);
    if (*st != AOL_OK) return true;
    const int per_sm = std::max(1, kernel_occupancy(reinterpret_cast<const void*>(kern), kSepThreads, smem));
    const int grid = int(std::max<int64_t>(1, std::min<int64_t>(sd.nunits, int64_t(dev.num_sms) * per_sm)));
    *st = launch_preflight(reinterpret_cast<const void*>(kern), kSepThreads, smem, "sep_chain_kernel");
    if (*st != AOL_OK) return true;
    kern<<<grid, kSepThreads, smem, s>>>(sd, d_in, d_out);
    note_launch("sep_chain_kernel");
    const cudaError_t e = cudaGetLastError();
    if (e != cudaSuccess) {
        set_error("launch of sep_chain_kernel failed: %s", cudaGetErrorString(e));
        *st = AOL_E_CUDA;
    }
    return true;
}

}  // namespace aol
