// sep_body.cuh -- the separable chain kernel (chain_sep.cu explains the class and the design), written once and
// compiled twice:
//   * statically into libaol.so (SEP_JIT undefined): every filter parameter is read from the SepDev argument --
//     window sums as dot products with 0/1 masks, the task's division by a magic number;
//   * per filter pair by NVRTC at run time (SEP_JIT defined, chain_sep.cu prepends the parameters as literal
//     constants): the masks fold away into plain sums of the window elements, the divisions by constant divisors
//     into multiply-shifts, the window dispatch and pattern lengths into straight-line code -- what the paper's
//     SaC compiler does for tilers known at compile time, done for descriptors known only at run time.
// Self-contained: no headers (NVRTC compiles it without the CUDA toolkit's include tree).
#ifndef AOL_SEP_BODY
#define AOL_SEP_BODY

constexpr int kSepNP = 16;    // pattern elements (L1, L2 <= 16)
constexpr int kSepNW = 8;     // windows per repetition
constexpr int kSepNB = 4;     // X row buffers (kSepNB - 1 rows in flight per CTA)
constexpr int kSepThreads = 256;

typedef int sep_i32;
typedef unsigned int sep_u32;
typedef long long sep_i64;

struct SepDev {
    sep_i32 HX, WX, HY, WY, HZ;
    sep_i32 p1, L1, nw1, o1r, o1c, R1;
    sep_i32 p2, L2, nw2, o2r, R2;
    sep_i32 d1, d2;
    sep_u32 d1_mul, d1_sh, d2_mul, d2_sh;
    sep_i32 nb, runs, nunits, planes;
    sep_i32 J, xstride, vec;   // staged row length, buffer stride (elements), 16-byte staging
    sep_i32 m1[kSepNW][kSepNP], m2[kSepNW][kSepNP];   // window masks (0/1)
};

#ifdef SEP_JIT
// NVRTC: SEP_NP1 .. SEP_D2, the array shapes SEP_HX .. SEP_O1C (literals) and the mask functors sep_m1 / sep_m2
// (constexpr, from the literal window starts) are defined ahead of this text
#define SEP_M1 sep_m1{}
#define SEP_M2 sep_m2{}
#define SEP_TASK(S, d, mul, sh) ((S) / (d) - (S) % (d))
#else
#define SEP_P1 sd.p1
#define SEP_L1 sd.L1
#define SEP_NW1 sd.nw1
#define SEP_P2 sd.p2
#define SEP_L2 sd.L2
#define SEP_NW2 sd.nw2
#define SEP_D1 sd.d1
#define SEP_D2 sd.d2
#define SEP_HX sd.HX
#define SEP_WX sd.WX
#define SEP_HY sd.HY
#define SEP_WY sd.WY
#define SEP_HZ sd.HZ
#define SEP_R1 sd.R1
#define SEP_J sd.J
#define SEP_XSTRIDE sd.xstride
#define SEP_VEC sd.vec
#define SEP_O1C sd.o1c
#define SEP_M1 [&](int k, int p) { return sd.m1[k][p]; }
#define SEP_M2 [&](int k, int p) { return sd.m2[k][p]; }
#define SEP_TASK(S, d, mul, sh) sep_task(S, d, mul, sh)
#endif

// C's S/d - S%d (truncating) = q (1 + d) - S, |S| / |d| by a magic number.
__device__ __forceinline__ sep_i32 sep_task(sep_i32 S, sep_i32 d, sep_u32 mul, sep_u32 sh) {
    const sep_u32 a = sep_u32(S < 0 ? -S : S);
    const sep_u32 qa = (__umulhi(a, mul) + a) >> sh;
    const sep_i32 q = ((S < 0) != (d < 0)) ? -sep_i32(qa) : sep_i32(qa);
    return q * (1 + d) - S;
}

// Window K's sum of a pattern held in registers: a dot product with the K-th 0/1 mask m(K, p).
template <int NP, int K, typename M>
__device__ __forceinline__ sep_i32 sep_dot(const sep_i32 (&x)[NP], const M& m) {
    sep_i32 S = 0;
#pragma unroll
    for (int p = 0; p < NP; ++p) S += x[p] * m(K, p);
    return S;
}

// out(k, window k's task value) for the first nw windows: a jump into a fall-through chain (nw is uniform), so
// only nw windows' multiply-adds issue (an unrolled loop guarded by k < nw was if-converted: all 8 issued).
#define SEP_W(K, NP, x, m, d, mul, sh, out) out(K, SEP_TASK((sep_dot<NP, K>(x, m)), d, mul, sh))
template <int NP, typename M, typename Out>
__device__ __forceinline__ void sep_windows(const sep_i32 (&x)[NP], M m, int nw, sep_i32 d, sep_u32 mul,
                                            sep_u32 sh, Out out) {
    switch (nw) {
        default:
        case 8: SEP_W(7, NP, x, m, d, mul, sh, out); [[fallthrough]];
        case 7: SEP_W(6, NP, x, m, d, mul, sh, out); [[fallthrough]];
        case 6: SEP_W(5, NP, x, m, d, mul, sh, out); [[fallthrough]];
        case 5: SEP_W(4, NP, x, m, d, mul, sh, out); [[fallthrough]];
        case 4: SEP_W(3, NP, x, m, d, mul, sh, out); [[fallthrough]];
        case 3: SEP_W(2, NP, x, m, d, mul, sh, out); [[fallthrough]];
        case 2: SEP_W(1, NP, x, m, d, mul, sh, out); [[fallthrough]];
        case 1: SEP_W(0, NP, x, m, d, mul, sh, out);
    }
}
#undef SEP_W

__device__ __forceinline__ void sep_cp_async16(sep_u32 saddr, const void* g) {
    asm volatile("cp.async.cg.shared.global [%0], [%1], 16;" ::"r"(saddr), "l"(g) : "memory");
}
__device__ __forceinline__ void sep_cp_async4(sep_u32 saddr, const void* g) {
    asm volatile("cp.async.ca.shared.global [%0], [%1], 4;" ::"r"(saddr), "l"(g) : "memory");
}
__device__ __forceinline__ void sep_cp_commit() { asm volatile("cp.async.commit_group;" ::: "memory"); }
template <int N>
__device__ __forceinline__ void sep_cp_wait() { asm volatile("cp.async.wait_group %0;" ::"n"(N) : "memory"); }
__device__ __forceinline__ sep_u32 sep_smem_u32(const void* p) {
    return sep_u32(__cvta_generic_to_shared(p));
}

// f1's pattern of repetition q from the staged X row (the row starts at column o1c, so repetition q's pattern
// is elements p1 q .. p1 q + NP1 - 1; elements past L1 are masked out by the window masks).
template <int NP1>
__device__ __forceinline__ void sep_load_pattern(const SepDev& sd, const sep_i32* xr, sep_i32 q, int tid,
                                                 sep_i32 (&x)[NP1]) {
    (void)sd;
    const sep_i32* xp = xr + SEP_P1 * q;
    if (NP1 % 4 == 0 && SEP_P1 % 4 == 0) {
        // 16-byte aligned pattern: NP1/4 LDS.128 (scalar loads at a stride of p1 words conflict p1/gcd-way on the
        // banks).  At p1 = 8 a quarter-warp's chunks v sit in every other 16-byte bank group: lanes with bit 2 set
        // take chunks 0 and 1 in the other order, which spreads both loads over all 8 groups (conflict-free).
        // (run-time specialised kernel only: with p1 read from the descriptor the swap costs the static kernel
        // more than the conflicts it saves -- 3.65 vs 3.14 ms on the d2 workload)
#ifdef SEP_JIT
        constexpr bool kSwap = true;
#else
        constexpr bool kSwap = false;
#endif
        const bool swp = kSwap && SEP_P1 == 8 && ((tid >> 2) & 1);
        const int4* xp4 = reinterpret_cast<const int4*>(xp);
        int4 c[NP1 / 4 > 0 ? NP1 / 4 : 1];
#pragma unroll
        for (int v = 0; v < NP1 / 4; ++v) c[v] = xp4[v];
        if (kSwap && NP1 >= 8) {
            const int4 L0 = xp4[swp ? 1 : 0], L1 = xp4[swp ? 0 : 1];   // load slots 0 and 1
            c[0] = swp ? L1 : L0;
            c[1] = swp ? L0 : L1;
        }
#pragma unroll
        for (int v = 0; v < NP1 / 4; ++v) {
            x[4 * v] = c[v].x;
            x[4 * v + 1] = c[v].y;
            x[4 * v + 2] = c[v].z;
            x[4 * v + 3] = c[v].w;
        }
    } else {
#pragma unroll
        for (int p = 0; p < NP1; ++p) x[p] = xp[p];
    }
}

// Stage one X row in shared memory: J elements from column o1c on (mod WX), by cp.async (16-byte chunks when the
// column origin and width allow).  (sd is only read by the static kernel: the JIT one has every parameter as a
// literal.)
__device__ __forceinline__ void sep_stage_row(const SepDev& sd, const sep_i32* src, sep_u32 dst, int tid) {
    (void)sd;
    // (one conditional subtraction when the staged span wraps at most once, o1c + J <= 2 WX: a literal in the
    // run-time specialised kernel; the static one keeps the plain loop)
#ifdef SEP_JIT
    const bool once = SEP_O1C + SEP_J <= 2 * SEP_WX;
#else
    constexpr bool once = false;
#endif
    if (SEP_VEC) {   // o1c, WX multiples of 4: every 16-byte chunk lies on one side of the wrap
        for (sep_i32 c = tid; 4 * c < SEP_J; c += kSepThreads) {
            sep_i32 col = SEP_O1C + 4 * c;
            if (once)
                col -= col >= SEP_WX ? SEP_WX : 0;
            else
                while (col >= SEP_WX) col -= SEP_WX;
            sep_cp_async16(dst + 16u * sep_u32(c), src + col);
        }
    } else {
        for (sep_i32 e = tid; e < SEP_J; e += kSepThreads) {
            sep_i32 col = SEP_O1C + e;
            if (once)
                col -= col >= SEP_WX ? SEP_WX : 0;
            else
                while (col >= SEP_WX) col -= SEP_WX;
            sep_cp_async4(dst + 4u * sep_u32(e), src + col);
        }
    }
}

template <int NP1, int NP2>
__device__ __forceinline__ void sep_chain_body(const SepDev& sd, const sep_i32* __restrict__ X,
                                               sep_i32* __restrict__ Z, sep_i32* sm) {
    sep_i32* ring = sm;                                             // [L2][WY]
    sep_i32* xb = sm + ((SEP_L2 * SEP_WY + 3) & ~3);                 // [kSepNB][xstride]
    const int tid = threadIdx.x;
    for (sep_i32 unit = blockIdx.x; unit < sd.nunits; unit += gridDim.x) {
        const sep_i32 plane = unit / sd.runs, run = unit - plane * sd.runs;
        const sep_i32 b0 = run * sd.nb, b1 = min(b0 + sd.nb, sd.R2);
        const sep_i32 nrows = (b1 - b0 - 1) * SEP_P2 + SEP_L2;
        const sep_i32* Xp = X + sep_i64(plane) * SEP_HX * SEP_WX;
        sep_i32* Zp = Z + sep_i64(plane) * SEP_HZ * SEP_WY;
        // X row of the next row to stage: Y row (o2r + p2 b0 + j) mod HY comes from X row (that + o1r) mod HX
        sep_i32 xrow_next = sep_i32((sep_i64(sd.o2r) + sep_i64(SEP_P2) * b0) % SEP_HY) + sd.o1r;
        if (xrow_next >= SEP_HX) xrow_next -= SEP_HX;
        sep_i32 staged = 0;

        auto issue = [&]() {
            if (staged < nrows) {
                const sep_i32* src = Xp + sep_i64(xrow_next) * SEP_WX;
                const sep_u32 dst = sep_smem_u32(xb + (staged % kSepNB) * SEP_XSTRIDE);
                sep_stage_row(sd, src, dst, tid);
                ++staged;
                if (++xrow_next == SEP_HX) xrow_next = 0;   // Y rows (and so X rows) advance by one, toroidally
            }
            sep_cp_commit();   // (empty groups keep the count uniform)
        };
#pragma unroll
        for (int i = 0; i < kSepNB - 1; ++i) issue();
        sep_i32 yslot = 0;                // ring slot of row j (= j mod L2)
        sep_i32 phase = -(SEP_L2 - 1);    // (j - (L2 - 1)) mod p2 once >= 0: 0 when row j completes a band
        sep_i32 band = b0;
        for (sep_i32 j = 0; j < nrows; ++j) {
            issue();
            sep_cp_wait<kSepNB - 1>();
            __syncthreads();   // row j staged by every thread; the previous band's ring reads are done
            // ---- f1: one Y row from the staged X row
            {
                const sep_i32* xr = xb + (j % kSepNB) * SEP_XSTRIDE;
                sep_i32* yr = ring + yslot * SEP_WY;
                for (sep_i32 q = tid; q < SEP_R1; q += kSepThreads) {
                    sep_i32 x[NP1];
                    sep_load_pattern<NP1>(sd, xr, q, tid, x);
                    sep_i32* yq = yr + SEP_NW1 * q;
                    sep_windows<NP1>(x, SEP_M1, SEP_NW1, SEP_D1, sd.d1_mul, sd.d1_sh,
                                     [&](int k, sep_i32 v) { yq[k] = v; });
                }
            }
            __syncthreads();   // the Y row is complete
            // ---- f2: the band whose last pattern row this was
            if (phase == 0) {
                sep_i32 roff[NP2];
                sep_i32 slot = yslot + 1 == SEP_L2 ? 0 : yslot + 1;   // oldest row of the ring = the band's row 0
#pragma unroll
                for (int i = 0; i < NP2; ++i) {
                    roff[i] = slot * SEP_WY;
                    if (++slot == SEP_L2) slot = 0;
                }
                sep_i32* zb = Zp + sep_i64(SEP_NW2) * band * SEP_WY;
                for (sep_i32 x = tid; x < SEP_WY; x += kSepThreads) {
                    sep_i32 y[NP2];
#pragma unroll
                    for (int i = 0; i < NP2; ++i) y[i] = i < SEP_L2 ? ring[roff[i] + x] : 0;
                    sep_windows<NP2>(y, SEP_M2, SEP_NW2, SEP_D2, sd.d2_mul, sd.d2_sh,
                                     [&](int k, sep_i32 v) { zb[sep_i64(k) * SEP_WY + x] = v; });
                }
                ++band;
            }
            if (++yslot == SEP_L2) yslot = 0;
            if (++phase == SEP_P2) phase = 0;
        }
        sep_cp_wait<0>();
        __syncthreads();   // the next unit restages the buffers and the ring
    }
}


#if defined(SEP_JIT) && defined(SEP_REG)
// Register-resident column filter (JIT only: it needs p2, L2 and the window masks as literals).  Thread t owns f1's
// repetitions q = t + 256 i (i < SEP_RPT) and so the Y columns nw1 q .. nw1 q + nw1 - 1 that f2 reads (f2 filters
// each column on its own): the f2 window sums accumulate in registers as the Y rows are produced -- the hand-WLF
// of the specialised K-5 kernel, here for any separable pair of run-time filters.  A Y row belongs to at most
// kRegNB = ceil(L2 / p2) bands; with the row loop unrolled over kRegNB p2 rows, a row's offset in each band and
// the band's accumulator slot are compile-time constants (the slot of band b is b mod kRegNB; a band's first row
// initialises its slot, its row L2 - 1 emits it).  One CTA barrier per row (the staged X row), no Y ring.
constexpr int kRegNB = (SEP_L2 + SEP_P2 - 1) / SEP_P2;
#ifndef SEP_NBUF
#define SEP_NBUF kSepNB
#endif
constexpr int kRegBuf = SEP_NBUF;   // X row buffers (kRegBuf - 1 rows in flight per CTA)
constexpr int kRegPeriod = kRegNB * SEP_P2;

#if SEP_VEC && !defined(SEP_NO_BULK) && defined(SEP_BULK_BYTES)
// TMA staging (16-byte-aligned rows): thread 0 copies a whole X row with 1-D bulk copies -- one per contiguous
// segment of the J elements from column o1c (mod WX), the last one rounded up to 16 bytes (within the row: WX and o1c
// are multiples of 4; the overhang lands in the buffer's slack) -- completing on the buffer's mbarrier, instead of
// every thread issuing 16-byte cp.async chunks: fewer, larger requests (HBM efficiency).
#define SEP_BULK 1
constexpr sep_u32 kSepBulkBytes = SEP_BULK_BYTES;   // bytes one row's copies deliver (host-computed expect-tx count)
__device__ __forceinline__ void sep_mbar_init(sep_u32 bar) {
    asm volatile("mbarrier.init.shared::cta.b64 [%0], 1;" ::"r"(bar) : "memory");
}
__device__ __forceinline__ void sep_bulk_row(const sep_i32* src_row, sep_u32 dst, sep_u32 bar) {
    asm volatile("{\n\t.reg .b64 st;\n\tmbarrier.arrive.expect_tx.shared::cta.b64 st, [%0], %1;\n\t}" ::"r"(bar),
                 "r"(kSepBulkBytes)
                 : "memory");
    sep_i32 col = SEP_O1C, left = SEP_J, off = 0;
#pragma unroll 1
    while (left > 0) {
        const sep_i32 len = left < SEP_WX - col ? left : SEP_WX - col;
        asm volatile("cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];" ::"r"(
                         dst + 4u * sep_u32(off)),
                     "l"(src_row + col), "r"(sep_u32((len + 3) / 4) * 16u), "r"(bar)
                     : "memory");
        off += len;
        left -= len;
        col = 0;
    }
}
__device__ __forceinline__ void sep_mbar_wait(sep_u32 bar, sep_u32 parity) {
    sep_u32 ok;
    do {
        asm volatile("{\n\t.reg .pred p;\n\tmbarrier.try_wait.parity.shared::cta.b64 p, [%1], %2;\n\t"
                     "selp.u32 %0, 1, 0, p;\n\t}"
                     : "=r"(ok)
                     : "r"(bar), "r"(parity)
                     : "memory");
    } while (!ok);
}
#endif

template <int NP1>
__device__ __forceinline__ void sep_reg_body(const SepDev& sd, const sep_i32* __restrict__ X, sep_i32* __restrict__ Z,
                                             sep_i32* sm) {
    sep_i32* xb = sm;   // [kRegBuf][xstride]
    const int tid = threadIdx.x;
#ifdef SEP_BULK
    // one mbarrier per row buffer after the buffers; a buffer's k-th use completes phase k
    const sep_u32 bars = sep_smem_u32(sm + kRegBuf * SEP_XSTRIDE);
    if (tid == 0) {
        for (int b = 0; b < kRegBuf; ++b) sep_mbar_init(bars + 8u * sep_u32(b));
        asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
    }
    __syncthreads();
    sep_u32 issued = 0, consumed = 0;   // rows staged / consumed by this CTA over all its units
#endif
    for (sep_i32 unit = blockIdx.x; unit < sd.nunits; unit += gridDim.x) {
        const sep_i32 plane = unit / sd.runs, run = unit - plane * sd.runs;
        const sep_i32 b0 = run * sd.nb, b1 = min(b0 + sd.nb, sd.R2);
        const sep_i32 nrows = (b1 - b0 - 1) * SEP_P2 + SEP_L2;
        const sep_i32* Xp = X + sep_i64(plane) * SEP_HX * SEP_WX;
        sep_i32* Zp = Z + sep_i64(plane) * SEP_HZ * SEP_WY;
        sep_i32 xrow_next = sep_i32((sep_i64(sd.o2r) + sep_i64(SEP_P2) * b0) % SEP_HY) + sd.o1r;
        if (xrow_next >= SEP_HX) xrow_next -= SEP_HX;
        sep_i32 staged = 0;
        auto issue = [&]() {
            if (staged < nrows) {
#ifdef SEP_BULK
                const sep_u32 b = issued % kRegBuf;
                if (tid == 0)
                    sep_bulk_row(Xp + sep_i64(xrow_next) * SEP_WX, sep_smem_u32(xb + b * SEP_XSTRIDE), bars + 8u * b);
                ++issued;
#else
                sep_stage_row(sd, Xp + sep_i64(xrow_next) * SEP_WX, sep_smem_u32(xb + (staged % kRegBuf) * SEP_XSTRIDE),
                              tid);
#endif
                ++staged;
                if (++xrow_next == SEP_HX) xrow_next = 0;
            }
#ifndef SEP_BULK
            sep_cp_commit();
#endif
        };
#pragma unroll
        for (int i = 0; i < kRegBuf - 1; ++i) issue();
        sep_i32 acc[kRegNB][SEP_NW2][SEP_RPT][SEP_NW1];
#pragma unroll
        for (int b = 0; b < kRegNB; ++b)
#pragma unroll
            for (int k2 = 0; k2 < SEP_NW2; ++k2)
#pragma unroll
                for (int i = 0; i < SEP_RPT; ++i)
#pragma unroll
                    for (int c = 0; c < SEP_NW1; ++c) acc[b][k2][i][c] = 0;
        for (sep_i32 j0 = 0; j0 < nrows; j0 += kRegPeriod) {
#pragma unroll
            for (int u = 0; u < kRegPeriod; ++u) {
                const sep_i32 j = j0 + u;
                if (j >= nrows) break;
#ifdef SEP_BULK
                const sep_u32 cb = consumed % kRegBuf;
                sep_mbar_wait(bars + 8u * cb, (consumed / kRegBuf) & 1u);   // row j has landed
                ++consumed;
                const sep_i32* xr = xb + cb * SEP_XSTRIDE;
#else
                sep_cp_wait<kRegBuf - 2>();
                const sep_i32* xr = xb + (j % kRegBuf) * SEP_XSTRIDE;
#endif
                // row j staged, and every thread is done with row j - 1: only now may its buffer take row
                // j + kRegBuf - 1 (this kernel has no second barrier per row to order that)
                __syncthreads();
                issue();
                sep_i32 y[SEP_RPT][SEP_NW1];
#pragma unroll
                for (int i = 0; i < SEP_RPT; ++i) {
                    // (threads past the last repetition compute a copy of it and store nothing)
                    const sep_i32 q = min(tid + kSepThreads * i, SEP_R1 - 1);
                    sep_i32 x[NP1];
                    sep_load_pattern<NP1>(sd, xr, q, tid, x);
#pragma unroll
                    for (int k = 0; k < SEP_NW1; ++k) {
                        sep_i32 S = 0;
#pragma unroll
                        for (int p = 0; p < NP1; ++p)
                            if (sep_m1{}(k, p)) S += x[p];
                        y[i][k] = SEP_TASK(S, SEP_D1, 0u, 0u);
                    }
                }
                // the row's offset in the band starting d band steps earlier: u % p2 + d p2 (all literals)
#pragma unroll
                for (int d = 0; d < kRegNB; ++d) {
                    const int t = u % SEP_P2 + d * SEP_P2;
                    const int slot = ((u / SEP_P2 - d) % kRegNB + kRegNB) % kRegNB;
                    if (t < SEP_L2) {
#pragma unroll
                        for (int k2 = 0; k2 < SEP_NW2; ++k2) {
                            const bool in = sep_m2{}(k2, t);
#pragma unroll
                            for (int i = 0; i < SEP_RPT; ++i)
#pragma unroll
                                for (int c = 0; c < SEP_NW1; ++c) {
                                    if (t == 0)
                                        acc[slot][k2][i][c] = in ? y[i][c] : 0;
                                    else if (in)
                                        acc[slot][k2][i][c] += y[i][c];
                                }
                        }
                    }
                    if (t == SEP_L2 - 1 && j >= SEP_L2 - 1) {   // band (j - L2 + 1) / p2 of the unit is complete
                        const sep_i32 band = b0 + (j - (SEP_L2 - 1)) / SEP_P2;
                        sep_i32* zb = Zp + sep_i64(SEP_NW2) * band * SEP_WY;
#pragma unroll
                        for (int i = 0; i < SEP_RPT; ++i) {
                            const sep_i32 q = tid + kSepThreads * i;
                            if (q < SEP_R1) {
#pragma unroll
                                for (int k2 = 0; k2 < SEP_NW2; ++k2)
#pragma unroll
                                    for (int c = 0; c < SEP_NW1; ++c)
                                        zb[sep_i64(k2) * SEP_WY + SEP_NW1 * q + c] =
                                            SEP_TASK(acc[slot][k2][i][c], SEP_D2, 0u, 0u);
                            }
                        }
                    }
                }
            }
        }
#ifndef SEP_BULK
        sep_cp_wait<0>();
#endif
        __syncthreads();   // the next unit restages the buffers
    }
}
#endif

#ifdef SEP_JIT
#ifdef SEP_REG
#define SEP_MIN_BLOCKS 4   // 64 registers: 4 CTAs of 256 threads per SM
#else
#define SEP_MIN_BLOCKS 1
#endif
extern "C" __global__ void __launch_bounds__(kSepThreads, SEP_MIN_BLOCKS) sep_chain_jit(const __grid_constant__ SepDev sd,
                                                                        const sep_i32* __restrict__ X,
                                                                        sep_i32* __restrict__ Z) {
    extern __shared__ __align__(16) sep_i32 sep_sm[];
#ifdef SEP_REG
    sep_reg_body<SEP_NP1>(sd, X, Z, sep_sm);
#else
    sep_chain_body<SEP_NP1, SEP_NP2>(sd, X, Z, sep_sm);
#endif
}
#endif

#endif  // AOL_SEP_BODY
