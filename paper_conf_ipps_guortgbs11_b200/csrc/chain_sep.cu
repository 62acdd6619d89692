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
#include <dlfcn.h>

#include <algorithm>
#include <atomic>
#include <cstdint>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <mutex>
#include <string>
#include <unordered_map>
#include <vector>

#include "common.h"
#include "ptx.cuh"

namespace aol {
namespace {

#include "sep_body.cuh"

template <int NP1, int NP2>
__global__ void __launch_bounds__(kSepThreads) sep_chain_kernel(const __grid_constant__ SepDev sd,
                                                                const int32_t* __restrict__ X,
                                                                int32_t* __restrict__ Z) {
    extern __shared__ __align__(16) int32_t sm[];
    sep_chain_body<NP1, NP2>(sd, X, Z, sm);
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

// Bands of f2 per work unit: up to `cap` (a unit re-reads L2 - p2 rows of its neighbour: 3 of every 9 nb rows for
// the paper's V filter), fewer when that leaves fewer than 4 units per SM.  AOL_SEP_BANDS overrides the cap (A/B).
void sep_set_bands(SepDev* sd, int cap, const DeviceInfo& dev) {
    static const int forced = [] {
        const char* e = std::getenv("AOL_SEP_BANDS");
        return e ? std::atoi(e) : 0;
    }();
    if (forced >= 1) cap = forced;
    int64_t nb = std::min<int64_t>(cap, sd->R2);
    while (nb > 1 && int64_t(sd->planes) * ((sd->R2 + nb - 1) / nb) < int64_t(dev.num_sms) * 4) --nb;
    sd->nb = int32_t(nb);
    sd->runs = int32_t((sd->R2 + nb - 1) / nb);
    sd->nunits = int32_t(int64_t(sd->planes) * sd->runs);
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
    sd->planes = int32_t(planes);
    sep_set_bands(sd, 8, dev);
    return true;
}

// ------------------------------------------------------------ run-time specialisation (NVRTC)
// The kernel body's text (sep_body.cuh, embedded by the build as a raw string literal).
const char kSepBodySrc[] =
#include "sep_body.inc"
    ;

// NVRTC entry points, resolved once with dlopen: libaol.so does not link NVRTC, and runs the static kernel when
// it is absent or a compilation fails.
struct Nvrtc {
    using Create = int (*)(void**, const char*, const char*, int, const char* const*, const char* const*);
    using Compile = int (*)(void*, int, const char* const*);
    using Size = int (*)(void*, size_t*);
    using Get = int (*)(void*, char*);
    using Destroy = int (*)(void**);
    Create create = nullptr;
    Compile compile = nullptr;
    Size cubin_size = nullptr, log_size = nullptr;
    Get cubin = nullptr, log = nullptr;
    Destroy destroy = nullptr;
    bool ok = false;
};

const Nvrtc& nvrtc() {
    static const Nvrtc n = [] {
        Nvrtc r;
        void* h = dlopen("libnvrtc.so.12", RTLD_NOW | RTLD_LOCAL);
        if (!h) h = dlopen("libnvrtc.so", RTLD_NOW | RTLD_LOCAL);
        if (!h) return r;
        r.create = reinterpret_cast<Nvrtc::Create>(dlsym(h, "nvrtcCreateProgram"));
        r.compile = reinterpret_cast<Nvrtc::Compile>(dlsym(h, "nvrtcCompileProgram"));
        r.cubin_size = reinterpret_cast<Nvrtc::Size>(dlsym(h, "nvrtcGetCUBINSize"));
        r.cubin = reinterpret_cast<Nvrtc::Get>(dlsym(h, "nvrtcGetCUBIN"));
        r.log_size = reinterpret_cast<Nvrtc::Size>(dlsym(h, "nvrtcGetProgramLogSize"));
        r.log = reinterpret_cast<Nvrtc::Get>(dlsym(h, "nvrtcGetProgramLog"));
        r.destroy = reinterpret_cast<Nvrtc::Destroy>(dlsym(h, "nvrtcDestroyProgram"));
        r.ok = r.create && r.compile && r.cubin_size && r.cubin && r.log_size && r.log && r.destroy;
        return r;
    }();
    return n;
}

// f1 repetitions per thread of the register-resident column filter (sep_reg_body), 0 when it does not apply: at
// most four repetitions per thread and 64 accumulators (AOL_SEP_REG=0 keeps the Y ring, for A/B measurements).
int sep_reg_rpt(const SepDev& sd) {
    static const bool enabled = [] {
        const char* e = std::getenv("AOL_SEP_REG");
        return !(e && e[0] == '0');
    }();
    const int rpt = (sd.R1 + kSepThreads - 1) / kSepThreads;
    const int nbl = (sd.L2 + sd.p2 - 1) / sd.p2;
    return enabled && rpt <= 4 && nbl * sd.nw2 * sd.nw1 * rpt <= 64 ? rpt : 0;
}

// Row staging of the register-resident kernel: 1-D bulk copies (TMA) when the rows are 16-byte aligned (sd.vec),
// else cp.async chunks; AOL_SEP_BULK=0 forces cp.async (A/B measurements).
bool sep_bulk(const SepDev& sd) {
    static const bool no_bulk = [] {
        const char* e = std::getenv("AOL_SEP_BULK");
        return e && e[0] == '0';
    }();
    return sd.vec && !no_bulk;
}

// X row buffers of the register-resident kernel: 4 with bulk copies (1.282 ms vs 1.330 at 3 and 1.370 at 6), 3 with
// cp.async (1.358 vs 1.364 at 4, 1.51 at 5-6; profiles/r02_f3_reg_sweep.jsonl).  AOL_SEP_NBUF overrides (A/B).
int sep_reg_nbuf(const SepDev& sd) {
    static const int forced = [] {
        const char* e = std::getenv("AOL_SEP_NBUF");
        const int v = e ? std::atoi(e) : 0;
        return v >= 2 && v <= 16 ? v : 0;
    }();
    return forced ? forced : sep_bulk(sd) ? 4 : 3;
}

// The literal parameters the specialised kernel is compiled for (also its cache key): the filters' patterns,
// windows and divisors, and the array shapes (a video's frame size is fixed; a new one compiles once more).
std::string sep_preamble(const aol_filter_t* f1, const aol_filter_t* f2, const SepDev& sd) {
    const int np1 = sd.p1 % 4 == 0 ? (sd.L1 + 3) / 4 * 4 : sd.L1;   // 16-byte pattern loads need NP1 % 4 == 0
    std::string s = "#define SEP_JIT 1\n";
    char b[256];
    std::snprintf(b, sizeof b,
                  "#define SEP_NP1 %d\n#define SEP_NP2 %d\n#define SEP_P1 %d\n#define SEP_L1 %d\n#define SEP_NW1 %d\n"
                  "#define SEP_P2 %d\n#define SEP_L2 %d\n#define SEP_NW2 %d\n#define SEP_D1 (%d)\n#define SEP_D2 (%d)\n",
                  np1, sd.L2, sd.p1, sd.L1, sd.nw1, sd.p2, sd.L2, sd.nw2, sd.d1, sd.d2);
    s += b;
    std::snprintf(b, sizeof b,
                  "#define SEP_HX %d\n#define SEP_WX %d\n#define SEP_HY %d\n#define SEP_WY %d\n#define SEP_HZ %d\n"
                  "#define SEP_R1 %d\n#define SEP_J %d\n#define SEP_XSTRIDE %d\n#define SEP_VEC %d\n#define SEP_O1C %d\n",
                  sd.HX, sd.WX, sd.HY, sd.WY, sd.HZ, sd.R1, sd.J, sd.xstride, sd.vec, sd.o1c);
    s += b;
    if (const int rpt = sep_reg_rpt(sd)) {
        std::snprintf(b, sizeof b, "#define SEP_REG 1\n#define SEP_RPT %d\n#define SEP_NBUF %d\n", rpt, sep_reg_nbuf(sd));
        s += b;
        if (!sep_bulk(sd)) s += "#define SEP_NO_BULK 1\n";
        // bytes one staged row's bulk copies deliver (the last contiguous segment rounded up to 16 bytes)
        int64_t col = sd.o1c, left = sd.J, total = 0;
        while (left > 0) {
            const int64_t len = std::min<int64_t>(left, sd.WX - col);
            total += (len + 3) / 4 * 16;
            left -= len;
            col = 0;
        }
        std::snprintf(b, sizeof b, "#define SEP_BULK_BYTES %lldu\n", static_cast<long long>(total));
        s += b;
    }
    for (int f = 0; f < 2; ++f) {
        const aol_filter_t* fl = f == 0 ? f1 : f2;
        const int L = f == 0 ? sd.L1 : sd.L2;
        std::string starts;
        for (int k = 0; k < fl->n_windows; ++k) {
            std::snprintf(b, sizeof b, "k == %d ? %d : ", k, fl->window_start[k]);
            starts += b;
        }
        s += "struct sep_m" + std::to_string(f + 1) +
             " { __device__ constexpr int operator()(int k, int p) const { return p >= (" + starts + "0) && p < (" +
             starts + "0) + " + std::to_string(fl->window_len) + " && p < " + std::to_string(L) + "; } };\n";
    }
    return s;
}

std::atomic<int> g_sep_jit{-1};   // -1: from AOL_CHAIN_JIT (default on); 0 / 1: set by aol_debug_set_chain_jit

bool sep_jit_enabled() {
    int v = g_sep_jit.load();
    if (v < 0) {
        const char* e = std::getenv("AOL_CHAIN_JIT");
        v = (e && e[0] == '0') ? 0 : 1;
    }
    return v != 0;
}

// NVRTC: the kernel body with the preamble's literals -> a cubin for sm_100a (false, the log in *note, on failure).
bool sep_nvrtc_compile(const std::string& pre, std::vector<char>* cubin, std::string* note) {
    const Nvrtc& nv = nvrtc();
    if (!nv.ok) {
        *note = "NVRTC not available";
        return false;
    }
    const std::string src = pre + kSepBodySrc;
    void* prog = nullptr;
    if (nv.create(&prog, src.c_str(), "aol_sep_chain.cu", 0, nullptr, nullptr) != 0) {
        *note = "nvrtcCreateProgram failed";
        return false;
    }
    const char* opts[] = {"--gpu-architecture=sm_100a", "-std=c++17", "-lineinfo"};
    bool ok = nv.compile(prog, 3, opts) == 0;
    if (ok) {
        size_t n = 0;
        nv.cubin_size(prog, &n);
        cubin->resize(n);
        nv.cubin(prog, cubin->data());
    } else {
        size_t n = 0;
        nv.log_size(prog, &n);
        std::string log(n, '\0');
        nv.log(prog, &log[0]);
        *note = "NVRTC: " + log;
    }
    nv.destroy(&prog);
    return ok;
}

// The specialised kernel for these filters: compiled on first use, then cached (per process; a library loaded
// through the runtime is available on every device).  nullptr: NVRTC missing or the compilation failed (the
// reason is kept for aol_last_error-free diagnostics in jit_note).
std::mutex g_jit_mu;
std::unordered_map<std::string, const void*> g_jit_cache;
std::string g_jit_note;

const void* sep_jit_kernel(const aol_filter_t* f1, const aol_filter_t* f2, const SepDev& sd) {
    if (!sep_jit_enabled()) return nullptr;
    const Nvrtc& nv = nvrtc();
    if (!nv.ok) return nullptr;
    const std::string pre = sep_preamble(f1, f2, sd);
    std::lock_guard<std::mutex> lock(g_jit_mu);
    auto it = g_jit_cache.find(pre);
    if (it != g_jit_cache.end()) return it->second;
    const void* kern = nullptr;
    std::vector<char> cubin;
    if (sep_nvrtc_compile(pre, &cubin, &g_jit_note)) {
        cudaLibrary_t lib = nullptr;
        cudaKernel_t k = nullptr;
        cudaError_t le = cudaLibraryLoadData(&lib, cubin.data(), nullptr, nullptr, 0, nullptr, nullptr, 0);
        if (le == cudaSuccess) le = cudaLibraryGetKernel(&k, lib, "sep_chain_jit");
        if (le == cudaSuccess)
            kern = reinterpret_cast<const void*>(k);   // the library stays loaded for the process
        else
            g_jit_note = std::string("loading the compiled kernel failed: ") + cudaGetErrorString(le);
        cudaGetLastError();
    }
    if (!kern && std::getenv("AOL_JIT_VERBOSE")) std::fprintf(stderr, "aol: chain JIT failed: %s\n", g_jit_note.c_str());
    g_jit_cache.emplace(pre, kern);   // failures are cached too: the static kernel serves those filters
    return kern;
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
    // the run-time specialised kernel when NVRTC is there, else the static one (same body, parameters read
    // from the descriptor)
    const void* jit = sep_jit_kernel(f1, f2, sd);
    const void* kern = jit ? jit : reinterpret_cast<const void*>(sep_kernel_for(sd.L1, sd.L2));
    const char* name = jit ? "sep_chain_jit" : "sep_chain_kernel";
    if (jit && sep_reg_rpt(sd)) {
        smem = int((4 * int64_t(sd.xstride) + 8) * sep_reg_nbuf(sd));   // row buffers + their mbarriers, no Y ring
        sep_set_bands(&sd, 24, dev);   // longer units: 1.358 ms at 24 bands vs 1.386 at 16 and 1.440 at 8
    }
    *st = kernel_smem(kern, smem);
    if (*st != AOL_OK) return true;
    const int per_sm = std::max(1, kernel_occupancy(kern, kSepThreads, smem));
    const int grid = int(std::max<int64_t>(1, std::min<int64_t>(sd.nunits, int64_t(dev.num_sms) * per_sm)));
    *st = launch_preflight(kern, kSepThreads, smem, name);
    if (*st != AOL_OK) return true;
    void* args[] = {&sd, const_cast<int32_t**>(&d_in), &d_out};
    const cudaError_t e = cudaLaunchKernel(kern, dim3(unsigned(grid)), dim3(kSepThreads), args, size_t(smem), s);
    note_launch(name);
    if (e != cudaSuccess) {
        set_error("launch of %s failed: %s", name, cudaGetErrorString(e));
        *st = AOL_E_CUDA;
    }
    return true;
}

// A single filter of the chain's shape runs as a chain with an identity partner (one pattern element, one window of
// length 1, divisor 1: T(S) = S/1 - S%1 = S): a row filter f as f -> identity column filter on its output, a
// column filter as identity row filter on its input -> f.  Only when the run-time specialised kernel is available:
// the statically compiled chain kernel is no faster than aol_filter_apply's own kernel for one repetition.
bool launch_sep_single(const aol_filter_t* f, const int32_t* d_in, int32_t* d_out, cudaStream_t s, aol_status_t* st) {
    if (!sep_jit_enabled() || !nvrtc().ok) return false;
    const int n = f->in.array_rank;
    if (n < 2 || f->in.pattern_rank != 1) return false;
    const int row = n - 2, col = n - 1;
    aol_filter_t id;
    std::memset(&id, 0, sizeof id);
    id.n_windows = 1;
    id.window_len = 1;
    id.divisor = 1;
    auto ident = [&](aol_tiler_t& t, const int64_t* shape, int fit_dim) {
        t.array_rank = t.rep_rank = n;
        t.pattern_rank = 1;
        t.pattern_shape[0] = 1;
        for (int a = 0; a < n; ++a) {
            t.array_shape[a] = t.rep_shape[a] = shape[a];
            t.paving[a][a] = 1;
            t.fitting[a][0] = a == fit_dim ? 1 : 0;
        }
    };
    if (f->in.fitting[col][0] == 1) {   // a row filter, then the identity down the columns of its output
        ident(id.in, f->out.array_shape, row);
        ident(id.out, f->out.array_shape, row);
        return launch_sep_chain(f, &id, d_in, d_out, s, st);
    }
    if (f->in.fitting[row][0] == 1) {   // the identity along the rows of its input, then a column filter
        ident(id.in, f->in.array_shape, col);
        ident(id.out, f->in.array_shape, col);
        return launch_sep_chain(&id, f, d_in, d_out, s, st);
    }
    return false;
}

void set_sep_jit(int on) { g_sep_jit.store(on ? 1 : 0); }

// CPU-testable: compile (not load) the run-time specialised kernel for a separable filter pair.
int sep_jit_compile_check(const aol_filter_t* f1, const aol_filter_t* f2, char* log, size_t cap) {
    DeviceInfo dev;
    if (device_info(&dev) != AOL_OK) dev = DeviceInfo{0, 148, 232448, 233472};   // no GPU: B200's figures
    cudaGetLastError();
    SepDev sd;
    int smem = 0;
    const char* why = "";
    if (!plan_sep(f1, f2, dev, &sd, &smem, &why)) {
        if (log && cap) std::snprintf(log, cap, "%s", why);
        return 0;
    }
    if (!nvrtc().ok) {
        if (log && cap) std::snprintf(log, cap, "NVRTC not available");
        return -1;
    }
    std::vector<char> cubin;
    std::string note;
    const bool ok = sep_nvrtc_compile(sep_preamble(f1, f2, sd), &cubin, &note);
    if (log && cap) std::snprintf(log, cap, "%s", ok ? (sep_reg_rpt(sd) ? "register-resident" : "ring") : note.c_str());
    return ok ? 1 : -2;
}

}  // namespace aol

extern "C" AOL_API void aol_debug_set_chain_jit(int on) { aol::set_sep_jit(on); }

extern "C" AOL_API int aol_debug_sep_jit_compile(const aol_filter_t* f1, const aol_filter_t* f2, char* log,
                                                 size_t cap) {
    if (!f1 || !f2) return 0;
    return aol::sep_jit_compile_check(f1, f2, log, cap);
}
