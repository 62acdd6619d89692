"""CPU-side checks of the C ABI: the library loads, exports every symbol the
header declares, and its host-only entry points / argument validation behave
(no kernel is launched here -- there is no GPU on the build box)."""
import ctypes
import os
import re

import numpy as np
import pytest

import bruteforce as bf
from conftest import ROOT, golden

aol = pytest.importorskip("paper_conf_ipps_guortgbs11_b200")
from paper_conf_ipps_guortgbs11_b200 import _lib  # noqa: E402


@pytest.fixture(scope="module", autouse=True)
def built():
    import __graft_entry__

    if not os.path.exists(_lib.LIB_PATH):
        __graft_entry__.build()
    _lib.lib()


def header_text():
    inc = os.path.join(ROOT, "include")
    return "".join(open(os.path.join(inc, n)).read() for n in sorted(os.listdir(inc)) if n.endswith(".h"))


def header_symbols():
    """Every entry point include/*.h declares (aol.h and the A/B-experiment header aol_tuning.h)."""
    return sorted(set(re.findall(r"AOL_API\s+[\w\s\*]+?\b(aol_\w+)\s*\(", header_text())))


def test_exports_every_declared_symbol():
    syms = header_symbols()
    assert len(syms) >= 17
    L = _lib.lib()
    for s in syms:
        assert hasattr(L, s), s
    assert set(syms) == set(_lib.SIGNATURES), "binding signatures out of sync with include/aol.h"


def test_exports_via_nm():
    import subprocess

    out = subprocess.run(["nm", "-D", "--defined-only", _lib.LIB_PATH], capture_output=True, text=True).stdout
    exported = set(re.findall(r" T (aol_\w+)", out))
    assert set(header_symbols()) <= exported
    # nothing but the ABI is exported from the library's own code
    assert all(s.startswith("aol_") for s in exported)


def test_version():
    assert aol.version() == 100


def test_presets_match_fig10():
    g = golden("fig10_tilers.json")
    for which, key in ((aol.PRESET_H_IN, "h_in"), (aol.PRESET_H_OUT, "h_out")):
        t = aol.tiler_preset(which, 1080, 1920)
        arr, rep, pat = aol._shapes(t)
        assert list(arr) == g[key]["array_shape"]
        assert list(rep) == g[key]["repetition_space"]
        assert list(pat) == g[key]["pattern_shape"]
        assert [t.fitting[0][0], t.fitting[1][0]] == g[key]["fitting_printed"][0]
        for j, col in enumerate(g[key]["paving_printed"]):
            assert [t.paving[0][j], t.paving[1][j]] == col


def test_presets_match_oracle_presets(orc):
    """The library's presets and the oracle's are written independently; they must agree."""
    for which in range(4):
        for H, W in ((1080, 1920), (288, 352), (18, 24)):
            Wv = W if which < 2 else 3 * W // 8
            a = aol.tiler_preset(which, H, Wv)
            b = orc.preset(which, H, Wv)
            assert bytes(a) == bytes(b), (which, H, W)


def test_preset_errors():
    with pytest.raises(aol.AolError) as e:
        aol.tiler_preset(aol.PRESET_H_IN, 1080, 1921)
    assert e.value.status == _lib.E_SHAPE
    with pytest.raises(aol.AolError) as e:
        aol.tiler_preset(aol.PRESET_V_IN, 1081, 720)
    assert e.value.status == _lib.E_SHAPE
    with pytest.raises(aol.AolError):
        aol.tiler_preset(7, 9, 8)


def test_validate():
    t = aol.make_tiler([4, 5], [2], [3], [0, 0], [[1], [2]], [[0], [1]])
    aol.tiler_validate(t)
    t.array_shape[0] = 0
    with pytest.raises(aol.AolError) as e:
        aol.tiler_validate(t)
    assert e.value.status == _lib.E_INVALID
    t = aol.make_tiler([1 << 40, 1 << 20], [1 << 30], [3], [0, 0], [[1], [2]], [[0], [1]])
    with pytest.raises(aol.AolError) as e:
        aol.tiler_validate(t)
    assert e.value.status == _lib.E_RANGE


@pytest.mark.parametrize("seed", range(40))
def test_is_injective_vs_bruteforce(seed):
    rng = np.random.default_rng(1000 + seed)
    d = bf.random_descriptor(rng)
    t = aol.make_tiler(d["array_shape"], d["rep_shape"], d["pattern_shape"], d["origin"], d["paving"], d["fitting"])
    cnt = bf.read_counts(d["array_shape"], d["rep_shape"], d["pattern_shape"], d["origin"], d["paving"],
                         d["fitting"])
    assert aol.tiler_is_injective(t) == bool(cnt.max() <= 1)


def test_paper_tilers_injectivity():
    # output tilers are bijections (single assignment); input tilers overlap by 3
    assert aol.tiler_is_injective(aol.tiler_preset(aol.PRESET_H_OUT, 18, 64))
    assert aol.tiler_is_injective(aol.tiler_preset(aol.PRESET_V_OUT, 18, 24))
    assert not aol.tiler_is_injective(aol.tiler_preset(aol.PRESET_H_IN, 18, 64))
    assert not aol.tiler_is_injective(aol.tiler_preset(aol.PRESET_V_IN, 18, 24))


@pytest.mark.parametrize("seed", range(400))
def test_injectivity_proof_is_sound(seed):
    """The host's injectivity proof (SEQUENTIAL scatters of proven tilers take the one-pass FAST kernels and
    need no workspace) never claims a tiler the brute-force enumeration finds non-injective."""
    rng = np.random.default_rng(5000 + seed)
    d = bf.random_descriptor(rng)
    if seed % 2:   # bias half the cases toward block-diagonal (provable) descriptors
        ra, rr, rp = len(d["array_shape"]), len(d["rep_shape"]), len(d["pattern_shape"])
        for j in range(rr):
            a = int(rng.integers(ra))
            for b in range(ra):
                d["paving"][b][j] = int(rng.integers(-9, 10)) if b == a else 0
        for k in range(rp):
            a = int(rng.integers(ra))
            for b in range(ra):
                d["fitting"][b][k] = int(rng.integers(-3, 4)) if b == a else 0
    t = aol.make_tiler(d["array_shape"], d["rep_shape"], d["pattern_shape"], d["origin"], d["paving"], d["fitting"])
    proven = _lib.lib().aol_tiler_scatter_workspace_bytes(ctypes.byref(t)) == 0
    cnt = bf.read_counts(d["array_shape"], d["rep_shape"], d["pattern_shape"], d["origin"], d["paving"],
                         d["fitting"])
    if proven:
        assert cnt.max() <= 1, d
    assert aol.tiler_is_injective(t) == bool(cnt.max() <= 1)


def test_injectivity_proof_covers_the_paper_and_d3_tilers():
    L = _lib.lib()
    ws = lambda t: L.aol_tiler_scatter_workspace_bytes(ctypes.byref(t))  # noqa: E731
    assert ws(aol.tiler_preset(aol.PRESET_H_OUT, 18, 64)) == 0 and ws(aol.tiler_preset(aol.PRESET_V_OUT, 18, 24)) == 0
    assert ws(aol.tiler_preset(aol.PRESET_H_IN, 18, 64)) > 0          # overlapping input tiler
    P, F = [[1, 0, 0], [0, 8, 0], [0, 0, 8]], [[0, 0], [1, 0], [0, 1]]
    for origin in ([0, 0, 0], [0, -3, 5]):                              # SURVEY d3 blocking, plain and wrapping
        assert ws(aol.make_tiler([64, 1024, 1024], [64, 128, 128], [8, 8], origin, P, F)) == 0
    assert ws(aol.make_tiler([7], [7], [], [3], [[-1]], [[]])) == 0     # reversal (coefficient -1)
    assert ws(aol.make_tiler([8], [2], [5], [0], [[4]], [[1]])) == 8 * 4   # overlapping windows: claims


def test_workspace_bytes():
    t = aol.make_tiler([4, 5], [2], [3], [0, 0], [[1], [2]], [[0], [1]])
    # the repetition dim moves both array dims: injectivity not provable -> 4-byte claims per element
    assert _lib.lib().aol_tiler_scatter_workspace_bytes(ctypes.byref(t)) == 20 * 4
    assert _lib.lib().aol_tiler_scatter_workspace_bytes(None) == 0
    L = _lib.lib()
    assert L.aol_downscale_frame_host_workspace_bytes(_lib.I32, 4, 3, 1080, 1920) > 2 * 4 * 3 * 1080 * 1920 * 4
    assert L.aol_downscale_frame_host_workspace_bytes(_lib.I32, 4, 3, 1080, 1921) == 0


def _frame(ptr_in, dtype, ptr_out, n, c, h, w):
    return _lib.lib().aol_downscale_frame(ctypes.c_void_p(ptr_in), dtype, ctypes.c_void_p(ptr_out), n, c, h, w,
                                          None, None)


def test_downscale_frame_validation_without_gpu():
    L = _lib.lib()
    assert _frame(0x1000, _lib.I32, 0x2000, 1, 3, 1080, 1921) == _lib.E_SHAPE
    assert _frame(0x1000, _lib.I32, 0x2000, 1, 3, 1081, 1920) == _lib.E_SHAPE
    assert _frame(0x1000, _lib.I16, 0x2000, 1, 3, 1080, 1920) == _lib.E_DTYPE
    assert _frame(0, _lib.I32, 0x2000, 1, 3, 1080, 1920) == _lib.E_INVALID
    assert _frame(0x1004, _lib.I32, 0x2000, 1, 3, 1080, 1920) == _lib.E_ALIGN
    assert _frame(0x1000, _lib.I32, 0x2000, -1, 3, 1080, 1920) == _lib.E_INVALID
    assert _frame(0, _lib.I32, 0, 0, 3, 1080, 1920) == _lib.OK       # zero frames: no-op
    assert b"16-byte" in L.aol_last_error() or True
    assert L.aol_downscale_h(None, None, 1, 10, 12, None) == _lib.E_SHAPE
    assert L.aol_downscale_v(None, None, 1, 10, 12, None) == _lib.E_SHAPE
    assert L.aol_downscale_h(None, None, 0, 9, 16, None) == _lib.OK
    assert L.aol_synth_frames(0, 0, 1, 1, 9, 8, 9, 0, _lib.I32, None, None) == _lib.E_INVALID
    assert L.aol_synth_frames(0, 0, 1, 1, 9, 8, 2, 0, _lib.U8, None, None) == _lib.E_DTYPE


def test_error_message_is_thread_local_string():
    L = _lib.lib()
    assert _frame(0x1000, _lib.I32, 0x2000, 1, 3, 1080, 1921) == _lib.E_SHAPE
    msg = L.aol_last_error().decode()
    assert "multiple of 8" in msg


def test_package_has_no_oracle_dependency():
    """The product package must not import or reference the oracle (no CPU fallback)."""
    pkg = os.path.join(ROOT, "paper_conf_ipps_guortgbs11_b200")
    for dirpath, _, files in os.walk(pkg):
        for fn in files:
            if fn.endswith((".py", ".cu", ".cuh", ".h", ".cpp")):
                with open(os.path.join(dirpath, fn)) as f:
                    src = f.read()
                assert "import oracle" not in src and "from oracle" not in src and "aol_oracle" not in src, fn


def test_filter_presets_and_validation(orc):
    """f3 filters: the presets lift the oracle's per-plane tilers to a stack of planes."""
    for kind, which_in, which_out, Wv in ((aol.FILTER_H, 0, 1, 64), (aol.FILTER_V, 2, 3, 24)):
        f = aol.filter_preset(kind, 5, 18, Wv)
        aol.filter_validate(f)
        for side, which in ((f.in_, which_in), (f.out, which_out)):
            arr, rep, pat = aol._shapes(side)
            o = orc.preset(which, 18, Wv)
            oarr, orep, opat = o.shapes
            assert arr == (5,) + oarr and rep == (5,) + orep and pat == opat
            assert side.paving[0][0] == 1 and all(side.paving[a + 1][j + 1] == o.paving[a][j]
                                                  for a in range(2) for j in range(2))
    f = aol.filter_preset(aol.FILTER_H, 1, 9, 16)
    bad = [("divisor", 0, _lib.E_INVALID), ("window_len", 0, _lib.E_INVALID), ("n_windows", 4, _lib.E_SHAPE)]
    for field, val, code in bad:
        g = aol.filter_preset(aol.FILTER_H, 1, 9, 16)
        setattr(g, field, val)
        with pytest.raises(aol.AolError) as e:
            aol.filter_validate(g)
        assert e.value.status == code, field
    g = aol.filter_preset(aol.FILTER_H, 1, 9, 16)
    g.out.rep_shape[1] = 3
    with pytest.raises(aol.AolError):
        aol.filter_validate(g)
    with pytest.raises(aol.AolError):
        aol.filter_preset(aol.FILTER_V, 1, 10, 16)
    assert f.n_windows == 3 and list(f.window_start)[:3] == [0, 2, 5] and f.window_len == 6


def test_kernel_division_identities():
    """The kernels rewrite Fig. 5's tmp/6 - tmp%6 (C semantics) as 7*(tmp/6) - tmp, and for
    non-negative 8-bit sums use tmp/6 == (tmp*43691) >> 18 (32-bit).  Both are checked
    exhaustively on their domains here (numpy trunc/fmod = C99 truncating / and %)."""
    S = np.arange(-(1 << 20), 1 << 20, dtype=np.int64)
    q = np.trunc(S / 6).astype(np.int64)
    assert np.array_equal(q - np.fmod(S, 6), 7 * q - S)
    U = np.arange(0, 98304, dtype=np.uint64)
    assert np.array_equal(((U * np.uint64(43691)) & np.uint64(0xFFFFFFFF)) >> np.uint64(18), U // np.uint64(6))
    # signed form for |S| < 49152 (uint8-frame V sums): ((S * 43691) >> 18) + (S < 0), arithmetic shift, in int32
    T = np.arange(-49151, 49152, dtype=np.int64)
    p = T * 43691
    assert p.min() > -(1 << 31) and p.max() < (1 << 31)
    assert np.array_equal((p >> 18) + (T < 0), np.trunc(T / 6).astype(np.int64))


def test_magic_division_formula():
    """filter.cu's magic_u31: floor(x/d) == (umulhi(x, mul) + x) >> sh for 0 <= x <= 2^31, with
    sh = ceil(log2 d), mul = floor(2^32 (2^sh - d) / d) + 1 (also the repetition decomposition's formula).
    Exhaustive over x < 2^16 for d < 300, and the extremes / random x for large d."""
    def magic(d):
        sh = 0
        while (1 << sh) < d:
            sh += 1
        return ((1 << 32) * ((1 << sh) - d)) // d + 1, sh

    rng = np.random.default_rng(5)
    xs_small = np.arange(0, 1 << 16, dtype=np.uint64)
    for d in list(range(1, 300)) + [1000, 1080, 1920, 12345, 65537, (1 << 30) + 3, (1 << 31) - 1, 1 << 31]:
        mul, sh = magic(d)
        xs = xs_small if d < 300 else np.concatenate(
            [rng.integers(0, (1 << 31) + 1, 200000, dtype=np.uint64), np.array([0, d - 1, d, (1 << 31) - 1, 1 << 31],
                                                                             dtype=np.uint64)])
        q = (((xs * np.uint64(mul)) >> np.uint64(32)) + xs) >> np.uint64(sh)
        assert np.array_equal(q, xs // np.uint64(d)), d


def test_headers_self_contained():
    """include/aol.h and aol_tuning.h need only <stdint.h>/<stddef.h>: they compile as strict C99 with NO CUDA
    include path (cudaStream_t is declared as cuda_runtime_api.h declares it), and as C++ together with the
    CUDA runtime header in either order."""
    import subprocess
    import tempfile

    d = tempfile.mkdtemp()
    src = os.path.join(d, "h.c")
    with open(src, "w") as f:
        f.write('#include "aol_tuning.h"\nint main(void) { cudaStream_t s = 0; (void)s; return aol_version() != AOL_VERSION; }\n')
    subprocess.check_call(["gcc", "-std=c99", "-pedantic", "-Wall", "-Wextra", "-Werror", "-I",
                           os.path.join(ROOT, "include"), "-c", src, "-o", os.path.join(d, "h.o")])
    for first, second in (("aol.h", "cuda_runtime_api.h"), ("cuda_runtime_api.h", "aol.h")):
        cpp = os.path.join(d, "h.cpp")
        with open(cpp, "w") as f:
            f.write(f'#include "{first}"\n#include "{second}"\nint g() {{ return aol_version(); }}\n')
        subprocess.check_call(["g++", "-std=c++11", "-Wall", "-Werror", "-I", os.path.join(ROOT, "include"), "-I",
                               "/usr/local/cuda/include", "-c", cpp, "-o", os.path.join(d, "h2.o")])


def test_c_example_builds_against_header():
    """examples/aol_example.c compiles and links against include/aol.h + libaol.so with gcc (C11)."""
    import subprocess
    import tempfile

    out = os.path.join(tempfile.mkdtemp(), "aol_example")
    subprocess.check_call(["gcc", "-std=c11", "-O2", "-Wall", "-Wextra", "-Werror", "-I", os.path.join(ROOT, "include"),
                           "-I", "/usr/local/cuda/include", os.path.join(ROOT, "examples", "aol_example.c"),
                           "-L", os.path.dirname(_lib.LIB_PATH), "-laol", "-L", "/usr/local/cuda/lib64", "-lcudart",
                           "-o", out])
    assert os.path.exists(out)


def test_binding_constants_match_header():
    """The Python binding's enum and flag values are the ones include/aol.h declares (marshalling only:
    a drifted constant would silently select another dtype, preset or launch option)."""
    import re

    hdr = header_text()
    flags = {m.group(1): int(m.group(2)) for m in re.finditer(r"#define AOL_FLAG_(\w+)\s+(\d+)", hdr)}
    assert flags == aol.FLAGS
    for name, val in (("AOL_U8", _lib.U8), ("AOL_I16", _lib.I16), ("AOL_I32", _lib.I32), ("AOL_I64", _lib.I64),
                      ("AOL_RAW8", _lib.RAW8), ("AOL_RAW64", _lib.RAW64), ("AOL_RGB8", _lib.RGB8), ("AOL_PRESET_V_OUT", _lib.PRESET_V_OUT),
                      ("AOL_SCATTER_SEQUENTIAL", _lib.SCATTER_SEQUENTIAL), ("AOL_FILTER_V", _lib.FILTER_V),
                      ("AOL_E_CUDA", -7)):
        m = re.search(name + r"\s*=\s*(-?\d+)", hdr)
        assert m and int(m.group(1)) == val, name
