"""CPU (no GPU): the run-time specialised separable chain kernel compiles with NVRTC for sm_100a -- the paper's
H -> V pair at several frame sizes and random separable pairs covering both kernel bodies (register-resident
column filter and Y ring), pattern loads on and off the 16-byte grid and wrapping origins.  A source the GPU box's
NVRTC would reject would otherwise only show up there, as the statically compiled fallback running instead."""
import ctypes

import numpy as np
import pytest

aol = pytest.importorskip("paper_conf_ipps_guortgbs11_b200")
from paper_conf_ipps_guortgbs11_b200 import _lib  # noqa: E402


def compile_pair(f1, f2):
    buf = ctypes.create_string_buffer(8192)
    rc = _lib.lib().aol_debug_sep_jit_compile(ctypes.byref(f1), ctypes.byref(f2), buf, len(buf))
    return rc, buf.value.decode(errors="replace")


def _need_nvrtc():
    rc, log = compile_pair(aol.filter_preset(aol.FILTER_H, 1, 9, 64), aol.filter_preset(aol.FILTER_V, 1, 9, 24))
    if rc == -1:
        pytest.skip("NVRTC not available")
    return rc, log


@pytest.mark.parametrize("shape", [(900, 1080, 1920), (3, 288, 352), (2, 27, 720), (192, 2160, 3840), (4, 36, 4800)])
def test_paper_pair_compiles(shape):
    _need_nvrtc()
    P, H, W = shape
    rc, log = compile_pair(aol.filter_preset(aol.FILTER_H, P, H, W), aol.filter_preset(aol.FILTER_V, P, H, 3 * W // 8))
    assert rc == 1, log
    # the register-resident body while 2 bands x 4 windows x 3 columns x repetitions per thread <= 64 accumulators
    assert log == ("register-resident" if W // 8 <= 512 else "ring"), log


def _eye(n, diag):
    return [[(diag[a] if a == j else 0) for j in range(n)] for a in range(n)]


@pytest.mark.parametrize("seed", range(12))
def test_random_separable_pairs_compile(seed):
    _need_nvrtc()
    rng = np.random.default_rng(4200 + seed)
    n = int(rng.integers(2, 4))
    lead = [int(rng.integers(1, 4)) for _ in range(n - 2)]
    HX, WX = int(rng.integers(1, 40)), int(rng.integers(4, 3000))
    if seed % 2 == 0:
        WX = 4 * int(rng.integers(1, 700))

    def windows(L):
        ln = int(rng.integers(1, L + 1))
        nw = int(rng.integers(1, 9))
        return [int(rng.integers(0, L - ln + 1)) for _ in range(nw)], ln, int(rng.choice([1, 3, 6, -7]))

    L1, p1 = int(rng.integers(1, 17)), int(rng.integers(1, 12))
    R1 = int(rng.integers(1, max(2, 2 * WX // p1)))
    st1, ln1, d1 = windows(L1)
    o1 = [0] * (n - 2) + [int(rng.integers(-2 * HX, 2 * HX + 1)), 4 * int(rng.integers(-WX, WX + 1)) if seed % 2 == 0
                          else int(rng.integers(-2 * WX, 2 * WX + 1))]
    nw1 = len(st1)
    L2 = int(rng.integers(1, 17))
    p2 = int(rng.integers(1, L2 + 1))
    R2 = int(rng.integers(1, 12))
    st2, ln2, d2 = windows(L2)
    nw2 = len(st2)
    ones = [1] * (n - 2)
    e_col = [[0]] * (n - 1) + [[1]]
    e_row = [[0]] * (n - 2) + [[1], [0]]
    ax, ay, az = lead + [HX, WX], lead + [HX, nw1 * R1], lead + [nw2 * R2, nw1 * R1]
    f1 = aol.make_filter(aol.make_tiler(ax, lead + [HX, R1], [L1], o1, _eye(n, ones + [1, p1]), e_col),
                         aol.make_tiler(ay, lead + [HX, R1], [nw1], [0] * n, _eye(n, ones + [1, nw1]), e_col),
                         st1, ln1, d1)
    f2 = aol.make_filter(aol.make_tiler(ay, lead + [R2, nw1 * R1], [L2], [0] * (n - 2) + [int(rng.integers(-HX, HX + 1)), 0],
                                        _eye(n, ones + [p2, 1]), e_row),
                         aol.make_tiler(az, lead + [R2, nw1 * R1], [nw2], [0] * n, _eye(n, ones + [nw2, 1]), e_row),
                         st2, ln2, d2)
    rc, log = compile_pair(f1, f2)
    assert rc in (0, 1), log   # 0: outside the class (e.g. rows too wide for shared memory)
