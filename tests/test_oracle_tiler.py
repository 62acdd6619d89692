"""Pins for the oracle's generic ArrayOL tiler (gather / scatter).

Each test pins oracle.gather / oracle.scatter to something other than the
oracle itself: pure-Python brute-force enumeration, numpy library routines for
special cases that reduce to them, and the constants printed in Fig. 10/11.
"""
import numpy as np
import pytest

import bruteforce as bf
from conftest import golden


def _tiler(orc, d):
    return orc.make_tiler(d["array_shape"], d["rep_shape"], d["pattern_shape"],
                          d["origin"], d["paving"], d["fitting"])


@pytest.mark.parametrize("seed", range(120))
def test_gather_scatter_vs_bruteforce(orc, seed):
    """Section IV P:L313-319 / Fig. 4 / Fig. 6 on random tiny descriptors."""
    rng = np.random.default_rng(seed)
    d = bf.random_descriptor(rng)
    dtype = [np.uint8, np.int16, np.int32, np.int64][seed % 4]
    A = rng.integers(0, 100, size=d["array_shape"]).astype(dtype)
    t = _tiler(orc, d)
    G = orc.gather(t, A)
    Gb = bf.gather(A, d["rep_shape"], d["pattern_shape"], d["origin"], d["paving"], d["fitting"])
    assert G.shape == Gb.shape
    assert np.array_equal(G, Gb)
    # scatter of random data into a random background: last writer wins (Fig. 6 order),
    # untouched cells keep their value (modarray)
    Gs = np.asarray(rng.integers(-50, 50, size=Gb.shape)).astype(dtype)
    bg = np.asarray(rng.integers(-50, 50, size=A.shape)).astype(dtype)
    S = orc.scatter(t, Gs, bg)
    Sb = bf.scatter(bg, Gs, d["rep_shape"], d["pattern_shape"], d["origin"], d["paving"], d["fitting"])
    assert np.array_equal(S, Sb)


def test_identity_copy(orc):
    """o=0, P=0, F=I, pattern = array shape -> the single tile is the array (numpy identity)."""
    A = np.arange(7 * 5, dtype=np.int32).reshape(7, 5)
    t = orc.make_tiler([7, 5], [], [7, 5], [0, 0], [[], []], [[1, 0], [0, 1]])
    assert np.array_equal(orc.gather(t, A), A)


@pytest.mark.parametrize("origin", [(0, 0), (3, 1), (-2, 4), (-15, -11), (40, -23)])
def test_roll(orc, origin):
    """F=I, pattern = array shape, origin o -> np.roll(A, -o) (toroidal arrays, reading Z4)."""
    A = np.arange(6 * 9, dtype=np.int32).reshape(6, 9)
    t = orc.make_tiler([6, 9], [], [6, 9], list(origin), [[], []], [[1, 0], [0, 1]])
    assert np.array_equal(orc.gather(t, A), np.roll(A, (-origin[0], -origin[1]), axis=(0, 1)))


def test_transpose(orc):
    """A permutation fitting matrix gives the numpy transpose."""
    A = np.arange(4 * 6 * 5, dtype=np.int64).reshape(4, 6, 5)
    F = [[0, 0, 1], [1, 0, 0], [0, 1, 0]]          # i = (i0,i1,i2) -> a = (i2, i0, i1)
    t = orc.make_tiler([4, 6, 5], [], [6, 5, 4], [0, 0, 0], [[], [], []], F)
    assert np.array_equal(orc.gather(t, A), A.transpose(1, 2, 0))


def test_blocks(orc):
    """P = diag(p), F = I, pattern p -> non-overlapping blocks (numpy reshape/transpose)."""
    A = np.arange(12 * 20, dtype=np.int32).reshape(12, 20)
    t = orc.make_tiler([12, 20], [3, 5], [4, 4], [0, 0], [[4, 0], [0, 4]], [[1, 0], [0, 1]])
    want = A.reshape(3, 4, 5, 4).transpose(0, 2, 1, 3)
    assert np.array_equal(orc.gather(t, A), want)


def test_overlapping_unfold_with_wrap(orc):
    """1-D pattern 11 every 8 (the H tiler along a row): numpy sliding windows of the
    row extended by its first 3 elements (the '% 1920' wrap of Fig. 11)."""
    W = 64
    A = np.arange(W, dtype=np.int32)
    t = orc.make_tiler([W], [W // 8], [11], [0], [[8]], [[1]])
    ext = np.concatenate([A, A[:3]])
    want = np.lib.stride_tricks.sliding_window_view(ext, 11)[::8]
    assert np.array_equal(orc.gather(t, A), want)


def test_fig10_presets(orc):
    """The H tilers are exactly Fig. 10; matrices per reading Z6."""
    g = golden("fig10_tilers.json")
    for which, key in ((orc.PRESET_H_IN, "h_in"), (orc.PRESET_H_OUT, "h_out")):
        t = orc.preset(which, 1080, 1920)
        arr, rep, pat = t.shapes
        spec = g[key]
        assert list(arr) == spec["array_shape"]
        assert list(pat) == spec["pattern_shape"]
        assert list(rep) == spec["repetition_space"]
        assert [t.origin[0], t.origin[1]] == spec["origin"]
        # printed fitting {{0,1}} is one column -> F[a][0]
        assert [t.fitting[0][0], t.fitting[1][0]] == spec["fitting_printed"][0]
        # printed paving {{1,0},{0,8}}: columns of P
        for j, col in enumerate(spec["paving_printed"]):
            assert [t.paving[0][j], t.paving[1][j]] == col
    assert g["bhf_repetition_space_text"]["value"] == g["h_in"]["repetition_space"]


def test_fig11_generated_gather_code(orc):
    """The oracle gather reproduces the GASPARD2-generated index code of Fig. 11
     for the listed work items (hand-evaluated in the fixture)."""
    g = golden("fig11_gather_code.json")
    t = orc.preset(orc.PRESET_H_IN, 1080, 1920)
    A = np.arange(1080 * 1920, dtype=np.int32).reshape(1080, 1920)   # value = flat offset
    G = orc.gather(t, A)
    assert G.shape == (1080, 240, 11)
    for case in g["cases"]:
        r0, r1 = case["tlIter"]
        assert list(G[r0, r1]) == case["flat"], case


def test_fig7_nongeneric_output_tiler(orc):
    """Fig. 7: out[i][j] = input[[i, j/3, j%3]] for the H output tiler."""
    H, W = 9, 48
    t = orc.preset(orc.PRESET_H_OUT, H, W)
    T = np.arange(H * (W // 8) * 3, dtype=np.int32).reshape(H, W // 8, 3)
    out = orc.scatter(t, T, np.full((H, 3 * W // 8), -7, np.int32))
    j = np.arange(3 * W // 8)
    want = T[:, j // 3, j % 3]
    assert np.array_equal(out, want)


def test_h_read_count_histogram(orc):
    """H gather over W=48: columns = 0,1,2 (mod 8) are read twice, the rest once
    (3 of 8 twice, 5 of 8 once); independent count via the brute force."""
    H, W = 2, 48
    t = orc.preset(orc.PRESET_H_IN, H, W)
    A = np.arange(H * W, dtype=np.int64).reshape(H, W)
    G = orc.gather(t, A)
    counts = np.bincount(G.reshape(-1), minlength=H * W).reshape(H, W)
    cb = bf.read_counts([H, W], [H, W // 8], [11], [0, 0], [[1, 0], [0, 8]], [[0], [1]])
    assert np.array_equal(counts, cb)
    assert np.bincount(counts[0]).tolist() == [0, 30, 18]
    assert all(counts[0, x] == (2 if x % 8 < 3 else 1) for x in range(W))


def test_v_read_count_histogram(orc):
    """V gather (reading Z1) over H=27: rows = 0,1,2 (mod 9) read twice, others once."""
    H, Wo = 27, 3
    t = orc.preset(orc.PRESET_V_IN, H, Wo)
    A = np.arange(H * Wo, dtype=np.int64).reshape(H, Wo)
    counts = np.bincount(orc.gather(t, A).reshape(-1), minlength=H * Wo).reshape(H, Wo)
    assert all(counts[y, 0] == (2 if y % 9 < 3 else 1) for y in range(H))
    assert np.bincount(counts[:, 0]).tolist() == [0, 18, 9]


@pytest.mark.parametrize("H,W,h_reps,v_reps", [
    (1080, 1920, 259200, 86400),     # HD: Fig. 10 repetition {1080,240}; V {120,720}
    (2160, 3840, 1036800, 345600),   # 4K, same ratios
    (288, 352, 12672, 4224),         # CIF, Section III
])
def test_pattern_counts(orc, H, W, h_reps, v_reps):
    _, rep, _ = orc.preset(orc.PRESET_H_IN, H, W).shapes
    assert rep[0] * rep[1] == h_reps
    _, rep, _ = orc.preset(orc.PRESET_V_IN, H, 3 * W // 8).shapes
    assert rep[0] * rep[1] == v_reps


def test_scatter_sequential_last_writer(orc):
    """Fig. 6: a colliding output tiler -- the last (r, i) in loop order wins,
    never-written cells keep their old value (modarray)."""
    # 1-D array of 10, rep 4, pattern 3, paving 2: cells 2,4,6 are written twice
    t = orc.make_tiler([10], [4], [3], [0], [[2]], [[1]])
    G = np.arange(100, 112, dtype=np.int32).reshape(4, 3)
    out = orc.scatter(t, G, np.full(10, -1, np.int32))
    # r=0 writes 0,1,2 ; r=1 writes 2,3,4 ; r=2 writes 4,5,6 ; r=3 writes 6,7,8 ; cell 9 untouched
    assert out.tolist() == [100, 101, 103, 104, 106, 107, 109, 110, 111, -1]


def test_invalid_arguments(orc):
    import ctypes
    t = orc.make_tiler([4], [2], [2], [0], [[2]], [[1]])
    t.array_shape[0] = 0
    buf = np.zeros(8, np.int32)
    p = buf.ctypes.data_as(ctypes.c_void_p)
    assert orc.lib().oracle_gather(ctypes.byref(t), 4, p, p) == -1
    t.array_shape[0] = 4
    assert orc.lib().oracle_gather(ctypes.byref(t), 3, p, p) == -1      # bad element size
    assert orc.lib().oracle_downscale_h(p, p, 1, 12) == -1              # W % 8 != 0
    assert orc.lib().oracle_downscale_v(p, p, 10, 3) == -1              # H % 9 != 0
