"""Pins for the oracle's filters (task, horizontal, vertical, whole downscaler, checksum).

Pins come from the paper's printed code and shapes (golden fixtures with
citations), hand-derived closed forms, C99 division tables, invariants
(constant frames, toroidal shift-equivariance, locality, channel/frame
independence) and special cases.  None re-derives its expectation by calling
the oracle's own formula.
"""
import numpy as np
import pytest

import synth
from conftest import golden


# ---------------------------------------------------------------- task (Fig. 5)

def test_task_h_windows_fig5(orc):
    """A unit impulse at pattern position p changes tile[k] iff p is in window k
    of Fig. 5: T(1) = -1, T(0) = 0 (C99 table)."""
    g = golden("fig5_task.json")
    L = g["h_pattern_len"]
    G = np.eye(L, dtype=np.int32)                         # rep p: impulse at position p
    T = orc.task_h(G)
    for p in range(L):
        for k, win in enumerate(g["h_windows"]):
            assert T[p, k] == (-1 if p in win else 0), (p, k)


def test_task_v_windows_reading(orc):
    """Same impulse probe for the V task (reading Z1/Z2 windows)."""
    g = golden("fig5_task.json")["v_reading"]
    L = g["v_pattern_len"]
    T = orc.task_v(np.eye(L, dtype=np.int32))
    for p in range(L):
        for k, win in enumerate(g["v_windows"]):
            assert T[p, k] == (-1 if p in win else 0), (p, k)


@pytest.mark.parametrize("task,key", [("task_h", None), ("task_v", "v_reading")])
def test_task_c99_table(orc, task, key):
    """T(S) = S/6 - S%6 with C99 truncation (reading Z3) on the hand-evaluated table;
    the sum S is placed on one tap p, so windows containing p give T(S), the
    others T(0) = 0."""
    g = golden("fig5_task.json")
    rows = g["c99_task_table"]["rows"]
    wins = g["h_windows"] if key is None else g[key]["v_windows"]
    L = g["h_pattern_len"] if key is None else g[key]["v_pattern_len"]
    for p in (5, 6):
        G = np.zeros((len(rows), L), np.int32)
        G[:, p] = [r[0] for r in rows]
        T = getattr(orc, task)(G)
        for (S, q, rem, t), out in zip(rows, T):
            assert q * 6 + rem == S and abs(rem) < 6 and (rem == 0 or (rem > 0) == (S > 0))
            assert list(out) == [t if p in w else 0 for w in wins], (S, p, list(out))


def test_task_matches_numpy_truncation(orc):
    """Library special case: C99 '/' and '%' are numpy trunc-divide and fmod."""
    rng = np.random.default_rng(5)
    G = rng.integers(-2000, 2000, size=(5000, 11)).astype(np.int32)
    T = orc.task_h(G)
    for k, s in enumerate((0, 2, 5)):
        S = G[:, s:s + 6].astype(np.int64).sum(1)
        q = np.trunc(S / 6).astype(np.int64)
        assert np.array_equal(T[:, k], q - np.fmod(S, 6))


# ------------------------------------------------------- horizontal filter

def test_ramp_closed_form_hd(orc):
    """Hand-derived closed form on the HD ramp (golden/ramp_h_hd.json)."""
    g = golden("ramp_h_hd.json")
    X = synth.frames(0, 0, 1, 1, 2, g["W"], "ramp")[0, 0]
    Y = orc.downscale_h(X)
    assert Y.shape == (2, 720)
    for y in range(2):
        assert list(Y[y, :9]) == g["first_outputs_any_row"]
        assert list(Y[y, -3:]) == g["last_rep_outputs_any_row"]
        r = np.arange(239)
        for k, off in enumerate((-1, 1, 4)):
            assert np.array_equal(Y[y, 3 * r + k], 8 * r + off)


@pytest.mark.parametrize("key", ["hd", "cif"])
def test_output_shapes(orc, key):
    """Fig. 2 (HD 1920x1080 -> 720x1080 -> 720x480) and Section III (CIF 352x288 -> 132x128)."""
    s = golden("shapes.json")[key]
    X = synth.frames(1, 0, 1, 1, s["H"], s["W"], "uniform")[0, 0]
    Y = orc.downscale_h(X)
    assert list(Y.shape) == s["Y"]
    Z = orc.downscale_v(Y)
    assert list(Z.shape) == s["Z"]


@pytest.mark.parametrize("c", [0, 1, 7, 100, 255, -3, -1000, 1 << 20, -(1 << 26)])
def test_constant_frame_invariant(orc, c):
    """X == c gives Z == c exactly (S = 6c, T(6c) = c - 0): pins divisor, window width
    and both stages."""
    X = synth.frames(0, 0, 1, 2, 18, 32, "constant", value=c)
    Z, _ = orc.downscale_frame(X)
    assert Z.shape == (1, 2, 8, 12)
    assert np.all(Z == c)


def test_h_shift_equivariance(orc):
    """Toroidal shift by one paving step: H(roll(X, 8, W)) = roll(H(X), 3, W')."""
    X = synth.planes(3, 1, 5, 64)[0]
    Y = orc.downscale_h(X)
    for m in (1, 2, 7):
        assert np.array_equal(orc.downscale_h(np.roll(X, 8 * m, axis=1)), np.roll(Y, 3 * m, axis=1))
    # rows are independent (fitting/paving never mix rows): row shift commutes
    assert np.array_equal(orc.downscale_h(np.roll(X, 2, axis=0)), np.roll(Y, 2, axis=0))


def test_v_shift_equivariance(orc):
    """V(roll(Y, 9, H)) = roll(V(Y), 4, H') (reading Z1), and columns commute."""
    Y = synth.planes(4, 1, 45, 6, "signed")[0] >> 8
    Z = orc.downscale_v(Y)
    for m in (1, 3):
        assert np.array_equal(orc.downscale_v(np.roll(Y, 9 * m, axis=0)), np.roll(Z, 4 * m, axis=0))
    assert np.array_equal(orc.downscale_v(np.roll(Y, 1, axis=1)), np.roll(Z, 1, axis=1))


def test_pipeline_shift_equivariance(orc):
    X = synth.frames(7, 0, 1, 1, 27, 48, "uniform")
    Z, _ = orc.downscale_frame(X)
    Zc = orc.downscale_frame(np.roll(X, (9, 16), axis=(2, 3)))[0]
    assert np.array_equal(Zc, np.roll(Z, (4, 6), axis=(2, 3)))


def test_locality(orc):
    """Changing one input pixel changes at most a 3-column x 3-row output neighbourhood
    (H windows overlap at most 2 per column, 3 columns per pixel; V rows likewise).
    T is many-to-one (T(S+7) = T(S) when S/6 steps by 1), so take the union over deltas."""
    H, W = 27, 48
    X = synth.frames(11, 0, 1, 1, H, W, "uniform")
    Z0, _ = orc.downscale_frame(X)
    for (y, x) in [(0, 0), (13, 21), (26, 47), (9, 8), (17, 45)]:
        changed = np.zeros_like(Z0, dtype=bool)
        for d in (1, 2, 3, 5, 50, -4):
            X2 = X.copy()
            X2[0, 0, y, x] += d
            changed |= orc.downscale_frame(X2)[0] != Z0
        ys, xs = np.nonzero(changed[0, 0])
        assert len(ys) > 0
        assert len(set(ys.tolist())) <= 3 and len(set(xs.tolist())) <= 3


def test_dark_frames_exercise_negative_branch(orc):
    """Dark [0,7] input drives H outputs negative (min -5) so V divides negative sums."""
    X = synth.frames(2, 0, 1, 1, 36, 64, "dark")
    Y = orc.downscale_h(X[0, 0])
    assert Y.min() < 0 and Y.min() >= -5 and Y.max() <= 7


def test_frames_and_channels_independent(orc):
    X = synth.frames(9, 0, 3, 3, 18, 24, "uniform")
    Z, cs = orc.downscale_frame(X)
    perm_f, perm_c = [2, 0, 1], [1, 2, 0]
    Zp, _ = orc.downscale_frame(X[perm_f][:, perm_c])
    assert np.array_equal(Zp, Z[perm_f][:, perm_c])
    # batch = per-frame
    for n in range(3):
        Zn, csn = orc.downscale_frame(X[n:n + 1])
        assert np.array_equal(Zn[0], Z[n]) and csn[0] == cs[n]


def test_frame_equals_h_then_v(orc):
    """downscale_frame = V o H per plane, H first (Fig. 2/3, reading Z13)."""
    X = synth.frames(12, 0, 2, 3, 18, 40, "uniform")
    Z, _ = orc.downscale_frame(X)
    assert np.array_equal(Z, orc.downscale_v(orc.downscale_h(X)))


def test_openmp_threads_same_result(orc):
    X = synth.frames(13, 0, 4, 3, 18, 32, "signed")
    a = orc.downscale_frame(X, nthreads=1)
    b = orc.downscale_frame(X, nthreads=4)
    assert np.array_equal(a[0], b[0]) and np.array_equal(a[1], b[1])


def test_h_and_v_do_not_commute(orc):
    """T is non-linear, so the stage order matters (reading Z13): a V-first pipeline
    differs from the oracle's H-first result on uniform content."""
    X = synth.planes(14, 1, 18, 32)[0]
    hv = orc.downscale_v(orc.downscale_h(X))
    # V first on the full-width plane, then H on the 8x32 result
    vh = orc.downscale_h(orc.downscale_v(X))
    assert hv.shape == vh.shape and not np.array_equal(hv, vh)


# ---------------------------------------------------------------- checksum

def test_checksum_hand_values(orc):
    """cs = sum (u32)z * (1 + (c*Ho + y)*Wo + x) mod 2^64, hand-evaluated."""
    Z = np.array([[[[1, -1]]]], np.int32)                  # weights 1 and 2
    assert int(orc.checksum(Z)[0]) == 1 + (2 ** 32 - 1) * 2
    Z = np.zeros((2, 3, 2, 5), np.int32)
    Z[1, 2, 1, 4] = 1                                       # weight 1 + (2*2+1)*5+4 = 30
    Z[1, 0, 0, 0] = 7                                       # weight 1
    cs = orc.checksum(Z)
    assert int(cs[0]) == 0 and int(cs[1]) == 30 + 7
    Z = np.full((1, 1, 1, 1), -(2 ** 31), np.int32)
    assert int(orc.checksum(Z)[0]) == 2 ** 31
    # wrap mod 2^64
    Z = np.full((1, 3, 480, 720), -1, np.int32)
    n = 3 * 480 * 720
    assert int(orc.checksum(Z)[0]) == ((2 ** 32 - 1) * (n * (n + 1) // 2)) % 2 ** 64
