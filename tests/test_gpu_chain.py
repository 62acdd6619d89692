"""f3 fused: two run-time repetitions chained in one kernel (aol_filter_chain_apply) against the oracle --
the paper's H then V filters (= the fused downscaler; a row filter then a column filter: the separable chain
kernel), random separable chains (any pattern lengths, paving steps, wrapping origins, windows, divisors, lead
dims), the reverse order and random general chains (the general chain kernel), and the two-launch fallback
through a workspace for chains that do not qualify."""
import numpy as np
import pytest
import torch

import synth

pytestmark = pytest.mark.gpu

aol = pytest.importorskip("paper_conf_ipps_guortgbs11_b200")


def _task_c(G, starts, L, d):
    """Fig. 5's task generalised (windows at `starts`, length L, divisor d): tmp/d - tmp%d in C semantics."""
    S = np.stack([G[..., s:s + L].astype(np.int64).sum(-1) for s in starts], -1)
    q = np.sign(S) * np.sign(d) * (np.abs(S) // abs(d))
    return (q - (S - q * d)).astype(np.int32)


@pytest.mark.parametrize("shape", [(2, 1080, 1920), (3, 288, 352), (2, 27, 720), (1, 9, 64), (2, 36, 1000),
                                   (1, 2160, 3840), (240, 1080, 1920)])
def test_chain_h_then_v_equals_fused_downscaler(orc, shape):
    """(240 HD planes: every SM busy with several CTAs for a while -- the staging ring's buffer reuse under load;
    a missing barrier between a row's reads and its buffer's next copy showed up only at this scale.)"""
    P, H, W = shape
    xh = synth.frames(51, 0, 1, P, H, W, "uniform")[0]
    x = torch.from_numpy(xh).cuda()
    fh = aol.filter_preset(aol.FILTER_H, P, H, W)
    fv = aol.filter_preset(aol.FILTER_V, P, H, 3 * W // 8)
    z = aol.filter_chain_apply(fh, fv, x)
    torch.cuda.synchronize()
    assert aol.last_kernel() == "sep_chain_jit"
    zf, _ = aol.downscale_frame(x.unsqueeze(1))
    assert torch.equal(z, zf[:, 0])
    if P * H * W <= 3 * 1080 * 1920:
        assert np.array_equal(z.cpu().numpy(), orc.downscale_v(orc.downscale_h(xh)))


@pytest.mark.parametrize("kind", ["dark", "signed"])
def test_chain_negative_sums(orc, kind):
    P, H, W = 2, 36, 256
    xh = synth.frames(52, 0, 1, P, H, W, kind)[0] >> (6 if kind == "signed" else 0)
    z = aol.filter_chain_apply(aol.filter_preset(aol.FILTER_H, P, H, W), aol.filter_preset(aol.FILTER_V, P, H, 96),
                               torch.from_numpy(xh).cuda())
    torch.cuda.synchronize()
    assert np.array_equal(z.cpu().numpy(), orc.downscale_v(orc.downscale_h(xh)))


def test_chain_v_then_h(orc):
    """The reverse order (V first): f1's window digits are the low digits of the row dim."""
    P, H, W = 2, 54, 512
    xh = synth.frames(53, 0, 1, P, H, W, "uniform")[0]
    fv = aol.filter_preset(aol.FILTER_V, P, H, W)
    fh = aol.filter_preset(aol.FILTER_H, P, 4 * H // 9, W)
    z = aol.filter_chain_apply(fv, fh, torch.from_numpy(xh).cuda())
    torch.cuda.synchronize()
    assert aol.last_kernel() == "chain_kernel"
    assert np.array_equal(z.cpu().numpy(), orc.downscale_h(orc.downscale_v(xh)))


@pytest.mark.parametrize("seed", range(40))
def test_random_chains(orc, seed):
    """f1: a random input tiler (wrapping, any sign), random windows and divisor, output [nrep1][n_out1] (a
    bijection, window digits low); f2: a random tiler over that array with its own windows and divisor,
    output [nrep2][n_out2].  Expected: the oracle's gather -> C task -> scatter, twice."""
    rng = np.random.default_rng(7000 + seed)

    def windows():
        n_in = int(rng.integers(1, 17))
        L = int(rng.integers(1, n_in + 1))
        n_out = int(rng.integers(1, 7))
        starts = [int(rng.integers(0, n_in - L + 1)) for _ in range(n_out)]
        d = int(rng.choice([1, 2, 3, 5, 6, 7, 9, 100, -1, -3, -6]))
        return n_in, L, n_out, starts, d

    n_in1, L1, n_out1, st1, d1 = windows()
    ra = int(rng.integers(1, 4))
    rep1 = [int(rng.integers(1, 7)) for _ in range(int(rng.integers(1, 3)))]
    arr_x = [int(rng.integers(2, 20)) for _ in range(ra)]
    o1 = [int(rng.integers(-2 * s, 2 * s + 1)) for s in arr_x]
    P1 = [[int(rng.integers(-4, 10)) for _ in rep1] for _ in range(ra)]
    F1 = [[int(rng.integers(-4, 10))] for _ in range(ra)]
    nrep1 = int(np.prod(rep1))
    arr_y = [nrep1, n_out1]
    strides = [int(np.prod(rep1[j + 1:])) for j in range(len(rep1))]
    P1o, F1o = [strides, [0] * len(rep1)], [[0], [1]]

    n_in2, L2, n_out2, st2, d2 = windows()
    rep2 = [int(rng.integers(1, 6)) for _ in range(int(rng.integers(1, 3)))]
    o2 = [int(rng.integers(-2 * s, 2 * s + 1)) for s in arr_y]
    P2 = [[int(rng.integers(-3, 6)) for _ in rep2] for _ in range(2)]
    F2 = [[int(rng.integers(-2, 3))] for _ in range(2)]
    nrep2 = int(np.prod(rep2))
    arr_z = [nrep2, n_out2]
    strides2 = [int(np.prod(rep2[j + 1:])) for j in range(len(rep2))]
    P2o, F2o = [strides2, [0] * len(rep2)], [[0], [1]]

    xh = np.asarray(rng.integers(-3000, 3000, size=arr_x)).astype(np.int32)
    y = orc.scatter(orc.make_tiler(arr_y, rep1, [n_out1], [0, 0], P1o, F1o),
                    _task_c(orc.gather(orc.make_tiler(arr_x, rep1, [n_in1], o1, P1, F1), xh), st1, L1, d1),
                    np.zeros(arr_y, np.int32))
    bg = np.full(arr_z, -7, np.int32)
    want = orc.scatter(orc.make_tiler(arr_z, rep2, [n_out2], [0, 0], P2o, F2o),
                       _task_c(orc.gather(orc.make_tiler(arr_y, rep2, [n_in2], o2, P2, F2), y), st2, L2, d2), bg)
    f1 = aol.make_filter(aol.make_tiler(arr_x, rep1, [n_in1], o1, P1, F1),
                         aol.make_tiler(arr_y, rep1, [n_out1], [0, 0], P1o, F1o), st1, L1, d1)
    f2 = aol.make_filter(aol.make_tiler(arr_y, rep2, [n_in2], o2, P2, F2),
                         aol.make_tiler(arr_z, rep2, [n_out2], [0, 0], P2o, F2o), st2, L2, d2)
    out = torch.from_numpy(bg.copy()).cuda()
    aol.filter_chain_apply(f1, f2, torch.from_numpy(xh).cuda(), out=out)
    torch.cuda.synchronize()
    assert aol.last_kernel() in ("chain_kernel", "sep_chain_kernel", "sep_chain_jit")
    assert np.array_equal(out.cpu().numpy(), want)


def _eye(n, diag):
    return [[(diag[a] if a == j else 0) for j in range(n)] for a in range(n)]


@pytest.mark.parametrize("seed", range(48))
def test_random_separable_chains(orc, seed):
    """A row filter then a column filter with every parameter random: lead dims (planes), pattern lengths <= 16,
    paving steps (patterns overlapping, abutting or leaving gaps along the row; p2 <= L2 down the columns),
    origins wrapping the row several times and shifting the rows, 1-8 windows, divisors of either sign, column
    origins on and off the 16-byte grid.  Expected: the oracle's gather -> C task -> scatter, twice.  Even seeds
    run the kernel specialised at run time (NVRTC), odd seeds the statically compiled one."""
    rng = np.random.default_rng(7700 + seed)
    n = int(rng.integers(2, 5))
    lead = [int(rng.integers(1, 4)) for _ in range(n - 2)]
    HX, WX = int(rng.integers(1, 40)), int(rng.integers(4, 300))
    if seed % 3 == 0:
        WX = 4 * int(rng.integers(1, 75))

    def windows(L):
        ln = int(rng.integers(1, L + 1))
        nw = int(rng.integers(1, 9))
        return nw, ln, [int(rng.integers(0, L - ln + 1)) for _ in range(nw)], int(rng.choice([1, 2, 3, 6, 7, -1, -6, 100]))

    L1 = int(rng.integers(1, 17))
    p1 = int(rng.integers(1, 12))
    R1 = int(rng.integers(1, max(2, 2 * WX // p1)))
    nw1, len1, st1, d1 = windows(L1)
    o1 = [0] * (n - 2) + [int(rng.integers(-2 * HX, 2 * HX + 1)), int(rng.integers(-2 * WX, 2 * WX + 1))]
    if seed % 3 == 0:
        o1[-1] = 4 * int(rng.integers(-WX // 2, WX // 2 + 1))
    WY = nw1 * R1
    L2 = int(rng.integers(1, 17))
    p2 = int(rng.integers(1, L2 + 1))
    R2 = int(rng.integers(1, 12))
    nw2, len2, st2, d2 = windows(L2)
    o2 = [0] * (n - 2) + [int(rng.integers(-2 * HX, 2 * HX + 1)), 0]
    ones = [1] * (n - 2)
    e_col = [[0]] * (n - 1) + [[1]]
    e_row = [[0]] * (n - 2) + [[1], [0]]
    ax, ay, az = lead + [HX, WX], lead + [HX, WY], lead + [nw2 * R2, WY]
    t1i = (ax, lead + [HX, R1], [L1], o1, _eye(n, ones + [1, p1]), e_col)
    t1o = (ay, lead + [HX, R1], [nw1], [0] * n, _eye(n, ones + [1, nw1]), e_col)
    t2i = (ay, lead + [R2, WY], [L2], o2, _eye(n, ones + [p2, 1]), e_row)
    t2o = (az, lead + [R2, WY], [nw2], [0] * n, _eye(n, ones + [nw2, 1]), e_row)
    xh = np.asarray(rng.integers(-3000, 3000, size=ax)).astype(np.int32)
    y = orc.scatter(orc.make_tiler(*t1o), _task_c(orc.gather(orc.make_tiler(*t1i), xh), st1, len1, d1),
                    np.zeros(ay, np.int32))
    bg = np.full(az, -7, np.int32)
    want = orc.scatter(orc.make_tiler(*t2o), _task_c(orc.gather(orc.make_tiler(*t2i), y), st2, len2, d2), bg)
    f1 = aol.make_filter(aol.make_tiler(*t1i), aol.make_tiler(*t1o), st1, len1, d1)
    f2 = aol.make_filter(aol.make_tiler(*t2i), aol.make_tiler(*t2o), st2, len2, d2)
    out = torch.from_numpy(bg.copy()).cuda()
    jit = seed % 2 == 0
    aol._lib.lib().aol_debug_set_chain_jit(int(jit))
    try:
        aol.filter_chain_apply(f1, f2, torch.from_numpy(xh).cuda(), out=out)
        torch.cuda.synchronize()
        assert aol.last_kernel() == ("sep_chain_jit" if jit else "sep_chain_kernel")
    finally:
        aol._lib.lib().aol_debug_set_chain_jit(1)
    assert np.array_equal(out.cpu().numpy(), want)


def test_unfusable_chain_needs_a_workspace(orc):
    """f1's output tiler with the window digit HIGH (column-major outputs) cannot be fused: without a
    workspace the call names the reason; with one, two launches give the oracle's result."""
    P, H, W = 1, 18, 64
    xh = synth.frames(54, 0, 1, P, H, W, "uniform")[0]
    fh = aol.filter_preset(aol.FILTER_H, P, H, W)
    # H output tiler writing window k to plane-row block k: Y [P][3H][W/8], y = k*H + row, x = r
    fh2 = aol.make_filter(fh.in_, aol.make_tiler([P, 3 * H, W // 8], [P, H, W // 8], [3], [0, 0, 0],
                                                 [[1, 0, 0], [0, 1, 0], [0, 0, 1]], [[0], [H], [0]]), [0, 2, 5], 6, 6)
    fv = aol.filter_preset(aol.FILTER_V, P, 3 * H, W // 8)
    x = torch.from_numpy(xh).cuda()
    with pytest.raises(aol.AolError) as e:
        aol.filter_chain_apply(fh2, fv, x)
    assert e.value.status == aol._lib.E_WORKSPACE and "low digits" in str(e.value)
    ws = torch.empty((P, 3 * H, W // 8), dtype=torch.int32, device="cuda")
    z = aol.filter_chain_apply(fh2, fv, x, workspace=ws)
    torch.cuda.synchronize()
    y = aol.filter_apply(fh2, x)
    assert torch.equal(z, aol.filter_apply(fv, y))


@pytest.mark.parametrize("seed", range(24))
def test_random_single_row_and_column_filters(orc, seed):
    """aol_filter_apply on ONE row filter or ONE column filter with random parameters (lead dims, pattern lengths,
    paving steps, wrapping origins, windows, divisors of either sign): these run the separable chain kernel,
    specialised at run time, with an identity partner filter.  Expected: the oracle's gather -> C task -> scatter."""
    rng = np.random.default_rng(9100 + seed)
    n = int(rng.integers(2, 5))
    lead = [int(rng.integers(1, 4)) for _ in range(n - 2)]
    H, W = int(rng.integers(1, 40)), int(rng.integers(4, 1200))
    if seed % 3 == 0:
        W = 4 * int(rng.integers(1, 300))
    L = int(rng.integers(1, 17))
    ln = int(rng.integers(1, L + 1))
    nw = int(rng.integers(1, 9))
    st = [int(rng.integers(0, L - ln + 1)) for _ in range(nw)]
    d = int(rng.choice([1, 2, 3, 6, 7, -1, -6, 100]))
    ones = [1] * (n - 2)
    e_col = [[0]] * (n - 1) + [[1]]
    e_row = [[0]] * (n - 2) + [[1], [0]]
    row_filter = seed % 2 == 0
    if row_filter:
        p = int(rng.integers(1, 12))
        R = int(rng.integers(1, max(2, 2 * W // p)))
        o = [0] * (n - 2) + [int(rng.integers(-2 * H, 2 * H + 1)), int(rng.integers(-2 * W, 2 * W + 1))]
        ax, ay = lead + [H, W], lead + [H, nw * R]
        ti = (ax, lead + [H, R], [L], o, _eye(n, ones + [1, p]), e_col)
        to = (ay, lead + [H, R], [nw], [0] * n, _eye(n, ones + [1, nw]), e_col)
    else:
        p = int(rng.integers(1, L + 1))
        R = int(rng.integers(1, 12))
        o = [0] * (n - 2) + [int(rng.integers(-2 * H, 2 * H + 1)), 0]
        ax, ay = lead + [H, W], lead + [nw * R, W]
        ti = (ax, lead + [R, W], [L], o, _eye(n, ones + [p, 1]), e_row)
        to = (ay, lead + [R, W], [nw], [0] * n, _eye(n, ones + [nw, 1]), e_row)
    xh = np.asarray(rng.integers(-3000, 3000, size=ax)).astype(np.int32)
    bg = np.full(ay, -7, np.int32)
    want = orc.scatter(orc.make_tiler(*to), _task_c(orc.gather(orc.make_tiler(*ti), xh), st, ln, d), bg)
    f = aol.make_filter(aol.make_tiler(*ti), aol.make_tiler(*to), st, ln, d)
    out = torch.from_numpy(bg.copy()).cuda()
    aol.filter_apply(f, torch.from_numpy(xh).cuda(), out=out)
    torch.cuda.synchronize()
    assert aol.last_kernel() == "sep_chain_jit"
    assert np.array_equal(out.cpu().numpy(), want)
