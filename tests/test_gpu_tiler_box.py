"""The round-2 wrapping-tiler kernels against the oracle: the footprint-staged box kernel (gathers and FAST
scatters whose array-side footprint per block of tiles is a dense box of whole rows) and the affine-piece kernel
(wrapping tilers split into a few affine sub-boxes of the index space, each walked with 16-byte vectors) -- the
paper's H / V input tilers (Fig. 10, reading Z1), d3's wrapping blockings, negative
coefficients, chunked blocks with a ragged last chunk, all element sizes.  Each case also checks which kernel ran
(aol_debug_last_kernel), so both paths are known to be exercised."""
import numpy as np
import pytest
import torch

pytestmark = pytest.mark.gpu

aol = pytest.importorskip("paper_conf_ipps_guortgbs11_b200")

DT = {1: torch.uint8, 2: torch.int16, 4: torch.int32, 8: torch.int64}
NP = {1: np.uint8, 2: np.int16, 4: np.int32, 8: np.int64}


def _arr(rng, shape, es):
    if es == 1:
        return rng.integers(0, 256, size=shape).astype(np.uint8)
    info = np.iinfo(NP[es])
    return rng.integers(info.min // 2, info.max // 2, size=shape, dtype=np.int64).astype(NP[es])


STAGED = ("tiler_box_kernel", "tiler_pieces_kernel")


def _run(orc, arr, rep, pat, origin, P, F, es=4, seed=0, scatter=None, expect_box=True, expect=STAGED,
         expect_scatter=None):
    rng = np.random.default_rng(seed)
    A = _arr(rng, arr, es)
    t = aol.make_tiler(arr, rep, pat, origin, P, F)
    to = orc.make_tiler(arr, rep, pat, origin, P, F)
    G = aol.tiler_gather(t, torch.from_numpy(A).cuda())
    torch.cuda.synchronize()
    kern = aol.last_kernel()
    want = orc.gather(to, A)
    assert np.array_equal(G.cpu().numpy(), want)
    if expect_box:
        assert kern in expect, kern
    if scatter:
        Gs = _arr(rng, tuple(rep) + tuple(pat), es)
        B0 = _arr(rng, arr, es)
        B = torch.from_numpy(B0).cuda()
        aol.tiler_scatter(t, torch.from_numpy(Gs).cuda(), B, mode="fast")
        torch.cuda.synchronize()
        if expect_box:
            assert aol.last_kernel() in (expect_scatter or expect), aol.last_kernel()
        assert np.array_equal(B.cpu().numpy(), orc.scatter(to, Gs, B0))
    return kern


@pytest.mark.parametrize("es", [1, 2, 4, 8])
@pytest.mark.parametrize("W", [64, 1920, 1000])
def test_h_input_tiler(orc, es, W):
    """Fig. 10's H input tiler over a stack of planes (wraps at the last repetition)."""
    H = 27
    _run(orc, [3, H, W], [3, H, W // 8], [11], [0, 0, 0], [[1, 0, 0], [0, 1, 0], [0, 0, 8]], [[0], [0], [1]], es=es)


@pytest.mark.parametrize("es", [1, 4])
def test_v_input_tiler(orc, es):
    """Reading Z1's V input tiler (pattern 12 every 9 rows, rows wrap at the last band) over 720-wide planes."""
    H, W = 36, 720
    _run(orc, [2, H, W], [2, H // 9, W], [12], [0, 0, 0], [[1, 0, 0], [0, 9, 0], [0, 0, 1]], [[0], [1], [0]], es=es)


@pytest.mark.parametrize("es", [1, 2, 4, 8])
@pytest.mark.parametrize("origin", [[0, -3, 5], [1, 7, -9], [0, 0, 3]])
def test_wrapping_blocking(orc, es, origin):
    """d3's 8x8 blocking, offset so tiles wrap in both image dims; gather and FAST scatter (exact cover)."""
    _run(orc, [3, 64, 256], [3, 8, 32], [8, 8], origin, [[1, 0, 0], [0, 8, 0], [0, 0, 8]],
         [[0, 0], [1, 0], [0, 1]], es=es, scatter=True)


def test_negative_coefficients(orc):
    """Reversed rows and columns (fitting -1, paving -8): signed steps, the box corner below the raw point."""
    _run(orc, [2, 32, 128], [2, 4, 16], [8, 8], [0, 5, -3], [[1, 0, 0], [0, -8, 0], [0, 0, 8]],
         [[0, 0], [-1, 0], [0, -1]], scatter=True)


def test_chunked_blocks_ragged_tail(orc):
    """Rows of 1000 elements: a block holds a chunk of the row dim (~12 rows), the last chunk is shorter;
    a pattern longer than the paving step (overlap) makes the box smaller than the tile block."""
    _run(orc, [50, 1000], [50, 125], [11], [3, -2], [[1, 0], [0, 8]], [[0], [1]])
    _run(orc, [50, 1000], [50, 125], [8], [-1, 4], [[1, 0], [0, 8]], [[0], [1]], scatter=True)


@pytest.mark.parametrize("seed", range(40))
def test_random_wrapping_descriptors(orc, seed):
    """Random block-diagonal wrapping tilers with long rows (box-eligible or not): always equal to the oracle;
    most take the box kernel."""
    rng = np.random.default_rng(9000 + seed)
    rows, cols = int(rng.integers(2, 40)), int(rng.integers(32, 600))
    pr, pc = int(rng.integers(1, 5)), int(rng.integers(1, 9))
    sr = int(rng.choice([pr, max(1, pr - 1), pr + 1]))
    sc = int(rng.choice([pc, max(1, pc - 2), pc + 2]))
    nr, nc = max(1, rows // sr), max(1, cols // sc)
    org = [int(rng.integers(-rows, rows)), int(rng.integers(-cols, cols))]
    sgn = int(rng.choice([1, -1]))
    es = int(rng.choice([1, 2, 4, 8]))
    _run(orc, [rows, cols], [nr, nc], [pr, pc], org, [[sr, 0], [0, sgn * sc]], [[1, 0], [0, sgn]], es=es,
         seed=seed, expect_box=False)


def test_box_path_taken_by_the_paper_tilers():
    """The d3 record's wrapping blocking runs as affine pieces (16-byte vectors; its array side is one element
    off the 16-byte grid and realigned across lanes), gather and FAST scatter; H_IN (11-element runs: no vectors)
    through the box kernel."""
    A = torch.zeros((2, 64, 256), dtype=torch.int32, device="cuda")
    t = aol.make_tiler([2, 64, 256], [2, 8, 32], [8, 8], [0, -3, 5], [[1, 0, 0], [0, 8, 0], [0, 0, 8]],
                       [[0, 0], [1, 0], [0, 1]])
    G = aol.tiler_gather(t, A)
    assert aol.last_kernel() == "tiler_pieces_kernel"
    aol.tiler_scatter(t, G, A, mode="fast")
    assert aol.last_kernel() == "tiler_pieces_kernel"
    X = torch.zeros((2, 36, 1920), dtype=torch.int32, device="cuda")
    th = aol.make_tiler([2, 36, 1920], [2, 36, 240], [11], [0, 0, 0], [[1, 0, 0], [0, 1, 0], [0, 0, 8]],
                        [[0], [0], [1]])
    aol.tiler_gather(th, X)
    assert aol.last_kernel() == "tiler_box_kernel"
    torch.cuda.synchronize()


@pytest.mark.parametrize("es", [1, 2, 4, 8])
@pytest.mark.parametrize("origin", [[0, -3, 5], [2, 13, -7], [0, 0, 1], [1, -8, 0]])
def test_affine_pieces(orc, es, origin):
    """Blockings shifted to wrap in one or both image dims split into affine pieces: gather and FAST scatter
    against the oracle.  Both take the piece kernel whenever a tile row holds whole 16-byte vectors (es >= 2;
    array-side starts off the 16-byte grid are realigned across neighbouring lanes), else the box kernel."""
    _run(orc, [3, 64, 256], [3, 8, 32], [8, 8], origin, [[1, 0, 0], [0, 8, 0], [0, 0, 8]],
         [[0, 0], [1, 0], [0, 1]], es=es, scatter=True, expect=("tiler_pieces_kernel",) if es >= 2 else STAGED)


@pytest.mark.parametrize("seed", range(48))
def test_affine_pieces_random_blockings(orc, seed):
    """Random blockings with random origins (on and off the 16-byte grid) and sizes, 2-, 4- and 8-byte
    elements: rows of tiles that end inside a warp, warps that straddle two rows."""
    rng = np.random.default_rng(9500 + seed)
    es = int(rng.choice([2, 4, 8]))
    br, bc = int(rng.choice([1, 2, 4, 8])), int(rng.choice([4, 8, 16]))
    nr, nc = int(rng.integers(1, 9)), int(rng.integers(2, 24))
    arr = [2, br * nr, bc * nc]
    org = [0, int(rng.integers(-br * nr, br * nr)), int(rng.integers(-bc * nc, bc * nc))]
    _run(orc, arr, [2, nr, nc], [br, bc], org, [[1, 0, 0], [0, br, 0], [0, 0, bc]], [[0, 0], [1, 0], [0, 1]],
         es=es, seed=seed, scatter=True, expect_box=False)
