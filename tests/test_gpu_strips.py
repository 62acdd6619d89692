"""Column strips of the fused TMA kernel (int32, W % 32 == 0): frames wider than one CTA's 992 consumer threads
(W > 7936, e.g. 8K DCI 8192) run as strips of <= 480 repetitions, each strip row loaded with the next
repetition's first 16 bytes (the pattern overlap; the row-wrapping strip's from column 0, Fig. 11's
toroidal '% W'), each band's output as 4 row segments.  Against the oracle, bit-exact, with checksums; the
flag AOL_FLAG_I32_STRIPS forces ~64-repetition strips at small widths, so several strips, a ragged last strip
and the wrap are exercised cheaply."""
import numpy as np
import pytest
import torch

import synth

pytestmark = pytest.mark.gpu

aol = pytest.importorskip("paper_conf_ipps_guortgbs11_b200")


def np_u64(t):
    return t.cpu().view(torch.int64).numpy().view(np.uint64)


def _check(orc, shape, opts, kind="signed", seed=41):
    N, C, H, W = shape
    xh = synth.frames(seed, 0, N, C, H, W, kind)
    zo, cso = orc.downscale_frame(xh, nthreads=16)
    x = torch.from_numpy(xh).cuda()
    z, cs = aol.downscale_frame(x, checksums=True, opts=opts)
    torch.cuda.synchronize()
    assert aol.last_kernel() == "fused_tma_kernel"
    assert np.array_equal(z.cpu().numpy(), zo), (shape, opts)
    assert np.array_equal(np_u64(cs), cso), (shape, opts)
    z2, _ = aol.downscale_frame(x, opts=opts)   # the instantiation without the checksum epilogue
    torch.cuda.synchronize()
    assert np.array_equal(z2.cpu().numpy(), zo), (shape, opts)


@pytest.mark.parametrize("shape", [(2, 3, 36, 1920), (1, 3, 27, 2048), (3, 1, 18, 1056), (1, 2, 9, 128),
                                   (2, 1, 45, 4096)])
def test_forced_strips(orc, shape):
    """1920: 4 strips of 64, the last 48 wide; 1056: strips of 64, 64, 4 (a 4-thread strip); 128: one strip."""
    N, C, H, W = shape
    o = {"kernel": 1, "flags": aol.FLAGS["I32_STRIPS"]}
    p = aol.downscale_frame_plan(N, C, H, W, opts=o)
    sr = p["block"] - 32
    nstrips = -(-(W // 8) // sr)
    assert p["kernel"] == 1 and sr % 32 == 0 and sr <= 64
    assert p["units"] % (N * C * nstrips) == 0
    _check(orc, shape, o)


@pytest.mark.parametrize("shape", [(1, 3, 18, 8192), (2, 1, 9, 7968), (1, 1, 27, 8000), (1, 1, 9, 15360)])
def test_wide_frames_take_strips(orc, shape):
    """Beyond W = 7936 the TMA kernel runs as strips by default (7968: 996 repetitions, just past one CTA)."""
    N, C, H, W = shape
    p = aol.downscale_frame_plan(N, C, H, W)
    assert p["kernel"] == 1 and p["block"] <= 512
    _check(orc, shape, None)


def test_8k_dci_frame(orc):
    """One 8K DCI frame (4320 x 8192, 3 channels) end to end."""
    _check(orc, (1, 3, 4320, 8192), None, kind="uniform", seed=43)


def test_wide_unaligned_width_uses_generic():
    """W % 32 != 0 beyond 7936: no strips (16-byte row segments need W % 32 == 0): the generic kernel."""
    assert aol.downscale_frame_plan(1, 1, 9, 8008)["kernel"] == 2
    assert aol.downscale_frame_plan(1, 1, 9, 8192, dtype=torch.uint8)["kernel"] == 2
