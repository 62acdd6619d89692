"""Persistent launch plans (aol_frame_plan_*): validation, planning and the TMA descriptor resolved once, each
call only the launches.  Against the oracle for every input type, across repeated launches, with new input
contents between launches, without checksums, and for a plan that falls back to the generic kernel."""
import ctypes

import numpy as np
import pytest
import torch

import synth

pytestmark = pytest.mark.gpu

aol = pytest.importorskip("paper_conf_ipps_guortgbs11_b200")


def np_u64(t):
    return t.cpu().view(torch.int64).numpy().view(np.uint64)


@pytest.mark.parametrize("shape", [(1, 3, 1080, 1920), (3, 3, 36, 128), (2, 1, 27, 720), (5, 3, 288, 352)])
@pytest.mark.parametrize("dtype", [torch.int32, torch.uint8])
def test_plan_matches_oracle_over_repeated_launches(orc, shape, dtype):
    N, C, H, W = shape
    xh = synth.frames(31, 0, N, C, H, W, "uniform")
    zo, cso = orc.downscale_frame(xh, nthreads=8)
    x = torch.from_numpy(xh.astype(np.uint8) if dtype == torch.uint8 else xh).cuda()
    plan = aol.FramePlan(x, checksums=True)
    assert plan.info()["kernel"] == 1
    for _ in range(4):   # every launch re-zeroes and recomputes the checksums
        z, cs = plan.launch()
        torch.cuda.synchronize()
        assert aol.last_kernel() == "fused_tma_kernel"
        assert np.array_equal(z.cpu().numpy(), zo)
        assert np.array_equal(np_u64(cs), cso)
    # new contents in the same buffers
    xh2 = synth.frames(32, 0, N, C, H, W, "dark")
    x.copy_(torch.from_numpy(xh2.astype(np.uint8) if dtype == torch.uint8 else xh2))
    zo2, cso2 = orc.downscale_frame(xh2, nthreads=8)
    z, cs = plan.launch()
    torch.cuda.synchronize()
    assert np.array_equal(z.cpu().numpy(), zo2) and np.array_equal(np_u64(cs), cso2)
    plan.close()


@pytest.mark.parametrize("out_dtype", [torch.int32, torch.int16])
def test_plan_packed_pixels_and_int16(orc, out_dtype):
    N, H, W = 2, 36, 256
    xp = synth.frames(33, 0, N, 3, H, W, "uniform")
    packed = torch.from_numpy(np.ascontiguousarray(np.transpose(xp, (0, 2, 3, 1))).astype(np.uint8)).cuda()
    zo, cso = orc.downscale_frame(xp, nthreads=8)
    plan = aol.FramePlan(packed, checksums=True, packed=True, out_dtype=out_dtype)
    for _ in range(2):
        z, cs = plan.launch()
        torch.cuda.synchronize()
        assert np.array_equal(z.cpu().numpy().astype(np.int32), zo) and np.array_equal(np_u64(cs), cso)
    x8 = torch.from_numpy(xp.astype(np.uint8)).cuda()
    plan2 = aol.FramePlan(x8, checksums=True, out_dtype=out_dtype)
    z, cs = plan2.launch()
    torch.cuda.synchronize()
    assert np.array_equal(z.cpu().numpy().astype(np.int32), zo) and np.array_equal(np_u64(cs), cso)


def test_plan_without_checksums_and_generic_fallback(orc):
    N, C, H, W = 2, 3, 18, 64
    xh = synth.frames(34, 0, N, C, H, W, "signed")
    zo, cso = orc.downscale_frame(xh, nthreads=8)
    x = torch.from_numpy(xh).cuda()
    p = aol.FramePlan(x)
    z, cs = p.launch()
    torch.cuda.synchronize()
    assert cs is None and np.array_equal(z.cpu().numpy(), zo)
    g = aol.FramePlan(x, checksums=True, opts={"kernel": 2})
    assert g.info()["kernel"] == 2
    z, cs = g.launch()
    torch.cuda.synchronize()
    assert np.array_equal(z.cpu().numpy(), zo) and np.array_equal(np_u64(cs), cso)


def test_plan_errors():
    L = aol._lib.lib()
    h = ctypes.c_void_p(0)
    x = torch.zeros((1, 3, 18, 60), dtype=torch.int32, device="cuda")   # W % 8 != 0
    z = torch.zeros((1, 3, 8, 21), dtype=torch.int32, device="cuda")
    st = L.aol_frame_plan_create(ctypes.c_void_p(x.data_ptr()), aol._lib.I32, ctypes.c_void_p(z.data_ptr()),
                                 aol._lib.I32, 1, 3, 18, 60, None, ctypes.byref(h))
    assert st == aol._lib.E_SHAPE and not h.value
    assert L.aol_frame_plan_launch(None, None, None) == aol._lib.E_INVALID
    assert L.aol_frame_plan_destroy(None) == aol._lib.OK
    x = torch.zeros((1, 3, 18, 64), dtype=torch.int32, device="cuda")
    p = aol.FramePlan(x, checksums=True)
    buf = torch.zeros(2, dtype=torch.int64, device="cuda")
    assert L.aol_frame_plan_launch(p._h, ctypes.c_void_p(buf.data_ptr() + 4), None) == aol._lib.E_ALIGN
    L.aol_debug_fail_next_launches(1)
    with pytest.raises(aol.AolError):
        p.launch()
    p.close()
