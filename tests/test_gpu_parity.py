"""GPU parity: every CUDA entry point against the CPU oracle, bit-exact.

The arithmetic is integer (Fig. 5, SaC `int`), so the bar is exact equality
(north_star: "bit-exact if the filter arithmetic is integer").  Inputs come from
synth/ (numpy) for the oracle side; the GPU side receives the same arrays, or
generates them with its own counter-based generator (checked equal first).
"""
import os

import numpy as np
import pytest
import torch

import bruteforce as bf
import synth

pytestmark = pytest.mark.gpu

aol = pytest.importorskip("paper_conf_ipps_guortgbs11_b200")


@pytest.fixture(scope="module", autouse=True)
def cuda_dev():
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    torch.cuda.set_device(0)
    aol.lib()
    yield


def np_u64(t: torch.Tensor) -> np.ndarray:
    return t.cpu().view(torch.int64).numpy().view(np.uint64)


# -------------------------------------------------------------- generator

@pytest.mark.parametrize("kind", ["uniform", "dark", "signed", "ramp", "constant"])
def test_synth_generator_matches_numpy(kind):
    a = aol.synth_frames(77, 5, 3, 3, 18, 64, kind, value=-11).cpu().numpy()
    b = synth.frames(77, 5, 3, 3, 18, 64, kind, value=-11)
    assert np.array_equal(a, b)


def test_synth_generator_u8():
    a = aol.synth_frames(3, 2, 2, 3, 9, 32, "uniform", dtype=torch.uint8).cpu().numpy()
    assert np.array_equal(a.astype(np.int32), synth.frames(3, 2, 2, 3, 9, 32, "uniform"))


# -------------------------------------------------------------- fused kernel

SHAPES = [
    (1, 3, 1080, 1920),   # d1: one HD frame (Fig. 2)
    (2, 3, 288, 352),     # CIF (Section III)
    (1, 1, 9, 32),        # one band: the V halo wraps onto its own rows
    (3, 2, 27, 64),
    (2, 3, 36, 256),
    (1, 2, 45, 3840),     # 4K width (480 reps, 15 consumer warps)
]
KINDS = ["uniform", "dark", "signed", "ramp", "constant"]


def run_oracle(orc, xh):
    return orc.downscale_frame(xh, nthreads=8)


@pytest.mark.parametrize("shape", SHAPES)
@pytest.mark.parametrize("kernel", [1, 2])
def test_fused_vs_oracle(orc, shape, kernel):
    N, C, H, W = shape
    for i, kind in enumerate(KINDS if H * W <= 64 * 1024 else ["uniform", "dark"]):
        xh = synth.frames(100 + i, 0, N, C, H, W, kind, value=-77)
        zo, cso = run_oracle(orc, xh)
        x = torch.from_numpy(xh).cuda()
        z, cs = aol.downscale_frame(x, checksums=True, opts={"kernel": kernel})
        torch.cuda.synchronize()
        got = z.cpu().numpy()
        assert np.array_equal(got, zo), (shape, kind, kernel, np.argwhere(got != zo)[:5])
        assert np.array_equal(np_u64(cs), cso), (shape, kind, kernel)


@pytest.mark.parametrize("opts", [
    {"bands_per_unit": 1}, {"bands_per_unit": 2}, {"bands_per_unit": 7}, {"bands_per_unit": 40},
    {"stages": 2}, {"stages": 3, "bands_per_unit": 5}, {"ctas_per_sm": 2}, {"ctas_per_sm": 2, "stages": 2},
    {"flags": 64}, {"flags": 64, "bands_per_unit": 1, "stages": 2}, {"ctas_per_sm": 4}, {"ctas_per_sm": 8, "stages": 2},
    {"flags": 128}, {"flags": 1024},
])
def test_fused_launch_options(orc, opts):
    """Unit boundaries, ring wrap-around and CTA residency do not change results."""
    N, C, H, W = 3, 3, 117, 512
    xh = synth.frames(9, 0, N, C, H, W, "uniform")
    zo, cso = run_oracle(orc, xh)
    x = torch.from_numpy(xh).cuda()
    o = dict(opts, kernel=1)
    z, cs = aol.downscale_frame(x, checksums=True, opts=o)
    plan = aol.downscale_frame_plan(N, C, H, W, opts=o)
    assert plan["kernel"] == 1
    torch.cuda.synchronize()
    assert np.array_equal(z.cpu().numpy(), zo)
    assert np.array_equal(np_u64(cs), cso)


@pytest.mark.parametrize("shape", [(1, 1, 9, 8), (2, 3, 18, 40), (1, 3, 36, 1000), (2, 3, 27, 720), (1, 2, 18, 2040),
                                   (1, 3, 18, 24), (2, 1, 27, 1448)])
def test_unaligned_width_shapes(orc, shape):
    """int32, W % 32 != 0 (e.g. 720-wide SD frames): the TMA kernel on linear rows (1-D bulk copies of the
    row triple, lane-rotated LDS.128), against the oracle and the generic kernel, with and without
    checksums."""
    N, C, H, W = shape
    xh = synth.frames(5, 0, N, C, H, W, "signed")
    zo, cso = run_oracle(orc, xh)
    assert aol.downscale_frame_plan(N, C, H, W)["kernel"] == 1
    x = torch.from_numpy(xh).cuda()
    for opts in (None, {"kernel": 1, "ctas_per_sm": 2, "bands_per_unit": 1},
                 {"kernel": 1, "ctas_per_sm": 3, "stages": 2}, {"kernel": 2}):
        z, cs = aol.downscale_frame(x, checksums=True, opts=opts)
        z2, _ = aol.downscale_frame(x, opts=opts)
        torch.cuda.synchronize()
        assert np.array_equal(z.cpu().numpy(), zo), opts
        assert np.array_equal(z2.cpu().numpy(), zo), opts
        assert np.array_equal(np_u64(cs), cso), opts


@pytest.mark.parametrize("shape", [(2, 3, 36, 128), (1, 3, 27, 1920), (1, 2, 18, 3840), (2, 1, 27, 720),
                                   (1, 1, 9, 4008)])
def test_row_and_triple_stages(orc, shape):
    """int32 ring stages of one row (AOL_FLAG_ROW_STAGES = 512; the default for W > 3271) and of one row
    triple (AOL_FLAG_TRIPLE_STAGES = 1024), on both smem layouts (+ AOL_FLAG_I32_LINEAR = 128) and with small
    rings: identical integers."""
    N, C, H, W = shape
    xh = synth.frames(8, 0, N, C, H, W, "signed")
    zo, cso = run_oracle(orc, xh)
    x = torch.from_numpy(xh).cuda()
    for flags in (512, 1024, 512 | 128, 1024 | 128):
        for extra in ({}, {"stages": 2, "bands_per_unit": 1}, {"ctas_per_sm": 2, "stages": 3}):
            o = dict(extra, kernel=1, flags=flags)
            try:
                z, cs = aol.downscale_frame(x, checksums=True, opts=o)
            except aol.AolError:
                assert W > 3271 and flags & 1024   # a triple ring may not fit next to 2 CTAs of wide frames
                continue
            torch.cuda.synchronize()
            assert np.array_equal(z.cpu().numpy(), zo), o
            assert np.array_equal(np_u64(cs), cso), o


@pytest.mark.parametrize("shape", [(2, 3, 36, 128), (1, 3, 27, 1920), (3, 1, 18, 352), (1, 1, 9, 32)])
def test_linear_rows_forced(orc, shape):
    """AOL_FLAG_I32_LINEAR (128): linear rows by 1-D bulk copies even when W % 32 == 0 (A/B against the
    default SWIZZLE_128B tensor loads): same integers."""
    N, C, H, W = shape
    xh = synth.frames(6, 0, N, C, H, W, "uniform")
    zo, cso = run_oracle(orc, xh)
    x = torch.from_numpy(xh).cuda()
    for opts in ({"kernel": 1, "flags": 128}, {"kernel": 1, "flags": 128, "ctas_per_sm": 2, "bands_per_unit": 2}):
        z, cs = aol.downscale_frame(x, checksums=True, opts=opts)
        torch.cuda.synchronize()
        assert np.array_equal(z.cpu().numpy(), zo), opts
        assert np.array_equal(np_u64(cs), cso), opts


@pytest.mark.parametrize("shape", [(1, 1, 9, 2056), (1, 2, 18, 4008), (1, 1, 9, 7432)])
def test_wide_unaligned_shapes(orc, shape):
    """int32, W % 32 != 0 and W > 2048: linear rows (one-row ring stages beyond W = 3271), against the
    oracle and the generic fused kernel; unknown flag bits (the removed SWIZZLE_32B layout's 256) are refused."""
    N, C, H, W = shape
    xh = synth.frames(5, 0, N, C, H, W, "signed")
    zo, cso = run_oracle(orc, xh)
    assert aol.downscale_frame_plan(N, C, H, W)["kernel"] == 1
    x = torch.from_numpy(xh).cuda()
    for opts in (None, {"kernel": 2}):
        z, cs = aol.downscale_frame(x, checksums=True, opts=opts)
        torch.cuda.synchronize()
        assert np.array_equal(z.cpu().numpy(), zo), opts
        assert np.array_equal(np_u64(cs), cso), opts
    with pytest.raises(aol.AolError):
        aol.downscale_frame(x, opts={"kernel": 1, "flags": 256})
    with pytest.raises(aol.AolError):
        aol.downscale_frame_plan(N, C, H, W, opts={"flags": 2})


@pytest.mark.parametrize("shape,kernel", [
    ((2, 3, 36, 128), 1), ((1, 3, 1080, 1920), 1), ((3, 3, 288, 352), 1), ((1, 1, 9, 16), 1),
    ((2, 2, 27, 3840), 1), ((1, 2, 18, 40), 2), ((2, 3, 36, 128), 2),
])
@pytest.mark.parametrize("kind", ["uniform", "dark", "ramp"])
def test_fused_u8_input(orc, shape, kernel, kind):
    """8-bit samples give the same integers, hence the same outputs (NEXT row f1)."""
    N, C, H, W = shape
    if kind == "ramp" and W > 256:
        kind = "uniform"
    xh = synth.frames(21, 0, N, C, H, W, kind)
    zo, cso = run_oracle(orc, xh)
    x8 = torch.from_numpy(xh.astype(np.uint8)).cuda()
    plan = aol.downscale_frame_plan(N, C, H, W, dtype=torch.uint8, opts={"kernel": kernel})
    assert plan["kernel"] == kernel
    z, cs = aol.downscale_frame(x8, checksums=True, opts={"kernel": kernel})
    torch.cuda.synchronize()
    assert np.array_equal(z.cpu().numpy(), zo)
    assert np.array_equal(np_u64(cs), cso)


def test_fused_u8_launch_options(orc):
    xh = synth.frames(22, 0, 3, 3, 117, 512, "uniform")
    zo, cso = run_oracle(orc, xh)
    x8 = torch.from_numpy(xh.astype(np.uint8)).cuda()
    for o in ({"bands_per_unit": 1}, {"stages": 2}, {"ctas_per_sm": 2}, {"ctas_per_sm": 4}, {"flags": 64},
              {"flags": 96, "bands_per_unit": 3}):
        z, cs = aol.downscale_frame(x8, checksums=True, opts=dict(o, kernel=1))
        torch.cuda.synchronize()
        assert np.array_equal(z.cpu().numpy(), zo), o
        assert np.array_equal(np_u64(cs), cso), o


@pytest.mark.parametrize("W", [1024, 1040, 1920, 2048, 3968])
def test_fused_u8_two_reps_per_thread(orc, W):
    """uint8 frames >= 1024 wide run two H repetitions per consumer thread (one LDS.128 for 16 samples);
    AOL_FLAG_U8_ONE_REP (32) forces one.  Both against the oracle, incl. W % 128 != 0 (1-D bulk copies),
    warps with idle lanes (W = 1040: 65 threads) and the row-wrapping repetition pair; with and without
    the checksum epilogue."""
    N, C, H = 2, 3, 36
    xh = synth.frames(23, 0, N, C, H, W, "uniform")
    xh[0, 1] = synth.frames(24, 0, 1, 1, H, W, "dark")[0, 0]   # negative V sums on one plane
    zo, cso = run_oracle(orc, xh)
    x8 = torch.from_numpy(xh.astype(np.uint8)).cuda()
    for flags in (0, 32, 64):
        o = {"kernel": 1, "flags": flags}
        plan = aol.downscale_frame_plan(N, C, H, W, dtype=torch.uint8, opts=o)
        z, cs = aol.downscale_frame(x8, checksums=True, opts=o)
        z2, _ = aol.downscale_frame(x8, opts=o)
        torch.cuda.synchronize()
        assert np.array_equal(z.cpu().numpy(), zo), flags
        assert np.array_equal(z2.cpu().numpy(), zo), flags
        assert np.array_equal(np_u64(cs), cso), flags
        # block = consumer threads (W/8 repetitions / reps-per-thread, whole warps) + 1 producer warp
        kr = 1 if flags == 32 else 2
        assert plan["block"] == ((W // 8 // kr) + 31) // 32 * 32 + 32, (flags, plan)


@pytest.mark.parametrize("shape,kernel", [
    ((1, 3, 1080, 1920), 1), ((2, 3, 288, 352), 1), ((2, 3, 36, 1040), 1), ((2, 3, 36, 128), 1),
    ((1, 2, 18, 40), 2), ((2, 3, 36, 128), 2), ((1, 3, 2160, 3840), 1), ((2, 1, 54, 4096), 1), ((3, 3, 90, 1920), 1),
])
def test_fused_u8_int16_output(orc, shape, kernel):
    """NEXT row f1's int16 output option: 8-bit samples give outputs in [-5, 255]; stored as int16 they are
    the oracle's integers, and the checksums equal the int32-output run's."""
    N, C, H, W = shape
    xh = synth.frames(25, 0, N, C, H, W, "uniform")
    xh[0, 0] = synth.frames(26, 0, 1, 1, H, W, "dark")[0, 0]   # negative outputs on one plane
    zo, cso = run_oracle(orc, xh)
    x8 = torch.from_numpy(xh.astype(np.uint8)).cuda()
    opts = {"kernel": kernel}
    plan = aol.downscale_frame_plan(N, C, H, W, dtype=torch.uint8, opts=opts, out_dtype=torch.int16)
    assert plan["kernel"] == kernel
    z, cs = aol.downscale_frame(x8, checksums=True, opts=opts, out_dtype=torch.int16)
    z2, _ = aol.downscale_frame(x8, opts=opts, out_dtype=torch.int16)
    torch.cuda.synchronize()
    if kernel == 1 and W in (1920, 3840, 4096):
        # the halo-last multi-CTA instantiations: 4 CTAs/SM of 160 threads (HD), 2 of 288 (4K, 4096)
        assert plan["ctas_per_sm"] == (4 if W == 1920 else 2), plan
    assert z.dtype == torch.int16
    assert np.array_equal(z.cpu().numpy().astype(np.int32), zo)
    assert np.array_equal(z2.cpu().numpy().astype(np.int32), zo)
    assert np.array_equal(np_u64(cs), cso)


def test_int16_output_needs_uint8_input():
    x = torch.zeros((1, 1, 9, 32), dtype=torch.int32, device="cuda")
    with pytest.raises(aol.AolError) as e:
        aol.downscale_frame(x, out_dtype=torch.int16)
    assert e.value.status == aol._lib.E_DTYPE


def test_no_checksum_and_zero_frames(orc):
    xh = synth.frames(1, 0, 1, 3, 18, 64)
    z, cs = aol.downscale_frame(torch.from_numpy(xh).cuda())
    assert cs is None
    assert np.array_equal(z.cpu().numpy(), run_oracle(orc, xh)[0])
    x0 = torch.empty((0, 3, 18, 64), dtype=torch.int32, device="cuda")
    z0, _ = aol.downscale_frame(x0, checksums=True)
    assert z0.shape == (0, 3, 8, 24)


# -------------------------------------------------------------- unfused stages

@pytest.mark.parametrize("shape", [(3, 1080, 1920), (2, 288, 352), (1, 9, 8), (4, 27, 1000)])
def test_downscale_h_v_vs_oracle(orc, shape):
    P, H, W = shape
    xh = synth.frames(31, 0, 1, P, H, W, "signed")[0] >> 4
    yo = orc.downscale_h(xh)
    x = torch.from_numpy(xh).cuda()
    y = aol.downscale_h(x)
    torch.cuda.synchronize()
    assert np.array_equal(y.cpu().numpy(), yo)
    zo = orc.downscale_v(yo)
    z = aol.downscale_v(y)
    torch.cuda.synchronize()
    assert np.array_equal(z.cpu().numpy(), zo)
    # cross-path: fused == v(h(x))
    zf, _ = aol.downscale_frame(x.unsqueeze(0))
    assert torch.equal(zf[0], z)


def test_frame_checksum_kernel(orc):
    z = torch.from_numpy(synth.frames(8, 0, 5, 3, 40, 30, "signed")).cuda()
    cs = aol.frame_checksum(z)
    assert np.array_equal(np_u64(cs), orc.checksum(z.cpu().numpy()))


# -------------------------------------------------------------- generic tilers

@pytest.mark.parametrize("seed", range(1000))   # seeds 0..999
def test_tiler_gather_scatter_vs_oracle(orc, seed):
    rng = np.random.default_rng(5000 + seed)
    d = bf.random_descriptor(rng)
    dtype = [np.uint8, np.int16, np.int32, np.int64][seed % 4]
    tdt = {np.uint8: torch.uint8, np.int16: torch.int16, np.int32: torch.int32, np.int64: torch.int64}[dtype]
    A = np.asarray(rng.integers(0, 120, size=d["array_shape"])).astype(dtype)
    ot = orc.make_tiler(d["array_shape"], d["rep_shape"], d["pattern_shape"], d["origin"], d["paving"],
                        d["fitting"])
    gt = aol.make_tiler(d["array_shape"], d["rep_shape"], d["pattern_shape"], d["origin"], d["paving"],
                        d["fitting"])
    Go = orc.gather(ot, A)
    G = aol.tiler_gather(gt, torch.from_numpy(A).cuda())
    torch.cuda.synchronize()
    assert np.array_equal(G.cpu().numpy(), Go)
    # SEQUENTIAL scatter == Fig. 6 oracle (collisions: last writer wins)
    Gs = np.asarray(rng.integers(0, 120, size=Go.shape)).astype(dtype)
    bg = np.asarray(rng.integers(0, 120, size=A.shape)).astype(dtype)
    So = orc.scatter(ot, Gs, bg)
    arr = torch.from_numpy(bg.copy()).cuda()
    aol.tiler_scatter(gt, torch.from_numpy(Gs).cuda().reshape(G.shape), arr, mode="sequential")
    torch.cuda.synchronize()
    assert np.array_equal(arr.cpu().numpy(), So)
    if aol.tiler_is_injective(gt):
        arr2 = torch.from_numpy(bg.copy()).cuda()
        aol.tiler_scatter(gt, torch.from_numpy(Gs).cuda().reshape(G.shape), arr2, mode="fast")
        torch.cuda.synchronize()
        assert np.array_equal(arr2.cpu().numpy(), So)


def test_tiler_d3_perf_instance_full_size(orc):
    """SURVEY 8(d) d3 at the size tools/bench_configs.py times: array {64,1024,1024} int32 (256 MB), rep
    {64,128,128}, pattern {8,8}, P = diag(1,8,8), F = [[0,0],[1,0],[0,1]] -- gather element by element
    against the C oracle, and the FAST scatter of the tiles back into a zeroed array rebuilds the input
    (the tiler is a bijection onto the array)."""
    arr, rep, pat = [64, 1024, 1024], [64, 128, 128], [8, 8]
    P, F = [[1, 0, 0], [0, 8, 0], [0, 0, 8]], [[0, 0], [1, 0], [0, 1]]
    A = synth.frames(77, 0, 1, 64, 1024, 1024, "signed")[0]
    ot = orc.make_tiler(arr, rep, pat, [0, 0, 0], P, F)
    gt = aol.make_tiler(arr, rep, pat, [0, 0, 0], P, F)
    Ad = torch.from_numpy(A).cuda()
    G = aol.tiler_gather(gt, Ad)
    torch.cuda.synchronize()
    assert np.array_equal(G.cpu().numpy(), orc.gather(ot, A))
    back = torch.zeros_like(Ad)
    aol.tiler_scatter(gt, G, back, mode="fast")
    torch.cuda.synchronize()
    assert torch.equal(back, Ad)


LINEAR_TILERS = [
    # (array, rep, pattern, origin, paving, fitting): no coordinate wraps -> affine offsets
    ([64, 96], [8, 12], [8, 8], [0, 0], [[8, 0], [0, 8]], [[1, 0], [0, 1]]),           # 8x8 blocks (vector path)
    ([4, 32, 64], [4, 4, 8], [8, 8], [0, 0, 0], [[1, 0, 0], [0, 8, 0], [0, 0, 8]], [[0, 0], [1, 0], [0, 1]]),
    ([50, 40], [6, 5], [3, 7], [2, 1], [[8, 0], [0, 8]], [[1, 0], [0, 1]]),             # offset, odd pattern
    ([37, 23], [23], [37], [0, 0], [[0], [1]], [[1], [0]]),                            # transpose column gather
    ([128], [15], [16], [0], [[8]], [[1]]),                                           # overlapping windows
]


@pytest.mark.parametrize("case", range(len(LINEAR_TILERS)))
@pytest.mark.parametrize("dtype", [np.uint8, np.int16, np.int32, np.int64])
def test_tiler_linear_paths(orc, case, dtype):
    """Affine (non-wrapping) tilers take the linear kernels, incl. 16-byte vector accesses."""
    arr, rep, pat, o, P, F = LINEAR_TILERS[case]
    rng = np.random.default_rng(case)
    A = np.asarray(rng.integers(0, 100, size=arr)).astype(dtype)
    ot = orc.make_tiler(arr, rep, pat, o, P, F)
    gt = aol.make_tiler(arr, rep, pat, o, P, F)
    Go = orc.gather(ot, A)
    G = aol.tiler_gather(gt, torch.from_numpy(A).cuda())
    torch.cuda.synchronize()
    assert np.array_equal(G.cpu().numpy(), Go)
    Gs = np.asarray(rng.integers(0, 100, size=Go.shape)).astype(dtype)
    bg = np.asarray(rng.integers(0, 100, size=A.shape)).astype(dtype)
    So = orc.scatter(ot, Gs, bg)
    for mode in (["fast", "sequential"] if aol.tiler_is_injective(gt) else ["sequential"]):
        arr_t = torch.from_numpy(bg.copy()).cuda()
        aol.tiler_scatter(gt, torch.from_numpy(Gs).cuda(), arr_t, mode=mode)
        torch.cuda.synchronize()
        assert np.array_equal(arr_t.cpu().numpy(), So), mode


@pytest.mark.parametrize("shape", [(3, 1080, 1920), (4, 288, 352), (2, 9, 8), (3, 27, 1000)])
def test_filter_presets_vs_oracle(orc, shape):
    """f3: the run-time generic repetition (gather + task + scatter in one kernel) with the paper's
    H and V descriptions equals the oracle's three-step filters."""
    P, H, W = shape
    xh = synth.frames(41, 0, 1, P, H, W, "signed")[0] >> 6
    x = torch.from_numpy(xh).cuda()
    y = aol.filter_apply(aol.filter_preset(aol.FILTER_H, P, H, W), x)
    torch.cuda.synchronize()
    yo = orc.downscale_h(xh)
    assert np.array_equal(y.cpu().numpy(), yo)
    z = aol.filter_apply(aol.filter_preset(aol.FILTER_V, P, H, 3 * W // 8), y)
    torch.cuda.synchronize()
    assert np.array_equal(z.cpu().numpy(), orc.downscale_v(yo))
    # cross-path: generic run-time repetitions == the specialised fused kernel
    zf, _ = aol.downscale_frame(x.unsqueeze(1))
    assert torch.equal(zf[:, 0], z)


@pytest.mark.parametrize("seed", range(60))
def test_filter_random_tilers_vs_oracle(orc, seed):
    """f3 with random input/output tilers and the paper's task windows: equal to the oracle's
    gather -> task_h/task_v -> scatter (Fig. 4, 5, 6) on the same descriptors."""
    rng = np.random.default_rng(900 + seed)
    n_in, starts, task = ((11, [0, 2, 5], orc.task_h) if seed % 2 == 0 else (12, [0, 2, 4, 6], orc.task_v))
    n_out = len(starts)
    ra = int(rng.integers(1, 4))
    rep = [int(rng.integers(1, 6)) for _ in range(int(rng.integers(1, 3)))]
    arr_in = [int(rng.integers(2, 17)) for _ in range(ra)]
    o_in = [int(rng.integers(-2 * s, 2 * s + 1)) for s in arr_in]
    P_in = [[int(rng.integers(-4, 10)) for _ in rep] for _ in range(ra)]
    F_in = [[int(rng.integers(-4, 10))] for _ in range(ra)]
    # injective output tiler: array [prod(rep), n_out], row = flattened rep, col = k
    nrep = int(np.prod(rep))
    arr_out = [nrep, n_out]
    strides = [int(np.prod(rep[j + 1:])) for j in range(len(rep))]
    P_out = [strides, [0] * len(rep)]
    F_out = [[0], [1]]
    xh = np.asarray(rng.integers(-300, 300, size=arr_in)).astype(np.int32)
    oti = orc.make_tiler(arr_in, rep, [n_in], o_in, P_in, F_in)
    oto = orc.make_tiler(arr_out, rep, [n_out], [0, 0], P_out, F_out)
    bg = np.full(arr_out, -99, np.int32)
    want = orc.scatter(oto, task(orc.gather(oti, xh)), bg)
    f = aol.make_filter(aol.make_tiler(arr_in, rep, [n_in], o_in, P_in, F_in),
                        aol.make_tiler(arr_out, rep, [n_out], [0, 0], P_out, F_out), starts, 6, 6)
    out = torch.from_numpy(bg.copy()).cuda()
    aol.filter_apply(f, torch.from_numpy(xh).cuda(), out=out)
    torch.cuda.synchronize()
    assert np.array_equal(out.cpu().numpy(), want)


def _task_c(G, starts, L, d):
    """Fig. 5's task generalised (windows at `starts`, length L, divisor d): tmp/d - tmp%d in C semantics."""
    S = np.stack([G[..., s:s + L].astype(np.int64).sum(-1) for s in starts], -1)
    q = np.sign(S) * np.sign(d) * (np.abs(S) // abs(d))
    return (q - (S - q * d)).astype(np.int32)


@pytest.mark.parametrize("seed", range(40))
def test_filter_random_windows_and_divisors(orc, seed):
    """f3 beyond the paper's two filters: random pattern sizes (1..20: register-pattern kernel up to 16,
    per-window kernel above), window sets and divisors of both signs.  Expected = oracle gather -> the
    task written out with C division -> oracle scatter."""
    rng = np.random.default_rng(1300 + seed)
    n_in = int(rng.integers(1, 21))
    L = int(rng.integers(1, n_in + 1))
    n_out = int(rng.integers(1, 9))
    starts = [int(rng.integers(0, n_in - L + 1)) for _ in range(n_out)]
    d = int(rng.choice([1, 2, 3, 5, 6, 7, 9, 100, 12345, -1, -3, -6, -77, (1 << 30) + 3]))
    contiguous = seed % 2 == 0
    if contiguous:   # pattern along the unit-stride dim of a wide array (128-bit loads), wrap only at row ends
        arr_in = [int(rng.integers(1, 4)), int(rng.integers(1, 5)), 8 * int(rng.integers(4, 40))]
        step = int(rng.integers(1, 9))
        rep = [arr_in[0], arr_in[1], arr_in[2] // step]
        o_in, P_in, F_in = [0, 0, int(rng.integers(0, 3))], [[1, 0, 0], [0, 1, 0], [0, 0, step]], [[0], [0], [1]]
    else:
        ra = int(rng.integers(1, 4))
        rep = [int(rng.integers(1, 6)) for _ in range(int(rng.integers(1, 3)))]
        arr_in = [int(rng.integers(2, 17)) for _ in range(ra)]
        o_in = [int(rng.integers(-2 * s, 2 * s + 1)) for s in arr_in]
        P_in = [[int(rng.integers(-4, 10)) for _ in rep] for _ in range(ra)]
        F_in = [[int(rng.integers(-4, 10))] for _ in range(ra)]
    nrep = int(np.prod(rep))
    arr_out = [nrep, n_out]
    strides = [int(np.prod(rep[j + 1:])) for j in range(len(rep))]
    P_out, F_out = [strides, [0] * len(rep)], [[0], [1]]
    xh = np.asarray(rng.integers(-5000, 5000, size=arr_in)).astype(np.int32)
    oti = orc.make_tiler(arr_in, rep, [n_in], o_in, P_in, F_in)
    oto = orc.make_tiler(arr_out, rep, [n_out], [0, 0], P_out, F_out)
    bg = np.full(arr_out, -99, np.int32)
    want = orc.scatter(oto, _task_c(orc.gather(oti, xh), starts, L, d), bg)
    f = aol.make_filter(aol.make_tiler(arr_in, rep, [n_in], o_in, P_in, F_in),
                        aol.make_tiler(arr_out, rep, [n_out], [0, 0], P_out, F_out), starts, L, d)
    out = torch.from_numpy(bg.copy()).cuda()
    aol.filter_apply(f, torch.from_numpy(xh).cuda(), out=out)
    torch.cuda.synchronize()
    assert np.array_equal(out.cpu().numpy(), want), (n_in, L, starts, d)


def test_tiler_paper_presets_on_gpu(orc):
    H, W = 27, 64
    xh = synth.planes(4, 1, H, W)[0]
    for which in (aol.PRESET_H_IN, aol.PRESET_V_IN):
        G = aol.tiler_gather(aol.tiler_preset(which, H, W), torch.from_numpy(xh).cuda())
        torch.cuda.synchronize()
        assert np.array_equal(G.cpu().numpy(), orc.gather(orc.preset(which, H, W), xh))


def test_tiler_batch_descriptor(orc):
    """The 4-D batch tiler (array {N,C,H,W}, rep {N,C,H,W/8}, pattern {11}) gathers the
    same patterns as the per-plane Fig. 10 tiler."""
    N, C, H, W = 2, 3, 9, 64
    xh = synth.frames(6, 0, N, C, H, W)
    P = [[1, 0, 0, 0], [0, 1, 0, 0], [0, 0, 1, 0], [0, 0, 0, 8]]
    F = [[0], [0], [0], [1]]
    t = aol.make_tiler([N, C, H, W], [N, C, H, W // 8], [11], [0, 0, 0, 0], P, F)
    G = aol.tiler_gather(t, torch.from_numpy(xh).cuda()).cpu().numpy()
    ot = orc.preset(orc.PRESET_H_IN, H, W)
    for n in range(N):
        for c in range(C):
            assert np.array_equal(G[n, c], orc.gather(ot, xh[n, c]))


# -------------------------------------------------------------- full-size configs

def _oracle_cs(orc, seed, index, C, H, W, chunk=16):
    """Oracle checksums of synthetic frames `index` (global frame indices), generated in chunks by the C form
    of the seeded generator."""
    index = list(index)
    out = np.empty(len(index), np.uint64)
    for k in range(0, len(index), chunk):
        idx = index[k:k + chunk]
        _, cs = orc.downscale_frame(synth.frames_c(seed, 0, len(idx), C, H, W, index=idx), nthreads=16)
        out[k:k + len(idx)] = cs
    return out


def test_bench_config_300_hd_frames(orc):
    """BASELINE configs[1]: 300 HD frames, the launch bench.py times.  EVERY frame's checksum against the
    oracle; frames {0, 149, 299} element by element; the fused epilogue against the
    stand-alone checksum kernel."""
    N, C, H, W = 300, 3, 1080, 1920
    x = aol.synth_frames(0, 0, N, C, H, W, "uniform")
    z, cs = aol.downscale_frame(x, checksums=True)
    cs2 = aol.frame_checksum(z)
    torch.cuda.synchronize()
    assert torch.equal(cs.view(torch.int64), cs2.view(torch.int64))
    for n in (0, 149, 299):
        xh = synth.frames(0, n, 1, C, H, W, "uniform")
        assert np.array_equal(x[n:n + 1].cpu().numpy(), xh)
        zo, cso = run_oracle(orc, xh)
        assert np.array_equal(z[n:n + 1].cpu().numpy(), zo), n
        assert np_u64(cs[n:n + 1])[0] == cso[0]
    got = np_u64(cs)
    want = _oracle_cs(orc, 0, range(N), C, H, W)
    bad = np.nonzero(got != want)[0]
    assert bad.size == 0, f"{bad.size} of 300 frame checksums differ from the oracle, first {bad[:8]}"


def test_4k_batch(orc):
    """BASELINE configs[3]: the 64-frame 3840x2160 batch bench.py's d4 record times.
    EVERY frame's checksum against the oracle; frames {0, 63} element by element."""
    N, C, H, W = 64, 3, 2160, 3840
    x = aol.synth_frames(1, 0, N, C, H, W, "uniform")
    z, cs = aol.downscale_frame(x, checksums=True)
    cs2 = aol.frame_checksum(z)
    torch.cuda.synchronize()
    assert torch.equal(cs.view(torch.int64), cs2.view(torch.int64))
    got = np_u64(cs)
    for n in (0, N - 1):
        zo, cso = run_oracle(orc, synth.frames(1, n, 1, C, H, W, "uniform"))
        assert np.array_equal(z[n:n + 1].cpu().numpy(), zo)
        assert got[n] == cso[0]
    del x, z
    torch.cuda.empty_cache()
    assert np.array_equal(got, _oracle_cs(orc, 1, range(N), C, H, W))


def test_d5_hd_stream_pool_512_frames(orc, tmp_path):
    """SURVEY 8(d) d5 at full HD size: a 512-frame stream through bench.py's strong-scaling mode with a device
    pool of 256 frames (two launches over the pool); the pool's 256 checksums against the oracle."""
    import json
    import subprocess
    import sys

    from conftest import ROOT

    dump = str(tmp_path / "cs.npy")
    r = subprocess.run([sys.executable, os.path.join(ROOT, "bench.py"), "--stream-frames", "512", "--pool", "256",
                        "--steps", "3", "--warmup", "3", "--no-cpu-baseline", "--dump-checksums", dump],
                       capture_output=True, text=True, timeout=900, cwd=ROOT)
    assert r.returncode == 0, r.stderr[-3000:]
    d = json.loads([l for l in r.stdout.splitlines() if l.startswith("{")][-1])
    assert d["scaling"] == "strong" and d["launch"]["launches_per_step"] == 2
    assert np.array_equal(np.load(dump), _oracle_cs(orc, 0, range(256), 3, 1080, 1920))


def test_cif_2000_frames(orc):
    """The paper's second workload (Section III): 2000 CIF frames 352x288 ->
    132x128 in the launch tools/bench_configs.py times (4 CTAs/SM).  EVERY frame's checksum against the
    oracle (one OpenMP oracle call over the whole batch), and frames {0, 999, 1999} element by element."""
    N, C, H, W = 2000, 3, 288, 352
    x = aol.synth_frames(4, 0, N, C, H, W, "uniform")
    z, cs = aol.downscale_frame(x, checksums=True)
    torch.cuda.synchronize()
    zo, cso = orc.downscale_frame(x.cpu().numpy(), nthreads=16)
    assert np.array_equal(np_u64(cs), cso)
    for n in (0, 999, 1999):
        assert np.array_equal(z[n].cpu().numpy(), zo[n]), n


def test_u8_300_hd_frames_int16_out(orc):
    """NEXT row f1 at bench size: 300 HD frames of 8-bit samples with int16 outputs (bench.py --dtype u8
    --out-dtype i16, 3 CTAs/SM) and with int32 outputs: the checksums of both equal the int32-input path's
    on the same integers, sampled frames element by element against the oracle."""
    N, C, H, W = 300, 3, 1080, 1920
    x8 = aol.synth_frames(0, 0, N, C, H, W, "uniform", dtype=torch.uint8)
    z16, cs16 = aol.downscale_frame(x8, checksums=True, out_dtype=torch.int16)
    z32, cs32 = aol.downscale_frame(x8, checksums=True)
    torch.cuda.synchronize()
    assert torch.equal(cs16.view(torch.int64), cs32.view(torch.int64))
    assert torch.equal(z16.to(torch.int32), z32)
    got = np_u64(cs16)
    for n in (0, 150, 299):
        zo, cso = run_oracle(orc, synth.frames(0, n, 1, C, H, W, "uniform"))
        assert np.array_equal(z16[n:n + 1].cpu().numpy().astype(np.int32), zo), n
        assert got[n] == cso[0], n
    del x8, z16, z32
    torch.cuda.empty_cache()


def test_host_streamed_matches_device(orc):
    N, C, H, W = 10, 3, 108, 256
    xh = synth.frames(12, 0, N, C, H, W)
    xpin = torch.from_numpy(xh).pin_memory()
    zh, csh = aol.downscale_frame_host(xpin, chunk_frames=3)
    zo, cso = run_oracle(orc, xh)
    assert np.array_equal(zh.numpy(), zo)
    assert np.array_equal(csh.view(torch.int64).numpy().view(np.uint64), cso)


@pytest.mark.parametrize("chunk", [1, 4, 7, 50])
def test_host_streamed_u8_and_ragged_chunks(orc, chunk):
    """uint8 samples from pageable and pinned host memory; chunk sizes that do not divide the batch."""
    N, C, H, W = 7, 3, 36, 256
    xh = synth.frames(13, 0, N, C, H, W)
    zo, cso = run_oracle(orc, xh)
    for pinned in (False, True):
        x8 = torch.from_numpy(xh.astype(np.uint8))
        if pinned:
            x8 = x8.pin_memory()
        zh, csh = aol.downscale_frame_host(x8, chunk_frames=chunk)
        assert np.array_equal(zh.numpy(), zo)
        assert np.array_equal(csh.view(torch.int64).numpy().view(np.uint64), cso)
    zh, csh = aol.downscale_frame_host(torch.from_numpy(xh), chunk_frames=chunk, checksums=False)
    assert csh is None and np.array_equal(zh.numpy(), zo)


# -------------------------------------------------------------- edge cases

@pytest.mark.parametrize("W,dtype,kernel", [(7680, torch.int32, 1), (7936, torch.int32, 1), (7944, torch.int32, 2),
                                            (7936, torch.uint8, 1), (8192, torch.uint8, 2), (16, torch.uint8, 1),
                                            (32, torch.int32, 1), (7432, torch.int32, 1)])
def test_width_limits(orc, W, dtype, kernel):
    """Widest frames the TMA kernel takes and the first widths that fall back to the generic kernel: both
    dtypes are capped by W/8 <= 992 consumer threads + 1 producer warp = 1024 (wide int32 frames stream one
    row per ring stage, so two stages + one 4-row output band fit in 227 KB of smem up to W = 7936).  Also
    the narrowest TMA widths."""
    N, C, H = 1, 1, 18
    xh = synth.frames(61, 0, N, C, H, W, "uniform")
    if dtype == torch.int32 and kernel == 1 and W > 3271:
        assert aol.downscale_frame_plan(N, C, H, W)["stages"] >= 2
    zo, cso = run_oracle(orc, xh)
    x = torch.from_numpy(xh.astype(np.uint8) if dtype == torch.uint8 else xh).cuda()
    assert aol.downscale_frame_plan(N, C, H, W, dtype=dtype)["kernel"] == kernel
    z, cs = aol.downscale_frame(x, checksums=True)
    torch.cuda.synchronize()
    assert np.array_equal(z.cpu().numpy(), zo)
    assert np.array_equal(np_u64(cs), cso)


def test_misaligned_and_noncontiguous_inputs():
    base = torch.zeros(1 * 3 * 18 * 64 + 4, dtype=torch.int32, device="cuda")
    x = base[1:1 + 3 * 18 * 64].view(1, 3, 18, 64)          # 4-byte offset: not 16-byte aligned
    with pytest.raises(aol.AolError) as e:
        aol.downscale_frame(x)
    assert e.value.status == aol._lib.E_ALIGN
    y = torch.zeros((1, 3, 18, 128), dtype=torch.int32, device="cuda")[..., ::2]
    with pytest.raises(ValueError):
        aol.downscale_frame(y)


def test_concurrent_streams_and_threads(orc):
    """The library is re-entrant: four host threads, four streams, interleaved launches."""
    import threading

    shapes = [(3, 3, 36, 256), (2, 3, 288, 352), (4, 1, 27, 1920), (2, 2, 18, 512)]
    inputs = [synth.frames(70 + i, 0, *s) for i, s in enumerate(shapes)]
    results, errors = [None] * 4, []

    def work(i):
        try:
            s = torch.cuda.Stream()
            with torch.cuda.stream(s):
                x = torch.from_numpy(inputs[i]).cuda()
                for _ in range(5):
                    z, cs = aol.downscale_frame(x, checksums=True, stream=s)
                s.synchronize()
                results[i] = (z.cpu().numpy(), np_u64(cs))
        except Exception as e:  # pragma: no cover - reported below
            errors.append(e)

    ts = [threading.Thread(target=work, args=(i,)) for i in range(4)]
    for t in ts:
        t.start()
    for t in ts:
        t.join()
    assert not errors, errors
    for i in range(4):
        zo, cso = run_oracle(orc, inputs[i])
        assert np.array_equal(results[i][0], zo) and np.array_equal(results[i][1], cso)


def test_binding_rejects_mismatched_buffers():
    """The Python binding checks caller-supplied outputs before the C call: the kernels write exactly the
    shape / dtype the ABI defines, so a smaller or differently typed buffer is refused (ValueError), never
    overrun."""
    x = aol.synth_frames(0, 0, 2, 3, 18, 64)
    with pytest.raises(ValueError):
        aol.downscale_frame(x, out=torch.empty((2, 3, 8, 23), dtype=torch.int32, device="cuda"))
    with pytest.raises(TypeError):   # int64 is not an output type at all
        aol.downscale_frame(x, out=torch.empty((2, 3, 8, 24), dtype=torch.int64, device="cuda"))
    with pytest.raises(ValueError):
        aol.downscale_frame(x, checksums=torch.empty(1, dtype=torch.uint64, device="cuda"))
    with pytest.raises(ValueError):
        aol.downscale_h(x, out=torch.empty((2, 3, 18, 23), dtype=torch.int32, device="cuda"))
    with pytest.raises(ValueError):
        aol.frame_checksum(x.to(torch.int64))
    t = aol.make_tiler([16, 24], [2, 3], [8, 8], [0, 0], [[8, 0], [0, 8]], [[1, 0], [0, 1]])
    A = torch.zeros((16, 24), dtype=torch.int32, device="cuda")
    with pytest.raises(ValueError):
        aol.tiler_gather(t, A, out=torch.empty((2, 3, 8, 7), dtype=torch.int32, device="cuda"))
    with pytest.raises(ValueError):
        aol.tiler_scatter(t, torch.zeros((2, 3, 8, 8), dtype=torch.int16, device="cuda"), A)
    # the right buffers still work
    z, cs = aol.downscale_frame(x, out=torch.empty((2, 3, 8, 24), dtype=torch.int32, device="cuda"),
                                checksums=torch.empty(2, dtype=torch.int64, device="cuda"))
    torch.cuda.synchronize()
    assert z.shape == (2, 3, 8, 24)


@pytest.mark.parametrize("dtype", [torch.uint8, torch.int32])
def test_interleaved_to_planar_via_tiler(orc, dtype):
    """SURVEY 8(f) f2's optional step: video frames arrive interleaved ([H][W][3], OpenCV's 24-bit BGR,
    P:L260 / P:L657-659); the split into the planar [3][H][W] layout the filters take is itself an ArrayOL
    tiler -- rep {3, H, W}, scalar pattern, paving mapping r = (c, y, x) to the array index (y, x, c).  The
    generic gather does it; the result equals numpy's transpose and downscales to the oracle's output."""
    H, W = 36, 64
    xi = synth.frames(12, 0, 1, 1, H, W * 3, "uniform")[0, 0].reshape(H, W, 3)   # [H][W][3] samples 0..255
    t = aol.make_tiler([H, W, 3], [3, H, W], [], [0, 0, 0], [[0, 1, 0], [0, 0, 1], [1, 0, 0]], [[], [], []])
    planar = aol.tiler_gather(t, torch.from_numpy(xi.astype(np.uint8) if dtype == torch.uint8 else xi).cuda())
    torch.cuda.synchronize()
    ref = np.ascontiguousarray(np.transpose(xi, (2, 0, 1)))
    assert np.array_equal(planar.cpu().numpy().astype(np.int32), ref)
    z, cs = aol.downscale_frame(planar.unsqueeze(0), checksums=True)
    zo, cso = orc.downscale_frame(ref[None].astype(np.int32))
    torch.cuda.synchronize()
    assert np.array_equal(z.cpu().numpy(), zo) and np.array_equal(np_u64(cs), cso)


@pytest.mark.parametrize("C,X,dtype", [(3, 64, np.uint8), (3, 1920, np.uint8), (2, 100, np.int16), (4, 5000, np.uint8),
                                       (3, 6000, np.int32), (8, 70, np.int64), (3, 16385, np.uint8)])
def test_deinterleave_tilers(orc, C, X, dtype):
    """Linear tilers whose innermost array dims are C interleaved channels inside tile-contiguous runs of X
    positions (the staged (de)interleave kernel; chunks of the run, ragged last chunk): gather == the C
    oracle, FAST scatter inverts it."""
    R = 3   # outer rows
    arr, rep = [R, X, C], [C, R, X]
    P = [[0, 1, 0], [0, 0, 1], [1, 0, 0]]
    rng = np.random.default_rng(C * 1000 + X)
    A = np.asarray(rng.integers(0, 100, size=arr)).astype(dtype)
    ot = orc.make_tiler(arr, rep, [], [0, 0, 0], P, [[], [], []])
    gt = aol.make_tiler(arr, rep, [], [0, 0, 0], P, [[], [], []])
    Ad = torch.from_numpy(A).cuda()
    G = aol.tiler_gather(gt, Ad)
    torch.cuda.synchronize()
    assert np.array_equal(G.cpu().numpy(), orc.gather(ot, A))
    back = torch.zeros_like(Ad)
    aol.tiler_scatter(gt, G, back, mode="fast")
    torch.cuda.synchronize()
    assert torch.equal(back, Ad)


@pytest.mark.parametrize("shape", [(2, 36, 128), (1, 9, 16), (3, 27, 352), (2, 18, 1040), (1, 1080, 1920),
                                   (1, 18, 3840)])
@pytest.mark.parametrize("out_dtype", [torch.int32, torch.int16])
def test_packed_rgb_frames(orc, shape, out_dtype):
    """Packed 24-bit pixels ([N][H][W][3], P:L260 as OpenCV delivers them) straight into the fused kernel
    (AOL_RGB8: the consumer gathers each channel's samples with byte permutes): planar outputs and checksums
    equal the oracle's on the transposed frames and the planar uint8 path's."""
    N, H, W = shape
    xp = synth.frames(21, 0, N, 3, H, W, "uniform")                      # planar int32 samples 0..255
    packed = torch.from_numpy(np.ascontiguousarray(np.transpose(xp, (0, 2, 3, 1))).astype(np.uint8)).cuda()
    zo, cso = run_oracle(orc, xp)
    z, cs = aol.downscale_frame_packed(packed, checksums=True, out_dtype=out_dtype)
    zp, csp = aol.downscale_frame(torch.from_numpy(xp.astype(np.uint8)).cuda(), checksums=True, out_dtype=out_dtype)
    torch.cuda.synchronize()
    assert np.array_equal(z.cpu().numpy().astype(np.int32), zo)
    assert np.array_equal(np_u64(cs), cso)
    assert torch.equal(z, zp) and torch.equal(cs.view(torch.int64), csp.view(torch.int64))
    for opts in ({"bands_per_unit": 1, "stages": 2}, {"ctas_per_sm": 2}):
        try:
            z2, cs2 = aol.downscale_frame_packed(packed, checksums=True, out_dtype=out_dtype, opts=opts)
        except aol.AolError:
            # two CTAs of a 4K frame's 3-plane staging + 2 ring stages do not fit one SM's shared memory
            assert W >= 3840 and opts.get("ctas_per_sm") == 2
            continue
        torch.cuda.synchronize()
        assert torch.equal(z2, z) and np.array_equal(np_u64(cs2), cso), opts


def test_packed_rgb_rejects():
    x = torch.zeros((1, 18, 40, 3), dtype=torch.uint8, device="cuda")   # W % 16 != 0
    with pytest.raises(aol.AolError):
        aol.downscale_frame_packed(x)


def test_packed_rgb_host_streamed(orc):
    """Packed 24-bit pixels from pinned HOST memory through the 3-stream pipeline (ragged last chunk):
    outputs and checksums equal the device path's and the oracle's."""
    N, H, W = 7, 36, 128
    xp = synth.frames(23, 0, N, 3, H, W, "uniform")
    packed = torch.from_numpy(np.ascontiguousarray(np.transpose(xp, (0, 2, 3, 1))).astype(np.uint8)).pin_memory()
    z, cs = aol.downscale_frame_host(packed, chunk_frames=3, packed=True)
    zo, cso = run_oracle(orc, xp)
    assert np.array_equal(z.numpy(), zo)
    assert np.array_equal(cs.view(torch.int64).numpy().view(np.uint64), cso)


@pytest.mark.parametrize("W,out_dtype,ok", [(6400, torch.int32, True), (6416, torch.int32, False),
                                            (6416, torch.int16, True), (7936, torch.int16, True)])
def test_packed_rgb_width_limit(orc, W, out_dtype, ok):
    """Packed 24-bit pixels: two 9W-byte ring stages plus the 3-plane output staging (18W bytes int32, 9W int16)
    fit the 227 KB opt-in up to W = 6400 with int32 outputs and W = 7936 with int16 outputs; the first width past
    the int32 limit is refused with a message naming that limit."""
    N, H = 1, 9
    xp = synth.frames(25, 0, N, 3, H, W, "uniform")
    packed = torch.from_numpy(np.ascontiguousarray(np.transpose(xp, (0, 2, 3, 1))).astype(np.uint8)).cuda()
    if not ok:
        with pytest.raises(aol.AolError) as e:
            aol.downscale_frame_packed(packed, out_dtype=out_dtype)
        assert e.value.status == aol._lib.E_SHAPE and "W <= 6400 with int32" in str(e.value)
        return
    z, cs = aol.downscale_frame_packed(packed, checksums=True, out_dtype=out_dtype)
    zo, cso = run_oracle(orc, xp)
    torch.cuda.synchronize()
    assert np.array_equal(z.cpu().numpy().astype(np.int32), zo) and np.array_equal(np_u64(cs), cso)


@pytest.mark.parametrize("kernel", [1, 2])
def test_failed_launch_enqueues_nothing(kernel):
    """A call that fails at its launch (forced by the test hook right before the first enqueue) returns
    AOL_E_CUDA and leaves the caller's output and checksum buffers untouched (include/aol.h: on error nothing
    has been enqueued); the next call works."""
    import ctypes

    N, C, H, W = 2, 3, 36, 128
    x = aol.synth_frames(3, 0, N, C, H, W)
    z = torch.full((N, C, 16, 48), -77, dtype=torch.int32, device="cuda")
    cs = torch.full((N,), 12345, dtype=torch.int64, device="cuda").view(torch.uint64)
    aol._lib.lib().aol_debug_fail_next_launches(1)
    with pytest.raises(aol.AolError) as e:
        aol.downscale_frame(x, out=z, checksums=cs, opts={"kernel": kernel})
    assert e.value.status == aol._lib.E_CUDA and "injected" in str(e.value)
    torch.cuda.synchronize()
    assert bool((z == -77).all()) and bool((cs.view(torch.int64) == 12345).all())
    aol.downscale_frame(x, out=z, checksums=cs, opts={"kernel": kernel})
    torch.cuda.synchronize()
    assert not bool((z == -77).any()) and not bool((cs.view(torch.int64) == 12345).any())


def test_misaligned_checksum_pointer_refused():
    """d_frame_checksums must be 8-byte aligned (a misaligned u64 atomic would be a sticky context fault):
    AOL_E_ALIGN from the fused call and from aol_frame_checksum, through the C ABI with raw pointers."""
    import ctypes

    L = aol._lib.lib()
    N, C, H, W = 1, 3, 18, 64
    x = aol.synth_frames(3, 0, N, C, H, W)
    z = torch.empty((N, C, 8, 24), dtype=torch.int32, device="cuda")
    buf = torch.zeros(4, dtype=torch.int64, device="cuda")
    bad = ctypes.c_void_p(buf.data_ptr() + 4)
    st = L.aol_downscale_frame(ctypes.c_void_p(x.data_ptr()), aol._lib.I32, ctypes.c_void_p(z.data_ptr()), N, C, H, W,
                               bad, ctypes.c_void_p(torch.cuda.current_stream().cuda_stream))
    assert st == aol._lib.E_ALIGN
    st = L.aol_frame_checksum(ctypes.c_void_p(z.data_ptr()), N, C, 8, 24, bad,
                              ctypes.c_void_p(torch.cuda.current_stream().cuda_stream))
    assert st == aol._lib.E_ALIGN
    torch.cuda.synchronize()
    assert bool((buf == 0).all())
