#!/usr/bin/env python
"""Small launches of every kernel, for compute-sanitizer (memcheck / racecheck / synccheck / initcheck).

Exits non-zero if any result differs from a second computation path, so a sanitizer run also checks
that instrumented execution still produces the right answer.
"""
import os
import sys

import torch

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import paper_conf_ipps_guortgbs11_b200 as aol  # noqa: E402


def main():
    import argparse
    ap = argparse.ArgumentParser()
    ap.add_argument("--dtypes", default="i32,u8")
    ap.add_argument("--kernels", default="1,2")
    ap.add_argument("--fused-only", action="store_true")
    ap.add_argument("--widths", default="", help="only these W values, e.g. 256")
    ap.add_argument("--chain-only", action="store_true", help="only the separable chain kernels (racecheck)")
    args = ap.parse_args()
    if args.chain_only:   # cp.async row staging + a shared-memory ring behind two barriers per row
        torch.cuda.set_device(0)
        P, H, W = 2, 36, 256
        x = aol.synth_frames(3, 0, 1, P, H, W, "uniform")[0]
        fh, fv = aol.filter_preset(aol.FILTER_H, P, H, W), aol.filter_preset(aol.FILTER_V, P, H, 3 * W // 8)
        want = aol.filter_apply(fv, aol.filter_apply(fh, x))
        ok = True
        for jit in (1, 0):
            aol._lib.lib().aol_debug_set_chain_jit(jit)
            ok &= torch.equal(aol.filter_chain_apply(fh, fv, x), want)
        torch.cuda.synchronize()
        print("sanitize workload (chain):", "OK" if ok else "MISMATCH")
        return 0 if ok else 1
    dts = [{"i32": torch.int32, "u8": torch.uint8}[d] for d in args.dtypes.split(",")]
    kernels = [int(k) for k in args.kernels.split(",")]
    torch.cuda.set_device(0)
    ok = True
    # W = 1040: uint8 two-repetitions-per-thread path with a partly idle warp and 1-D bulk copies
    # W = 40 / 1000: int32 rows with W % 32 != 0 (linear smem rows filled by 1-D bulk copies)
    shapes = [(2, 3, 27, 64), (1, 1, 9, 32), (1, 2, 18, 352), (2, 2, 18, 256), (1, 1, 18, 1040), (1, 2, 18, 40),
              (1, 1, 9, 1000)]
    if args.widths:
        shapes = [sh for sh in shapes if str(sh[3]) in args.widths.split(",")]
    for (N, C, H, W) in shapes:
        for dt in dts:
            x = aol.synth_frames(1, 0, N, C, H, W, "uniform", dtype=dt)
            ref = None
            all_opts = [{"kernel": 2}, {"kernel": 1}, {"kernel": 1, "stages": 2, "bands_per_unit": 1},
                        {"kernel": 1, "ctas_per_sm": 2}, {"kernel": 1, "flags": 64}]
            for opts in [o for o in all_opts if o["kernel"] in kernels]:
                try:
                    z, cs = aol.downscale_frame(x, checksums=True, opts=opts)
                except aol.AolError:
                    continue   # shape not eligible for this kernel
                torch.cuda.synchronize()
                if ref is None:
                    ref = (z.clone(), cs.clone())
                else:
                    ok &= torch.equal(z, ref[0]) and torch.equal(cs.view(torch.int64), ref[1].view(torch.int64))
        if W % 16 == 0 and C == 3:   # packed 24-bit pixels into the fused kernel == the planar uint8 path
            xu = aol.synth_frames(1, 0, N, C, H, W, "uniform", dtype=torch.uint8)
            zp, csp = aol.downscale_frame_packed(xu.permute(0, 2, 3, 1).contiguous(), checksums=True)
            zq, csq = aol.downscale_frame(xu, checksums=True)
            torch.cuda.synchronize()
            ok &= torch.equal(zp, zq) and torch.equal(csp.view(torch.int64), csq.view(torch.int64))
        if args.fused_only:
            continue
        x = aol.synth_frames(2, 0, N, C, H, W, "signed")
        y = aol.downscale_h(x)
        z = aol.downscale_v(y)
        zf, _ = aol.downscale_frame(x)
        ok &= torch.equal(z, zf)
        ok &= torch.equal(aol.frame_checksum(z).view(torch.int64),
                          aol.downscale_frame(x, checksums=True)[1].view(torch.int64))
    if args.fused_only:
        torch.cuda.synchronize()
        print("sanitize workload:", "OK" if ok else "MISMATCH")
        return 0 if ok else 1
    t = aol.make_tiler([16, 24], [2, 3], [8, 8], [0, 0], [[8, 0], [0, 8]], [[1, 0], [0, 1]])
    A = torch.arange(16 * 24, dtype=torch.int32, device="cuda").reshape(16, 24)
    G = aol.tiler_gather(t, A)
    B = torch.zeros_like(A)
    aol.tiler_scatter(t, G, B, mode="fast")
    ok &= torch.equal(A, B)
    B.zero_()
    aol.tiler_scatter(t, G, B, mode="sequential")
    ok &= torch.equal(A, B)
    tw = aol.make_tiler([9, 10], [4], [5, 3], [-3, 7], [[2], [3]], [[1, 0], [0, -1]])   # wrapping
    G2 = aol.tiler_gather(tw, A[:9, :10].contiguous())
    C2 = torch.zeros((9, 10), dtype=torch.int32, device="cuda")
    aol.tiler_scatter(tw, G2, C2, mode="sequential")
    # channel-interleaved runs: 3 x 8-bit (register transpose), 4 x 8-bit and 3 x 16-bit (smem-staged)
    for C, X, dt in ((3, 64, torch.uint8), (4, 80, torch.uint8), (3, 96, torch.int16)):
        ti = aol.make_tiler([2, X, C], [C, 2, X], [], [0, 0, 0], [[0, 1, 0], [0, 0, 1], [1, 0, 0]], [[], [], []])
        Ai = (torch.arange(2 * X * C, device="cuda") % 97).to(dt).reshape(2, X, C)
        Gi = aol.tiler_gather(ti, Ai)
        ok &= torch.equal(Gi, Ai.permute(2, 0, 1))
        Bi = torch.zeros_like(Ai)
        aol.tiler_scatter(ti, Gi, Bi, mode="fast")
        ok &= torch.equal(Ai, Bi)
    # a bijective blocking shifted to wrap in both dims (32-bit wrapping kernel): FAST scatter inverts the gather
    ts = aol.make_tiler([16, 24], [2, 3], [8, 8], [-3, 5], [[8, 0], [0, 8]], [[1, 0], [0, 1]])
    G3 = aol.tiler_gather(ts, A)
    D = torch.zeros_like(A)
    aol.tiler_scatter(ts, G3, D, mode="fast")
    ok &= torch.equal(A, D)
    # generic run-time filters (register-pattern kernel: 128-bit contiguous path, wrapping path, stepping)
    P, H, W = 2, 18, 256
    x = aol.synth_frames(3, 0, 1, P, H, W, "uniform")[0]
    y = aol.filter_apply(aol.filter_preset(aol.FILTER_H, P, H, W), x)
    z = aol.filter_apply(aol.filter_preset(aol.FILTER_V, P, H, 3 * W // 8), y)
    ok &= torch.equal(z, aol.downscale_frame(x.unsqueeze(1))[0][:, 0])
    # round 2: the fused chain of the same two filters (one kernel), the box tiler kernels (wrapping blocking
    # with 16-byte row copies and a ragged chunk; the paper's H input tiler), persistent plans
    z2 = aol.filter_chain_apply(aol.filter_preset(aol.FILTER_H, P, H, W), aol.filter_preset(aol.FILTER_V, P, H, 3 * W // 8), x)
    ok &= torch.equal(z, z2)
    Ab = torch.arange(3 * 64 * 256, dtype=torch.int32, device="cuda").reshape(3, 64, 256)
    tb = aol.make_tiler([3, 64, 256], [3, 8, 32], [8, 8], [1, 7, -9], [[1, 0, 0], [0, 8, 0], [0, 0, 8]], [[0, 0], [1, 0], [0, 1]])
    Gb = aol.tiler_gather(tb, Ab)
    Bb = torch.zeros_like(Ab)
    aol.tiler_scatter(tb, Gb, Bb, mode="fast")
    ok &= torch.equal(Ab, Bb)
    Ac = torch.arange(50 * 1000, dtype=torch.int32, device="cuda").reshape(50, 1000)
    tc = aol.make_tiler([50, 1000], [50, 125], [11], [3, -2], [[1, 0], [0, 8]], [[0], [1]])
    aol.tiler_gather(tc, Ac)
    # round 2, later: the separable chain statically compiled (the default above is the NVRTC-specialised one),
    # the general chain kernel (V then H), affine pieces with array sides off the 16-byte grid (gather + FAST
    # scatter, 2 / 4 / 8-byte elements), column strips of the fused kernel (forced at a small width)
    L = aol._lib.lib()
    L.aol_debug_set_chain_jit(0)
    z3 = aol.filter_chain_apply(aol.filter_preset(aol.FILTER_H, P, H, W), aol.filter_preset(aol.FILTER_V, P, H, 3 * W // 8), x)
    L.aol_debug_set_chain_jit(1)
    ok &= torch.equal(z, z3)
    xv = aol.synth_frames(5, 0, 1, 2, 54, 512, "uniform")[0]
    zvh = aol.filter_chain_apply(aol.filter_preset(aol.FILTER_V, 2, 54, 512), aol.filter_preset(aol.FILTER_H, 2, 24, 512), xv)
    yv = aol.filter_apply(aol.filter_preset(aol.FILTER_V, 2, 54, 512), xv)
    ok &= torch.equal(zvh, aol.filter_apply(aol.filter_preset(aol.FILTER_H, 2, 24, 512), yv))
    for dt in (torch.int16, torch.int32, torch.int64):
        Ap = torch.arange(3 * 64 * 256, device="cuda").reshape(3, 64, 256).to(dt)
        tp = aol.make_tiler([3, 64, 256], [3, 8, 32], [8, 8], [0, -3, 5], [[1, 0, 0], [0, 8, 0], [0, 0, 8]], [[0, 0], [1, 0], [0, 1]])
        Gp = aol.tiler_gather(tp, Ap)
        Bp = torch.zeros_like(Ap)
        aol.tiler_scatter(tp, Gp, Bp, mode="fast")
        ok &= torch.equal(Ap, Bp)
    xs = aol.synth_frames(6, 0, 2, 3, 27, 1056)
    zs, css = aol.downscale_frame(xs, checksums=True, opts={"kernel": 1, "flags": aol.FLAGS["I32_STRIPS"]})
    zt, cst = aol.downscale_frame(xs, checksums=True, opts={"kernel": 2})
    torch.cuda.synchronize()
    ok &= torch.equal(zs, zt) and torch.equal(css.view(torch.int64), cst.view(torch.int64))
    xp = aol.synth_frames(4, 0, 2, 3, 36, 256)
    pl = aol.FramePlan(xp, checksums=True)
    zp, csp = pl.launch()
    zq, csq = aol.downscale_frame(xp, checksums=True)
    torch.cuda.synchronize()
    ok &= torch.equal(zp, zq) and torch.equal(csp.view(torch.int64), csq.view(torch.int64))
    pl.close()
    torch.cuda.synchronize()
    print("sanitize workload:", "OK" if ok else "MISMATCH")
    return 0 if ok else 1


if __name__ == "__main__":
    sys.exit(main())
