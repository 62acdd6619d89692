#!/usr/bin/env python
"""Secondary measurements for every BASELINE.json config (bench.py times configs[1] only).

One JSON line per measurement (CUDA events on the launching stream, median of N,
after warm-up).  Algorithmic bytes: each input element read once, each output
element written once.

  d1   single HD frame, latency (warm L2 and cold L2 = 512 MB flush before each launch)
  d2x  300 HD frames: fused TMA kernel vs generic fused kernel vs unfused H -> V -> checksum
  d3   generic tiler perf instance: array {64,1024,1024} i32, rep {64,128,128}, pattern {8,8}
  d4   64 frames of 3840x2160 (4K), same ratios
  f1   300 HD frames with uint8 samples
  f4   CIF 352x288, 2000 frames (Section III)
  f1p  300 HD frames of packed 24-bit pixels (AOL_RGB8);  f2x interleaved -> planar split as a tiler gather
"""
import argparse
import json
import os
import statistics
import sys

import torch

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import paper_conf_ipps_guortgbs11_b200 as aol  # noqa: E402


def timed(fn, reps=20, warm=3, before=None, inner=1):
    """Median and min ms per call; `inner` calls back to back between the events (for ~0.1 ms kernels,
    where one call per event pair would mostly time the launch gap)."""
    s = torch.cuda.current_stream()
    for _ in range(warm):
        if before:
            before()
        fn()
    torch.cuda.synchronize()
    ts = []
    for _ in range(reps):
        if before:
            before()
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record(s)
        for _ in range(inner):
            fn()
        b.record(s)
        torch.cuda.synchronize()
        ts.append(a.elapsed_time(b) / inner)
    return statistics.median(ts), min(ts)


def peak():
    try:
        return float(json.load(open(os.path.join(ROOT, "MEASURED_PEAKS.json")))["hbm_gbs"])
    except Exception:
        return 6650.0


def emit(d):
    print(json.dumps(d), flush=True)


def frames_bytes(N, C, H, W, es=4, eo=4):
    return N * C * (H * W * es + (4 * (H // 9)) * (3 * (W // 8)) * eo)


def fused_line(name, N, C, H, W, dtype=torch.int32, opts=None, reps=20, out_dtype=torch.int32):
    x = aol.synth_frames(3, 0, N, C, H, W, "uniform", dtype=dtype)
    z = torch.empty((N, C, 4 * (H // 9), 3 * (W // 8)), dtype=out_dtype, device="cuda")
    cs = torch.empty(N, dtype=torch.uint64, device="cuda")
    call = lambda: aol.downscale_frame(x, out=z, checksums=cs, opts=opts)  # noqa: E731
    single, _ = timed(call, reps=reps)
    med, mn = timed(call, reps=reps, inner=5)   # back to back, as bench.py's consecutive steps
    b = frames_bytes(N, C, H, W, x.element_size(), z.element_size())
    plan = aol.downscale_frame_plan(N, C, H, W, dtype=dtype, opts=opts, out_dtype=out_dtype)
    emit({"config": name, "shape": [N, C, H, W], "dtype": str(dtype).split(".")[-1],
          "out_dtype": str(out_dtype).split(".")[-1], "timing": "5 calls back to back per event pair",
          "ms": med, "min_ms": mn, "ms_single_call": single,
          "frames_per_s": N / (med / 1e3), "GBps": b / (med / 1e3) / 1e9, "frac": b / (med / 1e3) / 1e9 / peak(),
          "kernel": plan["kernel"], "plan": plan})
    del x, z, cs
    torch.cuda.empty_cache()


def main():
    p = argparse.ArgumentParser()
    p.add_argument("--only", default="")
    a = p.parse_args()
    only = set(a.only.split(",")) if a.only else None

    def want(k):
        return only is None or k in only

    torch.cuda.set_device(0)
    if want("d1"):
        N, C, H, W = 1, 3, 1080, 1920
        x = aol.synth_frames(0, 0, N, C, H, W)
        z = torch.empty((N, C, 480, 720), dtype=torch.int32, device="cuda")
        cs = torch.empty(N, dtype=torch.uint64, device="cuda")
        flush = torch.empty(512 << 20, dtype=torch.uint8, device="cuda")
        # warm L2: a GPU-side sleep before each timed call keeps the host's ~18 us enqueue off the device
        # timeline (without it the event pair times the host, not the kernels)
        warm, _ = timed(lambda: aol.downscale_frame(x, out=z, checksums=cs), reps=50,
                        before=lambda: torch.cuda._sleep(200000))
        cold, _ = timed(lambda: aol.downscale_frame(x, out=z, checksums=cs), reps=50, before=lambda: flush.fill_(1))
        # host side of one call (validation, planning, tensor-map encode, launch) without waiting
        import time
        torch.cuda.synchronize()
        t0 = time.perf_counter()
        for _ in range(200):
            aol.downscale_frame(x, out=z, checksums=cs)
        host_us = (time.perf_counter() - t0) / 200 * 1e6
        torch.cuda.synchronize()
        # device time of one call with the host removed: CUDA graph of 20 calls, replayed
        g = torch.cuda.CUDAGraph()
        s = torch.cuda.Stream()
        s.wait_stream(torch.cuda.current_stream())
        with torch.cuda.stream(s):
            aol.downscale_frame(x, out=z, checksums=cs)
            torch.cuda.synchronize()
            with torch.cuda.graph(g, stream=s):
                for _ in range(20):
                    aol.downscale_frame(x, out=z, checksums=cs)
        torch.cuda.synchronize()
        graph_ms, _ = timed(lambda: g.replay(), reps=20)
        b = frames_bytes(N, C, H, W)
        emit({"config": "d1 single HD frame", "warm_l2_us": warm * 1e3, "cold_l2_us": cold * 1e3,
              "host_enqueue_us_per_call": host_us, "graph_replay_us_per_call": graph_ms * 1e3 / 20,
              "roofline_floor_us": b / peak() / 1e3, "cold_GBps": b / (cold / 1e3) / 1e9,
              "plan": aol.downscale_frame_plan(N, C, H, W)})
        del flush
    if want("d2x"):
        N, C, H, W = 300, 3, 1080, 1920
        fused_line("d2 fused TMA kernel", N, C, H, W)
        fused_line("d2 generic fused kernel (kernel=2)", N, C, H, W, opts={"kernel": 2}, reps=5)
        x = aol.synth_frames(0, 0, N, C, H, W)
        y = torch.empty((N, C, H, 720), dtype=torch.int32, device="cuda")
        z = torch.empty((N, C, 480, 720), dtype=torch.int32, device="cuda")
        cs = torch.empty(N, dtype=torch.uint64, device="cuda")

        def unfused():
            aol.downscale_h(x, out=y)
            aol.downscale_v(y, out=z)
            aol.frame_checksum(z, out=cs)

        med, _ = timed(unfused, reps=10)
        th, _ = timed(lambda: aol.downscale_h(x, out=y), reps=10)
        tv, _ = timed(lambda: aol.downscale_v(y, out=z), reps=10)
        b = frames_bytes(N, C, H, W)
        emit({"config": "d2 unfused H -> V -> checksum (Y through HBM)", "ms": med, "frames_per_s": N / (med / 1e3),
              "GBps_algorithmic": b / (med / 1e3) / 1e9, "h_ms": th, "v_ms": tv,
              "h_GBps": (x.numel() * 4 + y.numel() * 4) / (th / 1e3) / 1e9,
              "v_GBps": (y.numel() * 4 + z.numel() * 4) / (tv / 1e3) / 1e9})
        del x, y, z, cs
        torch.cuda.empty_cache()
    if want("d3"):
        t = aol.make_tiler([64, 1024, 1024], [64, 128, 128], [8, 8], [0, 0, 0],
                           [[1, 0, 0], [0, 8, 0], [0, 0, 8]], [[0, 0], [1, 0], [0, 1]])
        A = torch.randint(0, 1 << 30, (64, 1024, 1024), dtype=torch.int32, device="cuda")
        G = torch.empty((64, 128, 128, 8, 8), dtype=torch.int32, device="cuda")
        tg1, _ = timed(lambda: aol.tiler_gather(t, A, out=G))
        tg, _ = timed(lambda: aol.tiler_gather(t, A, out=G), inner=10)
        B = torch.empty_like(A)
        ts, _ = timed(lambda: aol.tiler_scatter(t, G, B, mode="fast"), inner=10)
        tc, _ = timed(lambda: B.copy_(A), inner=10)
        tq, _ = timed(lambda: aol.tiler_scatter(t, G, B, mode="sequential",
                                                workspace=torch.empty(A.numel() * 8, dtype=torch.uint8,
                                                                      device="cuda")), reps=5)
        nb = 2 * A.numel() * 4
        emit({"config": "d3 generic tiler {64,1024,1024} i32 -> 8x8 tiles", "timing": "10 calls back to back per event pair",
              "gather_ms": tg, "gather_GBps": nb / (tg / 1e3) / 1e9, "scatter_fast_ms": ts,
              "scatter_fast_GBps": nb / (ts / 1e3) / 1e9, "gather_ms_single_call": tg1,
              "torch_copy_GBps_same_arrays": nb / (tc / 1e3) / 1e9,
              "scatter_seq_ms": tq, "gather_frac": nb / (tg / 1e3) / 1e9 / peak(),
              "check_gather_is_blocking": bool(torch.equal(G[1, 2, 3], A[1, 16:24, 24:32]))})
        # the same blocking with origin (0, -3, 5): tiles wrap toroidally in both image dims (BASELINE configs[2]
        # "incl. modulo wrap-around"); and the paper's H input tiler (Fig. 10) over 64 HD planes
        tw = aol.make_tiler([64, 1024, 1024], [64, 128, 128], [8, 8], [0, -3, 5],
                            [[1, 0, 0], [0, 8, 0], [0, 0, 8]], [[0, 0], [1, 0], [0, 1]])
        twg, _ = timed(lambda: aol.tiler_gather(tw, A, out=G), inner=10)
        tws, _ = timed(lambda: aol.tiler_scatter(tw, G, B, mode="fast"), inner=10)
        emit({"config": "d3 generic tiler, wrapping in both dims (origin (0,-3,5))", "gather_ms": twg,
              "gather_GBps": nb / (twg / 1e3) / 1e9, "scatter_fast_ms": tws, "scatter_fast_GBps": nb / (tws / 1e3) / 1e9,
              "check_wrap": bool(torch.equal(G[0, 0, 0, 0], A[0, 1021, 5:13])), "roundtrip_ok": bool(torch.equal(A, B))})
        del A, G, B
        torch.cuda.empty_cache()
        X = aol.synth_frames(0, 0, 64, 1, 1080, 1920).reshape(64, 1080, 1920)
        th = aol.make_tiler([64, 1080, 1920], [64, 1080, 240], [11], [0, 0, 0],
                            [[1, 0, 0], [0, 1, 0], [0, 0, 8]], [[0], [0], [1]])
        GH = torch.empty((64, 1080, 240, 11), dtype=torch.int32, device="cuda")
        thg, _ = timed(lambda: aol.tiler_gather(th, X, out=GH), inner=5)
        emit({"config": "H_IN tiler (Fig. 10) gather over 64 HD planes", "gather_ms": thg,
              "gather_GBps": (X.numel() + GH.numel()) * 4 / (thg / 1e3) / 1e9,
              "check_wrap": bool(torch.equal(GH[0, 0, 239], torch.cat([X[0, 0, 1912:1920], X[0, 0, 0:3]])))})
        del X, GH
        torch.cuda.empty_cache()
    if want("f2x"):
        # f2's optional step: interleaved [N][H][W][3] 8-bit frames (OpenCV BGR) -> planar [N][3][H][W] as an
        # ArrayOL tiler gather (rep {N, 3, H, W}, scalar pattern), 64 HD frames
        N, H, W = 64, 1080, 1920
        xi = torch.randint(0, 256, (N, H, W, 3), dtype=torch.uint8, device="cuda")
        ti = aol.make_tiler([N, H, W, 3], [N, 3, H, W], [], [0, 0, 0, 0],
                            [[1, 0, 0, 0], [0, 0, 1, 0], [0, 0, 0, 1], [0, 1, 0, 0]], [[], [], [], []])
        xp = torch.empty((N, 3, H, W), dtype=torch.uint8, device="cuda")
        tg, _ = timed(lambda: aol.tiler_gather(ti, xi, out=xp), inner=5)
        emit({"config": "f2x interleaved -> planar split of 64 HD uint8 frames (tiler gather)", "ms": tg,
              "GBps": 2 * xi.numel() / (tg / 1e3) / 1e9, "frames_per_s": N / (tg / 1e3),
              "check": bool(torch.equal(xp[3, 1], xi[3, :, :, 1]))})
        del xi, xp
        torch.cuda.empty_cache()
    if want("f3"):
        # the paper's generic-vs-non-generic experiment on B200: run-time descriptors,
        # one fused gather+task+scatter kernel per filter, Y through HBM between the two filters
        N, C, H, W = 300, 3, 1080, 1920
        x = aol.synth_frames(0, 0, N, C, H, W).reshape(N * C, H, W)
        fh = aol.filter_preset(aol.FILTER_H, N * C, H, W)
        fv = aol.filter_preset(aol.FILTER_V, N * C, H, 720)
        y = torch.empty((N * C, H, 720), dtype=torch.int32, device="cuda")
        z = torch.empty((N * C, 480, 720), dtype=torch.int32, device="cuda")
        th, _ = timed(lambda: aol.filter_apply(fh, x, out=y), reps=5)
        tv, _ = timed(lambda: aol.filter_apply(fv, y, out=z), reps=5)
        zf, _ = aol.downscale_frame(x.reshape(N, C, H, W))
        b = frames_bytes(N, C, H, W)
        emit({"config": "f3 generic run-time filters H then V (300 HD frames)", "h_ms": th, "v_ms": tv,
              "frames_per_s": N / ((th + tv) / 1e3), "GBps_algorithmic": b / ((th + tv) / 1e3) / 1e9,
              "equals_fused": bool(torch.equal(zf.reshape(N * C, 480, 720), z))})
        del x, y, z, zf
        torch.cuda.empty_cache()
    if want("d5"):
        # configs[4] on one GPU: the 10,000-frame stream through bench.py's strong-scaling mode
        import subprocess
        r = subprocess.run([sys.executable, os.path.join(ROOT, "bench.py"), "--stream-frames", "10000", "--pool", "256",
                            "--steps", "5", "--warmup", "2", "--no-cpu-baseline"], capture_output=True, text=True)
        line = json.loads(r.stdout.strip().splitlines()[-1])
        emit({"config": "d5 10,000-frame HD stream, 1 GPU (pool 256)", "frames_per_s": line["value"],
              "ms_per_step": line["ms_per_step"], "GBps": line["roofline"]["achieved"],
              "launches_per_step": line["config"]["launches_per_step"], "scaling": line["scaling"]})
    if want("d4"):
        fused_line("d4 4K batch", 64, 3, 2160, 3840)
    if want("f1"):
        fused_line("f1 HD uint8 input", 300, 3, 1080, 1920, dtype=torch.uint8)
        fused_line("f1 HD uint8 input, int16 output", 300, 3, 1080, 1920, dtype=torch.uint8, out_dtype=torch.int16)
    if want("f4"):
        fused_line("f4 CIF 2000 frames", 2000, 3, 288, 352)
    if want("f1p"):
        # packed 24-bit pixels [N][H][W][3] straight into the fused kernel (AOL_RGB8)
        N, H, W = 300, 1080, 1920
        xp = aol.synth_frames(3, 0, N, 3, H, W, dtype=torch.uint8).permute(0, 2, 3, 1).contiguous()
        z = torch.empty((N, 3, 480, 720), dtype=torch.int32, device="cuda")
        cs = torch.empty(N, dtype=torch.uint64, device="cuda")
        med, mn = timed(lambda: aol.downscale_frame_packed(xp, out=z, checksums=cs), inner=5)
        b = frames_bytes(N, 3, H, W, 1, 4)
        emit({"config": "f1 HD packed 24-bit pixels (AOL_RGB8)", "shape": [N, H, W, 3], "timing": "5 calls back to back",
              "ms": med, "min_ms": mn, "frames_per_s": N / (med / 1e3), "GBps": b / (med / 1e3) / 1e9,
              "frac": b / (med / 1e3) / 1e9 / peak(), "plan": aol.downscale_frame_plan(N, 3, H, W, dtype="rgb8")})
        del xp, z, cs
        torch.cuda.empty_cache()


if __name__ == "__main__":
    main()
