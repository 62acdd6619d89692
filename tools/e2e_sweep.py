#!/usr/bin/env python
"""Host-streamed end-to-end rate (aol_downscale_frame_host) vs chunk size, int32 and uint8, 300 HD frames."""
import json
import os
import sys
import time

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_guortgbs11_b200 as aol  # noqa: E402

N, C, H, W = 300, 3, 1080, 1920
for dt in (torch.int32, torch.uint8):
    xd = aol.synth_frames(0, 0, N, C, H, W, dtype=dt)
    xh = torch.empty(xd.shape, dtype=dt, pin_memory=True)
    xh.copy_(xd)
    del xd
    zh = torch.empty((N, C, 480, 720), dtype=torch.int32, pin_memory=True)
    streams = [torch.cuda.Stream() for _ in range(3)]
    for chunk in (5, 10, 20, 50, 100):
        ws = torch.empty(aol.host_workspace_bytes(chunk, C, H, W, dt), dtype=torch.uint8, device="cuda")
        aol.downscale_frame_host(xh, out=zh, chunk_frames=chunk, workspace=ws, streams=streams)
        t0 = time.perf_counter()
        for _ in range(3):
            aol.downscale_frame_host(xh, out=zh, chunk_frames=chunk, workspace=ws, streams=streams)
        dt_s = (time.perf_counter() - t0) / 3
        print(json.dumps({"dtype": str(dt), "chunk": chunk, "frames_per_s": N / dt_s,
                          "h2d_GBps": xh.numel() * xh.element_size() / dt_s / 1e9}), flush=True)
        del ws
