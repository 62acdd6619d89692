#!/usr/bin/env python
"""Single-HD-frame latency (device time per call, CUDA graph of 20 calls) across launch options."""
import json
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_guortgbs11_b200 as aol  # noqa: E402


def graph_us(x, z, cs, opts, fn=None):
    g = torch.cuda.CUDAGraph()
    s = torch.cuda.Stream()
    s.wait_stream(torch.cuda.current_stream())
    with torch.cuda.stream(s):
        call = fn or (lambda: aol.downscale_frame(x, out=z, checksums=cs, opts=opts))
        call()
        torch.cuda.synchronize()
        with torch.cuda.graph(g, stream=s):
            for _ in range(20):
                call()
    torch.cuda.synchronize()
    ts = []
    for _ in range(10):
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record()
        g.replay()
        b.record()
        torch.cuda.synchronize()
        ts.append(a.elapsed_time(b) * 1000 / 20)
    return sorted(ts)[len(ts) // 2]


x = aol.synth_frames(0, 0, 1, 3, 1080, 1920)
z = torch.empty((1, 3, 480, 720), dtype=torch.int32, device="cuda")
cs = torch.empty(1, dtype=torch.uint64, device="cuda")
for opts in [None, {"flags": 64}, {"ctas_per_sm": 2}, {"ctas_per_sm": 2, "bands_per_unit": 1}, {"ctas_per_sm": 2, "bands_per_unit": 2},
             {"ctas_per_sm": 3, "bands_per_unit": 1}, {"bands_per_unit": 1}, {"bands_per_unit": 2}, {"stages": 3},
             {"flags": 512}, {"flags": 512, "stages": 8}, {"flags": 512, "ctas_per_sm": 2, "bands_per_unit": 1},
             {"flags": 512, "ctas_per_sm": 2, "bands_per_unit": 2}, {"flags": 512, "ctas_per_sm": 3, "bands_per_unit": 1},
             {"flags": 128}, {"flags": 128 | 512, "ctas_per_sm": 2, "bands_per_unit": 1}]:
    us = graph_us(x, z, cs, opts)
    print(json.dumps({"opts": opts, "us_per_call": us, "plan": aol.downscale_frame_plan(1, 3, 1080, 1920, opts=opts)}))

print(json.dumps({"opts": "no checksum", "us_per_call": graph_us(x, z, None, None), "plan": aol.downscale_frame_plan(1, 3, 1080, 1920)}))
print(json.dumps({"opts": "memset only", "us_per_call": graph_us(x, z, cs, None, fn=lambda: cs.zero_()), "plan": {}}))
xs = aol.synth_frames(0, 0, 1, 3, 36, 1920)
zs = torch.empty((1, 3, 16, 720), dtype=torch.int32, device="cuda")
print(json.dumps({"opts": "tiny frame 36x1920 no checksum", "us_per_call": graph_us(xs, zs, None, None), "plan": aol.downscale_frame_plan(1, 3, 36, 1920)}))
