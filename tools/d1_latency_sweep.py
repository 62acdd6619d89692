#!/usr/bin/env python
"""Single-HD-frame latency of ONE isolated call (CUDA events around it, a GPU sleep before so the host enqueue is
off the device timeline -- bench.py's d1 'warm' figure) across launch options; one JSON line per option."""
import json
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_guortgbs11_b200 as aol  # noqa: E402


def iso_us(fn, reps=60):
    for _ in range(5):
        fn()
    torch.cuda.synchronize()
    ts = []
    for _ in range(reps):
        torch.cuda._sleep(200000)
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record()
        fn()
        b.record()
        torch.cuda.synchronize()
        ts.append(a.elapsed_time(b) * 1000)
    ts.sort()
    return ts[len(ts) // 2]


x = aol.synth_frames(0, 0, 1, 3, 1080, 1920)
z = torch.empty((1, 3, 480, 720), dtype=torch.int32, device="cuda")
cs = torch.empty(1, dtype=torch.uint64, device="cuda")
for opts in [None, {"flags": 64}, {"ctas_per_sm": 2}, {"ctas_per_sm": 2, "bands_per_unit": 1},
             {"ctas_per_sm": 2, "bands_per_unit": 2}, {"ctas_per_sm": 3, "bands_per_unit": 1},
             {"bands_per_unit": 1}, {"bands_per_unit": 2}, {"stages": 3}, {"stages": 8}, {"flags": 512},
             {"flags": 512, "ctas_per_sm": 2, "bands_per_unit": 1}, {"ctas_per_sm": 4, "bands_per_unit": 1},
             {"flags": 2048}, {"flags": 2048, "bands_per_unit": 3}, {"flags": 2048, "bands_per_unit": 6}]:
    try:
        us = iso_us(lambda: aol.downscale_frame(x, out=z, checksums=cs, opts=opts))
        us0 = iso_us(lambda: aol.downscale_frame(x, out=z, opts=opts))
        print(json.dumps({"opts": opts, "iso_us": us, "iso_us_no_checksum": us0,
                          "plan": aol.downscale_frame_plan(1, 3, 1080, 1920, opts=opts)}), flush=True)
    except Exception as e:  # noqa: BLE001
        print(json.dumps({"opts": opts, "error": str(e)}), flush=True)
print(json.dumps({"opts": "empty call (memset of the checksum)", "iso_us": iso_us(lambda: cs.zero_())}), flush=True)
