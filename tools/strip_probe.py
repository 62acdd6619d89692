#!/usr/bin/env python
"""Column-strip fused kernel: frames/s and algorithmic TB/s for 8K DCI int32 frames (4320 x 8192 x 3) and, for
comparison, 4K (2160 x 3840) through the default kernel; one JSON line per case.  AOL_STRIP_REPS (env) sets the
strip width for A/B runs."""
import json
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_guortgbs11_b200 as aol  # noqa: E402


def t_ms(fn, reps=5, trials=9):
    for _ in range(3):
        fn()
    s, e = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    out = []
    for _ in range(trials):
        s.record()
        for _ in range(reps):
            fn()
        e.record()
        e.synchronize()
        out.append(s.elapsed_time(e) / reps)
    return sorted(out)[len(out) // 2]


for (N, H, W) in [(16, 4320, 8192), (64, 2160, 3840), (32, 4320, 7680)]:
    x = aol.synth_frames(0, 0, N, 3, H, W)
    z = torch.empty((N, 3, 4 * (H // 9), 3 * (W // 8)), dtype=torch.int32, device="cuda")
    cs = torch.empty(N, dtype=torch.uint64, device="cuda")
    p = aol.downscale_frame_plan(N, 3, H, W)
    ms = t_ms(lambda: aol.downscale_frame(x, out=z, checksums=cs))
    nbytes = x.numel() * 4 + z.numel() * 4
    print(json.dumps({"N": N, "H": H, "W": W, "ms": round(ms, 4), "fps": round(N / ms * 1e3, 1),
                      "TBps": round(nbytes / ms / 1e9, 3), "plan": p,
                      "strip_reps": os.environ.get("AOL_STRIP_REPS", "default")}), flush=True)
    del x, z
    torch.cuda.empty_cache()
