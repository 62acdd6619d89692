#!/usr/bin/env python
"""f3 measurements: the paper's H and V filters as run-time descriptors over 300 HD frames' planes --
two aol_filter_apply launches (Y through HBM) vs one fused aol_filter_chain_apply -- and the specialised
fused kernel, one JSON line each.  --ncu: one call of each (for ncu captures), then the d3 box tilers."""
import json
import os
import statistics
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_guortgbs11_b200 as aol  # noqa: E402


def timed(fn, reps=10, warm=2):
    for _ in range(warm):
        fn()
    torch.cuda.synchronize()
    ts = []
    for _ in range(reps):
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record()
        fn()
        b.record()
        torch.cuda.synchronize()
        ts.append(a.elapsed_time(b))
    return statistics.median(ts)


ncu = "--ncu" in sys.argv
N, C, H, W = 300, 3, 1080, 1920
P = N * C
x = aol.synth_frames(0, 0, N, C, H, W).reshape(P, H, W)
fh = aol.filter_preset(aol.FILTER_H, P, H, W)
fv = aol.filter_preset(aol.FILTER_V, P, H, 720)
y = torch.empty((P, H, 720), dtype=torch.int32, device="cuda")
z = torch.empty((P, 480, 720), dtype=torch.int32, device="cuda")
z2 = torch.empty_like(z)
if ncu:
    aol.filter_chain_apply(fh, fv, x, out=z2)
    torch.cuda.synchronize()
    sys.exit(0)
peak = float(json.load(open(os.path.join(os.path.dirname(os.path.dirname(os.path.abspath(__file__))), "MEASURED_PEAKS.json")))["hbm_gbs"])
b = N * C * (H * W + 480 * 720) * 4
t2 = timed(lambda: (aol.filter_apply(fh, x, out=y), aol.filter_apply(fv, y, out=z)))
tc = timed(lambda: aol.filter_chain_apply(fh, fv, x, out=z2))
chain_kernel = aol.last_kernel()
zf, _ = aol.downscale_frame(x.reshape(N, C, H, W))
tf = timed(lambda: aol.downscale_frame(x.reshape(N, C, H, W), out=zf))
same = bool(torch.equal(z, z2) and torch.equal(z2, zf.reshape(P, 480, 720)))
for name, t in (("f3 generic filters, two launches (Y through HBM)", t2),
                (f"f3 fused chain (one launch, {chain_kernel})", tc),
                ("d2 specialised fused kernel", tf)):
    print(json.dumps({"config": name, "frames": N, "ms": t, "frames_per_s": N / t * 1e3, "GBps": b / t / 1e6,
                      "frac": b / t / 1e6 / peak, "equal": same}), flush=True)
