#!/usr/bin/env python
"""Every d3 tiler kernel bench.py times, once each after one warm-up, for `ncu --set full` captures:
blocking 8x8 gather / FAST / SEQUENTIAL, the same wrapping (origin (0,-3,5)), the paper's H input tiler over
64 HD planes, and the f3 run-time filters (H then V presets over 300 HD frames' planes)."""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_guortgbs11_b200 as aol  # noqa: E402

which = sys.argv[1] if len(sys.argv) > 1 else "all"
arr, rep, pat = [64, 1024, 1024], [64, 128, 128], [8, 8]
P, F = [[1, 0, 0], [0, 8, 0], [0, 0, 8]], [[0, 0], [1, 0], [0, 1]]
A = torch.randint(0, 1 << 30, tuple(arr), dtype=torch.int32, device="cuda")
G = torch.empty(tuple(rep + pat), dtype=torch.int32, device="cuda")
B = torch.zeros_like(A)
for origin in ([0, 0, 0], [0, -3, 5]):
    t = aol.make_tiler(arr, rep, pat, origin, P, F)
    for _ in range(2):
        aol.tiler_gather(t, A, out=G)
        aol.tiler_scatter(t, G, B, mode="fast")
        aol.tiler_scatter(t, G, B, mode="sequential")
del A, G, B
torch.cuda.empty_cache()
X = aol.synth_frames(0, 0, 64, 1, 1080, 1920).reshape(64, 1080, 1920)
th = aol.make_tiler([64, 1080, 1920], [64, 1080, 240], [11], [0, 0, 0], [[1, 0, 0], [0, 1, 0], [0, 0, 8]],
                    [[0], [0], [1]])
GH = torch.empty((64, 1080, 240, 11), dtype=torch.int32, device="cuda")
for _ in range(2):
    aol.tiler_gather(th, X, out=GH)
del X, GH
torch.cuda.empty_cache()
if which == "all":
    N = 300 * 3
    x = aol.synth_frames(0, 0, 300, 3, 1080, 1920).reshape(N, 1080, 1920)
    fh = aol.filter_preset(aol.FILTER_H, N, 1080, 1920)
    fv = aol.filter_preset(aol.FILTER_V, N, 1080, 720)
    y = torch.empty((N, 1080, 720), dtype=torch.int32, device="cuda")
    z = torch.empty((N, 480, 720), dtype=torch.int32, device="cuda")
    for _ in range(2):
        aol.filter_apply(fh, x, out=y)
        aol.filter_apply(fv, y, out=z)
torch.cuda.synchronize()
print("ok")
