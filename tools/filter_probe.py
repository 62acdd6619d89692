#!/usr/bin/env python
"""f3 generic filter on 60 HD frames (for ncu)."""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_guortgbs11_b200 as aol  # noqa: E402

N, C, H, W = 60, 3, 1080, 1920
x = aol.synth_frames(0, 0, N, C, H, W).reshape(N * C, H, W)
fh = aol.filter_preset(aol.FILTER_H, N * C, H, W)
fv = aol.filter_preset(aol.FILTER_V, N * C, H, 720)
y = torch.empty((N * C, H, 720), dtype=torch.int32, device="cuda")
z = torch.empty((N * C, 480, 720), dtype=torch.int32, device="cuda")
for _ in range(2):
    aol.filter_apply(fh, x, out=y)
    aol.filter_apply(fv, y, out=z)
torch.cuda.synchronize()
print("ok")
