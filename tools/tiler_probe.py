#!/usr/bin/env python
"""The d3 perf instance, for ncu: array {64,1024,1024} i32 -> 8x8 tiles; 3 gathers + 3 FAST scatters."""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_guortgbs11_b200 as aol  # noqa: E402

t = aol.make_tiler([64, 1024, 1024], [64, 128, 128], [8, 8], [0, 0, 0],
                   [[1, 0, 0], [0, 8, 0], [0, 0, 8]], [[0, 0], [1, 0], [0, 1]])
A = torch.randint(0, 1 << 30, (64, 1024, 1024), dtype=torch.int32, device="cuda")
G = torch.empty((64, 128, 128, 8, 8), dtype=torch.int32, device="cuda")
for _ in range(3):
    aol.tiler_gather(t, A, out=G)
for _ in range(3):
    aol.tiler_scatter(t, G, A, mode="fast")
torch.cuda.synchronize()
print("ok")
