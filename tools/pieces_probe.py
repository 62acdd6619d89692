#!/usr/bin/env python
"""A/B probe for wrapping d3 blockings (array [64,1024,1024] int32, 8x8 tiles): gather and FAST scatter time
per origin and which kernel ran; run once with AOL_TILER_PIECES=0 (box kernel) and once without (the setting is
read once per process).  One JSON line per origin."""
import json
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_guortgbs11_b200 as aol  # noqa: E402

arr, rep, pat = [64, 1024, 1024], [64, 128, 128], [8, 8]
P, F = [[1, 0, 0], [0, 8, 0], [0, 0, 8]], [[0, 0], [1, 0], [0, 1]]
A = torch.randint(0, 1 << 30, tuple(arr), dtype=torch.int32, device="cuda")
G = torch.empty(tuple(rep + pat), dtype=torch.int32, device="cuda")
B = torch.zeros_like(A)
nbytes = 2 * A.numel() * 4


def t_ms(fn, reps=10, trials=15):
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


origins = [[0, 0, 0], [0, -3, 5], [0, -3, 4], [0, 0, 5], [0, -3, 0]]
if len(sys.argv) > 1 and sys.argv[1] == "--once":   # one gather + one FAST scatter per origin (ncu captures)
    for origin in origins[1:3]:
        t = aol.make_tiler(arr, rep, pat, origin, P, F)
        aol.tiler_gather(t, A, out=G)
        aol.tiler_scatter(t, G, B, mode="fast")
    torch.cuda.synchronize()
    sys.exit(0)
for origin in origins:
    for pieces in (os.environ.get("AOL_TILER_PIECES", "1"),):
        t = aol.make_tiler(arr, rep, pat, origin, P, F)
        g = t_ms(lambda: aol.tiler_gather(t, A, out=G))
        aol.tiler_gather(t, A, out=G)
        kg = aol.last_kernel()
        f = t_ms(lambda: aol.tiler_scatter(t, G, B, mode="fast"))
        aol.tiler_scatter(t, G, B, mode="fast")
        kf = aol.last_kernel()
        print(json.dumps({"origin": origin, "pieces": pieces, "gather_ms": round(g, 5), "gather_kernel": kg,
                          "gather_TBps": round(nbytes / g / 1e9, 3), "fast_ms": round(f, 5), "fast_kernel": kf,
                          "fast_TBps": round(nbytes / f / 1e9, 3)}), flush=True)
