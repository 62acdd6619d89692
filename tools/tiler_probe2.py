#!/usr/bin/env python
"""Generic tiler gather/scatter rates for a few linear descriptors on 256 MiB int32 arrays (d3 context):
identity (contiguous both sides), the d3 8x8 blocking, and a 32x32 blocking; plus torch's copy_ for scale."""
import json
import os
import statistics
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_guortgbs11_b200 as aol  # noqa: E402


def timed(fn, reps=20):
    for _ in range(3):
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


A = torch.randint(0, 1 << 30, (64, 1024, 1024), dtype=torch.int32, device="cuda")
nb = 2 * A.numel() * 4
B = torch.empty_like(A)
print(json.dumps({"case": "torch copy_", "ms": timed(lambda: B.copy_(A)), "GBps": nb / timed(lambda: B.copy_(A)) / 1e6}))
cases = {
    "identity": ([64, 1024, 1024], [64, 1024], [1024], [0, 0, 0], [[1, 0], [0, 1], [0, 0]], [[0], [0], [1]],
                 (64, 1024, 1024)),
    "d3 8x8 blocks": ([64, 1024, 1024], [64, 128, 128], [8, 8], [0, 0, 0], [[1, 0, 0], [0, 8, 0], [0, 0, 8]],
                      [[0, 0], [1, 0], [0, 1]], (64, 128, 128, 8, 8)),
    "32x32 blocks": ([64, 1024, 1024], [64, 32, 32], [32, 32], [0, 0, 0], [[1, 0, 0], [0, 32, 0], [0, 0, 32]],
                     [[0, 0], [1, 0], [0, 1]], (64, 32, 32, 32, 32)),
}
for name, (arr, rep, pat, o, P, F, gshape) in cases.items():
    t = aol.make_tiler(arr, rep, pat, o, P, F)
    G = torch.empty(gshape, dtype=torch.int32, device="cuda")
    tg = timed(lambda: aol.tiler_gather(t, A, out=G))
    ts = timed(lambda: aol.tiler_scatter(t, G, B, mode="fast"))
    print(json.dumps({"case": name, "gather_ms": tg, "gather_GBps": nb / tg / 1e6, "scatter_ms": ts,
                      "scatter_GBps": nb / ts / 1e6, "roundtrip_ok": bool(torch.equal(A, B))}))
