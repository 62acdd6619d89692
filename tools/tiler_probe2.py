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
    # origin (0, -3, 5): the d3 blocking shifted so that tiles wrap toroidally in both image dims
    "d3 8x8 blocks wrapping": ([64, 1024, 1024], [64, 128, 128], [8, 8], [0, -3, 5], [[1, 0, 0], [0, 8, 0], [0, 0, 8]],
                               [[0, 0], [1, 0], [0, 1]], (64, 128, 128, 8, 8)),
}
tag = {"wrap32": os.environ.get("AOL_TILER_WRAP32", "1"), "wraptab": os.environ.get("AOL_TILER_WRAPTAB", "1")}
for name, (arr, rep, pat, o, P, F, gshape) in cases.items():
    t = aol.make_tiler(arr, rep, pat, o, P, F)
    G = torch.empty(gshape, dtype=torch.int32, device="cuda")
    tg = timed(lambda: aol.tiler_gather(t, A, out=G))
    ts = timed(lambda: aol.tiler_scatter(t, G, B, mode="fast"))
    print(json.dumps({"case": name, **tag, "gather_ms": tg, "gather_GBps": nb / tg / 1e6, "scatter_ms": ts,
                      "scatter_GBps": nb / ts / 1e6, "roundtrip_ok": bool(torch.equal(A, B))}))
# uint8 elements (the d3 blocking on a 64 MiB byte array: 8-byte tile rows, no 16-byte vectors)
A8 = A.to(torch.uint8)
t = aol.make_tiler(*cases["d3 8x8 blocks"][:6])
G8 = torch.empty(cases["d3 8x8 blocks"][6], dtype=torch.uint8, device="cuda")
tg = timed(lambda: aol.tiler_gather(t, A8, out=G8))
print(json.dumps({"case": "d3 8x8 blocks u8", **tag, "gather_ms": tg, "gather_GBps": 2 * A8.numel() / tg / 1e6}))
# the paper's H input tiler (Fig. 10: pattern 11 every 8 columns, overlapping) over 64 HD planes
del B, G
X = torch.randint(0, 1 << 30, (64, 1080, 1920), dtype=torch.int32, device="cuda")
th = aol.make_tiler([64, 1080, 1920], [64, 1080, 240], [11], [0, 0, 0], [[1, 0, 0], [0, 1, 0], [0, 0, 8]],
                    [[0], [0], [1]])
GH = torch.empty((64, 1080, 240, 11), dtype=torch.int32, device="cuda")
tg = timed(lambda: aol.tiler_gather(th, X, out=GH))
print(json.dumps({"case": "H_IN tiler 64 HD planes", **tag, "gather_ms": tg,
                  "gather_GBps": (X.numel() + GH.numel()) * 4 / tg / 1e6}))
# the V input tiler (reading Z1: pattern 12 every 9 rows, wrapping at the last band) over 64 planes 1080 x 720
Y = X.view(-1)[: 64 * 1080 * 720].view(64, 1080, 720)
tv = aol.make_tiler([64, 1080, 720], [64, 120, 720], [12], [0, 0, 0], [[1, 0, 0], [0, 9, 0], [0, 0, 1]],
                    [[0], [1], [0]])
del GH
GV = torch.empty((64, 120, 720, 12), dtype=torch.int32, device="cuda")
tg = timed(lambda: aol.tiler_gather(tv, Y, out=GV))
print(json.dumps({"case": "V_IN tiler 64 planes 1080x720", **tag, "gather_ms": tg,
                  "gather_GBps": (Y.numel() + GV.numel()) * 4 / tg / 1e6}))
