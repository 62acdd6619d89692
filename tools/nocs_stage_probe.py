"""u8 -> int32 (planar and packed) without checksums: ring depth sweep (the no-checksum consumer runs ahead)."""
import json
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import bench  # noqa: E402
import paper_conf_ipps_guortgbs11_b200 as aol  # noqa: E402

x8 = aol.synth_frames(0, 0, 300, 3, 1080, 1920, dtype=torch.uint8)
xp = x8.permute(0, 2, 3, 1).contiguous()
z = torch.empty((300, 3, 480, 720), dtype=torch.int32, device="cuda")
cs = torch.empty(300, dtype=torch.uint64, device="cuda")
for name, fn, x in (("planar", aol.downscale_frame, x8), ("packed", aol.downscale_frame_packed, xp)):
    for st in (0, 2, 3, 4, 6, 8, 11):
        o = {"stages": st} if st else None
        for c in (None, cs):
            try:
                ms = bench.timed(lambda: fn(x, out=z, checksums=c, opts=o), inner=5)[0]
            except Exception as e:
                ms = str(e)[:80]
            print(json.dumps({"layout": name, "stages": st, "checksums": c is not None, "ms": ms}), flush=True)
