"""Cost of the fused checksum epilogue: the same launches with and without per-frame checksums, alternated."""
import json
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import bench  # noqa: E402
import paper_conf_ipps_guortgbs11_b200 as aol  # noqa: E402

for dt, odt, packed in ((torch.uint8, torch.int32, False), (torch.int32, torch.int32, False),
                        (torch.uint8, torch.int16, False), (torch.uint8, torch.int32, True)):
    x = aol.synth_frames(0, 0, 300, 3, 1080, 1920, dtype=dt)
    fn = aol.downscale_frame
    if packed:
        x = x.permute(0, 2, 3, 1).contiguous()
        fn = aol.downscale_frame_packed
    z = torch.empty((300, 3, 480, 720), dtype=odt, device="cuda")
    z2 = torch.empty_like(z)
    cs = torch.empty(300, dtype=torch.uint64, device="cuda")
    res = {"in": str(dt), "out": str(odt), "packed": packed, "checksum": [], "no_checksum": [], "no_checksum_1": []}
    for _ in range(3):
        res["checksum"].append(bench.timed(lambda: fn(x, out=z, checksums=cs), inner=5)[0])
        res["no_checksum"].append(bench.timed(lambda: fn(x, out=z2), inner=5)[0])
        res["no_checksum_1"].append(bench.timed(lambda: fn(x, out=z2), inner=1)[0])
    torch.cuda.synchronize()
    res["same_output"] = bool(torch.equal(z, z2))
    res["last_kernel"] = aol.last_kernel()
    print(json.dumps(res))
    del x, z, z2
    torch.cuda.empty_cache()
