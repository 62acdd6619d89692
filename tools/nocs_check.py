"""8-bit samples with int32 outputs, with and without checksums, HD and 4K (the no-checksum ring depth)."""
import json
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import bench  # noqa: E402
import paper_conf_ipps_guortgbs11_b200 as aol  # noqa: E402

for N, H, W in ((300, 1080, 1920), (64, 2160, 3840), (2000, 288, 352)):
    x = aol.synth_frames(0, 0, N, 3, H, W, dtype=torch.uint8)
    z = torch.empty((N, 3, 4 * H // 9, 3 * W // 8), dtype=torch.int32, device="cuda")
    z2 = torch.empty_like(z)
    cs = torch.empty(N, dtype=torch.uint64, device="cuda")
    a = bench.timed(lambda: aol.downscale_frame(x, out=z, checksums=cs), inner=5)[0]
    b = bench.timed(lambda: aol.downscale_frame(x, out=z2), inner=5)[0]
    torch.cuda.synchronize()
    print(json.dumps({"shape": [N, 3, H, W], "ms_checksum": a, "ms_no_checksum": b, "same": bool(torch.equal(z, z2))}))
    del x, z, z2
    torch.cuda.empty_cache()
