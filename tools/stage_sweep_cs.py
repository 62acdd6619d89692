"""Ring-depth sweep with checksums for 8-bit-sample configurations (HD / 4K / CIF, int32 / int16 outputs)."""
import json
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import bench  # noqa: E402
import paper_conf_ipps_guortgbs11_b200 as aol  # noqa: E402

for N, H, W in ((300, 1080, 1920), (64, 2160, 3840), (2000, 288, 352)):
    x = aol.synth_frames(0, 0, N, 3, H, W, dtype=torch.uint8)
    cs = torch.empty(N, dtype=torch.uint64, device="cuda")
    for odt in (torch.int32, torch.int16):
        z = torch.empty((N, 3, 4 * H // 9, 3 * W // 8), dtype=odt, device="cuda")
        for st in (0, 3, 4, 6, 8, 11, 16):
            o = {"stages": st} if st else None
            try:
                ms = bench.timed(lambda: aol.downscale_frame(x, out=z, checksums=cs, opts=o), inner=5)[0]
                plan = aol.downscale_frame_plan(N, 3, H, W, dtype=torch.uint8, opts=o, out_dtype=odt)
            except Exception as e:
                ms, plan = str(e)[:60], None
            print(json.dumps({"shape": [N, H, W], "out": str(odt), "stages_opt": st, "ms": ms,
                              "stages": plan and plan["stages"], "cps": plan and plan["ctas_per_sm"]}), flush=True)
        del z
    del x
    torch.cuda.empty_cache()
