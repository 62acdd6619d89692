"""One u8 -> int32 launch (300 HD frames) with or without checksums, for ncu (argv[1] = 'cs' or 'nocs')."""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_guortgbs11_b200 as aol  # noqa: E402

x = aol.synth_frames(0, 0, 300, 3, 1080, 1920, dtype=torch.uint8)
z = torch.empty((300, 3, 480, 720), dtype=torch.int32, device="cuda")
cs = torch.empty(300, dtype=torch.uint64, device="cuda") if sys.argv[1] == "cs" else None
for _ in range(4):
    aol.downscale_frame(x, out=z, checksums=cs)
torch.cuda.synchronize()
