"""Time the statically compiled separable chain (AOL_CHAIN_JIT=0) on the d2 workload (900 HD planes)."""
import json
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import bench  # noqa: E402
import paper_conf_ipps_guortgbs11_b200 as aol  # noqa: E402

P, H, W = 900, 1080, 1920
x = aol.synth_frames(0, 0, 300, 3, H, W).reshape(P, H, W)
fh = aol.filter_preset(aol.FILTER_H, P, H, W)
fv = aol.filter_preset(aol.FILTER_V, P, H, 3 * W // 8)
z = torch.empty((P, 4 * H // 9, 3 * W // 8), dtype=torch.int32, device="cuda")
aol.filter_chain_apply(fh, fv, x, out=z)
med, mn = bench.timed(lambda: aol.filter_chain_apply(fh, fv, x, out=z), inner=2, reps=10)
print(json.dumps({"lib": os.environ.get("AOL_LIB_PATH", "head"), "jit": os.environ.get("AOL_CHAIN_JIT", "1"),
                  "kernel": aol.last_kernel(), "ms": med}))
