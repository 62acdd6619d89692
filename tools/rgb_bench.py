import json, os, sys, statistics
sys.path.insert(0, os.getcwd())
import torch
import paper_conf_ipps_guortgbs11_b200 as aol
N, H, W = 300, 1080, 1920
xp = aol.synth_frames(0, 0, N, 3, H, W, dtype=torch.uint8)
packed = xp.permute(0, 2, 3, 1).contiguous()
z = torch.empty((N, 3, 480, 720), dtype=torch.int32, device="cuda")
cs = torch.empty(N, dtype=torch.uint64, device="cuda")
def t(fn, reps=20):
    for _ in range(3): fn()
    torch.cuda.synchronize()
    ts = []
    for _ in range(reps):
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record(); [fn() for _ in range(5)]; b.record(); torch.cuda.synchronize(); ts.append(a.elapsed_time(b) / 5)
    return statistics.median(ts)
ms_packed = t(lambda: aol.downscale_frame_packed(packed, out=z, checksums=cs))
cs1 = cs.clone()
ms_planar = t(lambda: aol.downscale_frame(xp, out=z, checksums=cs))
print(json.dumps({"packed_ms": ms_packed, "planar_u8_ms": ms_planar, "packed_fps": N / ms_packed * 1e3,
                  "same_checksums": bool(torch.equal(cs1.view(torch.int64), cs.view(torch.int64))),
                  "plan": aol.downscale_frame_plan(N, 3, H, W, dtype=torch.uint8)}))
