#!/usr/bin/env python
"""Practical HBM ceilings on this box for the downscaler's traffic mix (context for roofline.frac).

Times with CUDA events (median of 20, after warm-up):
  read   : int32 sum over the 7.46 GB input (torch reduction, read-only stream)
  write  : fill of a 1.24 GB int32 output (write-only stream)
  copy   : 1 GiB bf16 copy (the MEASURED_PEAKS.json definition, read+write)
  mix    : read 7.46 GB + write 1.24 GB in one pass (torch: z.copy_(x[..., :Wo-slice]) is not the same
           mix, so the mix ceiling is estimated as total / (read_time + write_time) -- a lower bound).
"""
import json
import statistics
import sys

import torch


def t_ms(fn, reps=20):
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


def main():
    x = torch.randint(0, 255, (300, 3, 1080, 1920), dtype=torch.int32, device="cuda")
    z = torch.empty((300, 3, 480, 720), dtype=torch.int32, device="cuda")
    a = torch.empty(1 << 30, dtype=torch.bfloat16, device="cuda")
    b = torch.empty_like(a)
    rb, wb = x.numel() * 4, z.numel() * 4
    xf = x.view(torch.float32)
    r = t_ms(lambda: xf.sum())
    r2 = t_ms(lambda: x.amax())
    w = t_ms(lambda: z.fill_(1))
    c = t_ms(lambda: b.copy_(a))
    out = {"read_GBps": rb / r / 1e6, "read_amax_GBps": rb / r2 / 1e6, "write_GBps": wb / w / 1e6, "copy_GBps": 2 * a.numel() * 2 / c / 1e6,
           "mix_lower_bound_GBps": (rb + wb) / (r + w) / 1e6, "read_ms": r, "write_ms": w,
           "downscale_floor_ms_at_read_write_rates": r + w}
    print(json.dumps(out))


if __name__ == "__main__":
    sys.exit(main())
