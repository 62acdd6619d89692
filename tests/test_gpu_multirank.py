"""The multi-rank bench path on one GPU: bench.py under torch.distributed.run with two ranks sharing the
box's single B200 over gloo (AOL_DIST_BACKEND=gloo; the driver's scaling runs use NCCL, one GPU per rank).
Covers the frame sharding (weak: disjoint 'frames per GPU' blocks; strong: the configs[4] stream split
into contiguous blocks cycling through per-rank device pools), the max-over-ranks timing and the checksum
gather, and checks every gathered checksum against the CPU oracle."""
import json
import os
import socket
import subprocess
import sys

import numpy as np
import pytest

import synth
from conftest import ROOT

pytestmark = pytest.mark.gpu

C, H, W = 3, 36, 256


def _port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def run2(tmp_path, *args):
    dump = str(tmp_path / "cs.npy")
    env = dict(os.environ, AOL_DIST_BACKEND="gloo")
    cmd = [sys.executable, "-m", "torch.distributed.run", "--nnodes=1", "--nproc-per-node", "2",
           "--master-addr", "127.0.0.1", "--master-port", str(_port()), os.path.join(ROOT, "bench.py"),
           "--gpus", "2", "--H", str(H), "--W", str(W), "--steps", "3", "--warmup", "3", "--no-cpu-baseline",
           "--dump-checksums", dump, *args]
    r = subprocess.run(cmd, capture_output=True, text=True, timeout=600, cwd=ROOT, env=env)
    assert r.returncode == 0, r.stderr[-3000:]
    lines = [l for l in r.stdout.strip().splitlines() if l.startswith("{")]
    assert len(lines) == 1, r.stdout
    return json.loads(lines[0]), np.load(dump)


def test_weak_two_ranks(orc, tmp_path):
    d, cs = run2(tmp_path, "--frames", "5")
    assert d["n_gpus"] == 2 and d["scaling"] == "weak" and d["gathered_checksums"] == 10
    assert d["value"] > 0 and d["e2e"]["checksums_match_device_path"] is True
    _, ref = orc.downscale_frame(synth.frames(0, 0, 10, C, H, W), nthreads=8)   # global frames 0..9
    assert np.array_equal(cs, ref)


def test_strong_stream_two_ranks(orc, tmp_path):
    # 23 stream frames: rank 0 owns global frames 0..11, rank 1 owns 12..22; pools of 4 frames per rank
    d, cs = run2(tmp_path, "--stream-frames", "23", "--pool", "4")
    assert d["scaling"] == "strong" and d["launch"]["launches_per_step"] == 3 and d["gpu_launches"] == 18
    _, ref0 = orc.downscale_frame(synth.frames(0, 0, 4, C, H, W), nthreads=8)
    _, ref1 = orc.downscale_frame(synth.frames(0, 12, 4, C, H, W), nthreads=8)
    assert np.array_equal(cs, np.concatenate([ref0, ref1]))


@pytest.mark.parametrize("mode", ["weak", "strong"])
def test_nccl_collectives_single_rank(orc, tmp_path, mode):
    """The NCCL code path of the multi-GPU bench (process group on the GPU, barrier, float64 MAX all-reduce,
    int64 checksum all-gather incl. the ragged strong-scaling gather) as a single rank on this one-GPU box
    (AOL_FORCE_DIST=1; NCCL cannot put two ranks on one GPU), checksums against the oracle."""
    dump = str(tmp_path / "cs.npy")
    env = dict(os.environ, AOL_FORCE_DIST="1")
    env.pop("AOL_DIST_BACKEND", None)
    extra = ["--frames", "4"] if mode == "weak" else ["--stream-frames", "7", "--pool", "3"]
    cmd = [sys.executable, "-m", "torch.distributed.run", "--nnodes=1", "--nproc-per-node", "1",
           "--master-addr", "127.0.0.1", "--master-port", str(_port()), os.path.join(ROOT, "bench.py"),
           "--H", str(H), "--W", str(W), "--steps", "3", "--warmup", "3", "--no-cpu-baseline",
           "--dump-checksums", dump, *extra]
    r = subprocess.run(cmd, capture_output=True, text=True, timeout=600, cwd=ROOT, env=env)
    assert r.returncode == 0, r.stderr[-3000:]
    d = json.loads([l for l in r.stdout.strip().splitlines() if l.startswith("{")][-1])
    n = 4 if mode == "weak" else 3
    assert d["gathered_checksums"] == n and d["value"] > 0
    _, ref = orc.downscale_frame(synth.frames(0, 0, n, C, H, W), nthreads=8)
    assert np.array_equal(np.load(dump), ref)
