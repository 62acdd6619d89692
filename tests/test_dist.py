"""Multi-process (gloo, world size 2, CPU) coverage of the frame-sharded path's host logic.

Each rank processes its own contiguous block of global frames (here with the
CPU oracle standing in for the GPU kernel -- the logic under test is the
sharding, the global frame indexing of the generator, and the gather), then the
ranks gather checksums and max elapsed time exactly as bench.py does.
"""
import os
import socket

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

from paper_conf_ipps_guortgbs11_b200 import shard


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _worker(rank, world, port, mode, total, result_q):
    import oracle
    import synth

    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        C, H, W = 3, 18, 32
        if mode == "weak":
            f0, n = shard.weak_range(rank, world, total)
            counts = None
        else:
            f0, n = shard.strong_range(rank, world, total)
            counts = [shard.strong_range(r, world, total)[1] for r in range(world)]
        x = synth.frames(42, f0, n, C, H, W)
        _, cs = oracle.downscale_frame(x)
        elapsed = 10.0 + rank  # stand-in for a device-timed region
        mx, allcs = shard.gather_results(torch.from_numpy(cs.view(np.int64)), elapsed, counts=counts)
        if rank == 0:
            result_q.put((mx, allcs.numpy().view(np.uint64).copy()))
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("mode,total", [("weak", 3), ("strong", 7)])
def test_sharded_checksums_match_single_process(mode, total):
    world = 2
    ctx = mp.get_context("spawn")
    q = ctx.SimpleQueue()
    port = _free_port()
    procs = [ctx.Process(target=_worker, args=(r, world, port, mode, total, q)) for r in range(world)]
    for p in procs:
        p.start()
    for p in procs:
        p.join(timeout=300)
        assert p.exitcode == 0
    mx, allcs = q.get()
    assert mx == 11.0                                   # max over ranks
    import oracle
    import synth

    n_all = world * total if mode == "weak" else total
    _, ref = oracle.downscale_frame(synth.frames(42, 0, n_all, 3, 18, 32))
    assert np.array_equal(allcs, ref)


def test_ranges_partition_the_stream():
    for world in (1, 2, 3, 4, 8):
        for total in (0, 1, 7, 300, 10000):
            blocks = [shard.strong_range(r, world, total) for r in range(world)]
            assert sum(n for _, n in blocks) == total
            pos = 0
            for f0, n in blocks:
                assert f0 == pos
                pos += n
            assert max(n for _, n in blocks) - min(n for _, n in blocks) <= 1
        assert [shard.weak_range(r, world, 300)[0] for r in range(world)] == [300 * r for r in range(world)]
    with pytest.raises(ValueError):
        shard.strong_range(2, 2, 10)


def test_gather_single_process():
    cs = torch.tensor([1, 2, 3], dtype=torch.int64)
    mx, out = shard.gather_results(cs, 5.0)
    assert mx == 5.0 and torch.equal(out, cs)
