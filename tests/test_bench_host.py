"""bench.py's host-side logic on CPU: sub-record selection, the shared config object of both arms, the
source-tree hash that guards quoted ncu captures, and the reference arm (the CPU oracle) end to end."""
import json
import os
import subprocess
import sys

import numpy as np

from conftest import ROOT

sys.path.insert(0, ROOT)
import bench  # noqa: E402


def test_extras_selection():
    assert bench.extras_of(bench.parse([])) == ["d1", "d3", "d4", "d5", "wide", "f1", "f3", "f4"]
    assert bench.extras_of(bench.parse(["--H", "36", "--W", "128"])) == []
    assert bench.extras_of(bench.parse(["--dtype", "u8"])) == []
    assert bench.extras_of(bench.parse(["--extras", "d1,d5"])) == ["d1", "d5"]
    assert bench.extras_of(bench.parse(["--extras", "none"])) == []
    assert bench.extras_of(bench.parse(["--H", "36", "--extras", "all"])) == ["d1", "d3", "d4", "d5", "wide", "f1", "f3", "f4"]


def test_src_hash_and_stale_capture_guard(tmp_path, monkeypatch):
    h = bench.src_hash()
    assert h == bench.src_hash() and len(h) == 16
    a = bench.parse([])
    plan = {"kernel": 1, "grid": 148, "block": 288, "smem_bytes": 1, "stages": 5, "bands_per_unit": 10,
            "ctas_per_sm": 1}
    prof = tmp_path / "profiles"
    prof.mkdir()
    entry = {"dram_bytes_per_launch": 8.7e9, "dram_pct_of_peak": 86.0, "tag": "t", "src_hash": h,
             "plan": bench.plan_key(plan)}
    (prof / "ncu_traffic.json").write_text(json.dumps({bench.traffic_key(a): entry}))
    monkeypatch.setattr(bench, "ROOT", str(tmp_path))
    monkeypatch.setattr(bench, "src_hash", lambda: h)
    assert bench.ncu_traffic(a, plan)[0] == 8.7e9
    assert bench.ncu_traffic(a, dict(plan, stages=6))[0] is None            # another launch plan
    monkeypatch.setattr(bench, "src_hash", lambda: "0" * 16)
    t, _, _, status = bench.ncu_traffic(a, plan)                             # another source tree
    assert t is None and "another source tree" in status


def test_bytes_per_frame_matches_survey():
    # 29,030,400 B per HD int32 frame; 116,121,600 per 4K frame
    assert bench.bytes_per_frame(bench.parse([])) == 29030400
    assert bench.frame_bytes(3, 2160, 3840) == 116121600
    assert bench.bytes_per_frame(bench.parse(["--dtype", "u8", "--out-dtype", "i16"])) == 3 * (1080 * 1920 + 480 * 720 * 2)


def test_reference_arm_runs_the_oracle_on_the_same_config():
    r = subprocess.run([sys.executable, os.path.join(ROOT, "bench.py"), "--impl", "reference", "--frames", "6",
                        "--H", "36", "--W", "128", "--steps", "3", "--warmup", "3"],
                       capture_output=True, text=True, timeout=600, cwd=ROOT)
    assert r.returncode == 0, r.stderr[-3000:]
    lines = [l for l in r.stdout.strip().splitlines() if l.startswith("{")]
    assert len(lines) == 1
    d = json.loads(lines[0])
    a = bench.parse(["--frames", "6", "--H", "36", "--W", "128"])
    assert d["impl"] == "reference" and d["value"] > 0 and d["steps"] == 3 and d["warmup"] == 3
    assert d["config"] == json.loads(json.dumps(bench.workload_config(a, 1)))   # same object as the GPU arm's
    assert d["cpu_baseline"]["value"] == d["value"] and d["cpu_baseline"]["kind"] == "oracle"
    assert d["e2e"] == {"value": d["value"], "unit": "frames/s", "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0}


def test_oracle_checksums_chunked_equals_one_call(orc):
    """The cpu_baseline leg's chunked oracle run (C generator, chunks of frames, an index list) gives the same
    checksums as one oracle call on the numpy generator's frames."""
    import synth

    idx = [3, 0, 7, 7, 2]
    cs, spent = bench.oracle_checksums(5, idx, 3, 18, 64, nthreads=2, chunk=2)
    x = np.concatenate([synth.frames(5, g, 1, 3, 18, 64) for g in idx])
    _, want = orc.downscale_frame(x)
    assert np.array_equal(cs, want) and spent > 0
