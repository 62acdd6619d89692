"""bench.py keeps its contract: one JSON line with the required keys, for the default (weak) mode, the
configs[4] stream mode and the reference arm.  Small shapes so this runs in seconds."""
import json
import os
import subprocess
import sys

import pytest

from conftest import ROOT

pytestmark = pytest.mark.gpu

REQUIRED = {"metric", "value", "unit", "n_gpus", "steps", "warmup", "ms_per_step", "higher_is_better", "scaling",
            "vs_baseline", "dtype", "data", "config", "roofline", "gpu_launches", "clocks"}


def run(*args):
    r = subprocess.run([sys.executable, os.path.join(ROOT, "bench.py"), *args], capture_output=True, text=True,
                       timeout=600, cwd=ROOT)
    assert r.returncode == 0, r.stderr[-3000:]
    lines = [l for l in r.stdout.strip().splitlines() if l.startswith("{")]
    assert len(lines) == 1, r.stdout
    return json.loads(lines[0])


def test_bench_default_contract():
    d = run("--frames", "12", "--H", "36", "--W", "128", "--steps", "5", "--warmup", "3", "--extras", "none")
    assert REQUIRED <= set(d)
    assert d["scaling"] == "weak" and d["n_gpus"] == 1 and d["higher_is_better"] is True
    assert d["value"] > 0 and d["gpu_launches"] == 10 and d["steps"] == 5 and d["warmup"] == 3
    r = d["roofline"]
    assert r["bound"] == "hbm" and r["unit"] == "GB/s" and abs(r["frac"] - r["achieved"] / r["peak"]) < 1e-9
    assert {"value", "unit", "h2d_bytes_per_step", "d2h_bytes_per_step"} <= set(d["e2e"])
    assert d["e2e"]["checksums_match_device_path"] is True
    assert 0.0 < d["e2e"]["frac_of_h2d_probe"] < 1.5
    cb = d["cpu_baseline"]
    assert cb["kind"] == "oracle" and cb["parity_all_frames"] is True and cb["frames_compared"] == 12
    assert cb["GBps_algorithmic"] > 0 and cb["cores"] >= 1
    assert d["config"]["workload"].startswith("12-frame 128x36")
    assert "records" not in d and d["roofline"]["traffic"] is None   # no capture of this workload


def test_bench_stream_mode():
    d = run("--stream-frames", "50", "--pool", "16", "--H", "36", "--W", "128", "--steps", "3", "--warmup", "3",
            "--no-cpu-baseline")
    assert d["scaling"] == "strong" and d["launch"]["launches_per_step"] == 4 and d["gpu_launches"] == 24


def test_bench_full_default_run_records_and_parity():
    """The driver's default command at bench size: the 300-frame HD headline plus the d1 / d3 / d4 / d5
    sub-records, every one with its oracle parity flag true -- all 300 d2 checksums (cpu_baseline leg), all
    64 4K checksums, all 10,000 stream-frame checksums, the d1 frame element by element, the tilers on a
    prefix plus the gather -> scatter identity."""
    d = run("--steps", "5", "--warmup", "3", "--cpu-baseline-seconds", "0")
    assert d["value"] > 100000 and d["config"]["frames_per_gpu"] == 300
    cb = d["cpu_baseline"]
    assert cb["parity_all_frames"] is True and cb["frames_compared"] == 300
    rec = d["records"]
    assert set(rec) == {"d1", "d3", "d4", "d5", "wide", "f1", "f3", "f4"}
    assert rec["d1"]["parity"] is True and rec["d1"]["graph_us_per_call"] > 0
    assert len(rec["d3"]) == 3 and all(r["parity"] is True for r in rec["d3"])
    assert rec["d4"]["parity"] is True and rec["d4"]["frames_per_s"] > 10000
    assert rec["wide"]["parity"] is True and rec["wide"]["kernel"] == "fused_tma_kernel"
    assert rec["f3"]["parity"] is True and rec["f3"]["two_launches_equal"] is True
    assert rec["f3"]["static"]["equal"] is True and rec["f3"]["static"]["kernel"] == "sep_chain_kernel"
    assert len(rec["f1"]) == 4 and all(r["parity"] is True for r in rec["f1"])
    assert rec["f4"]["parity"] is True and rec["f4"]["frames_per_s"] > 100000
    assert rec["d5"]["parity"] is True and rec["d5"]["scaling"] == "strong" and rec["d5"]["n_gpus"] == 1
    assert d["parity_all_records"] is True
