"""CPU checks of bench.py's contract that need no GPU: the reference arm (the
CPU oracle on a bounded sample) prints ONE JSON line with the contract keys,
on rank 0 only under a multi-rank launch."""
import json
import os
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _run(env_extra, *args):
    env = dict(os.environ, **env_extra)
    r = subprocess.run([sys.executable, os.path.join(ROOT, "bench.py"), "--impl", "reference", *args],
                       capture_output=True, text=True, env=env, timeout=300, cwd=ROOT)
    assert r.returncode == 0, r.stderr[-2000:]
    return [ln for ln in r.stdout.splitlines() if ln.strip()]


def test_reference_arm_json_line():
    lines = _run({}, "--steps", "2", "--warmup", "1", "--ref-log2n", "14")
    assert len(lines) == 1
    d = json.loads(lines[0])
    for k in ("metric", "value", "unit", "n_gpus", "steps", "warmup", "ms_per_step", "higher_is_better",
              "scaling", "vs_baseline", "dtype", "data", "config", "cpu_baseline", "e2e"):
        assert k in d, k
    assert d["impl"] == "reference" and d["unit"] == "tuples/s" and d["value"] > 0
    assert d["e2e"]["h2d_bytes_per_step"] == 0 and d["e2e"]["value"] == d["value"]
    assert d["cpu_baseline"]["kind"] == "oracle" and d["cpu_baseline"]["cores"] >= 1
    assert d["config"]["workload"].startswith("c2")


def test_reference_arm_multirank():
    # rank 0 of a 2-rank launch prints the line of the same c2 workload as N=1
    # (weak scaling at every N); rank 1 exits silently
    lines = _run({"WORLD_SIZE": "2", "RANK": "0"}, "--gpus", "2", "--steps", "1", "--warmup", "1",
                 "--ref-log2n", "14")
    d = json.loads(lines[0])
    assert d["scaling"] == "weak" and d["config"]["workload"].startswith("c2")
    assert _run({"WORLD_SIZE": "2", "RANK": "1"}, "--gpus", "2", "--steps", "1", "--warmup", "1") == []
