"""bench.py's launch plumbing (no GPU needed): `--gpus N` must launch N processes (one per
GPU) or fail loudly, never time one GPU and report it as N."""
import json
import os
import subprocess
import sys

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import bench  # noqa: E402


def test_launch_plan_single_gpu_runs_in_process():
    assert bench.launch_plan(1, {}, []) == ("run", None)
    assert bench.launch_plan(1, {"WORLD_SIZE": "1"}, []) == ("run", None)


def test_launch_plan_relaunches_under_torchrun():
    how, cmd = bench.launch_plan(8, {}, ["--gpus", "8", "--steps", "3"])
    assert how == "relaunch"
    assert cmd[1:3] == ["-m", "torch.distributed.run"]
    assert "--nproc-per-node=8" in cmd and "--master-addr=127.0.0.1" in cmd
    assert cmd[-3:] == ["--gpus", "8", "--steps", "3"][-3:]


def test_launch_plan_world_size_mismatch_is_an_error():
    how, msg = bench.launch_plan(2, {"WORLD_SIZE": "1"}, [])
    assert how == "error" and "WORLD_SIZE=1" in msg
    assert bench.launch_plan(4, {"WORLD_SIZE": "4"}, []) == ("run", None)
    assert bench.launch_plan(0, {}, [])[0] == "error"


def _run(args, env_extra=None):
    env = dict(os.environ)
    env.pop("WORLD_SIZE", None)
    env.update(env_extra or {})
    return subprocess.run([sys.executable, os.path.join(ROOT, "bench.py")] + args,
                          capture_output=True, text=True, timeout=600, env=env, cwd=ROOT)


def test_gpus_2_launches_two_ranks_reference_arm():
    """End to end on CPU: --gpus 2 re-executes under torch.distributed.run; the two ranks see
    WORLD_SIZE=2, rank 0 alone prints one line with n_gpus 2."""
    r = _run(["--gpus", "2", "--impl", "reference", "--steps", "1", "--warmup", "1",
              "--sf", "0.01"])
    assert r.returncode == 0, r.stderr[-3000:]
    lines = [json.loads(x) for x in r.stdout.splitlines() if x.startswith("{")]
    assert len(lines) == 1
    assert lines[0]["n_gpus"] == 2 and lines[0]["impl"] == "reference"
    assert lines[0]["config"]["sf_total"] == pytest.approx(0.02)


def test_mismatched_world_size_fails_loudly():
    r = _run(["--gpus", "2", "--impl", "reference", "--steps", "1", "--warmup", "1", "--sf", "0.01"],
             {"WORLD_SIZE": "1", "RANK": "0", "LOCAL_RANK": "0"})
    assert r.returncode == 2 and "WORLD_SIZE=1" in r.stderr
    assert not [x for x in r.stdout.splitlines() if x.startswith("{")]
