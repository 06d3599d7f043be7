"""bench.py host logic on CPU: the oracle's key slices partition the join, and the reference arm
(the CPU oracle, the only other place bench.py runs oracle/) prints a valid JSON line."""
import json
import os
import subprocess
import sys

import numpy as np
import pytest

import oracle
import workloads as W

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import bench  # noqa: E402

M64 = (1 << 64) - 1


def test_key_slices_partition_the_join():
    w = W.Workload("t", 1 << 13, 1 << 14, "zipf", keys="sparse", z=1.0, seed=210)
    cols = W.np_generate(w)
    full = oracle.hash_join(*cols)
    m = c = 0
    parts = bench.key_slices(w, *cols, 16)
    for p in parts:
        a, b = oracle.hash_join(*p)
        m, c = m + a, (c + b) & M64
    assert (m, c) == full
    assert sum(len(p[0]) for p in parts) == w.nR and sum(len(p[2]) for p in parts) == w.nS


def test_alg_bytes_model():
    kb, path = bench.alg_bytes(W.CONFIGS["c3"], 1 << 27)
    n = 1 << 28
    assert path == 40 * n + 8 * (1 << 27)  # 5 w n + 2 V matches
    assert kb["pass1"] == kb["pass2"] == 16 * n and kb["join"] == 8 * n + 8 * (1 << 27)


def test_reference_arm_runs_on_cpu():
    out = subprocess.run([sys.executable, os.path.join(ROOT, "bench.py"), "--impl", "reference", "--config", "c1",
                          "--steps", "2", "--warmup", "1"], capture_output=True, text=True, timeout=600)
    line = [l for l in out.stdout.splitlines() if l.startswith("{")][-1]
    d = json.loads(line)
    assert d["impl"] == "reference" and d["value"] > 0 and d["unit"] == "tuples/s"
    assert d["cpu_baseline"]["kind"] == "oracle" and d["cpu_baseline"]["cores"] == 1
    assert d["e2e"]["h2d_bytes_per_step"] == 0


@pytest.mark.gpu
@pytest.mark.parametrize("exchange", ["direct", "nccl"])
def test_bench_multi_rank_flow_on_one_gpu(exchange):
    """bench.py --gpus 2 under torchrun, both ranks on cuda:0 (--debug-one-device, gloo): the
    multi-rank flow the driver's scaling run uses -- row sharding, the exchange (direct: windows
    over CUDA IPC between the two processes), max-over-ranks timing, one JSON line from rank 0
    with the NVLink byte count -- with the closed-form check (matches = |S|) inside bench.py."""
    import json
    import socket
    import subprocess
    import sys

    import torch

    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    port = s.getsockname()[1]
    s.close()
    root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
    cmd = [sys.executable, "-m", "torch.distributed.run", "--nnodes=1", "--nproc-per-node", "2", "--master-addr",
           "127.0.0.1", "--master-port", str(port), os.path.join(root, "bench.py"), "--gpus", "2",
           "--debug-one-device", "--config", "c1", "--exchange", exchange, "--steps", "3", "--warmup", "3",
           "--no-e2e", "--no-cpu-baseline", "--clock-period", "0"]
    out = subprocess.run(cmd, capture_output=True, text=True, timeout=600, cwd=root)
    assert out.returncode == 0, out.stderr[-4000:]
    lines = [ln for ln in out.stdout.splitlines() if ln.startswith("{")]
    assert len(lines) == 1, out.stdout[-2000:]
    d = json.loads(lines[0])
    assert d["n_gpus"] == 2 and d["value"] > 0 and d["config"]["exchange"].startswith(exchange)
    assert d["nvlink"]["bytes_sent_per_gpu_per_step"] > 0
