"""The bench's N>1 path end to end on one GPU: two torchrun ranks (gloo
exchange; both ranks may share cuda:0) each run the Q1 fragment on their row
range, all-gather the partials and merge them in rank order.  The merged
result must equal the single-process run and the oracle (pin P8)."""
import json
import os
import socket
import subprocess
import sys

import pytest

import gen
import oracle

pytestmark = pytest.mark.gpu
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _bench(args, nproc=1):
    base = [sys.executable]
    if nproc > 1:
        base += ["-m", "torch.distributed.run", "--nnodes=1", f"--nproc-per-node={nproc}", "--master-addr",
                 "127.0.0.1", "--master-port", str(_port())]
    out = subprocess.run(base + [os.path.join(ROOT, "bench.py")] + args, capture_output=True, text=True,
                         timeout=900, cwd=ROOT)
    assert out.returncode == 0, out.stderr[-3000:]
    return json.loads(out.stdout.strip().splitlines()[-1])


@pytest.mark.parametrize("workload", ["q1", "q9"])
def test_two_ranks_merge_equals_one(workload):
    sf = 0.5
    common = ["--workload", workload, "--sf", str(sf), "--steps", "3", "--warmup", "1", "--no-cpu-baseline",
              "--no-e2e"]
    one = _bench(common)
    two = _bench(common + ["--gpus", "2", "--dist-backend", "gloo"], nproc=2)
    assert two["n_gpus"] == 2 and one["n_gpus"] == 1
    assert two["result"] == one["result"]
    assert two["result_digest"] == one["result_digest"] and two["result_groups"] == one["result_groups"]
    if workload == "q1":
        n = gen.lineitem_rows(sf)
        li = {k: gen.host(c, n, sf=sf, threads=8) for k, c in gen.LINEITEM_COLS.items()}
        exp = oracle.q1(li)
        got = {int(k): [int(x) for x in v[:6]] for k, v in one["result"].items()}
        assert got == exp


@pytest.mark.parametrize("workload", ["q1", "q6"])
def test_nccl_two_gpus_merge_equals_one(workload):
    """The production N>1 path: one rank per GPU over NCCL (all-gather of the
    partials captured in a CUDA graph with the device merge).  gpurun boxes
    have one GPU, so this runs only where two are visible."""
    import torch
    if torch.cuda.device_count() < 2:
        pytest.skip("needs two GPUs (NCCL over NVLink)")
    sf = 1.0
    common = ["--workload", workload, "--sf", str(sf), "--steps", "5", "--warmup", "3", "--no-cpu-baseline",
              "--no-e2e"]
    one = _bench(common)
    two = _bench(common + ["--gpus", "2"], nproc=2)
    assert two["n_gpus"] == 2 and two["cuda_graphs"] == "pipeline + (all-gather, merge)"
    assert two["result_digest"] == one["result_digest"]


@pytest.mark.parametrize("workload", ["q1", "q19"])
def test_graph_replay_equals_eager(workload):
    """The step captured as CUDA graphs (pipeline; all-gather + device merge)
    -- what N > 1 replays -- gives the eager step's result (N = 1 here, with
    --graph forcing the capture)."""
    common = ["--workload", workload, "--sf", "1", "--steps", "3", "--warmup", "3", "--no-cpu-baseline", "--no-e2e"]
    eager = _bench(common)
    graph = _bench(common + ["--graph"])
    assert graph["cuda_graphs"] == "pipeline + (all-gather, merge)", graph["cuda_graphs"]
    assert graph["result_digest"] == eager["result_digest"]
