#!/bin/bash
# multi-rank smoke on one GPU: 4 ranks (2x2 grid) and 8 ranks (2x4 grid) through torchrun; new runtime test
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 300 python -m pytest tests/test_gpu_runtime.py -q -p no:cacheprovider -x -k "concurrently" > gpurun_out/t79.log 2>&1; echo "exit $?" >> gpurun_out/t79.log
T="timeout 900 python -m torch.distributed.run --nnodes=1 --master-addr 127.0.0.1"
$T --nproc-per-node 4 --master-port 29551 bench.py --gpus 4 --steps 2 --warmup 3 --no-e2e > gpurun_out/b79_n4.log 2>&1; echo "exit $?" >> gpurun_out/b79_n4.log
$T --nproc-per-node 8 --master-port 29552 bench.py --gpus 8 --steps 2 --warmup 3 --no-e2e > gpurun_out/b79_n8.log 2>&1; echo "exit $?" >> gpurun_out/b79_n8.log
$T --nproc-per-node 4 --master-port 29553 bench.py --impl reference --gpus 4 --steps 1 --warmup 0 > gpurun_out/ref79_n4.log 2>&1; echo "exit $?" >> gpurun_out/ref79_n4.log
