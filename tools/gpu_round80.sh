#!/bin/bash
# multi-rank on one GPU after the leading step barrier: 8 ranks (2x4), 4 ranks (2x2), dist tests
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
T="timeout 900 python -m torch.distributed.run --nnodes=1 --master-addr 127.0.0.1"
$T --nproc-per-node 8 --master-port 29561 bench.py --gpus 8 --steps 2 --warmup 3 --no-e2e > gpurun_out/b80_n8.log 2>&1; echo "exit $?" >> gpurun_out/b80_n8.log
$T --nproc-per-node 4 --master-port 29562 bench.py --gpus 4 --steps 2 --warmup 3 --no-e2e > gpurun_out/b80_n4.log 2>&1; echo "exit $?" >> gpurun_out/b80_n4.log
timeout 600 python -m pytest tests/test_gpu_dist.py -q -p no:cacheprovider -x > gpurun_out/t80.log 2>&1; echo "exit $?" >> gpurun_out/t80.log
