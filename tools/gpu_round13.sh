#!/bin/bash
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_dist.py -m gpu -q -p no:cacheprovider -x > gpurun_out/gpu_dist.log 2>&1
echo "dist exit $?" >> gpurun_out/gpu_dist.log
timeout 1500 python -m pytest tests -m gpu -q -p no:cacheprovider > gpurun_out/gpu_tests.log 2>&1
echo "tests exit $?" >> gpurun_out/gpu_tests.log
timeout 900 python bench.py --steps 3 --warmup 3 --dump-log gpurun_out/bench_log.json > gpurun_out/bench_default.log 2>&1
timeout 900 python -m torch.distributed.run --nnodes=1 --nproc-per-node 2 --master-addr 127.0.0.1 --master-port 29511 bench.py --gpus 2 --steps 3 --warmup 2 > gpurun_out/bench_2rank.log 2>&1
echo "2rank exit $?" >> gpurun_out/bench_2rank.log
timeout 600 python bench.py --impl reference --steps 2 --warmup 1 > gpurun_out/bench_ref.log 2>&1
