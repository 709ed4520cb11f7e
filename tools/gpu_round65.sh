#!/bin/bash
# task pool + dist with bench config + torchrun 2-rank bench on one GPU + phases
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build65.log 2>&1
timeout 600 python -m pytest tests/test_gpu_dist.py tests/test_gpu_runtime.py -q -p no:cacheprovider -x > gpurun_out/t65.log 2>&1; echo "exit $?" >> gpurun_out/t65.log
timeout 300 python tools/step_phases.py --steps 3 > gpurun_out/phases65.log 2>&1
timeout 600 python -m torch.distributed.run --nnodes=1 --nproc-per-node 2 --master-addr 127.0.0.1 --master-port 29533 bench.py --gpus 2 --steps 3 --warmup 3 > gpurun_out/b65_n2.log 2>&1; echo "exit $?" >> gpurun_out/b65_n2.log
timeout 400 python bench.py --steps 5 --warmup 3 --no-e2e --no-cpu > gpurun_out/b65_def.log 2>&1
