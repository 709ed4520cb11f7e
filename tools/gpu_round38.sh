#!/bin/bash
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
nvidia-smi --query-gpu=timestamp,clocks.sm,power.draw,clocks_event_reasons.active --format=csv -lms 100 > gpurun_out/clk38.csv 2>&1 &
SMI=$!
timeout 120 ./tools/probe_tcf 1024 16 > gpurun_out/probe_tcf.log 2>&1
kill $SMI
