#!/bin/bash
# Timeline recipe for the multi-GPU overlap: run on a box with >= 2 GPUs and
# nsys (this image has no nsys; gpurun gives one GPU). The library marks its host phases
# with NVTX ranges ("tea_solve", "tea phase 1 (CG / presteps)", "tea phase 2 ...",
# "tea halo exchange", "tea reduce"); with --overlap on (auto across processes) the depth-d
# exchange of r (pack, ncclSend/ncclRecv, unpack) runs on the library's second stream
# while the first fused pass computes the block interior on the compute stream -- the CUDA
# rows of the timeline show the two streams overlapping. Loop mode 1 (chunked graphs) is
# what multi-process runs use, so the graph nodes appear as kernels under the graph launches.
#   bash tools/nsys_overlap.sh 4 4096
N=${1:-2}; MESH=${2:-4096}
mkdir -p gpurun_out
nsys profile --trace=cuda,nvtx,osrt --cuda-graph-trace=node -o gpurun_out/overlap_%q{RANK} \
  python -m torch.distributed.run --nnodes=1 --nproc-per-node $N --master-addr 127.0.0.1 \
  --master-port 29533 bench.py --gpus $N --n $MESH --steps 3 --warmup 3 --no-cpu --overlap 1
# then: nsys stats --report cuda_gpu_trace,nvtx_sum gpurun_out/overlap_0.nsys-rep
