SWEEP="C B" bash tools/gpu_quick.sh
bash tools/gpu_prof.sh xstatC C xstat
bash tools/gpu_prof.sh vec32C C vector32
