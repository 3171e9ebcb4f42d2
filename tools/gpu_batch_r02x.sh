# is dynamic tile scheduling still slower (bank-spread plan, PDL)?  per-cluster tails
cd $GRAFT_REPO_ROOT
O=gpurun_out/r02x; mkdir -p $O
for D in 0 1 0 1; do echo "dyn=$D" >> $O/gap.txt; SPMV_XPLAN_DYN=$D timeout 300 python tools/gap.py C rand >> $O/gap.txt 2>&1; done
for D in 0 1; do echo "dyn=$D" >> $O/gapB.txt; SPMV_XPLAN_DYN=$D timeout 300 python tools/gap.py B rand >> $O/gapB.txt 2>&1; done
